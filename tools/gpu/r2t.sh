# register diet (no inst / step0 fields, 32-bit counters and index): same-box A/B vs HEAD + parity subset
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000 t_end=10" "lv 100000" "schlogl 1000000 raw=0" "circadian 1250000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0" "vesicles 1000000 raw=0"; do
  CWC_DEVICE_SRC=tools/gpu/prev_kernel run "prev $c" $c reps=2
  run "new $c" $c reps=2
done
done
timeout 1500 python -m pytest tests -m gpu -q -x -k "crafted or tiny or lv_short or schedule or terminated or circadian_small or compartments_small or vesicles" 2>&1 | tail -2
