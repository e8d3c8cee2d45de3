# first wave spread over CTAs / schedulers: same-box A/B vs HEAD + parity subset
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 100000" "lv 125000" "lv 1000000 t_end=10" "schlogl 100000 raw=0" "circadian 100000 raw=0"; do
  CWC_DEVICE_SRC=tools/gpu/prev_kernel run "prev $c" $c reps=2
  run "new $c" $c reps=2
done
done
timeout 1500 python -m pytest tests -m gpu -q -x -k "schedule or tiny or lv_short or terminated or compact or staging or empty or zero_horizon" 2>&1 | tail -2
