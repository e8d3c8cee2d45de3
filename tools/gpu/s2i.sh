# regression check of the emission-heavy models vs the session-start kernel; current defaults
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0" "schlogl 1000000 raw=0" "circadian 1250000 raw=0" "lv 125000"; do
  CWC_DEVICE_SRC=tools/gpu/prev_kernel run "session-start $c" $c reps=2
  run "now $c" $c reps=2
  run "now D0 $c" $c draw_batch=0 reps=2
done
done
