# draw batch: deferred draw commit (default) vs per-step commit; parity subset of the default
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_crafted.py -q -x -k "schedule or tiny or lv_short or terminated or raw_staging or zero_horizon or circadian_small or compartments_small or vesicles or crafted or random" 2>&1 | tail -2
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 125000" "lv 1000000 t_end=10" "lv 100000" "circadian 1250000 raw=0" "schlogl 1000000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0"; do
  run "defer $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_DEFER_DRAW=0" run "step $c" $c reps=2
done
done
for rep in 1 2; do
  run "D0 lv 1000000" lv 1000000 draw_batch=0 reps=2
  run "defer lv 1000000" lv 1000000 reps=2
  for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0"; do
    CWC_DEVICE_SRC=tools/gpu/prev_kernel run "session-start kernel $c" $c reps=2
    run "now D0 $c" $c draw_batch=0 reps=2
  done
done
