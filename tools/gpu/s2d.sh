# draw batch (CWC_DRAW_BATCH = D draws per inner-loop trip) vs the per-step draw: parity subset + same-box A/B
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=2" timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "schedule or tiny or lv_short or terminated or raw_staging or zero_horizon or circadian_small or compartments_small" 2>&1 | tail -2
CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=3" timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "schedule or lv_short or terminated" 2>&1 | tail -1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000" "lv 125000" "lv 100000" "schlogl 1000000 raw=0" "circadian 1250000 raw=0"; do
  run "D0 $c" $c reps=2
  for D in 2 3 4; do CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=$D" run "D$D $c" $c reps=2; done
done
done
