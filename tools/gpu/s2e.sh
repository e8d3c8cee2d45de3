# draw batch with / without a warp reconvergence at the top of the inner loop (A/B)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "lv 125000" "lv 1000000 t_end=10" "circadian 1250000 raw=0" "schlogl 1000000 raw=0"; do
  run "D0 $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_LOOP_SYNCWARP=1" run "D0 sync $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=2" run "D2 $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=2;CWC_LOOP_SYNCWARP=1" run "D2 sync $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=4;CWC_LOOP_SYNCWARP=1" run "D4 sync $c" $c reps=2
done
