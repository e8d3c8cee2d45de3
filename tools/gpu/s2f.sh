# draw batch size sweep (with the inner-loop reconvergence) on every static model
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "lv 125000" "lv 1000000 t_end=10" "lv 100000" "circadian 1250000 raw=0" "schlogl 1000000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0"; do
  run "D0 $c" $c reps=2
  for D in 3 4 5 6 8; do CWC_KERNEL_DEFINES="CWC_DRAW_BATCH=$D;CWC_LOOP_SYNCWARP=1" run "D$D sync $c" $c reps=2; done
done
