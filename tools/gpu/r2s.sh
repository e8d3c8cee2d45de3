export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in vesicles compartments circadian neurospora schlogl; do
  n=1000000; [ $c = circadian ] && n=1250000
  run "$c smem" $c $n reps=2 raw=0
  run "$c global" $c $n reps=2 raw=0 smem_stats=0
done
run "lv1m smem" lv 1000000 t_end=10 reps=2
run "lv1m global" lv 1000000 t_end=10 reps=2 smem_stats=0
run "lv100k smem" lv 100000 reps=2
run "lv100k global" lv 100000 reps=2 smem_stats=0
