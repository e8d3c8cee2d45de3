# register budget with the draw batch: 1024 threads x 64 registers (8 warps / scheduler) vs 768 x 80
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
timeout 1200 python -m pytest tests/test_gpu_parity.py -q -x -k "bounds_checked or raw_staging" 2>&1 | tail -3
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000" "lv 500000" "lv 250000" "lv 125000" "lv 100000" "schlogl 1000000 raw=0" "circadian 1250000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0"; do
  run "768 $c" $c reps=2
  run "1024 $c" $c block_threads=1024 reps=2
done
done
for c in "lv 1000000" "lv 125000"; do
  run "1024 D3 $c" $c block_threads=1024 draw_batch=3 reps=2
  run "1024 D2 $c" $c block_threads=1024 draw_batch=2 reps=2
done
