export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for n in 125000 100000; do
  run "$n 768 auto" lv $n reps=2
  run "$n 896x1" lv $n reps=2 block_threads=896 min_blocks=1
  run "$n 864x1" lv $n reps=2 block_threads=864 min_blocks=1
done
run "125k 896x1 q16" lv 125000 reps=2 block_threads=896 min_blocks=1 quantum_samples=16
run "250k 768 auto" lv 250000 reps=2
run "250k 896x1" lv 250000 reps=2 block_threads=896 min_blocks=1
run "1M 768" lv 1000000 reps=1
run "1M 896x1" lv 1000000 reps=1 block_threads=896 min_blocks=1
