# 640 threads (96 registers) / 576 / 512 (128) vs 768 (80) with the draw batch, every config
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "lv 1000000" "lv 500000" "lv 250000" "schlogl 1000000 raw=0" "circadian 1250000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0" "vesicles 1000000 raw=0"; do
  run "768 $c" $c reps=2
  run "640 $c" $c block_threads=640 reps=2
  run "512 $c" $c block_threads=512 reps=2
done
for c in "lv 100000" "lv 125000"; do
  run "576 $c" $c block_threads=576 reps=2
  run "512 $c" $c block_threads=512 reps=2
done
