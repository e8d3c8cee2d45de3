# same-box A/B on the current kernel: register budget 64 (1024 threads) / 72 (896) vs 80 (768);
# seed-specialised round keys (seed_jit)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000" "lv 125000" "lv 100000"; do
  run "768 $c" $c reps=2
  run "1024 $c" $c block_threads=1024 reps=2
  run "896 $c" $c block_threads=896 reps=2
  run "768 seed_jit $c" $c seed_jit=1 reps=2
done
done
for c in "schlogl 1000000 raw=0" "circadian 1250000 raw=0" "compartments 1000000 raw=0"; do
  run "768 $c" $c reps=2
  run "1024 $c" $c block_threads=1024 reps=2
done
