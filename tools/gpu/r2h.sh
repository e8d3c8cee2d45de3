export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 600 python -m pytest tests -m gpu -q -x -k "pool_auto" 2>&1 | tail -3
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for q in 8 16; do run "q=$q 125k" lv 125000 reps=2 quantum_samples=$q; done
for q in 16 32; do run "q=$q 250k" lv 250000 reps=2 quantum_samples=$q; done
for q in 16 32 63; do run "q=$q 1M full" lv 1000000 reps=1 quantum_samples=$q; done
for c in schlogl compartments neurospora; do
  for q in 0 $( [ $c = schlogl ] && echo 32 || echo 13 ); do run "$c q=$q" $c 1000000 reps=2 quantum_samples=$q raw=0; done
done
for q in 0 7; do run "circadian q=$q" circadian 1250000 reps=2 quantum_samples=$q raw=0; done
run "896x1" lv 1000000 t_end=10 reps=2 block_threads=896 min_blocks=1
run "640x1" lv 1000000 t_end=10 reps=2 block_threads=640 min_blocks=1
run "ilp2 384" lv 1000000 t_end=10 reps=2 block_threads=384 min_blocks=1 ilp=2
run "ilp2 512" lv 1000000 t_end=10 reps=2 block_threads=512 min_blocks=1 ilp=2
run "ves default" vesicles 1000000 reps=2 raw=0
run "ves 384x151" vesicles 1000000 reps=2 raw=0 block_threads=384 min_blocks=1
run "ves 512x128" vesicles 1000000 reps=2 raw=0 block_threads=512 min_blocks=1
