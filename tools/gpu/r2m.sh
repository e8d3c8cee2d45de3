# compacted per-quantum launches: parity + A/B in the under-filled regime
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2m_build.txt 2>&1 || { cat gpurun_out/r2m_build.txt; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -k "compact or schedule or terminated or tiny_models or lv_short" > gpurun_out/r2m_tests.txt 2>&1
tail -3 gpurun_out/r2m_tests.txt
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
run "100k whole" lv 100000 reps=2 compact=0
for q in 0 32 128; do run "100k compact q=$q" lv 100000 reps=2 compact=1 quantum_samples=$q; done
run "125k quanta" lv 125000 reps=2 compact=0
run "125k compact" lv 125000 reps=2 compact=1
run "100k schlogl whole" schlogl 100000 reps=2 compact=0 raw=0
run "100k schlogl compact" schlogl 100000 reps=2 compact=1 raw=0
run "50k circadian whole" circadian 50000 reps=2 compact=0 raw=0
run "50k circadian compact" circadian 50000 reps=2 compact=1 raw=0
