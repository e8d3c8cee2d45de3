# full GPU suite on the new kernel (log on the high word, 32-bit step counter) + quantum sweep
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2g_build.txt 2>&1 || { cat gpurun_out/r2g_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q -x > gpurun_out/r2g_tests.txt 2>&1
tail -5 gpurun_out/r2g_tests.txt
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for q in 16 32; do run "q=$q 125k" lv 125000 reps=2 quantum_samples=$q; done
for q in 32 63 0; do run "q=$q 250k" lv 250000 reps=2 quantum_samples=$q; done
for q in 32 63; do run "q=$q 500k" lv 500000 t_end=20 reps=2 quantum_samples=$q; done
for q in 32 63 126; do run "q=$q 1M" lv 1000000 t_end=10 reps=2 quantum_samples=$q; done
