# draw batch as the default: full GPU tests, smoke, bench, vesicles batch A/B
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2g_build.txt 2>&1 || { tail gpurun_out/s2g_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/s2g_gpu_tests.log 2>&1; tail -3 gpurun_out/s2g_gpu_tests.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 900 python bench.py > gpurun_out/s2g_bench.json 2> gpurun_out/s2g_bench.err; echo "bench rc=$?"; cut -c1-300 gpurun_out/s2g_bench.json
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for D in 0 2 3 4; do run "ves D$D" vesicles 1000000 raw=0 draw_batch=$D reps=2; done
