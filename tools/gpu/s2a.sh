# HEAD re-verification after the container re-creation: build, GPU tests, smoke, default bench
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2a_build.txt 2>&1; echo "build rc=$?"
timeout 2400 python -m pytest tests -m gpu -q 2>&1 | tail -3 | tee gpurun_out/s2a_gpu_tests.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 900 python bench.py > gpurun_out/s2a_bench.json 2> gpurun_out/s2a_bench.err; echo "bench rc=$?"; cat gpurun_out/s2a_bench.json | cut -c1-400
