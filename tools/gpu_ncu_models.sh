export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { echo build failed; exit 1; }
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc $?"; tail -3 gpurun_out/pytest_gpu.log
timeout 900 ncu --set full --clock-control none --import-source on -k regex:cwc_ssa -s 1 -c 1 -o gpurun_out/ves_full python tools/quick_time.py vesicles 200000 reps=2 > gpurun_out/ncu_ves.log 2>&1; echo "ncu ves rc $?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:cwc_ssa -s 1 -c 1 -o gpurun_out/cmp_full python tools/quick_time.py compartments 1000000 reps=2 > gpurun_out/ncu_cmp.log 2>&1; echo "ncu cmp rc $?"
