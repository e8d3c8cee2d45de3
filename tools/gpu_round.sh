set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke rc $?
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc $?
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench rc $?
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_ncu.log 2>&1; echo ncu1 rc $?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:cwc_ssa -s 1 -c 1 -o gpurun_out/lv_full env PYTHONPATH=. python tools/quick_time.py lv 100000 reps=2 > gpurun_out/ncu_full.log 2>&1; echo ncu2 rc $?
tail -3 gpurun_out/pytest_gpu.log; tail -1 gpurun_out/bench.log
