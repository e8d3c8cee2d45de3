#!/bin/bash
# One GPU session: build, smoke, parity tests, optional A/B matrix (args), bench, ncu launch list
# and one ncu --set full capture of the SSA kernel (LV 100k).  Outputs under gpurun_out/.
export PYTHONPATH=$PWD
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc $?"; tail -1 gpurun_out/smoke.log
if [ -z "$SKIP_TESTS" ]; then
  timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc $?"; tail -2 gpurun_out/pytest_gpu.log
fi
if [ $# -gt 0 ]; then bash tools/exp_matrix.sh "$@" 2>&1 | tee gpurun_out/ab.log; fi
if [ -z "$SKIP_BENCH" ]; then
  timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo "bench rc $?"; tail -1 gpurun_out/bench.log
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_ncu.log 2>&1; echo "ncu launches rc $?"
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:cwc_ssa -s 1 -c 1 -o gpurun_out/lv_full python tools/quick_time.py lv 100000 reps=2 > gpurun_out/ncu_full.log 2>&1; echo "ncu full rc $?"
fi
