set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/lat_micro tools/lat_micro.cu && /tmp/lat_micro > gpurun_out/r2a_lat_micro.txt 2>&1
cat gpurun_out/r2a_lat_micro.txt
export PYTHONPATH=$PWD
python tools/quick_time.py lv 100000 reps=2 > gpurun_out/r2a_qt.txt 2>&1
python tools/quick_time.py lv 1000000 reps=2 >> gpurun_out/r2a_qt.txt 2>&1
python tools/quick_time.py lv 125000 reps=2 >> gpurun_out/r2a_qt.txt 2>&1
cat gpurun_out/r2a_qt.txt
timeout 900 ncu --metrics smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__warps_active.avg.per_cycle_active,smsp__warps_eligible.avg.per_cycle_active,smsp__inst_executed.sum,smsp__thread_inst_executed.sum,gpu__time_duration.sum,smsp__average_warp_latency_issue_stalled_wait.ratio,smsp__average_warp_latency_issue_stalled_barrier.ratio,smsp__average_warp_latency_issue_stalled_math_pipe_throttle.ratio,smsp__average_warp_latency_issue_stalled_dispatch_stall.ratio,smsp__average_warp_latency_issue_stalled_not_selected.ratio,sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active,sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active,sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active --clock-control none -k cwc_ssa_kernel python tools/quick_time.py lv 1000000 t_end=10 reps=1 > gpurun_out/r2a_ncu_lv1m_t10.txt 2>&1
tail -40 gpurun_out/r2a_ncu_lv1m_t10.txt
