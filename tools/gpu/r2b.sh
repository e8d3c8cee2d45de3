# micro: latency / pipe sharing; ncu pipe utilisation of the LV kernel at 1M (short horizon)
set -x
export PYTHONPATH=$PWD
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/lat_micro tools/lat_micro.cu && /tmp/lat_micro > gpurun_out/r2b_lat_micro.txt 2>&1
cat gpurun_out/r2b_lat_micro.txt
timeout 900 ncu --metrics "regex:sm__pipe_.*_cycles_active.avg.pct_of_peak_sustained_active,regex:sm__inst_executed_pipe_.*.avg.pct_of_peak_sustained_active,smsp__issue_active.avg.pct_of_peak_sustained_active,regex:smsp__pcsamp_warps_issue_stalled_.*" --clock-control none -k cwc_ssa_kernel python tools/quick_time.py lv 1000000 t_end=5 reps=1 fast_cut=0 > gpurun_out/r2b_ncu_pipes_lv1m.txt 2>&1
grep -v "^==" gpurun_out/r2b_ncu_pipes_lv1m.txt | tail -80
for v in "CWC_PIN_DRAW=0" "CWC_FAST_UNROLL=2" ""; do
  CWC_KERNEL_DEFINES="$v" python tools/quick_time.py lv 1000000 t_end=10 reps=2 fast_cut=0 2>&1 | sed "s/^/[$v] /"
done | tee gpurun_out/r2b_ab.txt
python tools/quick_time.py lv 1000000 t_end=10 reps=2 fast_cut=0 block_threads=1024 min_blocks=1 | sed "s/^/[1024x64reg] /" | tee -a gpurun_out/r2b_ab.txt
python tools/quick_time.py lv 1000000 t_end=10 reps=2 fast_cut=0 block_threads=512 min_blocks=2 | sed "s/^/[512x2x64reg] /" | tee -a gpurun_out/r2b_ab.txt
