# final tree: full GPU tests, smoke, compartments bench line and metrics (cooperative recording on)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2v_build.txt 2>&1 || { cat gpurun_out/s2v_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/s2v_gpu_tests.log 2>&1; tail -3 gpurun_out/s2v_gpu_tests.log
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 300 python tools/imin.py compartments > /dev/null 2>&1; cp profiles/imin_compartments.json gpurun_out/
python bench.py --config compartments --no-raw --steps 3 --no-cpu-baseline > gpurun_out/s2v_bench_compartments.json 2>&1
M=smsp__thread_inst_executed.sum,smsp__inst_executed.sum,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__warps_eligible.avg.per_cycle_active,smsp__warps_active.avg.per_cycle_active,gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum
timeout 900 ncu --metrics $M --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py compartments 1000000 raw=0 reps=1 2>/dev/null | grep cwc_ssa_kernel | awk -F'","' '{gsub(/"/,"",$15); print "[compartments] " $13 " " $15}' > gpurun_out/s2v_metrics.log
timeout 600 python bench.py > gpurun_out/s2v_bench_lv1m.json 2> gpurun_out/s2v_bench_lv1m.err
echo done
