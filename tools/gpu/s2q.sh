# auto CTA size: full GPU tests, smoke, bench lines (LV 1M default, LV 100k weak), timings
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2q_build.txt 2>&1 || { cat gpurun_out/s2q_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/s2q_gpu_tests.log 2>&1; tail -3 gpurun_out/s2q_gpu_tests.log
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "lv 100000" "lv 125000" "lv 50000" "lv 170000" "schlogl 100000 raw=0" "circadian 150000 raw=0"; do
  run "auto $c" $c reps=2
  run "768 $c" $c block_threads=768 reps=2
done
python bench.py --config lv --scaling weak --no-cpu-baseline > gpurun_out/s2q_bench_lv100k.json 2>&1
timeout 600 python bench.py > gpurun_out/s2q_bench_lv1m.json 2> gpurun_out/s2q_bench_lv1m.err
M=smsp__thread_inst_executed.sum,smsp__inst_executed.sum,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__warps_eligible.avg.per_cycle_active,smsp__warps_active.avg.per_cycle_active,gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum
eff() { name=$1; shift
  timeout 900 ncu --metrics $M --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py "$@" reps=1 2>/dev/null | grep cwc_ssa_kernel | awk -F'","' -v n=$name '{gsub(/"/,"",$15); print "[" n "] " $13 " " $15}'
}
{ eff lv125k lv 125000; eff lv100k lv 100000; } > gpurun_out/s2q_metrics.log
echo done
