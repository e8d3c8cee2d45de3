# final measurement pass after the sparse-recording unroll: tests, smoke, I_min, bench lines, metrics, launch list
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2w_build.txt 2>&1 || { cat gpurun_out/s2w_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/s2w_gpu_tests.log 2>&1; tail -3 gpurun_out/s2w_gpu_tests.log
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
for c in lv schlogl circadian compartments neurospora vesicles; do timeout 300 python tools/imin.py $c > /dev/null 2>&1; done
cp profiles/imin_*.json gpurun_out/
python bench.py > gpurun_out/s2w_bench_lv1m.json 2> gpurun_out/s2w_bench_lv1m.err
python bench.py --config lv --scaling weak --no-cpu-baseline > gpurun_out/s2w_bench_lv100k.json 2>&1
for c in schlogl compartments neurospora vesicles; do python bench.py --config $c --no-raw --steps 3 --no-cpu-baseline > gpurun_out/s2w_bench_$c.json 2>&1; done
python bench.py --config circadian --no-raw --steps 3 --no-cpu-baseline --instances 1250000 > gpurun_out/s2w_bench_circadian.json 2>&1
M=smsp__thread_inst_executed.sum,smsp__inst_executed.sum,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__warps_eligible.avg.per_cycle_active,smsp__warps_active.avg.per_cycle_active,gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum
eff() { name=$1; shift
  timeout 900 ncu --metrics $M --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py "$@" reps=1 2>/dev/null | grep cwc_ssa_kernel | awk -F'","' -v n=$name '{gsub(/"/,"",$15); print "[" n "] " $13 " " $15}'
}
{ eff lv1m lv 1000000; eff lv500k lv 500000; eff lv250k lv 250000; eff lv125k lv 125000; eff lv100k lv 100000
  eff schlogl schlogl 1000000 raw=0; eff circadian circadian 1250000 raw=0; eff compartments compartments 1000000 raw=0
  eff neurospora neurospora 1000000 raw=0; eff vesicles vesicles 1000000 raw=0; } > gpurun_out/s2w_metrics.log
head -3 gpurun_out/s2w_metrics.log
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/s2w_launches_bench_lv1m.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline > /dev/null 2>&1
echo done
