# raw-cut staging: parity (new test + raw-producing subset), same-box A/B and DRAM traffic
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/s2b_build.txt 2>&1 || { tail gpurun_out/s2b_build.txt; exit 1; }
timeout 1500 python -m pytest tests/test_gpu_parity.py -q -x -k "raw_staging or terminated or compacted or lv_ or vesicles or schedule or tiny or zero_horizon or full_size" > gpurun_out/s2b_tests.log 2>&1; tail -30 gpurun_out/s2b_tests.log
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1; do
for c in "lv 1000000" "lv 125000" "lv 100000"; do
  run "stage=0 $c" $c raw_stage=0 reps=2
  run "stage=1 $c" $c reps=2
done
done
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_srcunit_tex_op_write.sum
eff() { name=$1; shift
  timeout 900 ncu --metrics $M --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py "$@" reps=1 2>/dev/null | grep cwc_ssa_kernel | awk -F'","' -v n=$name '{gsub(/"/,"",$15); print "[" n "] " $13 " " $15}'
}
{ for st in 0 1; do eff lv1m_stage$st lv 1000000 raw_stage=$st; eff lv125k_stage$st lv 125000 raw_stage=$st; eff lv100k_stage$st lv 100000 raw_stage=$st; done; } > gpurun_out/s2b_traffic.log
cat gpurun_out/s2b_traffic.log
