export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for v in "" "CWC_BRANCHFREE=1"; do
  CWC_KERNEL_DEFINES="$v" run "1M $v" lv 1000000 t_end=10 reps=2
  CWC_KERNEL_DEFINES="$v" run "100k $v" lv 100000 reps=2
  CWC_KERNEL_DEFINES="$v" run "circ $v" circadian 1250000 reps=2 raw=0
done
timeout 1800 python tools/t3_ablation.py 1000000 2>&1 | tee gpurun_out/r2j_t3_schlogl.jsonl
for c in vesicles compartments circadian; do
  n=1000000; [ $c = circadian ] && n=1250000
  CWC_DEVICE_SRC=tools/gpu/prev_kernel run "$c prev (no smem bin 1)" $c $n reps=2 raw=0
  run "$c smem bin 1" $c $n reps=2 raw=0
done
# ncu: full set on a short-horizon LV 1M launch (same kernel, 101 cuts), DRAM traffic of the bench launch
timeout 1200 ncu --set full --import-source on --clock-control none -k cwc_ssa_kernel -c 1 -o gpurun_out/r2j_lv1m_t10_full -f python tools/quick_time.py lv 1000000 t_end=10 reps=1 > gpurun_out/r2j_ncu_full.log 2>&1
python tools/ncu_summary.py gpurun_out/r2j_lv1m_t10_full.ncu-rep > gpurun_out/r2j_lv1m_t10_ncu_summary.txt 2>&1
python tools/ncu_stalls.py gpurun_out/r2j_lv1m_t10_full.ncu-rep 0.5 > gpurun_out/r2j_lv1m_t10_stalls.txt 2>&1
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv 1000000 reps=1 > gpurun_out/r2j_traffic_lv1m.csv 2>&1
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv 125000 reps=1 > gpurun_out/r2j_traffic_lv125k.csv 2>&1
cat gpurun_out/r2j_lv1m_t10_ncu_summary.txt
