# full GPU suite on the current kernel + DRAM traffic by quantum count + 100k block sizes
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2k_build.txt 2>&1 || { cat gpurun_out/r2k_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q -x > gpurun_out/r2k_tests.txt 2>&1
tail -5 gpurun_out/r2k_tests.txt
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for q in 0 64 504; do
  run "1M q=$q" lv 1000000 reps=1 quantum_samples=$q
  timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv 1000000 reps=1 quantum_samples=$q 2>/dev/null | grep cwc_ssa | awk -F'","' '{print "[traffic 1M q='$q'] " $13 " " $15}'
done
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv 125000 reps=1 2>/dev/null | grep cwc_ssa | awk -F'","' '{print "[traffic 125k auto] " $13 " " $15}'
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv 100000 reps=1 2>/dev/null | grep cwc_ssa | awk -F'","' '{print "[traffic 100k auto] " $13 " " $15}'
for b in 768 736 704; do run "100k block $b" lv 100000 reps=2 block_threads=$b min_blocks=1; done
run "125k auto" lv 125000 reps=2
