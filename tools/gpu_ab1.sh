export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:cwc_ssa -s 1 -c 1 -o gpurun_out/lv_full python tools/quick_time.py lv 100000 reps=2 > gpurun_out/ncu_full.log 2>&1; echo ncu rc $?
bash tools/exp_matrix.sh "lv 100000" "DEF=CWC_FAST_UNROLL=2 lv 100000" "lv 100000 seed_jit=1" "lv 100000 block_threads=1024" "lv 1000000" "schlogl 1000000" > gpurun_out/ab1.log 2>&1
cat gpurun_out/ab1.log
