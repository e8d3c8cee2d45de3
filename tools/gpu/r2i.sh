# measurement of the current kernel: bench lines (LV 1M strong, LV 100k weak), I_min, launch list,
# ncu --set full of the LV 1M kernel (traffic + summary + per-instruction stalls)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 300 python tools/imin.py lv > gpurun_out/r2i_imin.txt 2>&1; cp profiles/imin_lotka_volterra.json gpurun_out/
python bench.py > gpurun_out/r2i_bench_lv1m.json 2> gpurun_out/r2i_bench_lv1m.err; tail -c 3000 gpurun_out/r2i_bench_lv1m.json
python bench.py --config lv --scaling weak --no-cpu-baseline > gpurun_out/r2i_bench_lv100k.json 2>&1; tail -c 600 gpurun_out/r2i_bench_lv100k.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r2i_launches_bench_lv1m.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline > /dev/null 2>&1
timeout 1500 ncu --set full --import-source on --clock-control none -k cwc_ssa_kernel -c 1 -o gpurun_out/r2i_lv1m_full -f python tools/quick_time.py lv 1000000 reps=1 > gpurun_out/r2i_ncu_full.log 2>&1
tail -2 gpurun_out/r2i_ncu_full.log
python tools/ncu_summary.py gpurun_out/r2i_lv1m_full.ncu-rep > gpurun_out/r2i_lv1m_ncu_summary.txt 2>&1
python tools/ncu_stalls.py gpurun_out/r2i_lv1m_full.ncu-rep 0.5 > gpurun_out/r2i_lv1m_stalls.txt 2>&1
cat gpurun_out/r2i_lv1m_ncu_summary.txt
