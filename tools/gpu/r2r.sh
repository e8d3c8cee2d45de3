# final-kernel measurement pass: GPU suite, smoke, bench lines (north star + BASELINE configs), launch list, I_min
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2r_build.txt 2>&1 || { cat gpurun_out/r2r_build.txt; exit 1; }
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/r2r_tests.txt 2>&1
tail -3 gpurun_out/r2r_tests.txt
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 300 python tools/imin.py lv > /dev/null 2>&1; cp profiles/imin_lotka_volterra.json gpurun_out/r2r_imin_lv.json
python bench.py > gpurun_out/r2r_bench_lv1m.json 2> gpurun_out/r2r_bench_lv1m.err; tail -c 700 gpurun_out/r2r_bench_lv1m.json
python bench.py --config lv --scaling weak --no-cpu-baseline > gpurun_out/r2r_bench_lv100k.json 2>&1
for c in schlogl circadian compartments; do python bench.py --config $c --no-raw --steps 3 --no-cpu-baseline $( [ $c = circadian ] && echo "--instances 1250000" ) > gpurun_out/r2r_bench_$c.json 2>&1; done
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r2r_launches_bench_lv1m.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline > /dev/null 2>&1
grep -c cwc_ssa gpurun_out/r2r_launches_bench_lv1m.csv
