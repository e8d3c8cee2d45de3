export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2u_build.txt 2>&1 || { cat gpurun_out/r2u_build.txt; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -k "staging or circadian_small or compartments_small or vesicles or tiny or neurospora or period or full_size_sub_ensemble_parity and (circadian or compartments)" 2>&1 | tail -3
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "circadian 1250000 raw=0" "neurospora 1000000 raw=0" "schlogl 1000000 raw=0" "lv 1000000 t_end=10"; do
  for m in 3 2; do run "$c smem=$m" $c reps=2 smem_stats=$m; done
done
