export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2v_build.txt 2>&1 || { cat gpurun_out/r2v_build.txt; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -k "staging or ticket or circadian_small or compartments_small or vesicles or tiny or neurospora or period or lv_short or schedule or imm_death" 2>&1 | tail -3
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "circadian 1250000 raw=0" "neurospora 1000000 raw=0" "schlogl 1000000 raw=0" "lv 1000000 t_end=10" "lv 100000"; do run "$c" $c reps=2; done
