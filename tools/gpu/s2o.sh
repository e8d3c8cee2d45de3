# cut emission inlined into its call sites vs out of line
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
CWC_KERNEL_DEFINES="CWC_EMIT_INLINE=1" timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "vesicles or compartments_small or circadian_small or tiny or lv_short" 2>&1 | tail -1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "circadian 1250000 raw=0" "neurospora 1000000 raw=0" "schlogl 1000000 raw=0" "lv 125000"; do
  run "noinline $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_EMIT_INLINE=1" run "inline $c" $c reps=2
done
done
