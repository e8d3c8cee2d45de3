# speculative batch (CWC_SPEC, cuts on the full-step path): parity subset + same-box A/B
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_crafted.py -q -x -k "lv_ or terminated or compacted or raw_staging or schedule or tiny or zero_horizon or circadian_small or compartments_small or crafted or random or full_size or bounds" 2>&1 | tail -2
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000" "lv 125000" "lv 100000" "circadian 1250000 raw=0" "schlogl 1000000 raw=0 fast_cut=0" "neurospora 1000000 raw=0 fast_cut=0"; do
  run "spec $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_SPEC=0" run "nospec $c" $c reps=2
done
done
