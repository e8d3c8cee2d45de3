# two-pass running sums in the fast step (CWC_TWO_PASS) vs one pass, models with >= 6 flat reactions
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
CWC_KERNEL_DEFINES="CWC_TWO_PASS=1" timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "tiny or circadian_small or compartments_small or vesicles or neurospora_rate" 2>&1 | tail -1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "circadian 1250000 raw=0" "neurospora 1000000 raw=0"; do
  run "tp0 $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_TWO_PASS=1" run "tp1 $c" $c reps=2
done
done
