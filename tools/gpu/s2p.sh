# cooperative cut recording: parity + same-box A/B
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1 || { echo BUILD FAILED; exit 1; }
timeout 1200 python -m pytest tests/test_gpu_parity.py -q -x -k "cooperative or vesicles or staging or tiny or bounds or compartments_small" 2>&1 | tail -3
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "vesicles 1000000 raw=0" "compartments 1000000 raw=0" "neurospora 1000000 raw=0" "schlogl 1000000 raw=0"; do
  CWC_KERNEL_DEFINES="CWC_COOP_EMIT=1" run "coop $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_COOP_EMIT=0" run "lane $c" $c reps=2
done
done
