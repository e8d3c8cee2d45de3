# pipelined speculative batch (next batch's draws in the same block as the state steps)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
CWC_KERNEL_DEFINES="CWC_SPEC=1;CWC_SPEC_PIPE=1;CWC_DRAW_BATCH=2" timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "lv_ or terminated or compacted or raw_staging or schedule" 2>&1 | tail -1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 1000000 t_end=10" "lv 125000" "circadian 1250000 raw=0"; do
  run "default $c" $c reps=2
  CWC_KERNEL_DEFINES="CWC_SPEC=1" run "spec $c" $c reps=2
  for D in 2 3 4; do CWC_KERNEL_DEFINES="CWC_SPEC=1;CWC_SPEC_PIPE=1;CWC_DRAW_BATCH=$D" run "spec-pipe D$D $c" $c reps=2; done
done
done
