export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for v in "" "CWC_PIPE_SPLIT=1" "" "CWC_PIPE_SPLIT=1"; do
  CWC_KERNEL_DEFINES="$v" run "1M $v" lv 1000000 t_end=10 reps=2
  CWC_KERNEL_DEFINES="$v" run "100k $v" lv 100000 reps=2
done
for v in "" "CWC_PIPE_SPLIT=1"; do
  CWC_KERNEL_DEFINES="$v" run "schlogl $v" schlogl 1000000 reps=2 raw=0
  CWC_KERNEL_DEFINES="$v" run "circ $v" circadian 1250000 reps=2 raw=0
done
timeout 600 python -m pytest tests -m gpu -q -x -k "crafted and random_injected_steps_match" > /tmp/t.txt 2>&1; tail -2 /tmp/t.txt
CWC_KERNEL_DEFINES="CWC_PIPE_SPLIT=1" timeout 600 python -m pytest tests -m gpu -q -x -k "crafted or lv_short or schedule_invariance" 2>&1 | tail -2
