#!/bin/bash
# GPU session: parity tests, every config at its BASELINE size (+ LV 1M), the bench line and the
# three compute-sanitizer tools on small runs of every model.  Outputs under gpurun_out/.
export PYTHONPATH=$PWD
SKIP_BENCH=1 bash tools/gpu_session.sh "lv 100000" "lv 1000000" "schlogl 1000000" "circadian 1250000" "compartments 1000000" "neurospora 1000000" "vesicles 1000000" "imm_death 1000000" "$@"
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo "bench rc $?"; tail -1 gpurun_out/bench.log
if [ -z "$SKIP_SAN" ]; then
for t in memcheck racecheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_run.py > gpurun_out/san_$t.log 2>&1; echo "$t rc $?"; tail -1 gpurun_out/san_$t.log; done
fi
