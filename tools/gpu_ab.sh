#!/bin/bash
# GPU A/B session: build, parity tests, then the timing matrix given as arguments (see exp_matrix.sh)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { echo build failed; tail gpurun_out/build.log; exit 1; }
if [ -z "$SKIP_TESTS" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc $?"; tail -3 gpurun_out/pytest_gpu.log
fi
bash tools/exp_matrix.sh "$@" 2>&1 | tee gpurun_out/ab.log
