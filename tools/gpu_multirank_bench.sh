#!/bin/bash
# Functional check of the multi-rank bench path on a one-GPU box: 2 torchrun ranks share the GPU
# (gloo for the all-reduce); rank 0 prints one JSON line; the reference arm runs on rank 0 only.
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { echo build failed; exit 1; }
timeout 900 python -m pytest tests -m gpu -x -q -k "empty_shard or many_cuts" > gpurun_out/pytest_new.log 2>&1; echo "pytest new rc $?"; tail -2 gpurun_out/pytest_new.log
CWC_DIST_BACKEND=gloo timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29517 bench.py --gpus 2 --steps 3 --warmup 3 --instances 50000 > gpurun_out/bench_2rank.log 2>&1; echo "bench 2 ranks rc $?"; grep '^{' gpurun_out/bench_2rank.log | cut -c1-400
timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29518 bench.py --impl reference --gpus 2 --steps 1 --warmup 3 --ref-step-s 5 > gpurun_out/bench_ref_2rank.log 2>&1; echo "reference 2 ranks rc $?"; grep '^{' gpurun_out/bench_ref_2rank.log | cut -c1-300
