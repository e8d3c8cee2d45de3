"""GPU: the multi-rank path end to end (torchrun, ranks sharing the available GPU(s)).

Rank shards + all-reduce of the packed statistics must equal the oracle's statistics of the
whole ensemble and one GPU run of it.  Uses NCCL when there is one GPU per rank, gloo otherwise (one B200 here).
"""
import os
import socket
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("nproc", [2, 3])
def test_torchrun_sharded_equals_whole(nproc):
    import torch
    env = dict(os.environ, PYTHONPATH=ROOT)
    if torch.cuda.device_count() < nproc:
        env["CWC_DIST_BACKEND"] = "gloo"
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={nproc}",
           "--master-addr", "127.0.0.1", "--master-port", str(_port()), os.path.join(ROOT, "tests", "workers", "dist_check.py")]
    r = subprocess.run(cmd, env=env, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    assert "DIST OK" in r.stdout, r.stdout[-3000:]
