"""GPU: steering and checkpoint robustness.

* terminate storm: cwc_cancel at random points of a small-count, many-quanta streaming run —
  every taken work item runs, so no quantum waits forever for a predecessor that was dropped;
* a checkpoint whose header was tampered with is rejected before any device memory is touched;
* NCCL world: dist.snapshot_sharded combines on a CPU (gloo) group, so it returns a partial
  snapshot (0 < cuts_final < T) while the persistent kernel still holds the GPU.
"""
import os
import socket
import subprocess
import sys

import numpy as np
import pytest

import workloads as W

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_cancel_storm_never_hangs():
    r = subprocess.run([sys.executable, os.path.join(ROOT, "tests", "workers", "cancel_storm.py"), "40"],
                       capture_output=True, text=True, timeout=300, env=dict(os.environ, PYTHONPATH=ROOT))
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-3000:]
    assert "CANCEL OK" in r.stdout


@pytest.mark.parametrize("field,offset,value", [
    ("qs = 0", 48, 0), ("qs > K + 1", 48, 10 ** 6), ("K != t_end/dt", 40, 7),
    ("first + count > n_total", 24, 90), ("count < 0", 32, -1)])
def test_tampered_checkpoint_header_is_rejected(field, offset, value):
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model.from_def(W.IMM_DEATH, hist_bins=64)
    m.simulate(100, 10.0, 1.0, 1)
    ck = m.checkpoint()
    bad = ck.copy()
    bad[offset:offset + 8] = np.frombuffer(np.int64(value).tobytes(), dtype=np.uint8)
    other = cwc.Model.from_def(W.IMM_DEATH, hist_bins=64)
    with pytest.raises(cwc.CWCError) as e:
        other.restore(bad)
    assert e.value.status == 1, field          # CWC_E_INVALID
    other.restore(ck)                           # the untouched checkpoint still restores
    assert other.finalize().finished == 100


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def test_nccl_snapshot_returns_while_kernel_runs():
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node=1", "--master-addr",
           "127.0.0.1", "--master-port", str(_port()), os.path.join(ROOT, "tests", "workers", "nccl_snapshot.py")]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=300, env=dict(os.environ, PYTHONPATH=ROOT))
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-3000:]
    assert "SNAPSHOT OK" in r.stdout
