"""Multi-process host logic of the multi-GPU path on CPU (gloo, world size 2 and 3).

Checks that dist.shard() partitions [0, N) into contiguous disjoint ranges, and that the SUM
all-reduce of per-rank packed statistics (here computed from the oracle's raw cuts of each
rank's range) equals the statistics of the whole ensemble — the property the NCCL path on
the B200 box relies on.
"""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

from helpers import numpy_stats


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _packed(raw, B, width):
    n, ssum, sqlo, sqhi, hist = numpy_stats(raw, [0] * raw.shape[1], [width] * raw.shape[1], B)
    return np.concatenate([n, ssum.ravel(), sqlo.ravel(), sqhi.ravel(), hist.ravel()]).astype(np.int64)


def _worker(rank, world, port, N, out_path):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    import torch
    import torch.distributed as dist

    import oracle
    import workloads as W
    from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import combine_stats, reduce_host_stats, shard

    dist.init_process_group("gloo", rank=rank, world_size=world)
    first, count = shard(N, rank, world)
    run = oracle.simulate(W.SCHLOGL, first, count, 2.0, 0.5, seed=11, nthreads=2)
    local = _packed(run.raw, 64, 16)
    total = reduce_host_stats(local)
    t = torch.from_numpy(local.copy())
    combine_stats(t)
    assert np.array_equal(t.numpy(), total)
    if rank == 0:
        np.save(out_path, total)
    dist.barrier()
    dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3])
def test_gloo_sharded_stats_equal_whole(tmp_path, world):
    import oracle
    import workloads as W
    N = 301
    out = str(tmp_path / "total.npy")
    mp.start_processes(_worker, args=(world, _free_port(), N, out), nprocs=world, join=True, start_method="spawn")
    total = np.load(out)
    whole = oracle.simulate(W.SCHLOGL, 0, N, 2.0, 0.5, seed=11, nthreads=4)
    assert np.array_equal(total, _packed(whole.raw, 64, 16))


def test_shard_partition():
    from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import shard
    for N in (0, 1, 7, 100, 1_000_003):
        for G in (1, 2, 3, 4, 8):
            ranges = [shard(N, r, G) for r in range(G)]
            assert ranges[0][0] == 0
            for (a, c), (b, _) in zip(ranges, ranges[1:]):
                assert a + c == b
            assert sum(c for _, c in ranges) == N
            assert max(c for _, c in ranges) - min(c for _, c in ranges) <= 1
    with pytest.raises(ValueError):
        shard(10, 2, 2)


def _partial_worker(rank, world, port, out_path):
    """On-line multi-rank streaming host rule: each rank's partial packed statistics of a prefix
    of its cuts (as a snapshot of a running shard would hold), SUM-combined, prefix MIN-reduced."""
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    import torch.distributed as dist

    import oracle
    import workloads as W
    from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import combine_partial, shard

    dist.init_process_group("gloo", rank=rank, world_size=world)
    N, T = 240, 5
    first, count = shard(N, rank, world)
    run = oracle.simulate(W.SCHLOGL, first, count, 2.0, 0.5, seed=5, nthreads=2)
    raw = run.raw.copy()
    cf_local = 2 + rank                      # this rank's shard has finished cuts [0, 2 + rank)
    raw[cf_local:, :, count // 2:] = -1      # later cuts: only part of its instances recorded
    packed, cf = combine_partial(_packed(raw, 64, 16), cf_local)
    assert cf == 2                           # the whole ensemble is final on the common prefix
    if rank == 0:
        np.save(out_path, packed)
    dist.barrier()
    dist.destroy_process_group()


def test_gloo_partial_snapshots_combine(tmp_path):
    import oracle
    import workloads as W
    world = 3
    out = str(tmp_path / "partial.npy")
    mp.start_processes(_partial_worker, args=(world, _free_port(), out), nprocs=world, join=True,
                       start_method="spawn")
    got = np.load(out)
    whole = _packed(oracle.simulate(W.SCHLOGL, 0, 240, 2.0, 0.5, seed=5, nthreads=2).raw, 64, 16)
    T, S, B = 5, 1, 64
    # the final prefix (cuts 0, 1) of every block of the packed layout equals the whole run's
    def blocks(p):
        n = p[:T]
        rest = p[T:]
        ts = T * S
        return [n, rest[:ts], rest[ts:2 * ts], rest[2 * ts:3 * ts], rest[3 * ts:].reshape(T, -1)]
    for a, b in zip(blocks(got), blocks(whole)):
        assert np.array_equal(a[:2], b[:2])
    assert (blocks(got)[0][2:] < 240).all()   # later cuts are partial
