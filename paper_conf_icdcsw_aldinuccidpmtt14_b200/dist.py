"""Multi-GPU sharding: one process per GPU, contiguous instance
ranges, ONE all-reduce of the packed int64 statistics.

Instances are independent Monte Carlo trajectories ("embarrassingly
parallel"); the paper runs one ff_mapCUDA node per GPU.  Here rank r of G
simulates global instances [floor(rN/G), floor((r+1)N/G)); because every trajectory's Philox
stream is keyed by its global id (R3) and the statistics are exact integer sums, the combined
result is bit-identical for any G.  The only device<->device exchange is
``torch.distributed.all_reduce(stats, SUM)`` (NCCL over NVLink on the B200 box; gloo on CPU
for the host-logic tests).
"""
from __future__ import annotations

from typing import Optional, Tuple


def shard(n_total: int, rank: int, world: int) -> Tuple[int, int]:
    """(first, count) of rank's contiguous share of [0, n_total)."""
    if world < 1 or not (0 <= rank < world) or n_total < 0:
        raise ValueError("bad shard arguments")
    first = (rank * n_total) // world
    last = ((rank + 1) * n_total) // world
    return first, last - first


def combine_stats(stats_tensor, group=None) -> None:
    """In-place SUM all-reduce of a packed stats tensor (int64) across the process group."""
    import torch.distributed as dist
    if dist.is_available() and dist.is_initialized() and dist.get_world_size(group) > 1:
        dist.all_reduce(stats_tensor, op=dist.ReduceOp.SUM, group=group)


class ShardedRun:
    """Per-rank state for repeated sharded simulations of one geometry (buffers reused)."""

    def __init__(self, model, n_total: int, t_end: float, sample_dt: float, group=None,
                 rank: Optional[int] = None, world: Optional[int] = None):
        import torch.distributed as dist
        from .api import DeviceBuffers
        if rank is None or world is None:
            if dist.is_available() and dist.is_initialized():
                rank, world = dist.get_rank(group), dist.get_world_size(group)
            else:
                rank, world = 0, 1
        self.model, self.n_total, self.t_end, self.dt, self.group = model, n_total, t_end, sample_dt, group
        self.rank, self.world = rank, world
        self.first, self.count = shard(n_total, rank, world)
        self.buffers = DeviceBuffers(model, self.count, t_end, sample_dt)

    def launch(self, seed: int, stream=None) -> None:
        """Enqueue this rank's shard and the all-reduce on ``stream`` (default: current)."""
        import torch
        s = stream if stream is not None else torch.cuda.current_stream()
        with torch.cuda.stream(s):
            self.model.simulate_range(self.n_total, self.first, self.count, self.t_end, self.dt, seed, stream=s)
            combine_stats(self.buffers.stats, self.group)

    def result(self):
        """Synchronise and finalise (the stats buffer now holds the whole ensemble)."""
        return self.model.finalize()


def simulate_sharded(model, n_total: int, t_end: float, sample_dt: float, seed: int, group=None):
    """Public multi-GPU call: every rank returns the statistics of the whole ensemble.  A run in
    which some rank found a compartment pool full (pool_full counter of the all-reduced statistics:
    the same on every rank) is repeated on every rank with doubled pool capacities (R20')."""
    while True:
        run = ShardedRun(model, n_total, t_end, sample_dt, group)
        run.launch(seed)
        res = run.result()
        if res.pool_full == 0 or not getattr(model, "pool_auto", False) or not model.grow_pools():
            return res


_HOST_GROUPS = {}


def host_group(group=None):
    """A CPU (gloo) process group over the ranks of ``group`` for host-resident buffers.

    Snapshots are host numpy arrays taken while each rank's SSA kernel still occupies its GPU:
    reducing them through NCCL would queue the collective behind that persistent kernel (and NCCL
    kernels cannot get SMs while it runs), so the on-line combine would only complete when the
    shard's whole simulation has ended.  A gloo group keeps them on the host.  Created once per
    group; collective on first use (every rank of the world calls combine_partial together)."""
    import torch.distributed as dist
    if dist.get_backend(group) == "gloo":
        return group
    key = None if group is None else tuple(dist.get_process_group_ranks(group))
    if key not in _HOST_GROUPS:
        _HOST_GROUPS[key] = dist.new_group(ranks=None if key is None else list(key), backend="gloo")
    return _HOST_GROUPS[key]


def combine_partial(packed, cuts_final: int, group=None):
    """SUM the packed statistics and MIN the final-cut prefixes across ranks (host numpy in,
    host numpy out): the combination rule of on-line multi-GPU streaming.  The reduction runs on
    a CPU (gloo) group (``host_group``): it never touches the device, so it completes while the
    ranks' kernels are still running."""
    import numpy as np
    import torch
    import torch.distributed as dist
    buf = torch.from_numpy(np.ascontiguousarray(packed, dtype=np.int64).copy())
    cf = torch.tensor([int(cuts_final)], dtype=torch.int64)
    if dist.is_available() and dist.is_initialized():
        hg = host_group(group)
        if dist.get_world_size(hg) > 1:
            dist.all_reduce(buf, op=dist.ReduceOp.SUM, group=hg)
            dist.all_reduce(cf, op=dist.ReduceOp.MIN, group=hg)
    return buf.numpy(), int(cf[0])


def snapshot_sharded(model, group=None):
    """On-line streaming over ranks: every rank snapshots its own
    running shard (copy engine, no synchronisation with its kernel), the packed statistics are
    summed and the final-cut prefixes min-reduced across ranks, and the combined partial result is
    loaded into ``model``.  Returns (cuts_final, EnsembleResult); cuts below cuts_final are the
    whole ensemble's exact statistics.  Collective: call it on every rank."""
    cf, _, _ = model.snapshot()
    packed, cf_all = combine_partial(model.stats_host(), cf, group)
    return cf_all, model.stats_load(packed, cf_all)


def reduce_host_stats(local_stats, group=None):
    """Host-side combine used by CPU (gloo) tests: SUM-all-reduce a numpy int64 buffer."""
    import numpy as np
    import torch
    import torch.distributed as dist
    t = torch.from_numpy(np.ascontiguousarray(local_stats, dtype=np.int64).copy())
    if dist.is_available() and dist.is_initialized() and dist.get_world_size(group) > 1:
        dist.all_reduce(t, op=dist.ReduceOp.SUM, group=group)
    return t.numpy()
