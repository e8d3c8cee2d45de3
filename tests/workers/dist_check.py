"""Worker of tests/test_gpu_dist.py: multi-rank check of the sharded path (dist.simulate_sharded).

    torchrun --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 tests/workers/dist_check.py

With CWC_DIST_BACKEND=gloo every rank may share one GPU (functional test of the multi-rank
code path when only one GPU is available); with the default nccl each rank needs its own GPU.
Rank 0 compares the all-reduced statistics with the ORACLE's statistics of the
whole ensemble (oracle.simulate + oracle.stats.ensemble_stats: integers n / sum / sumsq / hist
exact, mean / variance / quantiles bit-identical) and with a single-process GPU run, and prints
"DIST OK" (exit code 1 on a mismatch).
"""
import os
import sys

import numpy as np
import torch
import torch.distributed as dist

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import oracle  # noqa: E402
import workloads as W  # noqa: E402
from oracle.stats import ensemble_stats  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402
from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import simulate_sharded  # noqa: E402


def main():
    backend = os.environ.get("CWC_DIST_BACKEND", "nccl")
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if backend != "nccl":
        local %= torch.cuda.device_count()
    torch.cuda.set_device(local)
    if backend == "nccl":
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    else:
        dist.init_process_group(backend)
    rank, world = dist.get_rank(), dist.get_world_size()
    md, N, t_end, dt, seed = W.SCHLOGL, 20011, 2.0, 0.1, 99
    qs = (0.05, 0.25, 0.5, 0.75, 0.95)
    m = cwc.Model.from_def(md, hist_bins=512, device=local, quantiles=qs)
    res = simulate_sharded(m, N, t_end, dt, seed)
    ok = True
    if rank == 0:
        ref = cwc.Model.from_def(md, hist_bins=512, device=local, quantiles=qs).simulate(N, t_end, dt, seed)
        for name in ("n", "sum", "sqlo", "sqhi", "hist"):
            ok &= bool(np.array_equal(getattr(res, name), getattr(ref, name)))
        ok &= res.reactions == ref.reactions and res.finished == N
        # the combined statistics against the oracle's statistics of the whole ensemble
        orun = oracle.simulate(md, 0, N, t_end, dt, seed, nthreads=os.cpu_count() or 1)
        st = ensemble_stats(orun.raw, [0], [1], 512, qs)
        exact = res.sumsq_exact()
        ok_oracle = bool(np.array_equal(res.n, st.n) and np.array_equal(res.hist, st.hist))
        ok_oracle &= all(int(res.sum[k, 0]) == st.sum[k, 0] and exact[k, 0] == st.sumsq[k, 0]
                         for k in range(res.n.size))
        ok_oracle &= bool(np.array_equal(res.mean, st.mean, equal_nan=True) and
                          np.array_equal(res.var, st.var, equal_nan=True) and
                          np.array_equal(res.quantile, st.quantile, equal_nan=True))
        ok_oracle &= res.reactions == int(orun.reactions.sum())
        print(f"oracle comparison of the all-reduced statistics: {'equal' if ok_oracle else 'DIFFERENT'}",
              flush=True)
        ok &= ok_oracle
    # on-line streaming across ranks (dist.snapshot_sharded): combined partial results while the
    # shards run; the final-cut prefix of every combined snapshot equals the whole run's
    import time
    from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import shard, snapshot_sharded
    N2, t2 = 100_000, 10.0
    first, count = shard(N2, rank, world)
    m2 = cwc.Model.from_def(md, hist_bins=512, device=local, raw_samples=False, stream=1)
    m2.simulate_range(N2, first, count, t2, dt, seed)
    T2 = int(round(t2 / dt)) + 1
    snaps = []
    while True:
        cf, r2 = snapshot_sharded(m2)          # collective: same cf on every rank
        snaps.append((cf, {k: getattr(r2, k).copy() for k in ("n", "sum", "sqlo", "sqhi", "hist")}))
        if cf >= T2:
            break
        time.sleep(0.005)
    m2.finalize()
    if rank == 0:
        ref2 = cwc.Model.from_def(md, hist_bins=512, device=local, raw_samples=False).simulate(N2, t2, dt, seed)
        for cf, st in snaps:
            for name, v in st.items():
                ok &= bool(np.array_equal(v[:cf], getattr(ref2, name)[:cf]))
        partial = sorted({cf for cf, _ in snaps if 0 < cf < T2})
        print(f"streamed snapshots: final prefixes {partial[:8]}... of T={T2}", flush=True)
        print(("DIST OK" if ok else "DIST MISMATCH") + f" world={world} backend={backend} reactions={res.reactions}",
              flush=True)
    dist.barrier()
    dist.destroy_process_group()
    return 0 if ok else 1


if __name__ == "__main__":
    sys.exit(main())
