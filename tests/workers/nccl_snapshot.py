"""Worker of tests/test_gpu_steering.py, launched with torchrun over the NCCL backend: on-line
snapshots of a running shard are combined through dist.snapshot_sharded, whose reduction runs on
a CPU (gloo) group — so a combined snapshot with 0 < cuts_final < T is obtained WHILE the SSA
kernel still occupies the GPU (an NCCL all-reduce would queue behind the persistent kernel).
Prints "SNAPSHOT OK <cuts_final> <T>"."""
import os
import sys
import time

import torch
import torch.distributed as dist

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import workloads as W  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402
from paper_conf_icdcsw_aldinuccidpmtt14_b200.dist import shard, snapshot_sharded  # noqa: E402


def main():
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    rank, world = dist.get_rank(), dist.get_world_size()
    md, N, t_end, dt, seed = W.SCHLOGL, 1_000_000, 50.0, 0.1, 3
    T = int(round(t_end / dt)) + 1
    first, count = shard(N, rank, world)
    m = cwc.Model.from_def(md, hist_bins=1024, raw_samples=False, stream=1, device=local)
    m.simulate_range(N, first, count, t_end, dt, seed)
    t0 = time.time()
    seen = None
    while time.time() - t0 < 60:
        cf, res = snapshot_sharded(m)
        if 0 < cf < T:
            seen = cf
            break
        if cf >= T:
            break
        time.sleep(0.01)
    m.finalize()
    if rank == 0:
        ok = seen is not None
        print(("SNAPSHOT OK" if ok else "SNAPSHOT NOT PARTIAL") + f" {seen} {T} world={world} "
              f"backend={dist.get_backend()}", flush=True)
    dist.barrier()
    dist.destroy_process_group()
    return 0 if seen is not None else 1


if __name__ == "__main__":
    sys.exit(main())
