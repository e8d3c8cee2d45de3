"""Host-clock breakdown of the bench's end-to-end call (development aid)."""
import time
import torch
import workloads as W
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
from paper_conf_icdcsw_aldinuccidpmtt14_b200 import dist as cdist

cfg = W.CONFIGS["lv"]
N = cfg.n_instances
for rep in range(4):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, quantiles=cfg.quantiles)
    t1 = time.perf_counter()
    m.compile()
    t2 = time.perf_counter()
    run = cdist.ShardedRun(m, N, cfg.t_end, cfg.sample_dt)
    torch.cuda.synchronize()
    t3 = time.perf_counter()
    run.launch(cfg.seed)
    t4 = time.perf_counter()
    torch.cuda.synchronize()
    t5 = time.perf_counter()
    res = run.result()
    t6 = time.perf_counter()
    print(f"load {1e3*(t1-t0):.1f} ms  compile {1e3*(t2-t1):.1f}  buffers {1e3*(t3-t2):.1f}  launch {1e3*(t4-t3):.1f}  "
          f"kernel-wait {1e3*(t5-t4):.1f}  finalize {1e3*(t6-t5):.1f}  total {1e3*(t6-t0):.1f}  kernel_ms {res.kernel_ms:.1f}",
          flush=True)
    del run, m
