"""Quick device timing of one config (development aid, not the bench)."""
import sys, time
import torch
import workloads as W
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc

name = sys.argv[1] if len(sys.argv) > 1 else "lv"
cfg = W.CONFIGS[name]
N = int(sys.argv[2]) if len(sys.argv) > 2 else cfg.n_instances
opts = dict(a.split("=") for a in sys.argv[3:])
opts = {k: int(v) for k, v in opts.items()}
raw = bool(opts.pop("raw", 1))
t_end = float(opts.pop("t_end", cfg.t_end))
reps = int(opts.pop("reps", 3))
m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, raw_samples=raw, **opts)
bufs = cwc.DeviceBuffers(m, N, t_end, cfg.sample_dt)
s = torch.cuda.current_stream()
for it in range(reps):
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    m.simulate_range(N, 0, N, t_end, cfg.sample_dt, cfg.seed, stream=s)
    e1.record()
    torch.cuda.synchronize()
    res = m.finalize()
    ms = e0.elapsed_time(e1)
    print(f"{name} N={N} opts={opts} raw={raw}: {ms:.1f} ms  reactions={res.reactions:.4g}  "
          f"{res.reactions/ms*1e3:.4g} reactions/s  kernel_ms={res.kernel_ms:.1f} attrs={m.kernel_attributes()}", flush=True)
