"""Throughput of the SSA kernel against resident warps per scheduler (development aid).

    PYTHONPATH=. python tools/warp_curve.py [config] [t_end]

Static assignment (refill off, whole trajectories, thread slot s -> instance s): one CTA of
128 w threads per SM (blocks_per_sm = 1) and N = SMs x 128 w instances put exactly w busy warps
on every SM sub-partition (SMSP), w = 1, 2, 3, 6 (register budget <= 85 in every variant), plus
one single warp on the whole GPU.  Prints SMSP cycles per warp-step (32 reactions), the curve
that tools/sched_sim.py models.
"""
import sys

import torch

import workloads as W
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc

name = sys.argv[1] if len(sys.argv) > 1 else "lv"
t_end = float(sys.argv[2]) if len(sys.argv) > 2 else 5.0
cfg = W.CONFIGS[name]
props = torch.cuda.get_device_properties(0)
sms = props.multi_processor_count
extra = {k: int(v) for k, v in (a.split("=") for a in sys.argv[3:])}
for w in (0, 1, 2, 3, 6):
    n = 32 if w == 0 else sms * 128 * w
    bt = 32 if w == 0 else 128 * w
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, raw_samples=False,
                           refill=False, block_threads=bt, blocks_per_sm=1, **extra)
    m.simulate(n, t_end, cfg.sample_dt, cfg.seed)            # warm-up (compile, fast_cut choice)
    res = m.simulate(n, t_end, cfg.sample_dt, cfg.seed)
    f_mhz = 1965.0   # sustained SM clock of this pool under the SSA kernel (bench clocks line)
    cyc = res.kernel_ms * 1e-3 * f_mhz * 1e6
    warp_steps_per_smsp = res.reactions / 32 / (1 if w == 0 else sms * 4)
    print(f"{name} w={w} warps/SMSP ({'1 warp on the GPU' if w == 0 else 'every SMSP'}, "
          f"regs {m.kernel_attributes()['registers']}): {cyc / warp_steps_per_smsp:7.1f} SMSP cycles per warp-step "
          f"({cyc / warp_steps_per_smsp * max(w, 1):7.1f} per warp-iteration), kernel {res.kernel_ms:.1f} ms, "
          f"{res.reactions / res.kernel_ms * 1e3:.3g} reactions/s, clock {f_mhz:.0f} MHz", flush=True)
