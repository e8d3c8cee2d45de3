#!/usr/bin/env python
"""Benchmark: simulated reactions/s (whole box) and trajectories/s of the CWC ensemble SSA.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config lv] [--impl b200|reference]
    torchrun --nnodes=1 --nproc-per-node N --master-addr 127.0.0.1 bench.py --gpus N ...

One step = the whole hot path over one synthetic ensemble: instance
generation, SSA to t_end, sampling on the grid, fused on-line statistics, and (N > 1) the
NCCL all-reduce of the statistics.  Default workload: the north-star ensemble (BASELINE.json
north_star, config "lv1m"): Lotka-Volterra, 1,000,000 instances, t_end = 50, dt = 0.1,
STRONG scaling — the 1M instances are sharded over the N ranks (125k per GPU at N = 8), rank r
owning the contiguous global range [floor(rN/G), floor((r+1)N/G)).  ``--scaling weak`` keeps
the configured instances per GPU instead (e.g. ``--config lv --scaling weak``: BASELINE.json
configs[1], 100k per GPU).

Rank 0 prints ONE JSON line.  Timing: W warm-up steps, then K steps bracketed by barrier +
synchronize; each step is timed with CUDA events on the launching stream after a 256 MiB L2
flush (outside the events); ms_per_step is the max over ranks.  ``e2e`` repeats the metric
through the public API (dist.simulate_sharded: launch + all-reduce + device->host stats +
finalize), host wall clock, max over ranks.  ``cpu_baseline`` is the oracle (oracle/, plain C
SSA + Python stats) on this host's cores over a bounded sample of the same workload.
``--impl reference`` times that oracle alone (the "reference arm" of this tier).
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

import workloads as W  # noqa: E402

METRIC = "simulated reactions/sec (whole box)"
UNIT = "reactions/s"
PARAM_BYTES = 280   # sizeof(cwc_params): the __grid_constant__ launch parameter block (static_assert in runtime.cpp)
LOGTAB_BYTES = 3072  # CWC-log table uploaded once per model load (128 x {invc, logc, logclo})


# ---------------------------------------------------------------------------------- helpers
def measured_imin(model_name: str):
    """I_min of SURVEY §8(d): thread-instructions per reaction of a divergence-free single-warp
    run of this model's SSA kernel (tools/imin.py under ncu: smsp__inst_executed x 32 /
    reactions), committed as profiles/imin_<model>.json for the kernel revision it measured."""
    try:
        with open(os.path.join(ROOT, "profiles", f"imin_{model_name}.json")) as f:
            d = json.load(f)
        return float(d["imin_thread_inst_per_reaction"]), d
    except (OSError, KeyError, ValueError):
        return None, None


def algorithmic_instructions(info: dict) -> int:
    """Minimal thread-instruction count of one direct-method SSA step of this flat model on
    sm_100a (DESIGN.md §5 "algorithmic work"): the unit of the ALU roofline."""
    fixed = 40 + 6 + 29 + 8 + 4 + 2   # Philox, 2 uniforms, CWC-log, IEEE divide, t/cut/target, step++
    per_rule = 0
    orders = set()
    for j, rl in enumerate(info["reactants"]):
        per_rule += 1 + max(len(rl) - 1, 0) + (1 if j > 0 else 0) + 2   # k*h, factor products, cum, select
        for s, r in rl:
            orders.add((s, r))
    factors = sum({1: 1, 2: 4, 3: 8}[r] for _, r in orders)
    pairs = sum(1 for row in info["delta"] for d in row if d)
    touched = sum(1 for s in range(len(info["names"])) if any(row[s] for row in info["delta"]))
    inc = sum(1 for s in range(len(info["names"])) if any(row[s] > 0 for row in info["delta"]))
    return fixed + per_rule + factors + 2 * pairs + touched + 2 * inc


class ClockSampler:
    """nvidia-smi clocks / throttle reasons sampled every 200 ms during the timed region."""

    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, device_index: int):
        self.dev = device_index
        self.proc = None
        self.lines = []
        self.thread = None

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--id={self.dev}", f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "200"], stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except OSError:
            self.proc = None
            return
        self.thread = threading.Thread(target=self._read, daemon=True)
        self.thread.start()

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self) -> dict:
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except subprocess.TimeoutExpired:
            self.proc.kill()
        if self.thread:
            self.thread.join(timeout=2)
        sm, smax, reasons = [], [], set()
        names = ("hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap")
        for ln in self.lines:
            parts = [p.strip() for p in ln.split(",")]
            if len(parts) < 9:
                continue
            try:
                sm.append(float(parts[1]))
                smax.append(float(parts[2]))
            except ValueError:
                continue
            for name, v in zip(names, parts[5:9]):
                if v.lower() == "active":
                    reasons.add(name)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(smax) if smax else None,
                "reasons": sorted(reasons), "samples": len(sm)}


def host_cores() -> int:
    try:
        return len(os.sched_getaffinity(0))
    except AttributeError:
        return os.cpu_count() or 1


def oracle_sample(cfg, budget_s: float, first: int = 0):
    """Run the oracle (SSA + stats, as it stands) on growing instance batches of the same
    workload until ~budget_s seconds of CPU work; returns (reactions, instances, seconds, cores)."""
    import oracle
    from oracle.stats import ensemble_stats
    fm = oracle.flatten_def(cfg.model)
    cm = oracle.CModel(fm)
    cores = host_cores()
    S = len(fm.names)
    reactions = instances = 0
    spent = 0.0
    batch = cores
    nxt = first
    while spent < budget_s:
        t0 = time.perf_counter()
        run = oracle.simulate(cm, nxt, batch, cfg.t_end, cfg.sample_dt, cfg.seed, nthreads=cores)
        ensemble_stats(run.raw, [0] * S, [cfg.hist_width] * S, cfg.hist_bins, cfg.quantiles)
        dt = time.perf_counter() - t0
        spent += dt
        reactions += int(run.reactions.sum())
        instances += batch
        nxt += batch
        if dt < budget_s / 8:
            batch *= 2
    return reactions, instances, spent, cores


# ---------------------------------------------------------------------------------- reference arm
def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    cfg = W.CONFIGS[args.config]
    budget = args.ref_step_s
    for _ in range(args.warmup):
        oracle_sample(cfg, budget / 4)
    tot_r = tot_i = 0
    tot_s = 0.0
    cores = host_cores()
    for _ in range(args.steps):
        r, i, s, cores = oracle_sample(cfg, budget)
        tot_r, tot_i, tot_s = tot_r + r, tot_i + i, tot_s + s
    value = tot_r / tot_s
    line = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": args.gpus,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * tot_s / args.steps,
        "higher_is_better": True, "scaling": args.scaling, "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": {"workload": args.config, "description": cfg.description},
        "trajectories_per_s": tot_i / tot_s,
        "cpu_baseline": {"value": value, "unit": UNIT, "cores": cores, "kind": "oracle",
                         "sample": f"{tot_i} instances of '{args.config}' (full horizon t_end={cfg.t_end}) "
                                   f"over {args.steps} steps, SSA + stats"},
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


# ---------------------------------------------------------------------------------- B200 arm
def run_b200(args):
    import torch
    import torch.distributed as dist

    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import dist as cdist

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if world != args.gpus:
        print(f"--gpus {args.gpus} but WORLD_SIZE={world}: launch one process per GPU "
              f"(torchrun --nproc-per-node {args.gpus})", file=sys.stderr)
        return 2
    # one process per GPU; CWC_DIST_BACKEND=gloo lets a functional multi-rank run share one GPU —
    # such a line is tagged "shared_gpu" and is not a scaling point
    backend = os.environ.get("CWC_DIST_BACKEND", "nccl")
    ndev = max(1, torch.cuda.device_count())
    shared_gpu = world > ndev
    if shared_gpu and backend == "nccl":
        print(f"{world} ranks but {ndev} GPU(s): NCCL needs one GPU per rank", file=sys.stderr)
        return 2
    local = local % ndev
    torch.cuda.set_device(local)
    if world > 1:
        if backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))
        else:
            dist.init_process_group(backend)
    cfg = W.CONFIGS[args.config]
    if args.scaling == "strong":
        n_total = args.instances or cfg.n_instances
    else:
        n_total = (args.instances or cfg.n_instances) * world
    n_per = n_total // world

    t0 = time.perf_counter()
    model = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width,
                               quantiles=cfg.quantiles, raw_samples=not args.no_raw, device=local)
    model.compile()
    load_s = time.perf_counter() - t0
    info = model.info()
    run = cdist.ShardedRun(model, n_total, cfg.t_end, cfg.sample_dt, rank=rank, world=world)
    stream = torch.cuda.Stream()
    flush = torch.empty(256 * 1024 * 1024 // 4, dtype=torch.float32, device="cuda")

    def barrier():
        if world > 1:
            if backend == "nccl":
                dist.barrier(device_ids=[local])
            else:
                dist.barrier()

    for w in range(args.warmup):
        with torch.cuda.stream(stream):
            flush.zero_()
        run.launch(cfg.seed + w, stream)
        # finalise every warm-up run: the kernel variant (cut recording, runtime.cpp
        # choose_fast_cut) adapts to the measured reactions per cut, and its NVRTC compile must
        # happen here, not inside the first timed step
        res = run.result()
    torch.cuda.synchronize()

    clocks = ClockSampler(local)
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True),
           torch.cuda.Event(enable_timing=True)) for _ in range(args.steps)]
    clocks.start()
    barrier()
    torch.cuda.synchronize()
    reactions = []
    for i in range(args.steps):
        with torch.cuda.stream(stream):
            flush.zero_()
            e0, e1, e2 = ev[i]
            e0.record(stream)
            model.simulate_range(n_total, run.first, run.count, cfg.t_end, cfg.sample_dt, cfg.seed, stream=stream)
            e1.record(stream)
            cdist.combine_stats(run.buffers.stats)
            e2.record(stream)
    torch.cuda.synchronize()
    barrier()
    clk = clocks.stop()
    step_ms = [a.elapsed_time(c) for a, _, c in ev]
    kern_ms = [a.elapsed_time(b) for a, b, _ in ev]
    res = run.result()                      # totals over all ranks (stats all-reduced)
    total_reactions = res.reactions
    ms_local = sum(step_ms) / len(step_ms)
    kern_local = sum(kern_ms) / len(kern_ms)
    t = torch.tensor([ms_local, kern_local], dtype=torch.float64, device="cuda")
    if world > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    ms_per_step, kern_ms_max = float(t[0]), float(t[1])
    value = total_reactions / (ms_per_step / 1e3)
    traj_s = n_total / (ms_per_step / 1e3)

    # ---- e2e through the public API, host clock: model load from the host-side definition
    # (cwc_model_load: parse + flatten + codegen, NVRTC cubin from the cache, module upload),
    # device buffers, launch + all-reduce, D2H of the statistics + finalize
    e2e_ms = []
    n_stats = run.buffers.stats.numel()
    for i in range(1 + max(1, min(args.steps, 3))):   # first call untimed (allocator / module warm-up)
        torch.cuda.synchronize()
        barrier()
        h0 = time.perf_counter()
        m2 = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width,
                                quantiles=cfg.quantiles, raw_samples=not args.no_raw, device=local)
        r2 = cdist.simulate_sharded(m2, n_total, cfg.t_end, cfg.sample_dt, cfg.seed)
        if i > 0:
            e2e_ms.append(1e3 * (time.perf_counter() - h0))
        del m2
    te = torch.tensor([sum(e2e_ms) / len(e2e_ms)], dtype=torch.float64, device="cuda")
    if world > 1:
        dist.all_reduce(te, op=dist.ReduceOp.MAX)
    e2e_value = r2.reactions / (float(te[0]) / 1e3)
    cubin_bytes = model.kernel_image_bytes()

    # ---- roofline of the dominant (only) kernel: ALU issue bound
    props = torch.cuda.get_device_properties(local)
    sms = props.multi_processor_count
    peaks = {}
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            peaks = json.load(f)
    except OSError:
        pass
    f_max = float(peaks.get("sm_max_mhz", 1965.0)) * 1e6
    i_alg = algorithmic_instructions(info)
    i_min, imin_rec = measured_imin(cfg.model.name)
    i_unit = i_min if i_min is not None else float(i_alg)
    reactions_per_launch = total_reactions / world
    achieved = reactions_per_launch * i_unit / (kern_ms_max / 1e3) / 1e12
    peak = sms * 4 * 32 * f_max / 1e12
    raw_bytes = 0 if args.no_raw else res.n.size * len(info["names"]) * run.count * 4
    traffic = None   # DRAM bytes per launch from a committed ncu --set full capture of this launch
    import glob
    for path in sorted(glob.glob(os.path.join(ROOT, "profiles", "traffic_*.json"))):
        try:
            with open(path) as f:
                tr = json.load(f)
            if (tr.get("workload") == args.config and int(tr.get("instances", -1)) == run.count
                    and not args.no_raw):
                traffic = tr["dram_bytes_per_launch"]
        except (OSError, KeyError, ValueError):
            continue
    roof = {"bound": "alu", "achieved": achieved, "peak": peak, "unit": "Tinst/s", "frac": achieved / peak,
            "traffic": traffic,
            "detail": {"unit": "I_min thread-instructions per reaction x reactions per launch / kernel time "
                               "(SURVEY §8(d) useful fraction)" if i_min is not None else
                               "I_alg (hand count; no measured I_min for this model)",
                       "imin_thread_inst_per_reaction": i_min, "imin_source": (imin_rec or {}).get("source"),
                       "algorithmic_inst_per_reaction": i_alg, "sms": sms, "sm_clock_for_peak_mhz": f_max / 1e6,
                       "peak_source": "148 SMs x 4 schedulers x 32 lanes x sm_max_mhz (MEASURED_PEAKS.json)",
                       "frac_at_measured_clock": (achieved / (sms * 128 * clk["sm_mhz"] * 1e6 / 1e12))
                       if clk.get("sm_mhz") else None,
                       "kernel_ms": kern_ms_max,
                       "algorithmic_bytes_per_launch": raw_bytes + run.buffers.stats.numel() * 8,
                       "traffic_source": "profiles/traffic_*.json of this workload and per-rank instance count "
                                         "(ncu --set full, dram read+write of one launch)",
                       "sample_stream_gbs": (raw_bytes / (kern_ms_max / 1e3) / 1e9) if raw_bytes else 0.0}}

    # ---- CPU baseline: the oracle on this host's cores, rank 0 (every N)
    cpu = None
    if rank == 0 and not args.no_cpu_baseline:
        r_cpu, i_cpu, s_cpu, cores = oracle_sample(cfg, args.cpu_budget_s)
        cpu = {"value": r_cpu / s_cpu, "unit": UNIT, "cores": cores, "kind": "oracle",
               "sample": f"instances [0, {i_cpu}) of '{args.config}' at the full horizon, SSA + stats, "
                         f"{s_cpu:.1f} s", "trajectories_per_s": i_cpu / s_cpu}

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms_per_step, "higher_is_better": True, "scaling": args.scaling,
            "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": args.config, "description": cfg.description, "instances_per_gpu": n_per,
                       "instances_total": n_total, "t_end": cfg.t_end, "sample_dt": cfg.sample_dt,
                       "cuts": int(res.n.size), "species": len(info["names"]), "flat_reactions": len(info["rates"]),
                       "raw_samples": not args.no_raw, "parallelism": f"dp{world} (instance sharding)",
                       "shards": f"rank r simulates global instances [floor(r N/{world}), floor((r+1) N/{world}))",
                       "l2": "256 MiB buffer written before every timed step (outside the events)"},
            "trajectories_per_s": traj_s,
            "reactions_per_step": total_reactions,
            "kernel_ms": kern_ms_max,
            "gpu_launches": args.steps * res.launches,   # SSA (+ compaction) kernels of each step
            "roofline": roof,
            "cpu_baseline": cpu,
            "e2e": {"value": e2e_value, "unit": UNIT,
                    "h2d_bytes_per_step": PARAM_BYTES * r2.launches + LOGTAB_BYTES + cubin_bytes,
                    "d2h_bytes_per_step": n_stats * 8, "ms_per_step": float(te[0]),
                    "path": "Model.from_def + dist.simulate_sharded (public API): model load (host strings -> "
                            "flat model -> cached cubin -> module upload), buffers, launch + all-reduce, "
                            "D2H stats + finalize",
                    "h2d": "kernel image + CWC-log table + launch parameter block; instances are generated on the device "
                           "from the model's x0 and the seed (step a2)"},
            "clocks": clk,
            "kernel": {**model.kernel_attributes(), "load_s": load_s},
            "stats_check": {"finished": res.finished, "absorbed": res.absorbed, "overflowed": res.overflowed},
        }
        if shared_gpu:
            line["shared_gpu"] = True   # functional multi-rank run on fewer GPUs: not a scaling point
        print(json.dumps(line), flush=True)
    if world > 1:
        dist.destroy_process_group()
    return 0


def main(argv=None):
    ap = argparse.ArgumentParser(description=__doc__.split("\n\n")[0])
    ap.add_argument("--gpus", type=int, default=int(os.environ.get("WORLD_SIZE", "1")))
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--config", default="lv1m", choices=sorted(W.CONFIGS))
    ap.add_argument("--scaling", default="strong", choices=["strong", "weak"],
                    help="strong: the config's instances split over the ranks; weak: that many per rank")
    ap.add_argument("--impl", default="b200", choices=["b200", "reference"])
    ap.add_argument("--instances", type=int, default=0,
                    help="instances in total (strong) or per GPU (weak); default: the config's")
    ap.add_argument("--no-raw", action="store_true", help="do not keep raw samples (stats only)")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--cpu-budget-s", type=float, default=15.0)
    ap.add_argument("--ref-step-s", type=float, default=10.0)
    args = ap.parse_args(argv)
    if args.warmup < 3:
        print("warning: the bench contract asks for >= 3 warm-up steps", file=sys.stderr)
    if args.impl == "reference":
        return run_reference(args)
    return run_b200(args)


if __name__ == "__main__":
    sys.exit(main())
