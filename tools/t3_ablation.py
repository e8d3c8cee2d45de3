"""SURVEY §8(d) T3 on the GPU: scheduling ablation of the Schlogl ensemble (the paper's
divergence / load-balance stress case, Table I).

    PYTHONPATH=. python tools/t3_ablation.py [n_instances]          # GPU: timing + ncu per config

Configurations, each over the same ensemble (results bit-identical, R12):
  * refill on (this kernel): work items (quantum, instance) from the global queue, warp-level
    refill, Q/tau = 1, 10, 100 sample intervals per quantum, and auto;
  * refill off, per-quantum lockstep (the paper's GPU scheme): one launch per
    quantum, every lane runs quantum q of its own instance, launches as barriers; Q/tau = 1, 10, 100;
  * refill off, whole trajectories (static, one instance per lane at a time).
Per configuration: kernel time (CUDA events over all launches), reactions/s, and from ncu (summed
over the configuration's launches) warp execution efficiency = thread_inst / (32 inst) and issue
slots busy.  Prints one JSON line per configuration.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

CONFIGS = [("refill", q) for q in (1, 10, 100, 0)] + [("lockstep", q) for q in (1, 10, 100)] + [("static", 0)]
METRICS = ["smsp__thread_inst_executed.sum", "smsp__inst_executed.sum", "sm__cycles_active.sum",
           "smsp__issue_active.sum", "smsp__cycles_active.sum"]


def one(mode, q, n):
    import workloads as W
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS["schlogl"]
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, raw_samples=False, refill=(mode == "refill"),
                           quantum_samples=q)
    res = m.simulate(n, cfg.t_end, cfg.sample_dt, cfg.seed)
    return {"mode": mode, "q_over_tau": q, "n": n, "kernel_ms": res.kernel_ms, "reactions": res.reactions,
            "reactions_per_s": res.reactions / (res.kernel_ms / 1e3), "hist_checksum": int(res.hist.sum())}


def main():
    if len(sys.argv) > 1 and sys.argv[1] == "--one":
        mode, q, n = sys.argv[2], int(sys.argv[3]), int(sys.argv[4])
        one(mode, q, n)                     # warm-up (NVRTC, module)
        print(json.dumps(one(mode, q, n)), flush=True)
        return
    n = int(sys.argv[1]) if len(sys.argv) > 1 else 1_000_000
    for mode, q in CONFIGS:
        env = dict(os.environ, PYTHONPATH=ROOT)
        t = subprocess.run([sys.executable, os.path.abspath(__file__), "--one", mode, str(q), str(n)],
                           capture_output=True, text=True, env=env)
        rec = json.loads([ln for ln in t.stdout.splitlines() if ln.startswith("{")][-1])
        prof = subprocess.run(["ncu", "--metrics", ",".join(METRICS), "--csv", "-k", "cwc_ssa_kernel",
                               "--clock-control", "none", sys.executable, os.path.abspath(__file__), "--one", mode,
                               str(q), str(n)], capture_output=True, text=True, env=env).stdout
        rows = list(csv.reader(io.StringIO("\n".join(ln for ln in prof.splitlines() if ln.startswith('"')))))
        tot = {k: 0.0 for k in METRICS}
        if rows:
            h = rows[0]
            for r in rows[1:]:
                name = r[h.index("Metric Name")]
                if name in tot:
                    tot[name] += float(r[h.index("Metric Value")].replace(",", ""))
        # the profiled process simulates twice (warm-up + measured): halve the sums
        rec["warp_exec_efficiency"] = tot["smsp__thread_inst_executed.sum"] / (32 * tot["smsp__inst_executed.sum"]) \
            if tot["smsp__inst_executed.sum"] else None
        rec["issue_active"] = tot["smsp__issue_active.sum"] / tot["smsp__cycles_active.sum"] \
            if tot["smsp__cycles_active.sum"] else None
        rec["thread_inst_per_reaction"] = tot["smsp__thread_inst_executed.sum"] / (2 * rec["reactions"])
        print(json.dumps(rec), flush=True)


if __name__ == "__main__":
    main()
