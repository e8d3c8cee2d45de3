"""I_min of SURVEY §8(d): thread-instructions per reaction of a divergence-free single-warp run of
a model's SSA kernel (the unit of bench.py's useful roofline fraction).

    python tools/imin.py lv                 # GPU: runs itself under ncu, writes profiles/imin_<model>.json
    python tools/imin.py lv --worker        # (the profiled process)

One warp: 32 instances in 32-thread CTAs (the first warp to reach the work queue takes all 32
items), t_end = sample_dt (only the cuts at 0 and t_end, so no lane leaves the fast loop for a cut
in between).  I_min = smsp__thread_inst_executed.sum / reactions: executed thread-instructions,
so lanes whose trajectory ended early cost nothing.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

HORIZON = {"lotka_volterra": 4.0, "schlogl": 4.0, "circadian": 8.0, "compartments": 20.0, "neurospora": 24.0,
           "imm_death": 100.0, "vesicles": 50.0}


def _fast_cut():
    for a in sys.argv[2:]:
        if a.startswith("fast_cut="):
            return int(a.split("=")[1])
    return 0


def worker(cname):
    import workloads as W
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS[cname]
    t = HORIZON.get(cfg.model.name, 4.0)
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, block_threads=32,
                           fast_cut=_fast_cut())
    res = m.simulate(32, t, t, cfg.seed)
    print(json.dumps({"reactions": res.reactions, "t_end": t, "instances": 32}), flush=True)


def main():
    cname = sys.argv[1] if len(sys.argv) > 1 else "lv"
    if "--worker" in sys.argv:
        return worker(cname)
    cmd = ["ncu", "--metrics", "smsp__inst_executed.sum,smsp__thread_inst_executed.sum", "--csv", "-k",
           "cwc_ssa_kernel", "--clock-control", "none", sys.executable, os.path.abspath(__file__), cname, "--worker", f"fast_cut={_fast_cut()}"]
    out = subprocess.run(cmd, capture_output=True, text=True, env=dict(os.environ, PYTHONPATH=ROOT)).stdout
    run = json.loads([ln for ln in out.splitlines() if ln.startswith("{")][-1])
    rows = list(csv.reader(io.StringIO("\n".join(ln for ln in out.splitlines() if ln.startswith('"')))))
    hdr = rows[0]
    vals = {}
    for r in rows[1:]:
        vals[r[hdr.index("Metric Name")]] = float(r[hdr.index("Metric Value")].replace(",", ""))
    import workloads as W
    model = W.CONFIGS[cname].model.name
    rec = {
        "model": model,
        "imin_thread_inst_per_reaction": vals["smsp__thread_inst_executed.sum"] / run["reactions"],
        "warp_inst_per_warp_step": vals["smsp__inst_executed.sum"] * 32 / run["reactions"],
        "simt_efficiency": vals["smsp__thread_inst_executed.sum"] / (32 * vals["smsp__inst_executed.sum"]),
        "reactions": run["reactions"], "thread_inst": vals["smsp__thread_inst_executed.sum"],
        "warp_inst": vals["smsp__inst_executed.sum"],
        "source": f"tools/imin.py {cname}: ncu smsp__thread_inst_executed.sum of one cwc_ssa_kernel launch, 1 warp, "
                  f"32 instances, t_end = sample_dt = {run['t_end']} (no intermediate cuts), fast_cut={_fast_cut()}",
    }
    path = os.path.join(ROOT, "profiles", f"imin_{model}.json")
    with open(path, "w") as f:
        json.dump(rec, f, indent=1)
    print(json.dumps(rec))


if __name__ == "__main__":
    main()
