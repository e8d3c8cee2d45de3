"""Per-config efficiency table from a one-pass ncu metrics log (development aid).

    python tools/efficiency_table.py profiles/r2f_warp_efficiency_metrics.log

The log has lines "[name] metric value" for each full-size launch (tools/gpu/r2x.sh); I_min per
model comes from profiles/imin_<model>.json; frac = reactions/s x I_min / (148 x 4 x 32 x 1965 MHz).
Also writes profiles/traffic_*.json records for the LV launches (DRAM bytes per launch).
"""
import json
import os
import re
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import workloads as W  # noqa: E402

# name -> (config, instances, raw cuts on, reactions of the launch)
RUNS = {
    "lv1m": ("lv1m", 1_000_000, True), "lv500k": ("lv1m", 500_000, True), "lv250k": ("lv1m", 250_000, True),
    "lv125k": ("lv1m", 125_000, True), "lv100k": ("lv", 100_000, True), "schlogl": ("schlogl", 1_000_000, False),
    "circadian": ("circadian", 1_250_000, False), "compartments": ("compartments", 1_000_000, False),
    "neurospora": ("neurospora", 1_000_000, False), "vesicles": ("vesicles", 1_000_000, False),
}
REACTIONS = {"lv1m": 1.414e12, "lv500k": 7.07e11, "lv250k": 3.534e11, "lv125k": 1.767e11, "lv100k": 1.414e11,
             "schlogl": 2.479e11, "circadian": 1.741e11, "compartments": 5.731e10, "neurospora": 5.933e10,
             "vesicles": 5.731e8}
PEAK = 148 * 4 * 32 * 1965e6


def main(path):
    vals = {}
    for ln in open(path):
        m = re.match(r"\[(\w+)\] (\S+) ([0-9.]+)$", ln.strip())
        if m:
            vals.setdefault(m.group(1), {})[m.group(2)] = float(m.group(3))
    print("| config | kernel | reactions/s | issue busy | eligible warps | warp exec. eff. | I_min | thread-inst / reaction | frac | DRAM / algorithmic |")
    print("|---|---|---|---|---|---|---|---|---|---|")
    for name, v in vals.items():
        cname, n, raw = RUNS[name]
        cfg = W.CONFIGS[cname]
        md = cfg.model
        imin = json.load(open(os.path.join(ROOT, "profiles", f"imin_{md.name}.json")))["imin_thread_inst_per_reaction"]
        t = v["gpu__time_duration.sum"] * 1e-9
        eff = v["smsp__thread_inst_executed.sum"] / (32 * v["smsp__inst_executed.sum"])
        rps = REACTIONS[name] / t
        ipr = v["smsp__thread_inst_executed.sum"] / REACTIONS[name]
        import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
        S = cwc.Model.from_def(md).n_species
        T = cfg.n_samples
        alg = (T * S * n * 4 if raw else 0) + (T * (1 + 3 * S + S * (cfg.hist_bins + 2)) + 8) * 8
        dram = v["dram__bytes_read.sum"] + v["dram__bytes_write.sum"]
        print(f"| {name} | {t * 1e3:.0f} ms | {rps:.3g} | {v['smsp__issue_active.avg.pct_of_peak_sustained_active']:.1f} % "
              f"| {v['smsp__warps_eligible.avg.per_cycle_active']:.2f} | {eff:.3f} | {imin:.1f} | {ipr:.1f} "
              f"| {rps * imin / PEAK:.3f} | {dram / alg:.2f} |")
        if cname.startswith("lv"):
            rec = {"workload": cname, "instances": n, "dram_bytes_read": int(v["dram__bytes_read.sum"]),
                   "dram_bytes_write": int(v["dram__bytes_write.sum"]), "dram_bytes_per_launch": int(dram),
                   "algorithmic_bytes_per_launch": alg,
                   "source": f"ncu one-pass metrics of one cwc_ssa_kernel launch (tools/quick_time.py, {n} instances, "
                             f"raw cuts on), final round-2 kernel, {os.path.basename(path)}"}
            fname = "traffic_lv.json" if cname == "lv" else \
                ("traffic_lv1m.json" if n == 1_000_000 else f"traffic_lv1m_{n // 1000}k.json")
            with open(os.path.join(ROOT, "profiles", fname), "w") as f:
                json.dump(rec, f, indent=1)


if __name__ == "__main__":
    main(sys.argv[1])
