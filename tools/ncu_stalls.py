"""Per-SASS-instruction stall samples of the hottest loop from an ncu report (development aid).

    python tools/ncu_stalls.py report.ncu-rep [min_exec_fraction]
Prints, for every instruction executed at least min_exec_fraction (default 0.5) times as often as
the most executed one: address, warp-level execution count (normalised), stall samples by
reason, and the SASS text.
"""
import csv, subprocess, sys

path = sys.argv[1]
frac = float(sys.argv[2]) if len(sys.argv) > 2 else 0.5
out = subprocess.run(["ncu", "-i", path, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
ix = {k: i for i, k in enumerate(h)}
reasons = ["stall_wait", "stall_not_selected", "stall_dispatch", "stall_math", "stall_selected", "stall_short_sb",
           "stall_long_sb", "stall_branch_resolving", "stall_mio", "stall_barrier", "stall_no_inst"]
data = []
for r in rows[2:]:
    if len(r) < len(h):
        continue
    ex = float(r[ix["Instructions Executed"]] or 0)
    data.append((r[ix["Address"]], r[ix["Source"]], ex, {k: float(r[ix[k]] or 0) for k in reasons}))
mx = max(d[2] for d in data)
hot = [d for d in data if d[2] >= frac * mx]
tot = {k: sum(d[3][k] for d in hot) for k in reasons}
print(f"{len(hot)} hot instructions; stall samples: " + ", ".join(f"{k[6:]} {v:.0f}" for k, v in tot.items() if v))
print("addr   exec  " + " ".join(f"{k[6:12]:>6s}" for k in reasons) + "  sass")
for a, src, ex, st in hot:
    print(f"{a[-5:]} {ex / mx:5.2f} " + " ".join(f"{st[k]:6.0f}" for k in reasons) + "  " + src.strip()[:60])
