"""Per-SASS-instruction execution counts from an ncu report: the hot loop, normalised per step."""
import csv, subprocess, sys
from collections import Counter

path = sys.argv[1]
steps = float(sys.argv[2]) if len(sys.argv) > 2 else 1.0   # reactions (thread steps) for normalisation
out = subprocess.run(["ncu", "-i", path, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
hdr = rows[1]
ia, isrc, iex, ith, ism = (hdr.index("Address"), hdr.index("Source"), hdr.index("Instructions Executed"),
                           hdr.index("Thread Instructions Executed"), hdr.index("Warp Stall Sampling (All Samples)"))
tot_w = tot_t = 0
ops = Counter()
opt = Counter()
samples = Counter()
lines = []
for r in rows[2:]:
    if len(r) <= ith:
        continue
    w = float(r[iex] or 0); t = float(r[ith] or 0); smp = float(r[ism] or 0)
    tot_w += w; tot_t += t
    op = r[isrc].split()[0] if r[isrc].split() else "?"
    if op.startswith("@"):
        op = r[isrc].split()[1]
    ops[op.split(".")[0]] += w
    opt[op.split(".")[0]] += t
    samples[op.split(".")[0]] += smp
    lines.append((w, r[ia][-5:], r[isrc].strip(), smp))
print(f"total warp inst {tot_w:.4g}, thread inst {tot_t:.4g}; per step: warp-normalised {tot_t/steps:.1f} thread-inst")
for op, w in ops.most_common(40):
    print(f"{op:12s} {opt[op]/steps:8.2f} thread-inst/step  {100*w/tot_w:5.1f}% of warp inst   stall samples {samples[op]:.0f}")
if "--lines" in sys.argv:
    for w, a, s, smp in sorted(lines, reverse=True)[:int(sys.argv[sys.argv.index('--lines')+1])]:
        print(f"{w/tot_w*100:6.2f}%  {a} {smp:8.0f}  {s}")
if "--stalls" in sys.argv:
    n = int(sys.argv[sys.argv.index('--stalls') + 1])
    tot_s = sum(x[3] for x in lines)
    print(f"--- top {n} instructions by warp-stall samples (total {tot_s:.0f})")
    for w, a, s, smp in sorted(lines, key=lambda x: -x[3])[:n]:
        print(f"{smp/tot_s*100:6.2f}%  {a}  exec {w/tot_w*100:5.2f}%  {s}")
