"""Instruction mix of the SSA kernel's fast-step loop in a SASS dump (development aid).

    python tools/sass_loop.py kernel.sass      (cuobjdump -sass output; see tools/dump_sass.py)
Finds the innermost backward-branch loop that contains the Philox multiplies and prints its
instruction count by opcode class; instructions inside forward-branch-skipped sub-blocks of the
loop (the rare cut / slow paths) are listed separately when marked by a BSSY..BSYNC pair.
"""
import re, sys
from collections import Counter

lines = open(sys.argv[1]).read().splitlines()
ins = []
for ln in lines:
    m = re.match(r"\s*/\*([0-9a-f]{4,})\*/\s+(.*?);", ln)
    if m:
        ins.append((int(m.group(1), 16), m.group(2).strip()))
addr_idx = {a: i for i, (a, _) in enumerate(ins)}
best = None
for i, (a, txt) in enumerate(ins):
    m = re.search(r"BRA (0x[0-9a-f]+)", txt)
    if not m:
        continue
    tgt = int(m.group(1), 16)
    if tgt >= a or tgt not in addr_idx:
        continue
    body = ins[addr_idx[tgt]: i + 1]
    nw = sum(1 for _, t in body if "IMAD.WIDE.U32" in t)
    if nw >= 18 and (best is None or len(body) < len(best)):
        best = body
if best is None:
    sys.exit("no Philox loop found")
print(f"loop {best[0][0]:#x}..{best[-1][0]:#x}: {len(best)} instructions")


def cls(t):
    t = re.sub(r"^@!?U?P\w+\s+", "", t)
    op = t.split()[0]
    base = op.split(".")[0]
    if op.startswith("IMAD.WIDE"):
        return "IMAD.WIDE"
    if base in ("IMAD", "MOV") and (".MOV" in op or base == "MOV"):
        return "MOV"
    if base.startswith("U") or base in ("LDCU", "S2UR", "R2UR"):
        return "uniform"
    return base


c = Counter(cls(t) for _, t in best)
for k, v in sorted(c.items(), key=lambda kv: -kv[1]):
    print(f"  {k:12s} {v}")
if len(sys.argv) > 2:
    for a, t in best:
        print(f"{a:#06x}  {t}")
