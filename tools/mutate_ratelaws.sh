#!/bin/bash
# mutation check: each mutant of the oracle's rate laws (oracle/ssa.c propensity) must fail the
# stationary-law pins of tests/test_oracle_ratelaws.py (not only the formula restatement)
cd "$(dirname "$0")/.."
cp oracle/ssa.c /tmp/ssa.c.orig
run() {
  python - "$1" "$2" <<'PY'
import sys
s=open('/tmp/ssa.c.orig').read()
a,b=sys.argv[1],sys.argv[2]
assert s.count(a)==1, (a, s.count(a))
open('oracle/ssa.c','w').write(s.replace(a,b))
PY
  python -m pytest tests/test_oracle_ratelaws.py -q -k "stationary" 2>&1 | tail -1 | sed "s|^|[$3] |"
}
run 'if (law == 2) return (m->k[j] * Xn) / (Kn + Xn);' 'if (law == 2) return (m->k[j] * Kn) / (Kn + Xn);' "hill: K^n numerator"
run 'if (law == 2) return (m->k[j] * Xn) / (Kn + Xn);' 'if (law == 2) return (m->k[j] * X) / (Kn + Xn);' "hill: X^1 numerator"
run 'if (law == 1) return (m->k[j] * X) / (K + X);' 'if (law == 1) return (m->k[j] * K) / (K + X);' "mm: K numerator"
run 'if (law == 1) return (m->k[j] * X) / (K + X);' 'if (law == 1) return m->k[j] * X / K;' "mm: linear"
run 'for (int i = 1; i < n; ++i) r = r * y;' 'for (int i = 0; i < n; ++i) r = r * y;' "ipow: n+1"
run 'return (m->k[j] * Kn) / (Kn + Xn);' 'return (m->k[j] * Kn) / (Kn + X);' "hillr: X^1 denominator"
cp /tmp/ssa.c.orig oracle/ssa.c
python -c "import oracle; oracle.build(force=True)"
python -m pytest tests/test_oracle_ratelaws.py -q 2>&1 | tail -1
