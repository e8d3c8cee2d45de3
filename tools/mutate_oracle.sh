#!/bin/bash
# mutation check: each mutant of oracle/ssa.c must make tests/test_oracle_crafted.py fail
cd /root/repo
cp oracle/ssa.c /tmp/ssa.c.orig
run() {
  python - "$1" "$2" <<'PY'
import sys
s=open('/tmp/ssa.c.orig').read()
a,b=sys.argv[1],sys.argv[2]
assert s.count(a)==1, (a, s.count(a))
open('oracle/ssa.c','w').write(s.replace(a,b))
PY
  python -m pytest tests/test_oracle_crafted.py -q -x 2>&1 | tail -1 | sed "s|^|[$3] |"
}
run '(double)*k * jb->dt < t_next' '(double)*k * jb->dt <= t_next' "cut <="
run 'if (cum[j] > target)' 'if (cum[j] >= target)' "select >="
run 'for (int32_t j = M - 1; j >= 0; --j) if (a[j] > 0.0) { js = j; break; }' 'js = M - 1;' "hole: last rule"
run 'for (int32_t j = M - 1; j >= 0; --j) if (a[j] > 0.0) { js = j; break; }' 'js = 0;' "hole: first rule"
cp /tmp/ssa.c.orig oracle/ssa.c
python -c "import oracle; oracle.build(force=True)"
python -m pytest tests/test_oracle_crafted.py -q 2>&1 | tail -1
