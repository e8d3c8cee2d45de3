#!/bin/bash
# Development timing matrix (not the bench).  Each argument is one run:
#   "<config> <N> [opt=val ...]"            options passed to Model (ints)
#   "DEF=A=1;B=2 <config> <N> [opt=val]"     kernel #defines via CWC_KERNEL_DEFINES
export PYTHONPATH=$PWD
for spec in "$@"; do
  defs=""
  if [[ "$spec" == DEF=* ]]; then
    defs="${spec%% *}"; defs="${defs#DEF=}"; spec="${spec#* }"
  fi
  echo -n "[$defs] "
  CWC_KERNEL_DEFINES="$defs" timeout 300 python tools/quick_time.py $spec 2>&1 | tail -1
done
