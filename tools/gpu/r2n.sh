# warp execution efficiency / issue / eligible warps per config (one-pass metrics) + vesicles register budgets
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
M=smsp__thread_inst_executed.sum,smsp__inst_executed.sum,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__warps_eligible.avg.per_cycle_active,smsp__warps_active.avg.per_cycle_active,gpu__time_duration.sum
eff() { name=$1; shift
  timeout 900 ncu --metrics $M --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py "$@" reps=1 2>/dev/null | grep cwc_ssa_kernel | awk -F'","' -v n=$name '{gsub(/"/,"",$15); print "[" n "] " $13 " " $15}'
}
eff lv1m lv 1000000
eff lv125k lv 125000
eff lv100k lv 100000
eff schlogl schlogl 1000000 raw=0
eff circadian circadian 1250000 raw=0
eff compartments compartments 1000000 raw=0
eff neurospora neurospora 1000000 raw=0
eff vesicles vesicles 1000000 raw=0
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for b in 768 704 640 512; do run "ves $b" vesicles 1000000 reps=2 raw=0 block_threads=$b min_blocks=1; done
