# per-config ncu evidence: one launch of every BASELINE-shaped
# config at full size, ncu --set full (summary + per-instruction stalls)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
prof() { name=$1; shift
  timeout 1500 ncu --set full --import-source on --clock-control none -k cwc_ssa_kernel -c 1 -o gpurun_out/r2c_${name}_full -f python tools/quick_time.py "$@" reps=1 > gpurun_out/r2c_${name}_ncu.log 2>&1
  python tools/ncu_summary.py gpurun_out/r2c_${name}_full.ncu-rep > gpurun_out/r2c_${name}_ncu_summary.txt 2>&1
  python tools/ncu_stalls.py gpurun_out/r2c_${name}_full.ncu-rep 0.5 > gpurun_out/r2c_${name}_stalls.txt 2>&1
  rm -f gpurun_out/r2c_${name}_full.ncu-rep
  echo "== $name"; cat gpurun_out/r2c_${name}_ncu_summary.txt
}
prof schlogl schlogl 1000000 raw=0
prof circadian circadian 1250000 raw=0
prof compartments compartments 1000000 raw=0
prof neurospora neurospora 1000000 raw=0
prof vesicles vesicles 1000000 raw=0
prof lv100k lv 100000
prof lv125k lv 125000
for c in lv schlogl circadian compartments neurospora vesicles; do timeout 300 python tools/imin.py $c > /dev/null 2>&1; done
cp profiles/imin_*.json gpurun_out/
cat profiles/imin_*.json
