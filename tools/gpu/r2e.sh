# same-box A/B: r1 kernel (tools/gpu/r1_kernel) vs current; launch shapes at 100k / 125k / 1M
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for n in 1000000 125000 100000; do
  te=50; [ $n = 1000000 ] && te=10
  CWC_DEVICE_SRC=tools/gpu/r1_kernel run "r1 $n" lv $n t_end=$te reps=2
  run "new $n" lv $n t_end=$te reps=2
  run "new 1024x64 $n" lv $n t_end=$te reps=2 block_threads=1024 min_blocks=1
done
run "new q8 125000" lv 125000 reps=2 quantum_samples=63
run "new 1024x64 q8 125000" lv 125000 reps=2 quantum_samples=63 block_threads=1024 min_blocks=1
python tools/warp_curve.py lv 2 2>&1 | sed "s/^/[curve] /"
