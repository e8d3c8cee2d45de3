# fewer, fatter threads when instances < resident lanes (LV 100k / 125k): 704 / 640 threads per CTA
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for rep in 1 2; do
for c in "lv 100000" "lv 125000"; do
  run "768 $c" $c reps=2
  run "704 $c" $c block_threads=704 reps=2
  run "672 $c" $c block_threads=672 reps=2
  run "640 $c" $c block_threads=640 reps=2
done
done
