# single-warp latency: warp curve + ncu source-level stall samples of one warp running LV
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
python tools/warp_curve.py lv 2 2>&1 | tee gpurun_out/r2f_warp_curve.txt
cat > /tmp/one_warp.py <<'PY'
import workloads as W, paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
cfg = W.CONFIGS["lv"]
m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, raw_samples=False,
                       refill=False, block_threads=32, blocks_per_sm=1, fast_cut=0)
res = m.simulate(32, 4.0, 4.0, cfg.seed)
print("reactions", res.reactions, "kernel_ms", res.kernel_ms)
PY
timeout 600 ncu --set full --import-source on --clock-control none -k cwc_ssa_kernel -o gpurun_out/r2f_one_warp -f python /tmp/one_warp.py > gpurun_out/r2f_one_warp_ncu.log 2>&1
tail -3 gpurun_out/r2f_one_warp_ncu.log
python tools/ncu_stalls.py gpurun_out/r2f_one_warp.ncu-rep 0.5 > gpurun_out/r2f_one_warp_stalls.txt 2>&1
head -5 gpurun_out/r2f_one_warp_stalls.txt
run() { tag=$1; shift; python tools/quick_time.py "$@" 2>&1 | tail -1 | sed "s/^/[$tag] /"; }
for q in 32 63 126; do run "q=$q 125k" lv 125000 reps=2 quantum_samples=$q; done
run "q=63 100k" lv 100000 reps=2 quantum_samples=63
run "q=126 100k" lv 100000 reps=2 quantum_samples=126
