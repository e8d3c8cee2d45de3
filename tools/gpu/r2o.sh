# traffic of the per-rank shards of the strong-scaling run (N = 2, 4) + the multi-rank bench path
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for n in 500000 250000; do
  timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k cwc_ssa_kernel -c 1 --csv python tools/quick_time.py lv $n reps=1 2>/dev/null | grep cwc_ssa | awk -F'","' -v n=$n '{gsub(/"/,"",$15); print "[traffic " n "] " $13 " " $15}'
done
CWC_DIST_BACKEND=gloo timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 bench.py --gpus 2 --steps 3 --warmup 3 --cpu-budget-s 5 > gpurun_out/r2o_bench_2rank_shared.json 2> gpurun_out/r2o_bench_2rank_shared.err
tail -c 1500 gpurun_out/r2o_bench_2rank_shared.json; tail -5 gpurun_out/r2o_bench_2rank_shared.err
timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29534 bench.py --impl reference --gpus 2 --steps 2 --warmup 3 --ref-step-s 5 > gpurun_out/r2o_ref_2rank.json 2>&1
tail -c 800 gpurun_out/r2o_ref_2rank.json
