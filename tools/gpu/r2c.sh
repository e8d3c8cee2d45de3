# new GPU tests (crafted draws, steering, functional laws, dist vs oracle, full-size sub-ensembles) + I_min
set -x
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2c_build.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q -k "crafted or steering or functional_law or tiny or dist or full_size" > gpurun_out/r2c_tests.txt 2>&1
tail -30 gpurun_out/r2c_tests.txt
timeout 300 python tools/imin.py lv > gpurun_out/r2c_imin_lv.txt 2>&1; cat gpurun_out/r2c_imin_lv.txt
cp profiles/imin_*.json gpurun_out/ 2>/dev/null
