set -x
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/r2d_build.txt 2>&1
timeout 1800 python -m pytest tests -m gpu -q -k "crafted or steering or functional_law or tiny or dist or full_size" > gpurun_out/r2d_tests.txt 2>&1
tail -30 gpurun_out/r2d_tests.txt
python tools/warp_curve.py lv 5 > gpurun_out/r2d_warp_curve.txt 2>&1; cat gpurun_out/r2d_warp_curve.txt
