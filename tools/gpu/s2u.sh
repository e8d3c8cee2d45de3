# the whole GPU suite with the device bounds checks compiled into every kernel (CWC_CHECKS=1)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1 || { echo BUILD FAILED; exit 1; }
CWC_KERNEL_DEFINES="CWC_CHECKS=1" timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/s2u_gpu_tests_checked.log 2>&1; tail -3 gpurun_out/s2u_gpu_tests_checked.log
