# ncu --set full + per-instruction stalls of vesicles 1M (final kernel)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g._load_builder().build()" > /dev/null 2>&1
timeout 1200 ncu --set full --import-source on --clock-control none -k cwc_ssa_kernel -c 1 -o gpurun_out/s2m_ves_full -f python tools/quick_time.py vesicles 1000000 raw=0 reps=1 > /dev/null 2>&1
python tools/ncu_summary.py gpurun_out/s2m_ves_full.ncu-rep > gpurun_out/s2m_vesicles_ncu_summary.txt 2>&1
python tools/ncu_stalls.py gpurun_out/s2m_ves_full.ncu-rep 0.3 > gpurun_out/s2m_vesicles_stalls.txt 2>&1
rm -f gpurun_out/s2m_ves_full.ncu-rep
echo done
