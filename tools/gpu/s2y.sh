# compute-sanitizer on the final kernel (memcheck / racecheck / synccheck)
export PYTHONPATH=$PWD
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python tools/sanitize_run.py > gpurun_out/s2y_sanitize_$tool.log 2>&1
  echo "== $tool rc=$?"; tail -4 gpurun_out/s2y_sanitize_$tool.log
done
