"""Dump the NVRTC source + SASS of one workload's SSA kernel (development aid).

    PYTHONPATH=. python tools/dump_sass.py lv /tmp/sass_lv      -> /tmp/sass_lv/{kernel.cu,kernel.sass,ptxas.log}
Kernel variants: CWC_KERNEL_DEFINES="A=1;B=2" as for the runtime.
"""
import glob, os, subprocess, sys, tempfile

name = sys.argv[1] if len(sys.argv) > 1 else "lv"
out = sys.argv[2] if len(sys.argv) > 2 else f"/tmp/sass_{name}"
os.makedirs(out, exist_ok=True)
cache = tempfile.mkdtemp()
os.environ["CWC_CACHE_DIR"] = cache
import workloads as W  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402

cfg = W.CONFIGS[name]
opts = {k: int(v) for k, v in (a.split("=") for a in sys.argv[3:])}
m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, **opts)
src, log = m.compile()
open(f"{out}/kernel.cu", "w").write(src)
open(f"{out}/ptxas.log", "w").write(log)
cub = glob.glob(f"{cache}/*.cubin")[0]
sass = subprocess.run(["cuobjdump", "-sass", cub], capture_output=True, text=True).stdout
open(f"{out}/kernel.sass", "w").write(sass)
print(log)
print(f"{out}: {len(sass.splitlines())} SASS lines; attrs {m.kernel_attributes()}")
