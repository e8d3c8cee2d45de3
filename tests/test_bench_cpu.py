"""bench.py's contract on the host (no GPU): the reference arm's JSON line, the rank / GPU-count
check, and the committed I_min / traffic records it reads for the roofline object."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _bench(*args, env=None):
    return subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                          timeout=300, env=dict(os.environ, **(env or {})), cwd=ROOT)


def test_reference_arm_prints_one_json_line():
    r = _bench("--impl", "reference", "--config", "imm_death", "--steps", "1", "--warmup", "3", "--ref-step-s", "0.3")
    assert r.returncode == 0, r.stderr[-2000:]
    lines = [ln for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1
    d = json.loads(lines[0])
    for k in ("impl", "metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better",
              "scaling", "dtype", "data", "config", "cpu_baseline", "e2e"):
        assert k in d, k
    assert d["impl"] == "reference" and d["value"] > 0 and d["higher_is_better"] is True
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["e2e"]["value"] == d["value"]


def test_gpu_count_must_match_the_ranks():
    r = _bench("--gpus", "2", "--steps", "1", "--warmup", "3")
    assert r.returncode == 2 and "WORLD_SIZE=1" in r.stderr


def test_roofline_records_are_consistent():
    sys.path.insert(0, ROOT)
    import bench
    import workloads as W
    for cname in ("lv1m", "lv", "schlogl", "circadian", "compartments"):
        imin, rec = bench.measured_imin(W.CONFIGS[cname].model.name)
        assert imin is not None and 100 < imin < 400, cname
        assert "tools/imin.py" in rec["source"]
    for path in os.listdir(os.path.join(ROOT, "profiles")):
        if path.startswith("traffic_"):
            with open(os.path.join(ROOT, "profiles", path)) as f:
                tr = json.load(f)
            assert tr["dram_bytes_per_launch"] == tr["dram_bytes_read"] + tr["dram_bytes_write"]
            assert tr["workload"] in W.CONFIGS and tr["instances"] > 0
