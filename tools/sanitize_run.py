"""Small runs of every model for compute-sanitizer (memcheck / racecheck / synccheck):

    compute-sanitizer --tool memcheck python tools/sanitize_run.py

Exercises quanta + refill, raw cuts, overflow fill, absorption, period analysis, rate laws,
streaming snapshots and the shared-memory moment staging.
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import workloads as W  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402


def main():
    # sizes keep every run under ~1e6 reactions: the sanitizers slow kernels down 100-1000x
    runs = [
        (W.IMM_DEATH, 300, 10.0, 1.0, {}),
        (W.LOTKA_VOLTERRA, 300, 0.3, 0.05, {"quantum_samples": 2}),
        (W.LOTKA_VOLTERRA, 300, 0.3, 0.05, {"fast_cut": 1}),
        (W.SCHLOGL, 500, 0.5, 0.05, {"quantum_samples": 2, "block_threads": 128}),
        (W.CIRCADIAN, 200, 4.0, 0.5, {"period_species": "R", "period_lo": 100, "period_hi": 1000}),
        (W.COMPARTMENTS, 200, 2.0, 0.5, {"smem_stats": 0}),
        (W.NEUROSPORA, 200, 6.0, 0.5, {"period_species": "M", "period_lo": 100, "period_hi": 350}),
        (W.RUNAWAY, 100, 10.0, 0.5, {}),
        (W.DEAD, 100, 3.0, 0.5, {}),
        # round 2: dense staging, compacted per-quantum launches, the paper's lockstep launches
        (W.COMPARTMENTS, 200, 2.0, 0.5, {"smem_stats": 3}),
        (W.LOTKA_VOLTERRA, 300, 0.3, 0.05, {"compact": 1, "quantum_samples": 2}),
        (W.SCHLOGL, 500, 0.5, 0.05, {"refill": False, "quantum_samples": 3}),
        # round 2, second half: raw-cut staging with blocks cut by quanta (partial flushes), the
        # draw-batch loop (default) against the per-step draw, no staging
        (W.LOTKA_VOLTERRA, 300, 0.3, 0.05, {"quantum_samples": 3}),
        (W.LOTKA_VOLTERRA, 300, 0.3, 0.05, {"draw_batch": 0, "raw_stage": 0}),
        (W.CIRCADIAN, 200, 4.0, 0.5, {"draw_batch": 2}),
    ]
    for md, n, t_end, dt, opts in runs:
        m = cwc.Model.from_def(md, hist_bins=64, **opts)
        res = m.simulate(n, t_end, dt, 123)
        assert res.finished == n, md.name
        if "period_species" in opts:
            m.period_stats()
        print(f"{md.name}: {res.reactions} reactions ok", flush=True)
    m = cwc.Model.from_def(W.SCHLOGL, hist_bins=64, raw_samples=False)
    for cf, res in m.stream(2000, 0.5, 0.05, 7, poll_s=0.001):
        pass
    print("stream ok", flush=True)
    # terminate mid-run (cwc_cancel) and the LV path with cuts recorded outside the fast step
    m = cwc.Model.from_def(W.SCHLOGL, hist_bins=64, raw_samples=False)
    for cf, res in m.stream(4000, 1.0, 0.05, 9, poll_s=0.001, stop=lambda c, r: c > 0):
        pass
    print(f"cancel ok (cuts final {cf})", flush=True)
    m = cwc.Model.from_def(W.VESICLES, hist_bins=64, quantum_samples=3)
    res = m.simulate(300, 3.0, 0.5, 5)
    assert res.finished == 300
    print("vesicles (dynamic pools) ok", flush=True)
    # checkpoint / resume: terminate, save to host, restore into a fresh handle, resume
    m = cwc.Model.from_def(W.SCHLOGL, hist_bins=64)
    for cf, res in m.stream(4000, 1.0, 0.05, 11, poll_s=0.001, stop=lambda c, r: c > 0):
        pass
    ckpt = m.checkpoint()
    m2 = cwc.Model.from_def(W.SCHLOGL, hist_bins=64)
    m2.restore(ckpt)
    m2.resume()
    res = m2.finalize()
    assert res.finished == 4000
    print(f"checkpoint/resume ok (cuts final at stop {cf})", flush=True)
    # sparse staging with most items over the admission limit (the global overflow path)
    os.environ["CWC_KERNEL_DEFINES"] = "CWC_SPARSE_TICKETS=4"
    m = cwc.Model.from_def(W.CIRCADIAN, hist_bins=64, smem_stats=2)
    assert m.simulate(400, 4.0, 0.5, 13).finished == 400
    del os.environ["CWC_KERNEL_DEFINES"]
    print("sparse admission overflow ok", flush=True)
    # the injected-draw self-test kernel (both modes)
    m = cwc.Model.from_def(W.LOTKA_VOLTERRA, hist_bins=64)
    for mode in (0, 1):
        out = m.selftest_step([[1000, 1000]] * 64, [0.0] * 64, [1] * 64, 1.0, 0.1, [[0.5] * 8] * 64, [[0.3] * 8] * 64,
                              mode=mode)
        assert (out["n_done"] >= 1).all()
    print("self-test step ok", flush=True)


if __name__ == "__main__":
    main()
