"""Worker of tests/test_gpu_parity.py::test_bounds_checked_kernel (own process: a failed device
check traps and leaves the CUDA context unusable).  Every kernel here is compiled with
CWC_CHECKS=1 — each shared-memory and global index the SSA kernel forms (raw-cut staging rows
and their flushes, direct raw stores, sparse / dense statistics staging, item admissions) is
checked against its bounds and a violation traps — and every run is compared with the oracle
element by element.  The stand-in for compute-sanitizer, which the GPU pool does not run.
Prints "BOUNDS OK <runs>"."""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, ROOT)
os.environ["CWC_KERNEL_DEFINES"] = "CWC_CHECKS=1"

import oracle  # noqa: E402
import workloads as W  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402
from oracle.cwc_terms import flatten_def  # noqa: E402


def main():
    runs = [
        # (model, n, t_end, dt, seed, options)
        (W.LOTKA_VOLTERRA, 700, 50.0, 0.5, 7, {}),                                   # staging, absorb / overflow
        (W.LOTKA_VOLTERRA, 700, 50.0, 0.5, 7, {"quantum_samples": 5}),              # partial-block flushes
        (W.LOTKA_VOLTERRA, 700, 50.0, 0.5, 7, {"refill": False, "quantum_samples": 3}),
        (W.LOTKA_VOLTERRA, 700, 50.0, 0.5, 7, {"compact": 1, "fast_cut": 1}),
        (W.LOTKA_VOLTERRA, 700, 50.0, 0.5, 7, {"raw_stage": 0, "draw_batch": 0}),
        (W.SCHLOGL, 3000, 5.0, 0.1, 3, {"smem_stats": 3}),                           # dense staging
        (W.SCHLOGL, 3000, 5.0, 0.1, 3, {"smem_stats": 0, "block_threads": 256}),     # global statistics
        (W.CIRCADIAN, 800, 12.0, 0.5, 5, {"smem_stats": 2, "quantum_samples": 7}),   # sparse staging
        (W.COMPARTMENTS, 900, 20.0, 0.5, 9, {}),
        (W.VESICLES, 1200, 40.0, 0.5, 11, {"quantum_samples": 5}),                  # dynamic pools
        (W.IMM_DEATH, 300, 2000.0, 0.1, 77, {}),                                     # T = 20,001 (global moments)
    ]
    for md, n, t_end, dt, seed, opts in runs:
        m = cwc.Model.from_def(md, hist_bins=256, **opts)
        m.simulate_range(n, 0, n, t_end, dt, seed)
        res = m.finalize()
        raw = m.samples(0, n)
        flags, reactions, _ = m.records(0, n)
        ref = oracle.simulate(flatten_def(md), 0, n, t_end, dt, seed, nthreads=os.cpu_count() or 1)
        assert np.array_equal(raw, ref.raw), (md.name, opts)
        assert np.array_equal(flags, ref.flags) and np.array_equal(reactions, ref.reactions), (md.name, opts)
        assert res.reactions == int(ref.reactions.sum()), (md.name, opts)
    print(f"BOUNDS OK {len(runs)} runs", flush=True)


if __name__ == "__main__":
    main()
