"""Worker of tests/test_gpu_steering.py (own process, so a hang is killed by the test's timeout):
cancel a streaming simulation many times at random points of a small-count, many-quanta run.
Every terminated run must finish (no item waits forever), report an exact final-cut prefix, and
leave the handle usable.  Prints "CANCEL OK <runs>"."""
import os
import random
import sys
import time

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import workloads as W  # noqa: E402
import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc  # noqa: E402


def main():
    md, n, t_end, dt, seed = W.SCHLOGL, 3000, 20.0, 0.1, 5
    kw = dict(hist_bins=512, raw_samples=False, quantum_samples=1, stream=1)
    ref = cwc.Model.from_def(md, hist_bins=512, raw_samples=False).simulate(n, t_end, dt, seed)
    rng = random.Random(0)
    m = cwc.Model.from_def(md, **kw)
    runs = int(sys.argv[1]) if len(sys.argv) > 1 else 40
    stopped_early = 0
    for r in range(runs):
        m.simulate_range(n, 0, n, t_end, dt, seed)
        time.sleep(rng.random() * 0.03)
        m.cancel()
        res = m.finalize()
        cf = res.cuts_final
        T = res.n.size
        assert 0 <= cf <= T
        stopped_early += cf < T
        for name in ("n", "sum", "sqlo", "sqhi", "hist"):
            assert np.array_equal(getattr(res, name)[:cf], getattr(ref, name)[:cf]), (r, cf, name)
    again = m.simulate(n, t_end, dt, seed)       # the handle still runs to completion
    assert again.finished == n and np.array_equal(again.hist, ref.hist)
    print(f"CANCEL OK {runs} runs, {stopped_early} stopped before the horizon", flush=True)


if __name__ == "__main__":
    main()
