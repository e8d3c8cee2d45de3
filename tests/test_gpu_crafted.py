"""GPU: the SSA kernel's own step code driven by injected draws (cwc_selftest_step) against the
oracle's injected-draw step (oracle.step_with_draws), element by element.

The crafted cases of tests/test_oracle_crafted.py pin the oracle to readings R6-R9; here the
device reaches the same branches through the code the persistent kernel runs — the fast step
(mode 0: cwc_fast_compute / cwc_fast_commit / cwc_resolve, with cuts recorded inside the fast
step or on the full-step path: fast_cut 1 / 0) and the full step alone (mode 1) — and must give
the oracle's x, t, next cut, status, steps taken and emitted cuts.  Random reachable states
(cuts of oracle trajectories) with random lattice uniforms cover every workload model.
"""
import math

import numpy as np
import pytest

import oracle
import workloads as W
from oracle.cwc_terms import flatten, flatten_def

from test_oracle_crafted import A0, T0, U_MAX, find_u_tau, lattice

pytestmark = pytest.mark.gpu

# device status (cwc_ssa.cuh) -> oracle status (ssa.c)
DEV2ORA = {0: oracle.STEP_JUMP, 2: oracle.STEP_HORIZON, 3: oracle.STEP_ABSORBED, 4: oracle.STEP_OVERFLOWED}


def _model(species, rules, rates, term, fast_cut, x_cap=None):
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model(species, rules, rates, term, fast_cut=fast_cut)
    if x_cap is not None:
        m.set_option("x_cap", x_cap)
    return m


def _compare(m, fm, xs, ts, ks, K, dt, UT, US):
    """Run the device in both modes and the oracle on every trajectory; all outputs equal."""
    t_end = K * dt
    for mode in (0, 1):
        got = m.selftest_step(xs, ts, ks, t_end, dt, UT, US, mode=mode)
        for i in range(len(xs)):
            r = oracle.step_with_draws(fm, xs[i], ts[i], ks[i], K, dt, UT[i], US[i])
            ctx = (mode, i)
            assert DEV2ORA[int(got["status"][i])] == r.status, ctx
            assert int(got["n_done"][i]) == r.n_done, ctx
            assert np.array_equal(got["x"][i], r.x), ctx
            assert got["t"][i] == r.t, ctx
            assert int(got["k"][i]) == r.k, ctx
            assert np.array_equal(got["cuts"][i], r.cuts), ctx


@pytest.mark.parametrize("fast_cut", [0, 1])
def test_crafted_branches_match_oracle(fast_cut):
    cases = []
    # R7: event exactly on / just below / just above the grid point t_1 = 1.0
    fmb = flatten(["A"], ["top: . -> A"], [A0], "5*A")
    mb = _model(["A"], ["top: . -> A"], [A0], "5*A", fast_cut)
    far = lattice(1e-12)
    UT = [[find_u_tau(A0, T0, tt), far] for tt in (1.0, 1.0 - 2.0 ** -53, 1.0 + 2.0 ** -52)]
    US = [[0.5, 0.5]] * 3
    _compare(mb, fmb, [[5]] * 3, [T0] * 3, [1] * 3, 2, 1.0, UT, US)
    got = mb.selftest_step([[5]], [T0], [1], 2.0, 1.0, [UT[0]], [US[0]], mode=0)
    assert got["cuts"][0, 1, 0] == 6                   # the jump at t_1 is in cut 1 (R7)
    # R6 strict selection tie and its neighbour
    sp, ru, ra = ["A", "B", "C"], ["top: A -> A B", "top: A -> A C"], [1.0, 2.0]
    u_tie = 3002399751580331 * 2.0 ** -53
    _compare(_model(sp, ru, ra, "A", fast_cut), flatten(sp, ru, ra, "A"), [[1, 0, 0]] * 2, [0.0] * 2, [1] * 2, 1, 1.0,
             [[lattice(0.9)]] * 2, [[u_tie], [u_tie - 2 * 2.0 ** -53]])
    # R6 rounding hole (subnormal a0) with a trailing zero-propensity rule
    tiny = 5e-324
    sp, ru, ra = ["A", "B", "C", "D"], ["top: A -> A B", "top: A -> A D", "top: C -> ."], [tiny, tiny, 1.0]
    mh = _model(sp, ru, ra, "A", fast_cut)
    _compare(mh, flatten(sp, ru, ra, "A"), [[1, 0, 0, 0]], [0.0], [1], 2, 2.0 ** 1020, [[U_MAX]], [[U_MAX]])
    got = mh.selftest_step([[1, 0, 0, 0]], [0.0], [1], 2.0 ** 1021, 2.0 ** 1020, [[U_MAX]], [[U_MAX]])
    assert list(got["x"][0]) == [1, 0, 0, 1]
    # R8 absorbing, R9 overflow, several cuts in one step
    _compare(_model(["A", "B"], ["top: A -> B"], [1.0], "3*B", fast_cut), flatten(["A", "B"], ["top: A -> B"], [1.0], "3*B"),
             [[0, 3]], [0.4], [1], 4, 0.5, [[0.3, 0.3]], [[0.3, 0.3]])
    _compare(_model(["A"], ["top: A -> A A"], [1.0], "A", fast_cut, x_cap=10),
             flatten(["A"], ["top: A -> A A"], [1.0], "A", x_cap=10), [[10], [9]], [0.0, 0.0], [1, 1], 3, 1.0,
             [[lattice(0.9)] * 3] * 2, [[0.5] * 3] * 2)
    u = lattice(math.exp(-7.0))
    _compare(_model(["A"], ["top: . -> A"], [2.0], "5*A", fast_cut), flatten(["A"], ["top: . -> A"], [2.0], "5*A"),
             [[5]], [0.0], [0], 5, 1.0, [[u, far]], [[0.5, 0.5]])


def _random_cases(md, n, t_end, dt, seed, D):
    """Reachable states: cuts of oracle trajectories; draws: random R3-lattice uniforms."""
    fm = flatten_def(md)
    K = oracle.grid_K(t_end, dt)
    run = oracle.simulate(fm, 0, n, t_end, dt, seed, nthreads=8)
    rng = np.random.default_rng(seed)
    kc = rng.integers(0, K, n)
    xs = np.stack([run.raw[kc[i], :, i] for i in range(n)]).astype(np.int32)
    ok = (xs >= 0).all(axis=1)                          # skip frozen (missing) cuts
    xs, kc = xs[ok], kc[ok]
    ts = kc * dt + rng.random(len(kc)) * dt * 0.999     # inside (t_kc, t_kc+1)
    ks = kc + 1
    m52 = rng.integers(0, 2 ** 52, size=(len(kc), D, 2), dtype=np.int64)
    U = (2 * m52 + 1).astype(np.float64) * 2.0 ** -53   # exact: (2m+1) < 2^53
    return fm, xs, ts, ks, K, U[:, :, 0], U[:, :, 1]


@pytest.mark.parametrize("name", ["lv", "schlogl", "circadian", "compartments", "neurospora", "vesicles"])
def test_random_injected_steps_match_oracle(name):
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS[name]
    t_end = min(cfg.t_end, 5.0 if name in ("lv", "schlogl") else cfg.t_end / 4)
    t_end = round(t_end / cfg.sample_dt) * cfg.sample_dt
    fm, xs, ts, ks, K, UT, US = _random_cases(cfg.model, 300, t_end, cfg.sample_dt, 1234, 16)
    for fast_cut in (0, 1):
        m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, fast_cut=fast_cut)
        _compare(m, fm, xs, ts, ks, K, cfg.sample_dt, UT, US)


@pytest.mark.parametrize("name", sorted(W.TINY_MODELS))
def test_random_injected_steps_tiny_models(name):
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    md = W.TINY_MODELS[name]
    fm, xs, ts, ks, K, UT, US = _random_cases(md, 200, 4.0, 0.25, 99, 12)
    _compare(cwc.Model.from_def(md, hist_bins=64), fm, xs, ts, ks, K, 0.25, UT, US)
