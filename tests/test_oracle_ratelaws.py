"""Pins for the oracle's functional rate laws (reading R16').

* the propensity of every law equals its formula evaluated step by step (values that a
  dropped term, a wrong exponent or a swapped K would change);
* a law is inactive when its lhs is not available;
* a birth-death chain with Hill-repressed birth lambda(x) = k K^n / (K^n + x^n) and death mu x
  has the stationary law pi(x) ∝ prod_{i<x} lambda(i) / (mu (i+1)) (detailed balance); the
  oracle's long-time samples must fit it (chi-square).
"""
import math

import numpy as np

import oracle
import workloads as W
from oracle.cwc_terms import flatten, flatten_def


def test_law_propensities_formulas():
    fm = flatten(["A", "B", "C"],
                 ["top: A -> B @ mm(A, 7.5)", "top: . -> A @ hill(B, 4, 3)", "top: . -> C @ hillr(B, 4, 3)",
                  "top: C -> . @ mm(B, 2)"],
                 [2.0, 3.0, 5.0, 1.5], "2*A 5*B")
    cm = oracle.CModel(fm)
    for x in ([2, 5, 0], [0, 0, 3], [9, 1, 1], [4, 12, 7]):
        a, _ = cm.propensities(x)
        A, B, C = (float(v) for v in x)
        assert a[0] == ((2.0 * A) / (7.5 + A) if x[0] else 0.0)
        assert a[1] == (3.0 * (B * B * B)) / (64.0 + B * B * B)
        assert a[2] == (5.0 * 64.0) / (64.0 + B * B * B)
        # law on B but lhs C: inactive when C is absent
        assert a[3] == ((1.5 * B) / (2.0 + B) if x[2] else 0.0)


def test_autorepressor_stationary_law():
    from scipy.stats import chi2
    m = W.AUTOREPRESSOR
    k, mu = m.rates
    K, n = 30.0, 2
    xs = np.arange(0, 200)
    lam = k * K ** n / (K ** n + xs.astype(float) ** n)
    logp = np.concatenate([[0.0], np.cumsum(np.log(lam[:-1]) - np.log(mu * xs[1:]))])
    p = np.exp(logp - logp.max())
    p /= p.sum()
    N = 20000
    run = oracle.simulate(flatten_def(m), 0, N, 12.0, 12.0, seed=8, nthreads=8)   # t = 12/mu: mixed
    x = run.raw[-1, 0]
    obs = np.bincount(x, minlength=len(p))[: len(p)].astype(float)
    exp = p * N
    keep = exp >= 5
    stat = float((((obs - exp) ** 2) / exp)[keep].sum())
    assert chi2.sf(stat, keep.sum() - 1) > 1e-5, stat
    mean = float((xs * p).sum())
    var = float(((xs - mean) ** 2 * p).sum())
    assert abs(x.mean() - mean) <= 4 * math.sqrt(var / N)


def test_neurospora_oscillates_with_published_period():
    """The Leloup-Gonze-Goldbeter model with MM/Hill laws oscillates with a ~21.5 h period."""
    from oracle.period import finalize, period_stats
    fm = flatten_def(W.NEUROSPORA)
    run = oracle.simulate(fm, 0, 200, 96.0, 0.5, seed=1, nthreads=8)
    pa = W.PERIOD_ANALYSIS["neurospora"]
    ps = period_stats(run.raw, fm.names.index(pa["species"]), pa["lo"], pa["hi"])
    lp, ma, _ = finalize(ps, 0.5, pa["window"])
    assert 19.0 < lp[-1] < 24.0 and 19.0 < ma[-1] < 24.0
