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


def birth_death_law(lam, mu, xmax=400):
    """Stationary law of a birth-death chain with birth rate lam(x) and death rate mu(x) (x >= 1):
    detailed balance pi(x+1) mu(x+1) = pi(x) lam(x), i.e. pi(x) ∝ prod_{y<x} lam(y) / mu(y+1)."""
    xs = np.arange(0, xmax)
    lam_v = np.array([lam(float(y)) for y in xs])
    mu_v = np.array([mu(float(y)) for y in xs[1:]])
    logp = np.concatenate([[0.0], np.cumsum(np.log(lam_v[:-1]) - np.log(mu_v))])
    p = np.exp(logp - logp.max())
    return xs, p / p.sum()


def _fits_law(md, lam, mu, t_mix, seed, N=20000):
    from scipy.stats import chi2
    xs, p = birth_death_law(lam, mu)
    run = oracle.simulate(flatten_def(md), 0, N, t_mix, t_mix, seed=seed, nthreads=8)   # one cut at t_mix
    x = run.raw[-1, 0]
    obs = np.bincount(x, minlength=len(p))[: len(p)].astype(float)
    exp = p * N
    keep = exp >= 5
    stat = float((((obs - exp) ** 2) / exp)[keep].sum())
    assert chi2.sf(stat, keep.sum() - 1) > 1e-5, stat
    mean = float((xs * p).sum())
    var = float(((xs - mean) ** 2 * p).sum())
    assert abs(x.mean() - mean) <= 4 * math.sqrt(var / N)
    return mean


def test_autorepressor_stationary_law():
    """Hill-REPRESSED birth lambda(x) = k K^n / (K^n + x^n), linear death (law hillr)."""
    k, mu = W.AUTOREPRESSOR.rates
    K, n = 30.0, 2
    _fits_law(W.AUTOREPRESSOR, lambda x: k * K ** n / (K ** n + x ** n), lambda x: mu * x, 12.0, 8)


def test_hill_activated_birth_stationary_law():
    """Hill-ACTIVATED birth lambda(x) = k0 + k x^n / (K^n + x^n) (law hill, R16'), linear death.
    A dropped basal term, a swapped K^n / x^n or a wrong exponent moves the law far outside."""
    k0, k, mu = W.HILL_ACT.rates
    K, n = 15.0, 2
    mean = _fits_law(W.HILL_ACT, lambda x: k0 + k * x ** n / (K ** n + x ** n), lambda x: mu * x, 15.0, 21)
    assert 30.0 < mean < 40.0     # the positive feedback lifts the mean well above the basal 10


def test_michaelis_menten_death_stationary_law():
    """Constant birth k0, Michaelis-Menten death mu(x) = V x / (Km + x) (law mm, R16')."""
    k0, V = W.MM_DEATH.rates
    Km = 10.0
    mean = _fits_law(W.MM_DEATH, lambda x: k0, lambda x: V * x / (Km + x), 30.0, 22)
    assert 15.0 < mean < 40.0


def test_neurospora_oscillates_with_published_period():
    """The Leloup-Gonze-Goldbeter model with MM/Hill laws oscillates with a ~21.5 h period."""
    from oracle.period import finalize, period_stats
    fm = flatten_def(W.NEUROSPORA)
    run = oracle.simulate(fm, 0, 200, 96.0, 0.5, seed=1, nthreads=8)
    pa = W.PERIOD_ANALYSIS["neurospora"]
    ps = period_stats(run.raw, fm.names.index(pa["species"]), pa["lo"], pa["hi"])
    lp, ma, _ = finalize(ps, 0.5, pa["window"])
    assert 19.0 < lp[-1] < 24.0 and 19.0 < ma[-1] < 24.0
