"""Closed-form laws at GPU scale (north_star acceptance: "ensemble mean/variance are within 4
standard errors of the closed forms"), through the product path and its fused on-line
statistics (finalised mean / unbiased variance / histogram / quantiles, not raw samples).

With 1M instances the 4-SE bands are ~30x tighter than the oracle-size pins in
test_oracle_laws.py, so a slip anywhere in the path (propensities, waiting time, selection, the
cadlag cut, the integer moment accumulation, the variance finalisation) shows up here even
though the bit parity with the oracle is checked separately.  Laws:
  * immigration-death (config 1 model): x(t) ~ Poisson(lambda(t)), lambda = k/mu (1 - e^{-mu t})
  * Schlogl (config 3, full size): exact transient CME (scipy expm) — mean, variance,
    P(x >= 300) from the histogram, inverted-CDF quantiles
  * CWC transport into a nucleus (rule compiler path): S@nuc ~ Binomial(30, p(t))
  * Hill-repressed birth / linear death (functional rate law, R16'): stationary law by
    detailed balance
Fixed seeds: each check is deterministic; the 4-SE bands are the tolerance.
"""
import math

import numpy as np
import pytest

import workloads as W

from helpers import gpu_run

pytestmark = pytest.mark.gpu
Z = 4.0


def _check_mean_var(mean_emp, var_emp, n, mean, var, mu4, what):
    se_m = math.sqrt(var / n)
    se_v = math.sqrt(max(mu4 - var * var * (n - 3) / (n - 1), 1e-300) / n)
    assert abs(mean_emp - mean) <= Z * se_m, (what, "mean", mean_emp, mean, se_m)
    assert abs(var_emp - var) <= Z * se_v, (what, "var", var_emp, var, se_v)


def _pmf_moments(x, p):
    m = float((x * p).sum())
    v = float(((x - m) ** 2 * p).sum())
    mu4 = float(((x - m) ** 4 * p).sum())
    return m, v, mu4


def test_imm_death_poisson_1m():
    cfg = W.CONFIGS["imm_death"]
    kb, mu = cfg.model.rates
    N = 1_000_000
    res, *_ = gpu_run(cfg.model, N, 0, N, cfg.t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins, raw=False)
    assert res.finished == N and (res.n == N).all()
    for k in range(1, res.n.size):
        lam = kb / mu * (1 - math.exp(-mu * res.times[k]))
        _check_mean_var(res.mean[k, 0], res.var[k, 0], N, lam, lam, lam + 3 * lam * lam, f"t={res.times[k]}")


def test_schlogl_transient_cme_1m():
    from scipy.linalg import expm
    cfg = W.CONFIGS["schlogl"]
    c1, c2, c3, c4 = cfg.model.rates
    N = cfg.n_instances
    res, *_ = gpu_run(cfg.model, N, 0, N, cfg.t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins,
                      hist_width=cfg.hist_width, raw=False)
    assert res.finished == N
    n = 1501                                   # P(x > 1000) ~ 3e-28 on [0, 50]
    x = np.arange(n, dtype=np.float64)
    birth = c1 * x * (x - 1) / 2 + c3          # 2X -> 3X (R1: k * C(x, 2)) and 0 -> X
    death = c2 * x * (x - 1) * (x - 2) / 6 + c4 * x
    birth[-1] = 0.0
    Q = np.diag(-(birth + death)) + np.diag(birth[:-1], -1) + np.diag(death[1:], 1)
    E = expm(Q * cfg.sample_dt)
    p = np.zeros(n)
    p[250] = 1.0
    checks = {10, 50, 100, 500}                # t = 1, 5, 10, 50
    for k in range(1, max(checks) + 1):
        p = E @ p
        if k not in checks:
            continue
        m, v, mu4 = _pmf_moments(x, p)
        _check_mean_var(res.mean[k, 0], res.var[k, 0], N, m, v, mu4, f"t={res.times[k]}")
        # histogram (width 1 from 0): P(x >= 300) as a Bernoulli mean
        h = res.hist[k, 0]                     # [underflow, bins 0..1023, overflow]
        emp = h[301:].sum() / N
        pt = float(p[300:].sum())
        assert abs(emp - pt) <= Z * math.sqrt(pt * (1 - pt) / N), (k, emp, pt)
        # inverted-CDF quantiles: F(q - 1) < level and F(q) >= level, within the 4-SE band of F
        F = np.cumsum(p)
        for qi, level in enumerate(res.q):
            qv = int(res.quantile[k, 0, qi])
            band = Z * math.sqrt(level * (1 - level) / N)
            assert F[qv] >= level - band and (qv == 0 or F[qv - 1] < level + band), (k, level, qv)
    # the metastable transient at t = 50 is not the stationary law
    m50, _, _ = _pmf_moments(x, p)
    assert abs(m50 - 316.748) < 0.05


def test_transport_into_nucleus_binomial_1m():
    md = W.TINY_MODELS["transport"]            # S (out) <-> S@nuc via CWC compartment rules
    k_in, k_out = md.rates
    N, t_end, dt = 1_000_000, 4.0, 0.25
    res, *_ = gpu_run(md, N, 0, N, t_end, dt, 2024, hist_bins=64, raw=False)
    s_nuc = res.species.index("S@nuc")
    s_out = res.species.index("S")
    assert (res.sum[:, s_nuc] + res.sum[:, s_out] == 30 * N).all()      # conservation, exact
    for k in range(1, res.n.size):
        pin = k_in / (k_in + k_out) * (1 - math.exp(-(k_in + k_out) * res.times[k]))
        m, v = 30 * pin, 30 * pin * (1 - pin)
        mu4 = v * (1 + 3 * (30 - 2) * pin * (1 - pin))                   # Binomial 4th central moment
        _check_mean_var(res.mean[k, s_nuc], res.var[k, s_nuc], N, m, v, mu4, f"t={res.times[k]}")


def test_hill_autorepressor_stationary_1m():
    md = W.AUTOREPRESSOR                       # 0 -> P @ hillr(P, 30, 2), P -> 0
    k, K, nh = 60.0, 30.0, 2
    mu = md.rates[1]
    N = 1_000_000
    res, *_ = gpu_run(md, N, 0, N, 20.0, 5.0, 77, hist_bins=256, raw=False)
    # detailed balance: pi(x+1) / pi(x) = b(x) / d(x+1), b(x) = k K^n / (K^n + x^n), d(x) = mu x
    xs = np.arange(400)
    logpi = np.zeros(xs.size)
    for x in range(1, xs.size):
        b = k * K ** nh / (K ** nh + (x - 1) ** nh)
        logpi[x] = logpi[x - 1] + math.log(b / (mu * x))
    pi = np.exp(logpi - logpi.max())
    pi /= pi.sum()
    m, v, mu4 = _pmf_moments(xs.astype(np.float64), pi)
    for kk in (3, 4):                          # t = 15, 20: 15+ relaxation times from x0 = 0
        _check_mean_var(res.mean[kk, 0], res.var[kk, 0], N, m, v, mu4, f"t={res.times[kk]}")


def _birth_death_pi(lam, mu, xmax=600):
    """pi(x+1) / pi(x) = lam(x) / mu(x+1) (detailed balance of a birth-death chain)."""
    xs = np.arange(xmax)
    logpi = np.zeros(xs.size)
    for x in range(1, xs.size):
        logpi[x] = logpi[x - 1] + math.log(lam(x - 1) / mu(x))
    pi = np.exp(logpi - logpi.max())
    return xs.astype(np.float64), pi / pi.sum()


@pytest.mark.parametrize("name", ["hill_act", "mm_death"])
def test_functional_law_stationary_1m(name):
    """Hill-ACTIVATED birth and Michaelis-Menten death (R16') at 1M instances: the finalised mean
    and variance of the fused statistics within 4 SE of the detailed-balance stationary law."""
    md = W.TINY_MODELS[name]
    if name == "hill_act":
        k0, k, mu = md.rates
        xs, pi = _birth_death_pi(lambda x: k0 + k * x ** 2 / (15.0 ** 2 + x ** 2), lambda x: mu * x)
    else:
        k0, V = md.rates
        xs, pi = _birth_death_pi(lambda x: k0, lambda x: V * x / (10.0 + x))
    N = 1_000_000
    res, *_ = gpu_run(md, N, 0, N, 40.0, 10.0, 91, hist_bins=512, raw=False)
    m, v, mu4 = _pmf_moments(xs, pi)
    for kk in (3, 4):                          # t = 30, 40: far past the relaxation time
        _check_mean_var(res.mean[kk, 0], res.var[kk, 0], N, m, v, mu4, f"{name} t={res.times[kk]}")
