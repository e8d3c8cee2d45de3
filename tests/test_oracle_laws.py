"""Pins for the oracle SSA against laws the mathematics fixes (SURVEY.md §8(c) "what pins").

Each test is chosen so that a plausible slip in oracle/ssa.c fails it:
  * propensity convention (R1)      -> brute-force count of distinct reactant subsets
  * waiting-time law                -> A->0 from one molecule: P(x(t)=1) = exp(-mu t)
  * selection law / order           -> competing A->B, A->C: P(B) = k1/(k1+k2)
  * sampling convention (R7)        -> pure birth: x(t_k) ~ Poisson(k t_k) (an off-by-one
                                       sample is ~20 SE away)
  * whole path                      -> immigration-death Poisson(lambda(t)), isomerization
                                       Binomial, exact CME (scipy.linalg.expm) on tiny
                                       networks and on the Schlogl birth-death chain
  * absorbing / overflow (R8, R9)   -> dead model and runaway model
  * determinism                     -> thread count / range splitting invariance
Statistical checks use 4 standard errors (north_star acceptance).
"""
import itertools
import math

import numpy as np
import pytest

import oracle
import workloads as W
from oracle.cwc_terms import flatten, flatten_def

Z = 4.0


def _within(emp_mean, mean, var, n, z=Z):
    se = math.sqrt(max(var, 1e-300) / n)
    assert abs(emp_mean - mean) <= z * se, (emp_mean, mean, se)


def _var_se(var, n, mu4):
    # SE of the unbiased sample variance: sqrt((mu4 - var^2 (n-3)/(n-1)) / n)
    return math.sqrt(max(mu4 - var * var * (n - 3) / (n - 1), 1e-300) / n)


# ----------------------------------------------------------------------------- propensities
def _brute_h(x, reactants):
    """Number of distinct ways to pick the reactant multiset from labelled molecules."""
    mol = [s for s, n in enumerate(x) for _ in range(n)]
    need = {s: r for s, r in reactants}
    total = sum(need.values())
    cnt = 0
    for combo in itertools.combinations(range(len(mol)), total):
        got = {}
        for idx in combo:
            got[mol[idx]] = got.get(mol[idx], 0) + 1
        if got == need:
            cnt += 1
    return cnt


def test_propensities_brute_force():
    fm = flatten(["A", "B", "C"],
                 ["top: A A -> B", "top: A B -> C", "top: A A A -> .", "top: . -> A", "top: A B C -> A",
                  "top: B B C -> ."],
                 [1.0, 1.0, 1.0, 1.0, 1.0, 1.0], "4*A 2*B 1*C")
    cm = oracle.CModel(fm)
    rng = np.random.default_rng(7)
    states = [(4, 2, 1), (0, 0, 0), (1, 5, 2), (2, 2, 2), (3, 0, 4)] + \
             [tuple(int(v) for v in rng.integers(0, 6, 3)) for _ in range(20)]
    for x in states:
        a, cum = cm.propensities(x)
        for j, rl in enumerate(fm.reactants):
            assert a[j] == _brute_h(x, rl), (x, j)
        assert np.all(np.diff(cum) >= 0)
        assert cum[-1] == sum(a)  # small integers: left-to-right sum is exact


def test_dimer_first_rate():
    # 2A -> 0 with A0 = 4: first-jump rate exactly 6k (SURVEY §8(c) R1 pin)
    fm = flatten(["A"], ["top: A A -> ."], [0.25], "4*A")
    a, _ = oracle.CModel(fm).propensities([4])
    assert a[0] == 6 * 0.25


# ----------------------------------------------------------------------------- laws
def test_waiting_time_law():
    mu = 0.8
    fm = flatten(["A"], ["top: A -> ."], [mu], "A")
    N = 20000
    run = oracle.simulate(fm, 0, N, 5.0, 0.25, seed=11, nthreads=4)
    for k in range(1, 21):
        t = k * 0.25
        p = math.exp(-mu * t)
        frac = float((run.raw[k, 0] == 1).mean())
        _within(frac, p, p * (1 - p), N)
    # an instance whose molecule died is absorbed (R8); the others reached t_end
    dead = run.raw[-1, 0] == 0
    assert np.all(run.flags[dead] == oracle.FLAG_ABSORBED) and np.all(run.flags[~dead] == 0)
    assert np.array_equal(run.reactions, dead.astype(np.int64))


def test_selection_law():
    k1, k2, k3 = 0.3, 1.1, 0.6
    fm = flatten(["A", "B", "C", "D"], ["top: A -> B", "top: A -> C", "top: A -> D"], [k1, k2, k3], "A")
    N = 30000
    run = oracle.simulate(fm, 0, N, 40.0, 40.0, seed=5, nthreads=4)
    final = run.raw[-1]
    tot = k1 + k2 + k3
    for s, kk in ((1, k1), (2, k2), (3, k3)):
        p = kk / tot
        _within(float((final[s] == 1).mean()), p, p * (1 - p), N)


def test_pure_birth_poisson():
    m = W.PURE_BIRTH
    N = 10000
    run = oracle.simulate(m, 0, N, 10.0, 0.5, seed=3, nthreads=4)
    for k in range(run.K + 1):
        lam = m.rates[0] * k * 0.5
        x = run.raw[k, 0].astype(np.float64)
        _within(x.mean(), lam, lam, N)
        if lam > 0:
            v = x.var(ddof=1)
            assert abs(v - lam) <= Z * _var_se(lam, N, lam + 3 * lam * lam)


def test_imm_death_poisson_closed_form():
    cfg = W.CONFIGS["imm_death"]
    kb, mu = cfg.model.rates
    N = 4000
    run = oracle.simulate(cfg.model, 0, N, cfg.t_end, cfg.sample_dt, cfg.seed, nthreads=8)
    for k in (1, 2, 5, 10, 20, 50, 100):
        t = k * cfg.sample_dt
        lam = kb / mu * (1 - math.exp(-mu * t))
        x = run.raw[k, 0].astype(np.float64)
        _within(x.mean(), lam, lam, N)
        assert abs(x.var(ddof=1) - lam) <= Z * _var_se(lam, N, lam + 3 * lam * lam)
    # the paper-independent closed-form values of SURVEY §8(c)
    assert abs(kb / mu * (1 - math.exp(-mu * 1)) - 9.516258) < 1e-6
    assert abs(kb / mu * (1 - math.exp(-mu * 100)) - 99.995460) < 1e-6
    # ~1900 reactions per trajectory on [0, 100]: E = k*t + mu * int lambda = 1000 + 0.1*...
    expect = kb * 100 + kb * (100 - (1 - math.exp(-mu * 100)) / mu)
    assert abs(run.reactions.mean() - expect) < 0.01 * expect


def test_pure_death_binomial():
    m = W.PURE_DEATH
    x0, mu = 40, m.rates[0]
    N = 8000
    run = oracle.simulate(m, 0, N, 4.0, 0.5, seed=9, nthreads=4)
    for k in range(run.K + 1):
        p = math.exp(-mu * k * 0.5)
        x = run.raw[k, 0].astype(np.float64)
        _within(x.mean(), x0 * p, x0 * p * (1 - p), N)


def test_isomerization_binomial():
    m = W.ISOMERIZATION
    n0, k1, k2 = 20, 1.0, 0.5
    N = 8000
    run = oracle.simulate(m, 0, N, 3.0, 0.25, seed=21, nthreads=4)
    for k in range(run.K + 1):
        t = k * 0.25
        pinf = k1 / (k1 + k2)           # stationary fraction of B
        p = pinf * (1 - math.exp(-(k1 + k2) * t))
        xb = run.raw[k, 1].astype(np.float64)
        _within(xb.mean(), n0 * p, n0 * p * (1 - p), N)
        assert np.all(run.raw[k, 0] + run.raw[k, 1] == n0)


def _cme_generator(fm, states):
    idx = {s: i for i, s in enumerate(states)}
    n = len(states)
    Q = np.zeros((n, n))
    for s in states:
        for j, rl in enumerate(fm.reactants):
            h = 1
            for sp, r in rl:
                h *= math.comb(s[sp], r)
            a = fm.rates[j] * h
            if a == 0:
                continue
            nxt = tuple(v + d for v, d in zip(s, fm.delta[j]))
            Q[idx[nxt], idx[s]] += a
            Q[idx[s], idx[s]] -= a
    return Q


@pytest.mark.parametrize("mdl", [W.BINDING, W.DIMERISATION])
def test_tiny_cme(mdl):
    from scipy.linalg import expm
    fm = flatten_def(mdl)
    # reachable states by BFS
    start = tuple(fm.x0)
    states, frontier = {start}, [start]
    while frontier:
        s = frontier.pop()
        for j, rl in enumerate(fm.reactants):
            if all(s[sp] >= r for sp, r in rl):
                nxt = tuple(v + d for v, d in zip(s, fm.delta[j]))
                if nxt not in states:
                    states.add(nxt)
                    frontier.append(nxt)
    states = sorted(states)
    Q = _cme_generator(fm, states)
    N = 20000
    dt = 0.5
    run = oracle.simulate(fm, 0, N, 3.0, dt, seed=17, nthreads=8)
    p0 = np.zeros(len(states))
    p0[states.index(start)] = 1.0
    from scipy.stats import chi2
    for k in (1, 2, 4, 6):
        p = expm(Q * (k * dt)) @ p0
        samp = run.raw[k].T  # [N, S]
        obs = np.array([np.all(samp == np.array(s), axis=1).sum() for s in states], dtype=np.float64)
        assert obs.sum() == N  # every sample is a reachable state
        exp = p * N
        keep = exp >= 5
        stat = float((((obs - exp) ** 2) / exp)[keep].sum()) + \
            (float(((obs[~keep].sum() - exp[~keep].sum()) ** 2) / max(exp[~keep].sum(), 1e-9))
             if (~keep).any() else 0.0)
        dof = int(keep.sum()) - (0 if (~keep).any() else 1)
        # goodness of fit of the whole distribution against the exact CME, p > 1e-5
        assert chi2.sf(stat, max(dof, 1)) > 1e-5, (k, stat, dof)
        # and the mean of every species within 4 SE
        for s in range(samp.shape[1]):
            vals = np.array([st[s] for st in states], dtype=np.float64)
            mean = float((vals * p).sum())
            var = float(((vals - mean) ** 2 * p).sum())
            _within(samp[:, s].mean(), mean, var, N)


def test_schlogl_transient_cme():
    """Schlogl birth-death chain: exact transient CME on [0, 1500]."""
    from scipy.linalg import expm
    m = W.SCHLOGL
    c1, c2, c3, c4 = m.rates
    n = 1501
    x = np.arange(n, dtype=np.float64)
    birth = c1 * x * (x - 1) / 2 + c3
    death = c2 * x * (x - 1) * (x - 2) / 6 + c4 * x
    birth[-1] = 0.0
    Q = np.diag(-(birth + death)) + np.diag(birth[:-1], -1) + np.diag(death[1:], 1)
    E = expm(Q * 0.5)                      # one grid step of the exact CME
    p = np.zeros(n)
    p[250] = 1.0
    N = 3000
    run = oracle.simulate(m, 0, N, 2.0, 0.5, seed=31, nthreads=8)
    for k in (1, 2, 3, 4):
        p = E @ p
        mean = float((x * p).sum())
        var = float(((x - mean) ** 2 * p).sum())
        mu4 = float(((x - mean) ** 4 * p).sum())
        xs = run.raw[k, 0].astype(np.float64)
        _within(xs.mean(), mean, var, N)
        assert abs(xs.var(ddof=1) - var) <= Z * _var_se(var, N, mu4)
        if k == 2:
            # the survey's CME value at t = 1 (SURVEY.md §8(c) pins table): mean 257.698, var 5813.5
            assert abs(mean - 257.698) < 5e-3 and abs(var - 5813.5) < 0.5


# ----------------------------------------------------------------------------- R8 / R9
def test_dead_model_absorbed():
    run = oracle.simulate(W.DEAD, 0, 50, 10.0, 1.0, seed=1)
    assert np.all(run.flags == oracle.FLAG_ABSORBED)
    assert np.all(run.reactions == 0)
    assert np.all(run.raw[:, 0, :] == 7) and np.all(run.raw[:, 1, :] == 3)


def test_runaway_overflow_freezes():
    run = oracle.simulate(W.RUNAWAY, 0, 200, 20.0, 0.5, seed=2)
    assert np.all(run.flags == oracle.FLAG_OVERFLOWED)
    for i in range(200):
        col = run.raw[:, 0, i]
        miss = col == -1
        first = int(np.argmax(miss))
        assert miss.any() and np.all(miss[first:]) and not miss[:first].any()
        assert np.all(col[:first] <= 10) and np.all(np.diff(col[:first]) >= 0)
        # each birth increments by one: 9 births reach 10, the 10th overflows
        assert run.reactions[i] == 10


def test_zero_horizon():
    run = oracle.simulate(W.LOTKA_VOLTERRA, 0, 16, 0.0, 0.1, seed=4)
    assert run.raw.shape == (1, 2, 16)
    assert np.all(run.raw[0] == 1000) and np.all(run.reactions == 0)


def test_invalid_grid():
    with pytest.raises(oracle.CWCError):
        oracle.simulate(W.IMM_DEATH, 0, 4, 1.05, 0.1, seed=1)


# ----------------------------------------------------------------------------- determinism
def test_thread_and_range_invariance():
    m = W.SCHLOGL
    a = oracle.simulate(m, 0, 64, 1.0, 0.1, seed=99, nthreads=1)
    b = oracle.simulate(m, 0, 64, 1.0, 0.1, seed=99, nthreads=5)
    c1 = oracle.simulate(m, 0, 23, 1.0, 0.1, seed=99, nthreads=2)
    c2 = oracle.simulate(m, 23, 41, 1.0, 0.1, seed=99, nthreads=3)
    assert np.array_equal(a.raw, b.raw) and np.array_equal(a.reactions, b.reactions)
    assert np.array_equal(a.raw, np.concatenate([c1.raw, c2.raw], axis=2))
    d = oracle.simulate(m, 0, 64, 1.0, 0.1, seed=100, nthreads=1)
    assert not np.array_equal(a.raw, d.raw)


# ----------------------------------------------------------------------------- invariants
def test_circadian_invariants():
    cfg = W.CONFIGS["circadian"]
    fm = flatten_def(cfg.model)
    run = oracle.simulate(fm, 0, 40, 48.0, 0.5, cfg.seed, nthreads=8)
    n = fm.names
    assert np.all(run.raw[:, n.index("DA"), :] + run.raw[:, n.index("DAp"), :] == 1)
    assert np.all(run.raw[:, n.index("DR"), :] + run.raw[:, n.index("DRp"), :] == 1)
    assert np.all(run.raw >= 0)
    # oscillation: the repressor R peaks at ~1000-2000 molecules within 48 h
    assert run.raw[:, n.index("R"), :].max() > 500
