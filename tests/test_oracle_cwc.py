"""Pins for the oracle's CWC tree matching / flattening (oracle/cwc_terms.py).

The expected tables below were flattened BY HAND from the CWC semantics stated in
PAPER.md P:L203-215 (§IV) and the flattening readings of DESIGN.md §3 (species = (region,
atom) in region pre-order then alphabet order; one flat reaction per (rule, context,
injective compartment assignment), R15).  The transport model is pinned by its closed
form: every molecule moves independently, so S@nuc(t) ~ Binomial(30, p(t)).
"""
import math

import numpy as np
import pytest

import oracle
import workloads as W
from oracle.cwc_terms import CWCError, flatten, flatten_def


def _sparse(fm):
    return [(fm.reactants[j], {s: d for s, d in enumerate(fm.delta[j]) if d}, fm.rates[j])
            for j in range(len(fm.rates))]


def test_model_E_hand_flattened():
    fm = flatten_def(W.COMPARTMENTS)
    assert fm.names == ["L", "R@cell.wrap", "RL@cell.wrap", "S@cell", "M@cell", "P@cell",
                        "S@cell/nuc", "G@cell/nuc", "M@cell/nuc"]
    assert fm.x0 == [500, 100, 0, 0, 0, 0, 0, 2, 0]
    expect = [
        ([(0, 1), (1, 1)], {0: -1, 1: -1, 2: 1}, 0.01),
        ([(2, 1)], {2: -1, 0: 1, 1: 1}, 1.0),
        ([(2, 1)], {2: -1, 1: 1, 3: 1}, 0.5),
        ([(3, 1)], {3: -1, 6: 1}, 0.2),
        ([(6, 1)], {6: -1, 3: 1}, 0.1),
        ([(6, 1), (7, 1)], {8: 1}, 0.05),
        ([(8, 1)], {8: -1, 4: 1}, 1.0),
        ([(4, 1)], {5: 1}, 2.0),
        ([(4, 1)], {4: -1}, 0.2),
        ([(5, 1)], {5: -1}, 0.05),
        ([(3, 1)], {3: -1}, 0.1),
        ([], {0: 1}, 50.0),
        ([(0, 1)], {0: -1}, 0.1),
        ([(6, 1)], {6: -1}, 0.1),
    ]
    assert _sparse(fm) == expect


def test_two_cells_hand_flattened():
    fm = flatten_def(W.TWO_CELLS)
    assert fm.names == ["A", "B", "A@cell#0", "B@cell#0", "B@cell#1.wrap", "A@cell#1", "B@cell#1"]
    assert fm.x0 == [20, 0, 3, 0, 2, 0, 0]
    expect = [
        ([(0, 1)], {0: -1, 2: 1}, 0.05),
        ([(0, 1)], {0: -1, 5: 1}, 0.05),
        ([(2, 1)], {2: -1, 3: 1}, 1.0),
        ([(5, 1)], {5: -1, 6: 1}, 1.0),
        ([(3, 1)], {3: -1, 1: 1}, 0.5),
        ([(6, 1)], {6: -1, 1: 1}, 0.5),
    ]
    assert _sparse(fm) == expect
    assert fm.rule_of == [0, 0, 1, 1, 2, 2]


def test_flat_models_are_identity():
    fm = flatten_def(W.LOTKA_VOLTERRA)
    assert fm.names == ["Y1", "Y2"] and fm.x0 == [1000, 1000] and fm.x_cap == 100_000
    assert _sparse(fm) == [([(0, 1)], {0: 1}, 10.0), ([(0, 1), (1, 1)], {0: -1, 1: 1}, 0.01),
                           ([(1, 1)], {1: -1}, 10.0)]
    fm = flatten_def(W.SCHLOGL)
    assert _sparse(fm) == [([(0, 2)], {0: 1}, 0.03), ([(0, 3)], {0: -1}, 1e-4), ([], {0: 1}, 200.0),
                           ([(0, 1)], {0: -1}, 3.5)]
    fm = flatten_def(W.CIRCADIAN)
    assert fm.names == list(W.CIRCADIAN.species) and len(fm.rates) == 16


def test_default_cap_keeps_counts_exact():
    # order 3 in one species: C(cap, 3) < 2^53 <= C(cap + 1, 3)
    cap = flatten_def(W.SCHLOGL).x_cap
    assert math.comb(cap, 3) < 2 ** 53 <= math.comb(cap + 1, 3)
    # heterodimer: cap^2 < 2^53
    cap = flatten_def(W.CIRCADIAN).x_cap
    assert cap * cap < 2 ** 53 <= (cap + 1) ** 2
    assert flatten_def(W.IMM_DEATH).x_cap == 1 << 30
    with pytest.raises(CWCError):
        flatten(["A"], ["top: A A A -> ."], [1.0], "A", x_cap=10 ** 6)


@pytest.mark.parametrize("rules,rates,term,kind", [
    (["top: Q -> ."], [1.0], "A", "invalid"),                       # unknown atom
    (["top: A ."], [1.0], "A", "parse"),                             # no arrow
    (["A -> ."], [1.0], "A", "parse"),                               # no label
    (["top: A -> ."], [-1.0], "A", "invalid"),                       # negative rate
    (["top: A -> ."], [float("nan")], "A", "invalid"),
    (["top: A -> (. $x | $X)^c"], [1.0], "A", "unsupported"),        # compartment creation
    (["top: A -> (.|B)^c (.|B)^c"], [1.0], "A", "unsupported"),    # two creations in one rule (R20)
    (["top: A ($x | $X)^c -> A $X ($x | $X)^c"], [1.0], "A", "unsupported"),  # release, not destroyed
    (["top: A -> (.|B)^c", "c: B -> (.|A)^d"], [1.0, 1.0], "A", "unsupported"),  # nested dynamic
    (["top: ($x | $X)^c -> ."], [1.0], "(. | (.|.)^d)^c", "unsupported"),  # dynamic with nested compartment
    (["top: A A A A -> ."], [1.0], "A", "unsupported"),              # order > 3
    (["top: (A | $X)^c -> (. | $X)^c"], [1.0], "A (A|.)^c", "unsupported"),  # closed wrap
    (["top: (. $x | $X)^c (. $y | $Y)^c -> (. $y | $X)^c (. $x | $Y)^c"], [1.0],
     "(.|.)^c (.|.)^c", "unsupported"),                              # variables moved
    (["top: A -> B"], [1.0], "(A | .)^top", "invalid"),              # reserved label
])
def test_rejections(rules, rates, term, kind):
    with pytest.raises(CWCError) as e:
        flatten(["A", "B"], rules, rates, term)
    assert e.value.kind == kind


def test_transport_binomial_closed_form():
    fm = flatten_def(W.TRANSPORT)
    assert fm.names == ["S", "S@nuc"]
    kin, kout = W.TRANSPORT.rates
    N = 8000
    run = oracle.simulate(fm, 0, N, 4.0, 0.5, seed=77, nthreads=8)
    for k in range(run.K + 1):
        t = k * 0.5
        p = kin / (kin + kout) * (1 - math.exp(-(kin + kout) * t))
        x = run.raw[k, 1].astype(np.float64)
        se = math.sqrt(max(30 * p * (1 - p), 1e-12) / N)
        assert abs(x.mean() - 30 * p) <= 4 * se
        assert np.all(run.raw[k, 0] + run.raw[k, 1] == 30)


def test_model_E_conservation():
    fm = flatten_def(W.COMPARTMENTS)
    run = oracle.simulate(fm, 0, 64, 20.0, 0.5, seed=5, nthreads=8)
    n = fm.names
    assert np.all(run.raw[:, n.index("R@cell.wrap")] + run.raw[:, n.index("RL@cell.wrap")] == 100)
    assert np.all(run.raw[:, n.index("G@cell/nuc")] == 2)
    assert np.all(run.raw >= 0)


def test_two_cells_conservation():
    fm = flatten_def(W.TWO_CELLS)
    run = oracle.simulate(fm, 0, 64, 20.0, 0.5, seed=5, nthreads=8)
    # A + B over all regions except the fixed membrane B is conserved; the membrane B stays 2
    free = run.raw[:, [0, 1, 2, 3, 5, 6], :].sum(axis=1)
    assert np.all(free == 23) and np.all(run.raw[:, 4] == 2)
