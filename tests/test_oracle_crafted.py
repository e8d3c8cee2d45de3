"""Pins of the oracle's rare branches with crafted draws ("event forced onto a grid
point (unit test with crafted u)"; readings R6, R7, R8, R9 in DESIGN.md §3).

No Philox stream reaches these branches on demand, so the oracle exposes its step with injected
uniforms (``oracle.step_with_draws``, ssa.c ``oracle_step_with_draws``; ``oracle.simulate`` runs
the very same ``ssa_step`` with Philox draws).  Each expected value below follows from the
reading itself, not from the oracle:

* R7 ("cut ... at a given simulation time"; cadlag): the cut at t_k holds every jump
  with time <= t_k — an event exactly ON the grid point belongs to that cut.  Fails if ssa.c's cut
  test ``t_k < t_next`` becomes ``<=``.
* R6 (selection): j* = min{j : cum_j > target} — strictly greater, so a target equal to cum_j
  selects j+1.  Fails under ``>=``.
* R6 (rounding hole): when no cum_j exceeds the rounded target (only possible for a subnormal
  a0: fl(u a0) = a0), the LAST POSITIVE a_j is selected, never a trailing zero-propensity rule.
* R8 absorbing, R9 overflow, horizon and several cuts in one step.
"""
import math

import numpy as np
import pytest

import oracle
from oracle.cwc_terms import flatten

U_MAX = 1.0 - 2.0 ** -53          # the largest uniform (R3 lattice (2m+1) 2^-53)


def lattice(u: float) -> float:
    """The R3 uniform nearest to u: an odd multiple of 2^-53."""
    m = round(u * 2.0 ** 53)
    if m % 2 == 0:
        m += 1
    return m * 2.0 ** -53


def birth_model(rate=1.0):
    return flatten(["A"], ["top: . -> A"], [rate], "5*A")


def find_u_tau(a0: float, t: float, t_target: float) -> float:
    """An R3 uniform u with fl(t + fl(-CWC-log(u) / a0)) == t_target (searched with the oracle's
    own log, itself pinned against mpmath in test_oracle_rng_log.py)."""
    u0 = lattice(math.exp(-(t_target - t) * a0))
    for d in range(0, 64):
        for u in (u0 + 2 * d * 2.0 ** -53, u0 - 2 * d * 2.0 ** -53):
            if (t + (-oracle.cwclog(u) / a0)) == t_target:
                return u
    raise AssertionError("no lattice uniform lands exactly on the grid point")


# a0 = 16 and t0 = 1 - 1/16: consecutive uniforms move t_next by less than half an ulp of 1.0,
# so every representable t_next near t_1 = 1.0 is reachable
A0, T0 = 16.0, 0.9375


def test_event_exactly_on_a_grid_point_belongs_to_that_cut():
    fm = birth_model(A0)                                # a0 = 16 exactly, whatever x
    t0, dt, K = T0, 1.0, 2
    u_on = find_u_tau(A0, t0, 1.0)                      # the birth happens at t = 1.0 = t_1
    u_far = lattice(1e-12)                              # second step: far beyond t_K
    r = oracle.step_with_draws(fm, [5], t0, 1, K, dt, [u_on, u_far], [0.5, 0.5])
    assert r.js[0] == 0 and r.status == oracle.STEP_HORIZON and r.n_done == 2
    # the jump at exactly t_1 is in cut 1 (x = 6), not the state before it (x = 5)
    assert r.cuts[1, 0] == 6 and r.cuts[2, 0] == 6
    assert r.cuts[0, 0] == -2                            # cut 0 was done before this state


def test_event_just_before_and_after_a_grid_point():
    fm = birth_model(A0)
    t0, dt, K = T0, 1.0, 2
    below = 1.0 - 2.0 ** -53
    u_below = find_u_tau(A0, t0, below)
    u_far = lattice(1e-12)
    r = oracle.step_with_draws(fm, [5], t0, 1, K, dt, [u_below, u_far], [0.5, 0.5])
    assert r.cuts[1, 0] == 6                             # jump before t_1: in cut 1
    above = 1.0 + 2.0 ** -52
    u_above = find_u_tau(A0, t0, above)
    r = oracle.step_with_draws(fm, [5], t0, 1, K, dt, [u_above, u_far], [0.5, 0.5])
    assert r.cuts[1, 0] == 5 and r.cuts[2, 0] == 6        # jump after t_1: cut 1 holds x before it
    assert r.t == above and r.k == 3


def test_selection_tie_is_strict():
    # a = (1, 2): a0 = 3, cum = (1, 3); u with fl(3u) == 1.0 exactly -> target == cum_0
    fm = flatten(["A", "B", "C"], ["top: A -> A B", "top: A -> A C"], [1.0, 2.0], "A")
    u_tie = 3002399751580331 * 2.0 ** -53              # 3u = 1 + 2^-53 -> rounds (to even) to 1.0
    assert 3.0 * u_tie == 1.0 and u_tie == lattice(u_tie)
    r = oracle.step_with_draws(fm, [1, 0, 0], 0.0, 1, 1, 1.0, [lattice(0.9)], [u_tie])
    assert list(r.js) == [1] and list(r.x) == [1, 0, 1]  # cum_0 = target is NOT > target
    u_below = u_tie - 2 * 2.0 ** -53
    assert 3.0 * u_below < 1.0
    r = oracle.step_with_draws(fm, [1, 0, 0], 0.0, 1, 1, 1.0, [lattice(0.9)], [u_below])
    assert list(r.js) == [0] and list(r.x) == [1, 1, 0]


def test_rounding_hole_selects_the_last_positive_rule():
    # a = (2^-1074, 2^-1074, 0): a0 = 2^-1073 (subnormal) and fl(u_sel * a0) == a0 for the largest
    # uniform, so no cum_j exceeds the target (the R6 hole); the fallback takes the last rule with
    # a_j > 0 (rule 1), never the trailing zero-propensity rule 2 (no C) nor simply rule 0
    tiny = 5e-324
    assert tiny == 2.0 ** -1074 and U_MAX * (2 * tiny) == 2 * tiny
    fm = flatten(["A", "B", "C", "D"], ["top: A -> A B", "top: A -> A D", "top: C -> ."], [tiny, tiny, 1.0], "A")
    dt = 2.0 ** 1020                                      # tau = -log(u)/a0 ~ 2^-53 * 2^1073 = 2^1020
    r = oracle.step_with_draws(fm, [1, 0, 0, 0], 0.0, 1, 2, dt, [U_MAX], [U_MAX])
    assert r.n_done == 1 and r.status == oracle.STEP_JUMP
    assert list(r.js) == [1] and list(r.x) == [1, 0, 0, 1]
    # the same rules with normal rates: the target stays below a0 and j* = rule 1 without the hole
    fm2 = flatten(["A", "B", "C", "D"], ["top: A -> A B", "top: A -> A D", "top: C -> ."], [3.0, 3.0, 1.0], "A")
    r = oracle.step_with_draws(fm2, [1, 0, 0, 0], 0.0, 1, 2, 1.0, [lattice(0.9)], [U_MAX])
    assert list(r.js) == [1] and list(r.x) == [1, 0, 0, 1]


def test_absorbing_state_holds_and_consumes_no_draw():
    fm = flatten(["A", "B"], ["top: A -> B"], [1.0], "3*B")
    r = oracle.step_with_draws(fm, [0, 3], 0.4, 1, 4, 0.5, [0.3, 0.3], [0.3, 0.3])
    assert r.status == oracle.STEP_ABSORBED and r.n_done == 1 and list(r.js) == [-1]
    assert (r.cuts[1:, 0] == 0).all() and (r.cuts[1:, 1] == 3).all() and r.k == 5 and r.t == 0.4


def test_overflow_freezes_and_marks_missing():
    fm = flatten(["A"], ["top: A -> A A"], [1.0], "A", x_cap=10)
    r = oracle.step_with_draws(fm, [10], 0.0, 1, 3, 1.0, [lattice(0.9)], [0.5])
    assert r.status == oracle.STEP_OVERFLOWED and list(r.x) == [11]
    assert (r.cuts[1:, 0] == -1).all()


def test_several_cuts_in_one_step_and_horizon():
    fm = birth_model(2.0)                                # a0 = 2
    u = lattice(math.exp(-7.0))                          # next jump near t = 3.5: cuts 0..3 before it
    assert 3.0 < -oracle.cwclog(u) / 2.0 < 4.0
    r = oracle.step_with_draws(fm, [5], 0.0, 0, 5, 1.0, [u, lattice(1e-12)], [0.5, 0.5])
    assert list(r.cuts[:4, 0]) == [5, 5, 5, 5] and list(r.cuts[4:, 0]) == [6, 6]
    assert r.status == oracle.STEP_HORIZON and list(r.x) == [6]


def test_injected_philox_draws_reproduce_simulate():
    """Feeding the step the instance's own Philox draws (R3) reproduces oracle.simulate."""
    import workloads as W
    from oracle.cwc_terms import flatten_def
    fm = flatten_def(W.LOTKA_VOLTERRA)
    seed, inst, t_end, dt = 0x5EED0002, 12345, 0.5, 0.1
    K = oracle.grid_K(t_end, dt)
    ref = oracle.simulate(fm, inst, 1, t_end, dt, seed)
    n = int(ref.reactions[0]) + 1
    ut, us = [], []
    for step in range(n):
        w = oracle.philox4x32_10([step & 0xFFFFFFFF, step >> 32, inst & 0xFFFFFFFF, inst >> 32],
                                 [seed & 0xFFFFFFFF, seed >> 32])
        ut.append(oracle.u01(w[0], w[1]))
        us.append(oracle.u01(w[2], w[3]))
    r = oracle.step_with_draws(fm, fm.x0, 0.0, 0, K, dt, ut, us)
    assert r.status == oracle.STEP_HORIZON and r.n_done == n
    assert np.array_equal(r.cuts, ref.raw[:, :, 0])


@pytest.mark.parametrize("k,K,dt", [(-1, 2, 1.0), (0, 2, 0.0), (0, -1, 1.0), (4, 2, 1.0)])
def test_rejects_bad_arguments(k, K, dt):
    with pytest.raises(oracle.CWCError):
        oracle.step_with_draws(birth_model(), [1], 0.0, k, K, dt, [0.5], [0.5])
