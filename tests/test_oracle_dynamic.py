"""Pins for the oracle's dynamic compartments (reading R20).

The flattening into bounded pools (oracle/cwc_terms.py) and the oracle SSA's gates, slot
placement and transfers (oracle/ssa.c) are checked against an independent statement of the
CWC semantics (terms are multisets of atoms and compartments; rules
rewrite them, creating and destroying compartments): for each tiny model the transitions
are written BY HAND on terms below (no parser, no flattening), the chemical master equation
is built on the reachable terms, and

  * the CME of the flat model, lumped onto terms (a term = top atoms + the multiset of its
    compartments; a full pool = the absorbing "overflow" state), must give the same
    distribution at every time (exact up to expm rounding) — flattening and lumpability;
  * oracle SSA ensembles must match the term-level law (4-SE bands on means, chi^2 on a
    marginal) — the SSA's gates / placement / transfers.
"""
import math
from collections import Counter

import numpy as np
import pytest
import scipy.linalg

import oracle
import workloads as W
from oracle.cwc_terms import GATE_POSITIVE, flatten_def

pytestmark = pytest.mark.filterwarnings("ignore::RuntimeWarning")

FULL = "FULL"


def canon(top: Counter, comps):
    """Canonical term: (sorted top atoms, sorted tuple of (label, wrap, content))."""
    ms = lambda c: tuple(sorted((k, v) for k, v in c.items() if v))  # noqa: E731
    return (ms(top), tuple(sorted((l, ms(w), ms(c)) for l, w, c in comps)))


def uncanon(t):
    top, comps = t
    return Counter(dict(top)), [(l, Counter(dict(w)), Counter(dict(c))) for l, w, c in comps]


# ---------------------------------------------------------------- term-level semantics (by hand)
def ves_tiny_moves(t, cap=3):
    """VES_TINY: top: A -> A (.|B)^v (1.0);  v: B -> . (0.7);  top: ($x|$X)^v -> $X (0.5);
    top: B -> . (0.3).  Creation beyond `cap` vesicles -> overflow."""
    top, comps = uncanon(t)
    out = []
    if top["A"]:
        if len(comps) < cap:
            out.append((1.0 * top["A"], canon(top, comps + [("v", Counter(), Counter(B=1))])))
        else:
            out.append((1.0 * top["A"], FULL))
    for i, (l, w, c) in enumerate(comps):
        if c["B"]:
            c2 = Counter(c)
            c2["B"] -= 1
            out.append((0.7 * c["B"], canon(top, comps[:i] + [(l, w, c2)] + comps[i + 1:])))
        top2 = top + c           # dissolution releases the content ($X); the wrap ($x) vanishes
        out.append((0.5, canon(top2, comps[:i] + comps[i + 1:])))
    if top["B"]:
        top2 = Counter(top)
        top2["B"] -= 1
        out.append((0.3 * top["B"], canon(top2, comps)))
    return out


def cell_kill_moves(t, cap=2):
    """CELL_KILL: top: K -> K (2*R | S)^c (0.8);  top: (R $x|$X)^c -> $x (0.4 per R);
    c: . -> S (0.6, only inside an existing c);  top: (. $x | S $X)^c -> . (0.3 per S);
    top: R -> . (0.5)."""
    top, comps = uncanon(t)
    out = []
    if top["K"]:
        if len(comps) < cap:
            out.append((0.8 * top["K"], canon(top, comps + [("c", Counter(R=2), Counter(S=1))])))
        else:
            out.append((0.8 * top["K"], FULL))
    for i, (l, w, c) in enumerate(comps):
        rest = comps[:i] + comps[i + 1:]
        if w["R"]:
            w2 = Counter(w)
            w2["R"] -= 1
            out.append((0.4 * w["R"], canon(top + w2, rest)))   # wrap rest released, content gone
        c2 = Counter(c)
        c2["S"] += 1
        out.append((0.6, canon(top, comps[:i] + [(l, w, c2)] + comps[i + 1:])))
        if c["S"]:
            out.append((0.3 * c["S"], canon(top, rest)))         # everything removed
    if top["R"]:
        top2 = Counter(top)
        top2["R"] -= 1
        out.append((0.5 * top["R"], canon(top2, comps)))
    return out


def bounded(t, limit):
    if t == FULL:
        return True
    top, comps = t
    return all(v <= limit for _, v in top) and all(v <= limit for _, w, c in comps for _, v in w + c)


def term_cme(x0, moves, limit, times):
    """Distribution over terms at `times` (states beyond `limit` molecules are truncated: the
    probability lost there is returned and must be negligible)."""
    idx, states, frontier = {x0: 0}, [x0], [x0]
    trans = []
    while frontier:
        nxt = []
        for s in frontier:
            if s == FULL:
                continue
            for rate, t in moves(s):
                if not bounded(t, limit):
                    trans.append((idx[s], -1, rate))
                    continue
                if t not in idx:
                    idx[t] = len(states)
                    states.append(t)
                    nxt.append(t)
                trans.append((idx[s], idx[t], rate))
        frontier = nxt
    n = len(states)
    Q = np.zeros((n, n))
    for a, b, r in trans:
        Q[a, a] -= r
        if b >= 0:
            Q[a, b] += r
    p0 = np.zeros(n)
    p0[0] = 1.0
    return states, [p0 @ scipy.linalg.expm(Q * t) for t in times]


# ---------------------------------------------------------------- flat model side
def flat_moves(fm):
    """Transitions of the flat network (R1 propensities x R20 gate; delta, then placement into
    the first free slot, then transfers) on flat states."""
    def moves(x):
        out = []
        for j, rate in enumerate(fm.rates):
            h = 1
            for s, r in fm.reactants[j]:
                h *= math.comb(x[s], r) if x[s] >= r else 0
            g = fm.gate_species[j]
            if g >= 0 and (x[g] < 1 if fm.gate_kind[j] == GATE_POSITIVE else x[g] != 0):
                h = 0
            if h == 0 or rate == 0:
                continue
            y = [a + d for a, d in zip(x, fm.delta[j])]
            for alive, adds in fm.place[j]:
                if y[alive] == 0:
                    for s, n in adds:
                        y[s] += n
                    break
            for src, dst in fm.transfer[j]:
                if dst >= 0:
                    y[dst] += y[src]
                y[src] = 0
            out.append((rate * h, tuple(y)))
        return out
    return moves


def lump(fm, x, label_of_slot):
    """Flat state -> canonical term (or FULL)."""
    if fm.sentinel >= 0 and x[fm.sentinel] > 0:
        return FULL
    top = Counter()
    slots = {}
    for s, name in enumerate(fm.names):
        if name.startswith("#") or x[s] == 0 and "@" not in name:
            continue
        if "@" not in name:
            top[name] += x[s]
            continue
        atom, where = name.split("@", 1)
        slot = where.split(".")[0]
        ent = slots.setdefault(slot, [Counter(), Counter()])
        ent[1 if not where.endswith(".wrap") else 0][atom] += x[s]
    comps = []
    for s, name in enumerate(fm.names):
        if name.startswith("#alive@") and x[s] == 1:
            slot = name.split("@", 1)[1]
            w, c = slots.get(slot, [Counter(), Counter()])
            comps.append((label_of_slot(slot), w, c))
    return canon(top, comps)


def flat_cme_lumped(fm, limit, times):
    x0 = tuple(fm.x0)
    moves = flat_moves(fm)
    ok = lambda y: all(v <= limit for s, v in enumerate(y) if not fm.names[s].startswith("#"))  # noqa: E731
    idx, states, frontier = {x0: 0}, [x0], [x0]
    trans = []
    while frontier:
        nxt = []
        for s in frontier:
            if fm.sentinel >= 0 and s[fm.sentinel] > 0:
                continue
            for rate, t in moves(s):
                if not ok(t):
                    trans.append((idx[s], -1, rate))
                    continue
                if t not in idx:
                    idx[t] = len(states)
                    states.append(t)
                    nxt.append(t)
                trans.append((idx[s], idx[t], rate))
        frontier = nxt
    n = len(states)
    Q = np.zeros((n, n))
    for a, b, r in trans:
        Q[a, a] -= r
        if b >= 0:
            Q[a, b] += r
    p0 = np.zeros(n)
    p0[0] = 1.0
    label = lambda slot: slot.split("/")[-1].split("[")[0]  # noqa: E731
    out = []
    for t in times:
        p = p0 @ scipy.linalg.expm(Q * t)
        d = Counter()
        for st, pr in zip(states, p):
            d[lump(fm, st, label)] += pr
        out.append(d)
    return out


CASES = [
    (W.VES_TINY, ves_tiny_moves, 6),
    (W.CELL_KILL, cell_kill_moves, 9),
]


@pytest.mark.parametrize("md,moves,limit", CASES, ids=[c[0].name for c in CASES])
def test_flat_pools_lump_to_term_cme(md, moves, limit):
    """Exact: the flat (pooled) CTMC lumped onto terms is the term-level CTMC (R20)."""
    fm = flatten_def(md)
    top, comps = Counter(), []
    # the initial term of both models: one atom at the top and one compartment
    for s, name in enumerate(fm.names):
        if "@" not in name and not name.startswith("#") and fm.x0[s]:
            top[name] += fm.x0[s]
    x0 = lump(fm, tuple(fm.x0), lambda slot: slot.split("[")[0])
    times = [0.3, 1.0, 2.5]
    states, pt = term_cme(x0, moves, limit, times)
    flat = flat_cme_lumped(fm, limit, times)
    for p, d in zip(pt, flat):
        term_d = {s: pr for s, pr in zip(states, p)}
        keys = set(term_d) | set(d)
        err = max(abs(term_d.get(k, 0.0) - d.get(k, 0.0)) for k in keys)
        assert err < 1e-10, err
        assert 1.0 - sum(term_d.values()) < 1e-4       # truncation negligible (same on both sides)
        assert sum(d.values()) > 1 - 1e-4
    # the full-pool state is reached with positive probability (the overflow path is exercised)
    assert flat[-1][FULL] > 1e-4


@pytest.mark.parametrize("md,moves,limit", CASES, ids=[c[0].name for c in CASES])
def test_oracle_ssa_matches_term_law(md, moves, limit):
    """Statistical: oracle SSA ensembles follow the term-level law (counts of compartments and
    of top-level atoms at the cuts; overflow fraction)."""
    fm = flatten_def(md)
    x0 = lump(fm, tuple(fm.x0), lambda slot: slot.split("[")[0])
    t_end, dt, n = 2.5, 0.5, 20000
    times = [dt * k for k in range(1, 6)]
    states, pt = term_cme(x0, moves, limit, times)
    run = oracle.simulate(fm, 0, n, t_end, dt, 0x5EED00DD, nthreads=8)
    alive = [s for s, nm in enumerate(fm.names) if nm.startswith("#alive@")]
    tops = [s for s, nm in enumerate(fm.names) if "@" not in nm and not nm.startswith("#")]
    for k, p in zip(range(1, 6), pt):
        raw = run.raw[k]                                  # [S][n]
        live = raw[0] >= 0
        n_full = int((~live).sum())
        p_full = sum(pr for s, pr in zip(states, p) if s == FULL)
        se = np.sqrt(max(p_full * (1 - p_full), 1e-12) / n)
        assert abs(n_full / n - p_full) < 4 * se + 1e-9
        ncomp = raw[alive][:, live].sum(axis=0)
        # conditional law given "not full"
        mass = {s: pr for s, pr in zip(states, p) if s != FULL}
        z = sum(mass.values())
        m1 = sum(pr * len(s[1]) for s, pr in mass.items()) / z
        m2 = sum(pr * len(s[1]) ** 2 for s, pr in mass.items()) / z
        sd = np.sqrt(max(m2 - m1 * m1, 1e-12))
        assert abs(ncomp.mean() - m1) < 4 * sd / np.sqrt(live.sum())
        for s in tops:
            atom = fm.names[s]
            v = raw[s][live]
            e1 = sum(pr * dict(st[0]).get(atom, 0) for st, pr in mass.items()) / z
            e2 = sum(pr * dict(st[0]).get(atom, 0) ** 2 for st, pr in mass.items()) / z
            sd = np.sqrt(max(e2 - e1 * e1, 1e-12))
            assert abs(v.mean() - e1) < 4 * sd / np.sqrt(live.sum()) + 1e-12, (atom, k)
    # chi^2 on the number of compartments at the last cut
    p = pt[-1]
    raw = run.raw[5]
    live = raw[0] >= 0
    ncomp = raw[alive][:, live].sum(axis=0)
    mass = Counter()
    for s, pr in zip(states, p):
        if s != FULL:
            mass[len(s[1])] += pr
    z = sum(mass.values())
    obs = Counter(ncomp.tolist())
    chi2 = sum((obs[c] - live.sum() * pr / z) ** 2 / (live.sum() * pr / z) for c, pr in mass.items() if pr / z > 1e-3)
    dof = sum(1 for pr in mass.values() if pr / z > 1e-3) - 1
    assert chi2 < dof + 6 * np.sqrt(2 * dof) + 10


def test_pool_layout_and_capacity_option():
    """Names, order and initial values of the pooled species (R20 layout)."""
    fm = flatten_def(W.VES_TINY)
    assert fm.names == ["A", "B", "#free:v", "#full", "B@v[0]", "#alive@v[0]", "B@v[1]", "#alive@v[1]",
                        "B@v[2]", "#alive@v[2]"]
    assert fm.x0 == [1, 0, 2, 0, 1, 1, 0, 0, 0, 0]
    assert fm.sentinel == 3 and fm.flag == [n.startswith("#alive") for n in fm.names]
    # creation: gated on a free slot, placed into the first free slot; pool full -> "#full"
    assert (fm.gate_species[0], fm.gate_kind[0]) == (2, GATE_POSITIVE)
    assert fm.place[0] == [(5, [(4, 1), (5, 1)]), (7, [(6, 1), (7, 1)]), (9, [(8, 1), (9, 1)])]
    assert {s: d for s, d in enumerate(fm.delta[1]) if d} == {3: 1} and fm.gate_kind[1] == 2
    # dissolution of slot 1: frees it, moves B@v[1] to the top
    j = [j for j in range(len(fm.rates)) if fm.rule_of[j] == 2][1]
    assert fm.transfer[j] == [(6, 1)]
    assert {s: d for s, d in enumerate(fm.delta[j]) if d} == {2: 1, 7: -1}
