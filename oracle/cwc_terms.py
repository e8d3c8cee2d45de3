"""ORACLE (test infrastructure only) — CWC terms, patterns and their tree matching.

Plain-Python reading of the Calculus of Wrapped Compartments as PAPER.md states it
(§IV): terms are multisets of atoms and compartments; a compartment is a
membrane (wrap) multiset plus a content term plus a label; rewrite rules are local to a
compartment label (or the top level) and may involve nested compartments.  The oracle
enumerates every occurrence ("tree matching") of every rule in the initial
term; because the structure is static (no compartment is created or destroyed — reading
R15/R16 in DESIGN.md) the set of match sites never changes, so each (rule, context,
assignment) is one flat reaction of a mass-action network.

This module shares no code with the product's C++ rule compiler
(paper_conf_icdcsw_aldinuccidpmtt14_b200/csrc/compiler.cpp); both implement the
DESIGN.md §3 "input syntax" and "flattening" readings independently.

Pins: tests/test_oracle_cwc.py checks the flattening of App. B model E and of a
two-compartment model against tables flattened by hand, and the transport model
against its Binomial closed form.
"""
from __future__ import annotations

import itertools
import math
import re
from collections import Counter
from dataclasses import dataclass, field
from typing import Dict, List, Optional, Sequence, Tuple


class CWCError(ValueError):
    """Raised for invalid / unparsable / unsupported model input."""

    def __init__(self, kind: str, msg: str):
        super().__init__(f"{kind}: {msg}")
        self.kind = kind  # "invalid" | "parse" | "unsupported"


# ------------------------------------------------------------------------------------------
# Terms (initial state) and patterns (rule sides)
# ------------------------------------------------------------------------------------------

@dataclass
class Compartment:
    label: str
    wrap: Counter
    content: "Term"


@dataclass
class Term:
    atoms: Counter = field(default_factory=Counter)
    comps: List[Compartment] = field(default_factory=list)


@dataclass
class PatComp:
    label: str
    wrap: Counter
    wrap_var: Optional[str]
    content: Counter
    content_var: Optional[str]


@dataclass
class Pattern:
    atoms: Counter
    comps: List[PatComp]


_TOKEN = re.compile(r"\s*(?:(->)|(\d+)\s*\*|(\$[A-Za-z_][A-Za-z0-9_]*)|([A-Za-z_][A-Za-z0-9_]*)|(\S))")


def _tokens(text: str) -> List[Tuple[str, str]]:
    out = []
    pos = 0
    text = text.strip()
    while pos < len(text):
        m = _TOKEN.match(text, pos)
        if not m or m.end() == pos:
            break
        pos = m.end()
        if m.group(1):
            out.append(("arrow", "->"))
        elif m.group(2):
            out.append(("mult", m.group(2)))
        elif m.group(3):
            out.append(("var", m.group(3)))
        elif m.group(4):
            out.append(("name", m.group(4)))
        else:
            out.append(("sym", m.group(5)))
    return out


class _Parser:
    def __init__(self, text: str, alphabet: Sequence[str], allow_vars: bool):
        self.toks = _tokens(text)
        self.i = 0
        self.alphabet = set(alphabet)
        self.allow_vars = allow_vars
        self.text = text

    def peek(self):
        return self.toks[self.i] if self.i < len(self.toks) else ("eof", "")

    def take(self):
        t = self.peek()
        self.i += 1
        return t

    def expect(self, kind, val=None):
        t = self.take()
        if t[0] != kind or (val is not None and t[1] != val):
            raise CWCError("parse", f"expected {val or kind} in {self.text!r}, got {t[1]!r}")
        return t

    def atom(self, name):
        if name not in self.alphabet:
            raise CWCError("invalid", f"unknown atom {name!r}")
        return name

    def seq(self, stop, nested: bool, multi_var: bool = False):
        """atoms / n*A / '.' / vars / (compartments if nested) until a stop symbol.  With
        multi_var (a rule's right-hand side at rule level) the variables come back as a list."""
        atoms: Counter = Counter()
        comps = []
        var = [] if multi_var else None
        while True:
            kind, val = self.peek()
            if kind == "eof" or (kind == "sym" and val in stop) or kind == "arrow":
                break
            self.take()
            if kind == "sym" and val == ".":
                continue
            if kind == "mult":
                n = int(val)
                _, name = self.expect("name")
                atoms[self.atom(name)] += n
            elif kind == "name":
                atoms[self.atom(val)] += 1
            elif kind == "var":
                if not self.allow_vars:
                    raise CWCError("parse", f"variable {val} in a term")
                if multi_var:
                    if val in var:
                        raise CWCError("unsupported", f"variable {val} released twice: {self.text!r}")
                    var.append(val)
                    continue
                if var is not None:
                    raise CWCError("unsupported", f"two variables in one multiset: {self.text!r}")
                var = val
            elif kind == "sym" and val == "(":
                if not nested:
                    raise CWCError("unsupported", f"nested compartment in a pattern compartment: {self.text!r}")
                comps.append(self.compartment())
            else:
                raise CWCError("parse", f"unexpected {val!r} in {self.text!r}")
        return atoms, comps, var

    def compartment(self):
        wrap, wcomps, wvar = self.seq(("|",), nested=False)
        if wcomps:
            raise CWCError("parse", "compartment inside a membrane")
        self.expect("sym", "|")
        if self.allow_vars:
            content, ccomps, cvar = self.seq((")",), nested=False)
        else:
            content, ccomps, cvar = self.seq((")",), nested=True)
        self.expect("sym", ")")
        self.expect("sym", "^")
        _, label = self.expect("name")
        if label == "top":
            raise CWCError("invalid", "'top' is reserved for the outermost level")
        if self.allow_vars:
            return PatComp(label, wrap, wvar, content, cvar)
        return Compartment(label, wrap, Term(content, ccomps))


def parse_term(text: str, alphabet: Sequence[str]) -> Term:
    p = _Parser(text, alphabet, allow_vars=False)
    atoms, comps, _ = p.seq((), nested=True)
    if p.peek()[0] != "eof":
        raise CWCError("parse", f"trailing input in term {text!r}")
    return Term(atoms, comps)


LAW_MASS_ACTION, LAW_MM, LAW_HILL, LAW_HILLR = 0, 1, 2, 3
_LAWS = {"mm": LAW_MM, "hill": LAW_HILL, "hillr": LAW_HILLR}


@dataclass
class Rule:
    label: str
    lhs: Pattern
    rhs: Pattern
    rate: float
    law: int = LAW_MASS_ACTION   # reading R16': functional rate laws
    law_atom: Optional[str] = None
    law_K: float = 0.0
    law_n: int = 1
    # reading R20 (dynamic compartments): for every lhs pattern compartment, the index of the
    # rhs compartment it persists as, or None when the rule destroys it; the rhs compartment
    # the rule creates (ground, at most one) or None; the rule-level variables the rhs releases
    keep: List[Optional[int]] = field(default_factory=list)
    create: Optional[int] = None
    release: List[str] = field(default_factory=list)


def parse_law(text: str, alphabet: Sequence[str]):
    """'mm(X, K)' | 'hill(X, K, n)' | 'hillr(X, K, n)' -> (law, atom, K, n)."""
    m = re.fullmatch(r"\s*(mm|hill|hillr)\s*\(\s*([A-Za-z_][A-Za-z0-9_]*)\s*,\s*([^,()]+?)\s*(?:,\s*([0-9]+)\s*)?\)\s*",
                     text)
    if not m:
        raise CWCError("parse", f"bad rate law {text!r}")
    law = _LAWS[m.group(1)]
    atom = m.group(2)
    if atom not in alphabet:
        raise CWCError("invalid", f"unknown atom {atom!r} in rate law")
    try:
        K = float(m.group(3))
    except ValueError:
        raise CWCError("parse", f"bad constant in rate law {text!r}")
    if not math.isfinite(K) or K <= 0:
        raise CWCError("invalid", f"rate-law constant must be finite and > 0: {text!r}")
    if law == LAW_MM:
        if m.group(4) is not None:
            raise CWCError("parse", f"mm takes (species, K): {text!r}")
        n = 1
    else:
        if m.group(4) is None:
            raise CWCError("parse", f"{m.group(1)} takes (species, K, n): {text!r}")
        n = int(m.group(4))
        if not 1 <= n <= 8:
            raise CWCError("invalid", f"Hill exponent must be in [1, 8]: {text!r}")
    return law, atom, K, n


def parse_rule(text: str, alphabet: Sequence[str], rate: float) -> Rule:
    if not isinstance(rate, (int, float)) or not math.isfinite(rate) or rate < 0:
        raise CWCError("invalid", f"rate {rate!r} of rule {text!r}")
    if ":" not in text:
        raise CWCError("parse", f"rule without label: {text!r}")
    label, body = text.split(":", 1)
    label = label.strip()
    law = (LAW_MASS_ACTION, None, 0.0, 1)
    if "@" in body:
        body, law_txt = body.split("@", 1)
        law = parse_law(law_txt, alphabet)
    if not re.fullmatch(r"[A-Za-z_][A-Za-z0-9_]*", label):
        raise CWCError("parse", f"bad rule label {label!r}")
    if body.count("->") != 1:
        raise CWCError("parse", f"rule must contain exactly one '->': {text!r}")
    ltxt, rtxt = body.split("->")
    sides = []
    release: List[str] = []
    for k, side in enumerate((ltxt, rtxt)):
        p = _Parser(side, alphabet, allow_vars=True)
        atoms, comps, var = p.seq((), nested=True, multi_var=(k == 1))
        if p.peek()[0] != "eof":
            raise CWCError("parse", f"trailing input in {side!r}")
        if k == 0 and var is not None:
            raise CWCError("unsupported", f"variable at rule level: {text!r}")
        if k == 1:
            release = var
        sides.append(Pattern(atoms, comps))
    lhs, rhs = sides
    # Structure (readings R15, R20): an rhs compartment with the variables of an lhs pattern
    # compartment is that compartment (same label); an rhs compartment without variables is
    # created (at most one per rule); an lhs compartment that does not reappear is destroyed,
    # and its variables may be released at rule level on the rhs.
    seen = set()
    for a in lhs.comps:
        if a.wrap_var is None or a.content_var is None:
            raise CWCError("unsupported", f"pattern compartment without $wrap/$content variables: {text!r}")
        for v in (a.wrap_var, a.content_var):
            if v in seen:
                raise CWCError("unsupported", f"variable {v} used twice: {text!r}")
            seen.add(v)
    keep: List[Optional[int]] = [None] * len(lhs.comps)
    create = None
    for bi, b in enumerate(rhs.comps):
        if b.wrap_var is None and b.content_var is None:
            if create is not None:
                raise CWCError("unsupported", f"more than one compartment created: {text!r}")
            create = bi
            continue
        match = [ai for ai, a in enumerate(lhs.comps) if (a.wrap_var, a.content_var) == (b.wrap_var, b.content_var)]
        if not match or keep[match[0]] is not None:
            raise CWCError("unsupported", f"variables moved between compartments: {text!r}")
        if lhs.comps[match[0]].label != b.label:
            raise CWCError("unsupported", f"relabelling a compartment: {text!r}")
        keep[match[0]] = bi
    gone = {v for a, kp in zip(lhs.comps, keep) if kp is None for v in (a.wrap_var, a.content_var)}
    for v in release:
        if v not in gone:
            raise CWCError("unsupported", f"variable {v} released but its compartment is not destroyed: {text!r}")
    return Rule(label, lhs, rhs, float(rate), *law, keep=keep, create=create, release=list(release))


# ------------------------------------------------------------------------------------------
# Regions and flattening
# ------------------------------------------------------------------------------------------

DEFAULT_CAPACITY = 8  # slots per dynamic-compartment pool (reading R20)


@dataclass
class Region:
    name: str            # "" for top content, "cell", "cell.wrap", "cell/nuc", "ves[2]", ...
    owner_label: str     # label of the compartment owning the region ("top" for top)
    is_wrap: bool
    atoms: Counter       # initial multiset
    children: List[int]  # indices (into regions) of the *content* regions of child compartments
    child_wraps: List[int]
    slot: Optional[Tuple[int, int]] = None  # (pool, slot) for the regions of a pool slot


@dataclass
class Pool:
    """Reading R20: the C_l slots for the dynamic compartments of label l in one region."""
    parent: int
    label: str
    slots: List[Tuple[int, int]]   # (wrap region, content region) per slot
    occupied: int                  # slots filled by the initial term (0 .. occupied-1)


def regions_of(term: Term, dynamic=frozenset(), creators=frozenset(), capacity=None):
    """Pre-order list of regions: top content, then for each static compartment (in order of
    appearance, depth first) its wrap region and its content region, then the pools of
    dynamic compartments of the region (label order; slot by slot: wrap, content).  Returns
    (regions, pools); creators = {(context label, created label)} of the rules."""
    capacity = capacity or {}
    regions: List[Region] = []
    pools: List[Pool] = []

    def visit_content(t: Term, name: str, label: str) -> int:
        idx = len(regions)
        regions.append(Region(name, label, False, Counter(t.atoms), [], []))
        static = [c for c in t.comps if c.label not in dynamic]
        counts = Counter(c.label for c in static)
        seen: Counter = Counter()
        for c in static:
            seg = c.label if counts[c.label] == 1 else f"{c.label}#{seen[c.label]}"
            seen[c.label] += 1
            path = seg if name == "" else f"{name}/{seg}"
            widx = len(regions)
            regions.append(Region(path + ".wrap", c.label, True, Counter(c.wrap), [], []))
            cidx = visit_content(c.content, path, c.label)
            regions[idx].children.append(cidx)
            regions[idx].child_wraps.append(widx)
        dyn_init = [c for c in t.comps if c.label in dynamic]
        for c in dyn_init:
            if c.content.comps:
                raise CWCError("unsupported", f"dynamic compartment {c.label!r} with nested compartments")
        labels = sorted({c.label for c in dyn_init} | {l for (ctx, l) in creators if ctx == label})
        for l in labels:
            init = [c for c in dyn_init if c.label == l]
            cap = int(capacity.get(l, DEFAULT_CAPACITY))
            if cap < 1 or len(init) > cap:
                raise CWCError("invalid", f"capacity of {l!r} must be >= 1 and hold the initial compartments")
            pool = Pool(idx, l, [], len(init))
            pid = len(pools)
            pools.append(pool)
            for k in range(cap):
                path = f"{l}[{k}]" if name == "" else f"{name}/{l}[{k}]"
                w = Counter(init[k].wrap) if k < len(init) else Counter()
                ct = Counter(init[k].content.atoms) if k < len(init) else Counter()
                widx = len(regions)
                regions.append(Region(path + ".wrap", l, True, w, [], [], (pid, k)))
                cidx = len(regions)
                regions.append(Region(path, l, False, ct, [], [], (pid, k)))
                regions[idx].children.append(cidx)
                regions[idx].child_wraps.append(widx)
                pool.slots.append((widx, cidx))
        return idx

    visit_content(term, "", "top")
    return regions, pools


@dataclass
class FlatModel:
    """The oracle's flat network. Species = (region, atom); reactions in canonical order."""

    species: List[Tuple[int, str]]       # (region index, atom or flag pseudo-atom)
    names: List[str]
    x0: List[int]
    rates: List[float]
    reactants: List[List[Tuple[int, int]]]   # per reaction: [(species, order)], species ascending
    delta: List[List[int]]                   # per reaction: dense net change [S]
    rule_of: List[int]                       # originating CWC rule index
    x_cap: int
    law: List[int] = field(default_factory=list)          # per reaction: LAW_* (R16')
    law_species: List[int] = field(default_factory=list)  # species the law reads (-1: none)
    law_K: List[float] = field(default_factory=list)
    law_n: List[int] = field(default_factory=list)
    # reading R20 (dynamic compartments)
    gate_species: List[int] = field(default_factory=list)  # per reaction: -1 or the gating species
    gate_kind: List[int] = field(default_factory=list)     # GATE_POSITIVE: x >= 1, GATE_ZERO: x == 0
    place: List[List[Tuple[int, List[Tuple[int, int]]]]] = field(default_factory=list)
    #   per reaction: candidate slots in order, (alive species, [(species, added count)]); the
    #   first slot whose alive species is 0 receives its additions (a creation)
    transfer: List[List[Tuple[int, int]]] = field(default_factory=list)
    #   per reaction: (src, dst) applied after delta: x[dst] += x[src] (dst >= 0), x[src] = 0
    sentinel: int = -1                   # species "#full": > 0 means a pool overflowed (R9, R20)
    flag: List[bool] = field(default_factory=list)  # per species: a 0/1 slot-occupancy flag


GATE_NONE, GATE_POSITIVE, GATE_ZERO = 0, 1, 2


def _species_name(region: Region, atom: str) -> str:
    return atom if region.name == "" else f"{atom}@{region.name}"


def max_safe_cap(reactant_lists: Sequence[Sequence[Tuple[int, int]]], limit: int = 1 << 30) -> int:
    """Largest cap <= limit with prod_s C(cap, r_s) < 2^53 for every reaction (reading R9:
    every propensity count h_j is then exact in a double)."""
    def ok(cap: int) -> bool:
        for rl in reactant_lists:
            h = 1
            for _, r in rl:
                h *= math.comb(cap, r)
            if h >= (1 << 53):
                return False
        return True

    lo, hi = 1, limit
    if ok(hi):
        return hi
    while lo < hi:
        mid = (lo + hi + 1) // 2
        if ok(mid):
            lo = mid
        else:
            hi = mid - 1
    return lo


ALIVE, FULL = "#alive", "#full"


def _free(label: str) -> str:
    return "#free:" + label


def flatten(alphabet: Sequence[str], rules: Sequence[str], rates: Sequence[float],
            initial_term: str, x_cap: Optional[int] = None, capacity=None) -> FlatModel:
    alphabet = list(alphabet)
    if len(set(alphabet)) != len(alphabet) or not alphabet:
        raise CWCError("invalid", "alphabet must be non-empty and without duplicates")
    for a in alphabet:
        if not re.fullmatch(r"[A-Za-z_][A-Za-z0-9_]*", a) or a == "top":
            raise CWCError("invalid", f"bad atom name {a!r}")
    if len(rules) != len(rates):
        raise CWCError("invalid", "one rate per rule")
    term = parse_term(initial_term, alphabet)
    parsed = [parse_rule(r, alphabet, k) for r, k in zip(rules, rates)]
    # reading R20: a label is dynamic when some rule creates or destroys a compartment of it
    dynamic = set()
    creators = set()
    for rule in parsed:
        if rule.create is not None:
            dynamic.add(rule.rhs.comps[rule.create].label)
            creators.add((rule.label, rule.rhs.comps[rule.create].label))
        for a, kp in zip(rule.lhs.comps, rule.keep):
            if kp is None:
                dynamic.add(a.label)
    for ctx, l in creators:
        if ctx in dynamic:
            raise CWCError("unsupported", f"compartment {l!r} created inside dynamic compartment {ctx!r}")
    regions, pools = regions_of(term, frozenset(dynamic), frozenset(creators), capacity)
    pool_of = {(pl.parent, pl.label): i for i, pl in enumerate(pools)}

    def alive(ri: int):
        pid, k = regions[ri].slot
        return (pools[pid].slots[k][1], ALIVE)

    # --- tree matching: enumerate (rule, context, assignment) in canonical order -----------
    raw_reactions = []  # dicts: rule, rate, react, delta, ctx, gate, place, destroyed
    for ri, rule in enumerate(parsed):
        for ci, ctx in enumerate(regions):
            if ctx.is_wrap or ctx.owner_label != rule.label:
                continue
            m = len(rule.lhs.comps)
            for assign in itertools.permutations(range(len(ctx.children)), m):
                if any(regions[ctx.children[a]].owner_label != pc.label
                       for a, pc in zip(assign, rule.lhs.comps)):
                    continue
                react: Counter = Counter()
                prod: Counter = Counter()
                destroyed = []  # (wrap region, content region, release wrap, release content)
                for atom, n in rule.lhs.atoms.items():
                    react[(ci, atom)] += n
                for atom, n in rule.rhs.atoms.items():
                    prod[(ci, atom)] += n
                if ctx.slot is not None:          # inside a pool slot: only while it is occupied
                    react[alive(ci)] += 1
                    prod[alive(ci)] += 1
                for a, pc, kp in zip(assign, rule.lhs.comps, rule.keep):
                    wi, cci = ctx.child_wraps[a], ctx.children[a]
                    for atom, n in pc.wrap.items():
                        react[(wi, atom)] += n
                    for atom, n in pc.content.items():
                        react[(cci, atom)] += n
                    if regions[cci].slot is not None:
                        react[alive(cci)] += 1
                    if kp is not None:
                        qc = rule.rhs.comps[kp]
                        for atom, n in qc.wrap.items():
                            prod[(wi, atom)] += n
                        for atom, n in qc.content.items():
                            prod[(cci, atom)] += n
                        if regions[cci].slot is not None:
                            prod[alive(cci)] += 1
                    else:                          # destroyed (R20): the slot is freed
                        pid = regions[cci].slot[0]
                        prod[(pools[pid].parent, _free(pools[pid].label))] += 1
                        destroyed.append((wi, cci, pc.wrap_var in rule.release, pc.content_var in rule.release))
                if sum(n for (r_, at), n in react.items() if at != ALIVE) > 3:
                    raise CWCError("unsupported", f"reaction order > 3 in rule {ri}")
                delta = Counter(prod)
                delta.subtract(react)
                base = dict(rule=ri, rate=rule.rate, react=react, delta=delta, ctx=ci, gate=None, place=None,
                            destroyed=destroyed)
                if rule.create is None:
                    raw_reactions.append(base)
                    continue
                # creation (R20): into the lowest free slot of the pool, else the pool is full
                qc = rule.rhs.comps[rule.create]
                pid = pool_of[(ci, qc.label)]
                fkey = (ci, _free(qc.label))
                place = []
                for wi, cci in pools[pid].slots:
                    adds = Counter({(cci, ALIVE): 1})
                    for atom, n in qc.wrap.items():
                        adds[(wi, atom)] += n
                    for atom, n in qc.content.items():
                        adds[(cci, atom)] += n
                    place.append(((cci, ALIVE), adds))
                d_place = Counter(delta)
                d_place[fkey] -= 1
                raw_reactions.append(dict(base, delta=d_place, gate=(fkey, GATE_POSITIVE), place=place))
                raw_reactions.append(dict(base, react=Counter(react), delta=Counter({(0, FULL): 1}),
                                          gate=(fkey, GATE_ZERO), place=None, destroyed=[]))

    # --- species: referenced (region, atom) pairs, region pre-order then alphabet order, then
    # the flags of the region: "#alive" (a slot's content region), "#free:<label>" (pool
    # parent, label order), "#full" (top) --------------------------------------------------
    used = set()
    for ri_, reg in enumerate(regions):
        for atom, n in reg.atoms.items():
            if n > 0:
                used.add((ri_, atom))
    for pl in pools:
        used.add((pl.parent, _free(pl.label)))
        for wi, cci in pl.slots:
            used.add((cci, ALIVE))
    has_full = any(r["gate"] is not None and r["gate"][1] == GATE_ZERO for r in raw_reactions)
    if has_full:
        used.add((0, FULL))
    for r in raw_reactions:
        used.update(r["react"].keys())
        used.update(r["delta"].keys())
        if r["gate"] is not None:
            used.add(r["gate"][0])
        for _, adds in r["place"] or []:
            used.update(adds.keys())
        if parsed[r["rule"]].law != LAW_MASS_ACTION:
            used.add((r["ctx"], parsed[r["rule"]].law_atom))
    # transfers of destroyed compartments: every atom species of the slot's regions
    for r in raw_reactions:
        xfer = []
        for wi, cci, rel_w, rel_c in r["destroyed"]:
            for reg, rel in ((wi, rel_w), (cci, rel_c)):
                for (sr, atom) in sorted(k for k in used if k[0] == reg and k[1] in alphabet):
                    dst = (r["ctx"], atom) if rel else None
                    xfer.append(((sr, atom), dst))
                    if dst is not None:
                        used.add(dst)
        r["xfer"] = xfer
    aidx = {a: i for i, a in enumerate(alphabet)}

    def order(ra):
        reg, atom = ra
        if atom in aidx:
            return (reg, 0, aidx[atom], "")
        if atom == ALIVE:
            return (reg, 1, 0, "")
        if atom.startswith("#free:"):
            return (reg, 2, 0, atom)
        return (reg, 3, 0, "")

    species = sorted(used, key=order)
    sidx = {sp: i for i, sp in enumerate(species)}
    S = len(species)
    if S == 0:
        raise CWCError("invalid", "model has no species")
    names = [_species_name(regions[r], a) for r, a in species]
    x0 = []
    for r, a in species:
        if a == ALIVE:
            pid, k = regions[r].slot
            x0.append(1 if k < pools[pid].occupied else 0)
        elif a.startswith("#free:"):
            pl = pools[pool_of[(r, a[6:])]]
            x0.append(len(pl.slots) - pl.occupied)
        elif a == FULL:
            x0.append(0)
        else:
            x0.append(regions[r].atoms.get(a, 0))
    flag = [a == ALIVE for _, a in species]

    reactants, deltas, rates_f, rule_of = [], [], [], []
    law, law_sp, law_K, law_n = [], [], [], []
    gate_s, gate_k, place_l, xfer_l = [], [], [], []
    for r in raw_reactions:
        rl = parsed[r["rule"]]
        law.append(rl.law)
        law_sp.append(sidx[(r["ctx"], rl.law_atom)] if rl.law != LAW_MASS_ACTION else -1)
        law_K.append(rl.law_K)
        law_n.append(rl.law_n)
        reactants.append(sorted((sidx[sp], n) for sp, n in r["react"].items() if n > 0))
        d = [0] * S
        for sp, n in r["delta"].items():
            d[sidx[sp]] += n
        deltas.append(d)
        rates_f.append(r["rate"])
        rule_of.append(r["rule"])
        gate_s.append(sidx[r["gate"][0]] if r["gate"] is not None else -1)
        gate_k.append(r["gate"][1] if r["gate"] is not None else GATE_NONE)
        place_l.append([(sidx[al], sorted((sidx[sp], n) for sp, n in adds.items() if n))
                        for al, adds in (r["place"] or [])])
        xfer_l.append(sorted((sidx[src], sidx[dst] if dst is not None else -1) for src, dst in r["xfer"]))

    # flags are 0/1 and do not limit the exact propensity range (R9)
    cap_max = max_safe_cap([[(sp, n) for sp, n in rl if not flag[sp]] for rl in reactants])
    if x_cap is None:
        x_cap = cap_max
    elif not (1 <= x_cap <= cap_max):
        raise CWCError("invalid", f"x_cap {x_cap} outside [1, {cap_max}]")
    if any(v > x_cap for v in x0):
        raise CWCError("invalid", "initial count above x_cap")
    return FlatModel(species, names, x0, rates_f, reactants, deltas, rule_of, x_cap, law, law_sp, law_K, law_n,
                     gate_s, gate_k, place_l, xfer_l, sidx.get((0, FULL), -1), flag)


def flatten_def(model) -> FlatModel:
    """Flatten a workloads.ModelDef."""
    return flatten(model.species, model.rules, model.rates, model.initial_term, model.x_cap,
                   dict(getattr(model, "capacity", ()) or ()))
