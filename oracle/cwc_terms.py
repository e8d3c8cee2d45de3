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

    def seq(self, stop, nested: bool):
        """atoms / n*A / '.' / vars / (compartments if nested) until a stop symbol."""
        atoms: Counter = Counter()
        comps = []
        var = None
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
    for side in (ltxt, rtxt):
        p = _Parser(side, alphabet, allow_vars=True)
        atoms, comps, var = p.seq((), nested=True)
        if p.peek()[0] != "eof":
            raise CWCError("parse", f"trailing input in {side!r}")
        if var is not None:
            raise CWCError("unsupported", f"variable at rule level: {text!r}")
        sides.append(Pattern(atoms, comps))
    lhs, rhs = sides
    # static structure: rhs compartments correspond to lhs compartments one to one, in order,
    # with the same label and the same (present) variables (reading R15/R16).
    if len(lhs.comps) != len(rhs.comps):
        raise CWCError("unsupported", f"compartment creation/destruction: {text!r}")
    seen = set()
    for a, b in zip(lhs.comps, rhs.comps):
        if a.label != b.label:
            raise CWCError("unsupported", f"relabelling a compartment: {text!r}")
        if a.wrap_var is None or a.content_var is None:
            raise CWCError("unsupported", f"pattern compartment without $wrap/$content variables: {text!r}")
        if (a.wrap_var, a.content_var) != (b.wrap_var, b.content_var):
            raise CWCError("unsupported", f"variables moved between compartments: {text!r}")
        for v in (a.wrap_var, a.content_var):
            if v in seen:
                raise CWCError("unsupported", f"variable {v} used twice: {text!r}")
            seen.add(v)
    return Rule(label, lhs, rhs, float(rate), *law)


# ------------------------------------------------------------------------------------------
# Regions and flattening
# ------------------------------------------------------------------------------------------

@dataclass
class Region:
    name: str            # "" for top content, "cell", "cell.wrap", "cell/nuc", ...
    owner_label: str     # label of the compartment owning the region ("top" for top)
    is_wrap: bool
    atoms: Counter       # initial multiset
    children: List[int]  # indices (into regions) of the *content* regions of child compartments
    child_wraps: List[int]


def regions_of(term: Term) -> List[Region]:
    """Pre-order list of regions: top content, then for each compartment (in order of
    appearance, depth first) its wrap region and its content region."""
    regions: List[Region] = []

    def visit_content(t: Term, name: str, label: str) -> int:
        idx = len(regions)
        regions.append(Region(name, label, False, Counter(t.atoms), [], []))
        counts = Counter(c.label for c in t.comps)
        seen: Counter = Counter()
        for c in t.comps:
            seg = c.label if counts[c.label] == 1 else f"{c.label}#{seen[c.label]}"
            seen[c.label] += 1
            path = seg if name == "" else f"{name}/{seg}"
            widx = len(regions)
            regions.append(Region(path + ".wrap", c.label, True, Counter(c.wrap), [], []))
            cidx = visit_content(c.content, path, c.label)
            regions[idx].children.append(cidx)
            regions[idx].child_wraps.append(widx)
        return idx

    visit_content(term, "", "top")
    return regions


@dataclass
class FlatModel:
    """The oracle's flat network. Species = (region, atom); reactions in canonical order."""

    species: List[Tuple[int, str]]       # (region index, atom)
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


def flatten(alphabet: Sequence[str], rules: Sequence[str], rates: Sequence[float],
            initial_term: str, x_cap: Optional[int] = None) -> FlatModel:
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
    regions = regions_of(term)

    # --- tree matching: enumerate (rule, context, assignment) in canonical order -----------
    raw_reactions = []  # (rule index, rate, reactants {(region, atom): order}, delta {(region, atom): n})
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
                for atom, n in rule.lhs.atoms.items():
                    react[(ci, atom)] += n
                for atom, n in rule.rhs.atoms.items():
                    prod[(ci, atom)] += n
                for a, pc, qc in zip(assign, rule.lhs.comps, rule.rhs.comps):
                    wi, cci = ctx.child_wraps[a], ctx.children[a]
                    for atom, n in pc.wrap.items():
                        react[(wi, atom)] += n
                    for atom, n in pc.content.items():
                        react[(cci, atom)] += n
                    for atom, n in qc.wrap.items():
                        prod[(wi, atom)] += n
                    for atom, n in qc.content.items():
                        prod[(cci, atom)] += n
                if sum(react.values()) > 3:
                    raise CWCError("unsupported", f"reaction order > 3 in rule {ri}")
                delta = Counter(prod)
                delta.subtract(react)
                raw_reactions.append((ri, rule.rate, react, delta, ci))

    # --- species: referenced (region, atom) pairs, region pre-order then alphabet order -----
    used = set()
    for ri_, reg in enumerate(regions):
        for atom, n in reg.atoms.items():
            if n > 0:
                used.add((ri_, atom))
    for ri, _, react, delta, ci in raw_reactions:
        used.update(react.keys())
        used.update(key for key, v in delta.items())
        if parsed[ri].law != LAW_MASS_ACTION:
            used.add((ci, parsed[ri].law_atom))
    aidx = {a: i for i, a in enumerate(alphabet)}
    species = sorted(used, key=lambda ra: (ra[0], aidx[ra[1]]))
    sidx = {sp: i for i, sp in enumerate(species)}
    S = len(species)
    if S == 0:
        raise CWCError("invalid", "model has no species")
    names = [_species_name(regions[r], a) for r, a in species]
    x0 = [regions[r].atoms.get(a, 0) for r, a in species]

    reactants, deltas, rates_f, rule_of = [], [], [], []
    law, law_sp, law_K, law_n = [], [], [], []
    for ri, rate, react, delta, ci in raw_reactions:
        rl = parsed[ri]
        law.append(rl.law)
        law_sp.append(sidx[(ci, rl.law_atom)] if rl.law != LAW_MASS_ACTION else -1)
        law_K.append(rl.law_K)
        law_n.append(rl.law_n)
        reactants.append(sorted((sidx[sp], n) for sp, n in react.items() if n > 0))
        d = [0] * S
        for sp, n in delta.items():
            d[sidx[sp]] += n
        deltas.append(d)
        rates_f.append(rate)
        rule_of.append(ri)

    cap_max = max_safe_cap(reactants)
    if x_cap is None:
        x_cap = cap_max
    elif not (1 <= x_cap <= cap_max):
        raise CWCError("invalid", f"x_cap {x_cap} outside [1, {cap_max}]")
    if any(v > x_cap for v in x0):
        raise CWCError("invalid", "initial count above x_cap")
    return FlatModel(species, names, x0, rates_f, reactants, deltas, rule_of, x_cap, law, law_sp, law_K, law_n)


def flatten_def(model) -> FlatModel:
    """Flatten a workloads.ModelDef."""
    return flatten(model.species, model.rules, model.rates, model.initial_term, model.x_cap)
