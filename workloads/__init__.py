"""Synthetic workloads (inputs only) shared by the product path, the oracle and the bench.

This module holds *inputs*: CWC model definitions (alphabet, rule strings, rates,
initial term), run configurations (instances, horizon, sample grid, seed, histogram
layout) and nothing of the method's arithmetic.  It is the one module both sides may
import (task rule ③: "only the seeded input generators serve both").

The paper gives no model parameters (PAPER.md L323-327 only cites [18], [20]); the
models below are the synthetic "shaped like" workloads fixed in SURVEY.md Appendix B
(reading R17 in DESIGN.md).  Rule order is selection order (reading R6).
"""
from dataclasses import dataclass, field
from typing import Dict, List, Optional, Sequence, Tuple

DEFAULT_QUANTILES = (0.05, 0.25, 0.5, 0.75, 0.95)


@dataclass(frozen=True)
class ModelDef:
    """A CWC model as the C ABI receives it (cwc_model_load)."""

    name: str
    species: Tuple[str, ...]          # the alphabet of atoms, in order (species order within a region)
    rules: Tuple[str, ...]            # "label: lhs -> rhs" strings, selection order
    rates: Tuple[float, ...]          # one rate per rule
    initial_term: str
    x_cap: Optional[int] = None       # reading R9; None = model default (largest safe cap <= 2^30)
    capacity: Tuple[Tuple[str, int], ...] = ()  # reading R20: slots per dynamic-compartment pool


@dataclass(frozen=True)
class RunConfig:
    """One BASELINE.json config, made concrete."""

    cid: int
    model: ModelDef
    n_instances: int
    t_end: float
    sample_dt: float
    seed: int
    hist_bins: int
    hist_width: int
    hist_lo: int = 0
    quantiles: Tuple[float, ...] = DEFAULT_QUANTILES
    description: str = ""

    @property
    def n_samples(self) -> int:
        return int(round(self.t_end / self.sample_dt)) + 1


# --- App. B models -------------------------------------------------------------------

IMM_DEATH = ModelDef(
    name="imm_death",
    species=("A",),
    rules=("top: . -> A", "top: A -> ."),
    rates=(10.0, 0.1),
    initial_term=".",
)

# Gillespie 1977 Lotka reactions with X-bar folded into c1.
LOTKA_VOLTERRA = ModelDef(
    name="lotka_volterra",
    species=("Y1", "Y2"),
    rules=("top: Y1 -> Y1 Y1", "top: Y1 Y2 -> Y2 Y2", "top: Y2 -> ."),
    rates=(10.0, 0.01, 10.0),
    initial_term="1000*Y1 1000*Y2",
    x_cap=100_000,
)

SCHLOGL = ModelDef(
    name="schlogl",
    species=("X",),
    rules=("top: X X -> X X X", "top: X X X -> X X", "top: . -> X", "top: X -> ."),
    rates=(0.03, 1e-4, 200.0, 3.5),
    initial_term="250*X",
)

# Vilar, Kueh, Barkai, Leibler (PNAS 2002) genetic oscillator; DAp/DRp = DA'/DR'.
CIRCADIAN = ModelDef(
    name="circadian",
    species=("DA", "DR", "DAp", "DRp", "MA", "MR", "A", "R", "C"),
    rules=(
        "top: DAp -> DA A",
        "top: DA A -> DAp",
        "top: DRp -> DR A",
        "top: DR A -> DRp",
        "top: DAp -> DAp MA",
        "top: DA -> DA MA",
        "top: DRp -> DRp MR",
        "top: DR -> DR MR",
        "top: MA -> MA A",
        "top: MR -> MR R",
        "top: A R -> C",
        "top: C -> R",
        "top: A -> .",
        "top: R -> .",
        "top: MA -> .",
        "top: MR -> .",
    ),
    rates=(50.0, 1.0, 100.0, 1.0, 500.0, 50.0, 50.0, 0.01, 50.0, 5.0, 2.0, 1.0, 1.0, 0.2, 10.0, 0.5),
    initial_term="DA DR",
)

# Depth-2 compartments: top ⊃ cell ⊃ nuc, receptor binding on the cell membrane,
# transport across the nuclear membrane (SURVEY.md App. B model E).
COMPARTMENTS = ModelDef(
    name="compartments",
    species=("L", "R", "RL", "S", "G", "M", "P"),
    rules=(
        "top: L (R $x | $X)^cell -> (RL $x | $X)^cell",
        "top: (RL $x | $X)^cell -> L (R $x | $X)^cell",
        "top: (RL $x | $X)^cell -> (R $x | S $X)^cell",
        "cell: S ($y | $Y)^nuc -> ($y | S $Y)^nuc",
        "cell: ($y | S $Y)^nuc -> S ($y | $Y)^nuc",
        "nuc: S G -> S G M",
        "cell: ($y | M $Y)^nuc -> M ($y | $Y)^nuc",
        "cell: M -> M P",
        "cell: M -> .",
        "cell: P -> .",
        "cell: S -> .",
        "top: . -> L",
        "top: L -> .",
        "nuc: S -> .",
    ),
    rates=(0.01, 1.0, 0.5, 0.2, 0.1, 0.05, 1.0, 2.0, 0.2, 0.05, 0.1, 50.0, 0.1, 0.1),
    initial_term="500*L (100*R | (. | 2*G)^nuc)^cell",
)

MODELS: Dict[str, ModelDef] = {
    m.name: m for m in (IMM_DEATH, LOTKA_VOLTERRA, SCHLOGL, CIRCADIAN, COMPARTMENTS)
}

# --- BASELINE.json configs ------------------------------------------

SEED_BASE = 0x5EED0000

CONFIGS: Dict[str, RunConfig] = {
    "imm_death": RunConfig(1, IMM_DEATH, 1_000, 100.0, 1.0, SEED_BASE + 1, 256, 1,
                           description="immigration-death, 1,000 instances, t_end=100, dt=1"),
    "lv": RunConfig(2, LOTKA_VOLTERRA, 100_000, 50.0, 0.1, SEED_BASE + 2, 1024, 128,
                    description="Lotka-Volterra, 100k instances, t_end=50, dt=0.1"),
    # the north-star run (BASELINE.json north_star: "a 1M-instance Lotka-Volterra ensemble"): the
    # bench headline, strong-scaled over 1/2/4/8 GPUs (125k instances per GPU at 8)
    "lv1m": RunConfig(2, LOTKA_VOLTERRA, 1_000_000, 50.0, 0.1, SEED_BASE + 2, 1024, 128,
                      description="Lotka-Volterra, 1M instances (north-star ensemble), t_end=50, dt=0.1"),
    "schlogl": RunConfig(3, SCHLOGL, 1_000_000, 50.0, 0.1, SEED_BASE + 3, 1024, 1,
                         description="Schlogl bistable, 1M instances, t_end=50, dt=0.1"),
    "circadian": RunConfig(4, CIRCADIAN, 10_000_000, 48.0, 0.5, SEED_BASE + 4, 1024, 4,
                           description="Vilar circadian oscillator, 10M instances (8 GPUs), t_end=48h, dt=0.5h"),
    "compartments": RunConfig(5, COMPARTMENTS, 1_000_000, 100.0, 0.5, SEED_BASE + 5, 1024, 1,
                              description="CWC cell+nucleus (depth 2, transport), 1M instances, t_end=100, dt=0.5"),
}

# --- tiny models for closed-form / CME pins -------------------------------------------------

PURE_BIRTH = ModelDef("pure_birth", ("A",), ("top: . -> A",), (3.0,), ".")
PURE_DEATH = ModelDef("pure_death", ("A",), ("top: A -> .",), (0.5,), "40*A")
ISOMERIZATION = ModelDef("isomerization", ("A", "B"), ("top: A -> B", "top: B -> A"), (1.0, 0.5), "20*A")
BINDING = ModelDef("binding", ("A", "B", "C"), ("top: A B -> C", "top: C -> A B"), (0.3, 1.0), "5*A 5*B")
DIMERISATION = ModelDef("dimerisation", ("A", "B"), ("top: A A -> B", "top: B -> A A"), (0.2, 1.0), "10*A")
DEAD = ModelDef("dead", ("A", "B"), ("top: A -> B", "top: B -> A"), (0.0, 0.0), "7*A 3*B")
RUNAWAY = ModelDef("runaway", ("A",), ("top: A -> A A",), (1.0,), "1*A", x_cap=10)
# transport in and out of a nucleus: S@top <-> S@nuc, a Binomial law (SURVEY.md §8(c) pins)
TRANSPORT = ModelDef(
    "transport", ("S",),
    ("top: S ($y | $Y)^nuc -> ($y | S $Y)^nuc", "top: ($y | S $Y)^nuc -> S ($y | $Y)^nuc"),
    (0.7, 0.3), "30*S (. | .)^nuc",
)
# two compartments with the same label (reading R15: one flat reaction per assignment)
TWO_CELLS = ModelDef(
    "two_cells", ("A", "B"),
    ("top: A (. $x | $X)^cell -> (. $x | A $X)^cell", "cell: A -> B", "top: (. $x | B $X)^cell -> B (. $x | $X)^cell"),
    (0.05, 1.0, 0.5), "20*A (. | 3*A)^cell (2*B | .)^cell",
)

TINY_MODELS = {m.name: m for m in (PURE_BIRTH, PURE_DEATH, ISOMERIZATION, BINDING, DIMERISATION,
                                   DEAD, RUNAWAY, TRANSPORT, TWO_CELLS)}

# --- functional rate laws ------------------------------------------------------
# The paper's own workload is the Neurospora circadian model of [20] (PAPER.md P:L323-327,
# L541-543), whose kinetics are Michaelis-Menten / Hill, not mass action.  Its parameters are
# not in PAPER.md; these are the published deterministic values of Leloup, Gonze & Goldbeter
# (J. Biol. Rhythms 1999) [ext], converted to molecule numbers with a system size of 100
# molecules per nM (the usual stochastic version, Gonze et al. PNAS 2002 [ext]):
#   dM/dt  = vs KI^n/(KI^n + FN^n) - vm M/(Km + M)
#   dFC/dt = ks M - vd FC/(Kd + FC) - k1 FC + k2 FN,   dFN/dt = k1 FC - k2 FN
# vs 1.6, vm 0.505, vd 1.4 nM/h; ks 0.5, k1 0.5, k2 0.6 /h; Km 0.5, Kd 0.13, KI 1 nM; n 4.
NEUROSPORA = ModelDef(
    name="neurospora",
    species=("M", "FC", "FN"),
    rules=(
        "top: . -> M @ hillr(FN, 100, 4)",     # frq transcription, repressed by nuclear FRQ
        "top: M -> . @ mm(M, 50)",             # frq mRNA degradation
        "top: M -> M FC",                      # translation
        "top: FC -> . @ mm(FC, 13)",           # cytosolic FRQ degradation
        "top: FC -> FN",                       # nuclear import
        "top: FN -> FC",                       # nuclear export
    ),
    rates=(160.0, 50.5, 0.5, 140.0, 0.5, 0.6),
    initial_term=".",
)
MODELS[NEUROSPORA.name] = NEUROSPORA
CONFIGS["neurospora"] = RunConfig(
    6, NEUROSPORA, 1_000_000, 96.0, 0.5, SEED_BASE + 6, 1024, 1,
    description="Neurospora circadian model (Leloup-Gonze-Goldbeter, MM/Hill kinetics, 100 molecules/nM), "
                "1M instances, t_end=96h, dt=0.5h, period analysis on M")
# period analysis of the paper's experiment: oscillation events of frq mRNA
PERIOD_ANALYSIS = {"neurospora": dict(species="M", lo=100, hi=350, window=48),
                   "circadian": dict(species="R", lo=100, hi=1000, window=48)}

# a birth-death chain with Hill-repressed birth and linear death: its stationary law is known in
# closed form (detailed balance), pinning the functional-rate path of the oracle
AUTOREPRESSOR = ModelDef("autorepressor", ("P",), ("top: . -> P @ hillr(P, 30, 2)", "top: P -> ."),
                         (60.0, 1.0), ".")
TINY_MODELS[AUTOREPRESSOR.name] = AUTOREPRESSOR
# Hill-ACTIVATED birth (positive feedback, unimodal: lambda'(x*) ~ 0.22 < 1) on top of a basal birth,
# linear death; and constant birth with Michaelis-Menten death.  Both are birth-death chains
# whose stationary laws follow from detailed balance (tests/test_oracle_ratelaws.py)
HILL_ACT = ModelDef("hill_act", ("P",), ("top: . -> P", "top: . -> P @ hill(P, 15, 2)", "top: P -> ."),
                    (10.0, 30.0, 1.0), ".")
MM_DEATH = ModelDef("mm_death", ("P",), ("top: . -> P", "top: P -> . @ mm(P, 10)"), (20.0, 30.0), ".")
TINY_MODELS[HILL_ACT.name] = HILL_ACT
TINY_MODELS[MM_DEATH.name] = MM_DEATH

# --- dynamic compartments (reading R20, bounded pools) ------------------------
# Vesicle traffic shaped like the paper's compartment creation/destruction: a
# budding site A creates vesicles loaded with 20 cargo B; cargo is processed to C inside;
# vesicles fuse with the top level releasing their content; B and C are degraded at the top.
# Vesicle number is an immigration-death process, Poisson(0.2/0.1 = 2) at stationarity; the
# pool holds 8 (P(N > 8) ~ 2e-4; a full pool freezes the instance as OVERFLOWED, R9).
VESICLES = ModelDef(
    name="vesicles",
    species=("A", "B", "C"),
    rules=(
        "top: A -> A (. | 20*B)^ves",   # budding
        "ves: B -> C",                  # processing inside a vesicle
        "top: ($x | $X)^ves -> $X",     # fusion: the content is released to the top level
        "top: B -> .",
        "top: C -> .",
    ),
    rates=(0.2, 0.2, 0.1, 0.05, 0.05),
    initial_term="A",
    capacity=(("ves", 8),),
)
MODELS[VESICLES.name] = VESICLES
CONFIGS["vesicles"] = RunConfig(
    7, VESICLES, 1_000_000, 100.0, 0.5, SEED_BASE + 7, 1024, 1,
    description="vesicle traffic with dynamic compartments (R20, 8-slot pool), 1M instances, t_end=100, dt=0.5")

# tiny dynamic models for the term-level CME pin (tests/test_oracle_dynamic.py): creation with
# cargo, internal decay, dissolution releasing the content, destruction without release
VES_TINY = ModelDef(
    "ves_tiny", ("A", "B"),
    ("top: A -> A (. | B)^v", "v: B -> .", "top: ($x | $X)^v -> $X", "top: B -> ."),
    (1.0, 0.7, 0.5, 0.3), "A (. | B)^v", capacity=(("v", 3),))
CELL_KILL = ModelDef(
    "cell_kill", ("K", "R", "S"),
    ("top: K -> K (2*R | S)^c", "top: (R $x | $X)^c -> $x", "c: . -> S", "top: (. $x | S $X)^c -> .",
     "top: R -> ."),
    (0.8, 0.4, 0.6, 0.3, 0.5), "K (2*R | S)^c", capacity=(("c", 2),))
TINY_MODELS[VES_TINY.name] = VES_TINY
TINY_MODELS[CELL_KILL.name] = CELL_KILL
