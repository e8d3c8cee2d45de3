"""CPU-side checks of the C ABI library (no GPU): it loads, exports every symbol include/cwc.h
declares, its rule compiler agrees with the oracle's independent flattening on every workload,
it rejects what DESIGN.md §3 says it must reject with the right status, and NVRTC compiles the
model-specialised SSA kernel for sm_100a without spilling.
"""
import ctypes
import os
import re

import pytest

import workloads as W
from oracle.cwc_terms import CWCError as OracleError
from oracle.cwc_terms import flatten, flatten_def

import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
from paper_conf_icdcsw_aldinuccidpmtt14_b200 import _lib

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared_functions():
    with open(os.path.join(ROOT, "include", "cwc.h")) as f:
        text = f.read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    return sorted(set(re.findall(r"\b(cwc_[a-z0-9_]+)\s*\(", text)))


def test_library_exports_every_declared_symbol():
    so = ctypes.CDLL(_lib.SO_PATH)
    names = _declared_functions()
    assert len(names) >= 20
    for n in names:
        assert hasattr(so, n), n
    assert set(names) == set(_lib.SIGNATURES), "binding and header disagree"
    assert b"sm_100a" in _lib.lib.cwc_version()


@pytest.mark.parametrize("name", sorted(W.MODELS) + sorted(W.TINY_MODELS))
def test_compiler_matches_oracle_flattening(name):
    md = W.MODELS.get(name) or W.TINY_MODELS[name]
    m = cwc.Model.from_def(md)
    info = m.info()
    fm = flatten_def(md)
    assert info["names"] == fm.names
    assert info["x0"] == fm.x0
    assert info["rates"] == fm.rates
    assert info["reactants"] == [list(r) for r in fm.reactants]
    assert info["delta"] == fm.delta
    assert info["rule_of"] == fm.rule_of
    assert info["x_cap"] == fm.x_cap
    assert info["n_rules"] == len(md.rules)
    assert info["law"] == fm.law and info["law_species"] == fm.law_species
    assert info["law_K"] == fm.law_K and info["law_n"] == fm.law_n
    # reading R20 (dynamic compartments): gates, placements, transfers, sentinel, flags
    assert info["gate_species"] == fm.gate_species and info["gate_kind"] == fm.gate_kind
    assert info["place"] == [[(a, list(ad)) for a, ad in p] for p in fm.place]
    assert info["transfer"] == [list(t) for t in fm.transfer]
    assert info["sentinel"] == fm.sentinel and info["flag"] == fm.flag


def test_capacity_option_reflattens():
    """capacity.<label> re-flattens the model (R20) exactly as the oracle does."""
    m = cwc.Model.from_def(W.VES_TINY)
    for cap in (1, 5):
        m.set_option("capacity.v", cap)
        fm = flatten(W.VES_TINY.species, W.VES_TINY.rules, W.VES_TINY.rates, W.VES_TINY.initial_term,
                     capacity={"v": cap})
        info = m.info()
        assert info["names"] == fm.names and info["delta"] == fm.delta and info["x0"] == fm.x0
        assert info["place"] == [[(a, list(ad)) for a, ad in p] for p in fm.place]
    with pytest.raises(cwc.CWCError):
        m.set_option("capacity.nosuch", 4)      # not a dynamic label
    with pytest.raises(cwc.CWCError):
        m.set_option("capacity.v", 0)
    assert len(m.info()["names"]) == len(flatten(W.VES_TINY.species, W.VES_TINY.rules, W.VES_TINY.rates,
                                                 W.VES_TINY.initial_term, capacity={"v": 5}).names)


REJECT = [
    (["top: Q -> ."], [1.0], "A", 1),
    (["top: A ."], [1.0], "A", 2),
    (["A -> ."], [1.0], "A", 2),
    (["top: A -> ."], [-1.0], "A", 1),
    (["top: A -> ."], [float("nan")], "A", 1),
    (["top: A -> ."], [float("inf")], "A", 1),
    (["top: A -> (. $x | $X)^c"], [1.0], "A", 3),
    (["top: A -> (.|B)^c (.|B)^c"], [1.0], "A", 3),                # two creations (R20)
    (["top: A ($x | $X)^c -> A $X ($x | $X)^c"], [1.0], "A", 3),   # release of a kept compartment
    (["top: A -> (.|B)^c", "c: B -> (.|A)^d"], [1.0, 1.0], "A", 3),  # nested dynamic compartments
    (["top: ($x | $X)^c -> ."], [1.0], "(. | (.|.)^d)^c", 3),        # dynamic with nested content
    (["top: A A A A -> ."], [1.0], "A", 3),
    (["top: (A | $X)^c -> (. | $X)^c"], [1.0], "A (A|.)^c", 3),
    (["top: (. $x | $X)^c (. $y | $Y)^c -> (. $y | $X)^c (. $x | $Y)^c"], [1.0], "(.|.)^c (.|.)^c", 3),
    (["top: A -> B"], [1.0], "(A | .)^top", 1),
    (["top: A -> B"], [1.0], "(A | .", 2),
    (["top: A -> B"], [1.0], "3 A", 2),
    (["top: A -> B @ mm(A)"], [1.0], "A", 2),                       # rate laws (R16')
    (["top: A -> B @ hill(A, 3)"], [1.0], "A", 2),
    (["top: A -> B @ foo(A, 3)"], [1.0], "A", 2),
    (["top: A -> B @ mm(Q, 3)"], [1.0], "A", 1),
    (["top: A -> B @ mm(A, -3)"], [1.0], "A", 1),
    (["top: A -> B @ hill(A, 3, 9)"], [1.0], "A", 1),
    (["top: A -> B @ hillr(A, 3, 0)"], [1.0], "A", 1),
    (["top: A -> B @ mm(A, 3"], [1.0], "A", 2),
]


@pytest.mark.parametrize("rules,rates,term,status", REJECT)
def test_rejections_match_oracle(rules, rates, term, status):
    with pytest.raises(cwc.CWCError) as e:
        cwc.Model(["A", "B"], rules, rates, term)
    assert e.value.status == status, str(e.value)
    kind = {1: "invalid", 2: "parse", 3: "unsupported"}[status]
    with pytest.raises(OracleError) as oe:
        flatten(["A", "B"], rules, rates, term)
    assert oe.value.kind == kind


def test_options_validation():
    m = cwc.Model.from_def(W.SCHLOGL)
    cap = m.info()["x_cap_max"]
    with pytest.raises(cwc.CWCError):
        m.set_option("x_cap", cap + 1)
    with pytest.raises(cwc.CWCError):
        m.set_option("x_cap", 100)          # below x0 = 250
    with pytest.raises(cwc.CWCError):
        m.set_option("nope", 1)
    with pytest.raises(cwc.CWCError):
        m.set_option("block_threads", 100)
    with pytest.raises(cwc.CWCError):
        m.set_option("hist_width.Q", 2)
    m.set_option("hist_width.X", 4)
    m.set_option("hist_lo", -3)
    assert m.info()["hist_width"] == [4] and m.info()["hist_lo"] == [-3]
    with pytest.raises(cwc.CWCError):
        m.set_quantiles([0.5, 1.5])


def test_state_errors_before_simulate():
    m = cwc.Model.from_def(W.IMM_DEATH)
    with pytest.raises(cwc.CWCError) as e:
        m.stats()
    assert e.value.status == 6
    with pytest.raises(cwc.CWCError) as e:
        m.samples(0, 1)
    assert e.value.status == 6
    with pytest.raises(cwc.CWCError) as e:
        m.buffer_sizes(10, 1.05, 0.1)
    assert e.value.status == 1


def test_buffer_sizes_layout():
    m = cwc.Model.from_def(W.LOTKA_VOLTERRA, hist_bins=1024)
    n_stats, n_raw, n_scratch = m.buffer_sizes(1000, 50.0, 0.1)
    T, S, B = 501, 2, 1024
    assert n_stats == T * (1 + 3 * S + S * (B + 2)) + _lib.N_CTR
    assert n_raw == -(-T // 8) * 8 * S * 1000   # time-blocked [ceil(T/8)][S][count][8]
    assert n_scratch >= 1000 * (S * 4 + 8 + 8 + 8 + 4 + 4)
    m.set_option("raw_samples", 0)
    assert m.buffer_sizes(1000, 50.0, 0.1)[1] == 0


@pytest.mark.parametrize("name", sorted(W.MODELS))
def test_nvrtc_compiles_for_sm100a(name):
    m = cwc.Model.from_def(W.MODELS[name])
    src, log = m.compile()
    assert "cwc_ssa_kernel" in src and "__dmul_rn" in src
    attrs = m.kernel_attributes()
    # spills only around the out-of-line cut emission / slow path are tolerated; pooled
    # dynamic-compartment models (R20: ~30 species, ~20 running sums) spill a few in the loop
    assert attrs["local_bytes"] <= (2048 if W.MODELS[name].capacity else 512), log
    assert 0 < attrs["registers"] <= 255
    # the image is an sm_100a ELF cubin (what the module upload sends to the device)
    import ctypes
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import _lib
    img, n = ctypes.c_void_p(), ctypes.c_size_t()
    assert _lib.lib.cwc_kernel_image(m._h, ctypes.byref(img), ctypes.byref(n)) == 0
    assert n.value == m.kernel_image_bytes() > 1024 and ctypes.string_at(img, 4) == b"\x7fELF"
    # the species state is indexed by compile-time constants only
    body = src[src.index("generated model section"):]
    assert "x[j]" not in body and "x[s]" not in body.split("cwc_bin")[0]


def test_simulate_without_gpu_fails_loudly():
    torch = pytest.importorskip("torch")
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    m = cwc.Model.from_def(W.IMM_DEATH)
    with pytest.raises(cwc.CWCError) as e:
        m.simulate(10, 1.0, 1.0, 1)
    assert e.value.status == 4


def test_steering_and_checkpoint_calls_out_of_order():
    """Terminate / resume / checkpoint / host-stats calls before any simulation are state errors
    (no device needed); a restore of garbage is rejected as invalid input."""
    import numpy as np
    m = cwc.Model.from_def(W.IMM_DEATH)
    for call in (m.cancel, m.resume, m.checkpoint, m.stats_host):
        with pytest.raises(cwc.CWCError) as e:
            call()
        assert e.value.status == 6, call
    with pytest.raises(cwc.CWCError) as e:
        m.stats_load(np.zeros(10, dtype=np.int64), 0)
    assert e.value.status == 6
    with pytest.raises(cwc.CWCError) as e:
        m.restore(np.zeros(64, dtype=np.uint8))
    assert e.value.status == 1


def test_pool_growth_reflattens_and_keeps_options():
    """Reading R20': Model.grow_pools doubles every compartment-pool capacity, re-flattens the model
    and re-applies the model's options (host only: flattening needs no GPU)."""
    import dataclasses
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    md = dataclasses.replace(W.VESICLES, capacity=(("ves", 3),))
    m = cwc.Model.from_def(md, hist_bins=77, hist_width={"A": 2}, x_cap=5000)
    assert m.pool_capacities() == {"ves": 3}
    s3 = m.n_species
    assert m.grow_pools() and m.pool_capacities() == {"ves": 6}
    info = m.info()
    assert m.n_species > s3 and sum(n.startswith("#alive") for n in info["names"]) == 6
    assert info["hist_bins"] == 77 and info["x_cap"] == 5000
    assert info["hist_width"][info["names"].index("A")] == 2
    # the flat network at the grown capacity is the oracle's flattening at that capacity
    from oracle.cwc_terms import flatten_def
    fm = flatten_def(dataclasses.replace(md, capacity=(("ves", 6),)))
    assert info["names"] == fm.names
    static = cwc.Model.from_def(W.LOTKA_VOLTERRA)
    assert static.pool_capacities() == {} and not static.grow_pools()
