"""GPU parity: the CUDA path (through the C ABI) against the oracle, element by element.

Bar (north_star): integer species counts at every cut identical to the oracle
(we require 100 %: both sides follow R3-R7 bit for bit), identical per-instance flags and
reaction counts, and finalised statistics bit-identical to the oracle's statistics of the
oracle's samples.  Sizes span several CTAs and a ragged tail; the bench-size runs are checked
on sampled instances plus the raw-vs-stats property that holds at any size.
"""
import numpy as np
import pytest

import oracle
import workloads as W
from oracle.cwc_terms import flatten_def

from helpers import assert_matches_oracle_stats, assert_stats_match_raw, gpu_run

pytestmark = pytest.mark.gpu

QS = (0.05, 0.25, 0.5, 0.75, 0.95)


def _oracle(md, first, count, t_end, dt, seed, nthreads=16):
    return oracle.simulate(flatten_def(md), first, count, t_end, dt, seed, nthreads=nthreads)


# ------------------------------------------------------------------ device primitives
def test_device_philox_matches_oracle():
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import selftest_philox
    rng = np.random.default_rng(1)
    n = 50000
    ctr = rng.integers(0, 2 ** 32, size=(n, 4), dtype=np.uint64).astype(np.uint32)
    key = rng.integers(0, 2 ** 32, size=(n, 2), dtype=np.uint64).astype(np.uint32)
    ctr[0], key[0] = 0, 0
    ctr[1], key[1] = 0xFFFFFFFF, 0xFFFFFFFF
    ctr[2], key[2] = [0x243F6A88, 0x85A308D3, 0x13198A2E, 0x03707344], [0xA4093822, 0x299F31D0]
    out = selftest_philox(ctr, key)
    assert list(out[0]) == [0x6627E8D5, 0xE169C58D, 0xBC57AC4C, 0x9B00DBD8]
    for i in range(0, n, 97):
        assert tuple(int(v) for v in out[i]) == oracle.philox4x32_10([int(v) for v in ctr[i]],
                                                                    [int(v) for v in key[i]])


def test_device_u01_matches_oracle():
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import selftest_u01
    rng = np.random.default_rng(2)
    w = rng.integers(0, 2 ** 32, size=(20000, 2), dtype=np.uint64).astype(np.uint32)
    w[0] = [0, 0]
    w[1] = [0xFFFFFFFF, 0xFFFFFFFF]
    out = selftest_u01(w)
    for i in range(len(w)):
        assert out[i] == oracle.u01(int(w[i, 0]), int(w[i, 1]))


def test_device_log_bit_identical_to_oracle():
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import selftest_log
    rng = np.random.default_rng(3)
    u = np.concatenate([rng.random(200000), np.exp2(-rng.random(100000) * 53.0),
                        [2.0 ** -53, 1 - 2.0 ** -53, 0.5, 0.6875, 0.999, 1 - 1 / 256]])
    u = u[(u >= 2.0 ** -53) & (u < 1.0)]
    got = selftest_log(u)
    ref = np.array([oracle.cwclog(float(v)) for v in u])
    assert np.array_equal(got.view(np.uint64), ref.view(np.uint64))


# ------------------------------------------------------------------ whole-path parity
def _parity(md, n, t_end, dt, seed, *, first=0, hist_bins=256, hist_width=1, **opts):
    res, raw, flags, reactions, m = gpu_run(md, first + n, first, n, t_end, dt, seed, hist_bins=hist_bins,
                                            hist_width=hist_width, quantiles=QS, **opts)
    orun = _oracle(md, first, n, t_end, dt, seed)
    assert raw.shape == orun.raw.shape
    same = np.all(raw == orun.raw, axis=(0, 1))
    assert same.mean() == 1.0, f"{(~same).sum()} of {n} instances differ"
    assert np.array_equal(flags, orun.flags)
    assert np.array_equal(reactions, orun.reactions)
    assert res.reactions == int(orun.reactions.sum())
    assert res.absorbed == int((orun.flags == oracle.FLAG_ABSORBED).sum())
    assert res.overflowed == int((orun.flags == oracle.FLAG_OVERFLOWED).sum())
    assert res.finished == n
    assert_matches_oracle_stats(res, orun.raw, QS)
    return res, raw, m


def test_config1_imm_death_full():
    cfg = W.CONFIGS["imm_death"]
    _parity(cfg.model, cfg.n_instances, cfg.t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins,
            hist_width=cfg.hist_width)


@pytest.mark.parametrize("fast_cut", [-1, 0, 1])
def test_lv_short_horizon_ragged(fast_cut):
    # LV has ~3,000 reactions per cut: auto (-1) records cuts on the full-step path (0)
    cfg = W.CONFIGS["lv"]
    _parity(cfg.model, 1537, 2.0, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width,
            fast_cut=fast_cut)


def test_terminated_instances_under_quanta():
    """Absorbed / overflowed instances end in an early quantum; every later quantum item of the
    instance must be skipped (regression: the third quantum waited forever)."""
    cfg = W.CONFIGS["lv"]
    res, *_ = _parity(cfg.model, 400, 50.0, 0.5, cfg.seed + 7, hist_bins=cfg.hist_bins, hist_width=cfg.hist_width,
                      quantum_samples=4)
    assert res.overflowed > 0 and res.absorbed > 0


@pytest.mark.parametrize("q", [0, 16])
def test_compacted_launches_drop_finished_instances(q):
    """Compacted per-quantum launches (option compact): instances that absorb or overflow leave
    the launch lists; every instance's cuts, flags and reactions still equal the oracle's."""
    cfg = W.CONFIGS["lv"]
    res, raw, m = _parity(cfg.model, 700, 50.0, 0.5, cfg.seed + 7, hist_bins=cfg.hist_bins,
                          hist_width=cfg.hist_width, compact=1, quantum_samples=q)
    assert res.overflowed > 0 and res.absorbed > 0 and res.launches > 2


def test_lv_long_horizon_absorb_and_overflow():
    # long horizon: predator extinction, prey runaway past X_cap (R9) and full extinction (R8)
    cfg = W.CONFIGS["lv"]
    res, raw, m = _parity(cfg.model, 300, 50.0, 0.5, cfg.seed + 7, hist_bins=cfg.hist_bins,
                          hist_width=cfg.hist_width)
    assert res.overflowed > 0


def test_schlogl_small_quanta():
    cfg = W.CONFIGS["schlogl"]
    _parity(cfg.model, 3001, 5.0, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins, quantum_samples=3)


def test_circadian_small():
    cfg = W.CONFIGS["circadian"]
    _parity(cfg.model, 700, 12.0, cfg.sample_dt, cfg.seed, first=123_456, hist_bins=cfg.hist_bins,
            hist_width=cfg.hist_width)


def test_compartments_small():
    cfg = W.CONFIGS["compartments"]
    _parity(cfg.model, 900, 20.0, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins)


def test_vesicles_dynamic_compartments():
    """SURVEY §8(f)-4 (reading R20): creation into pool slots, dissolution releasing the
    content, processing inside slots; ragged size, nonzero first."""
    cfg = W.CONFIGS["vesicles"]
    _parity(cfg.model, 1500, 40.0, cfg.sample_dt, cfg.seed, first=77_777, hist_bins=cfg.hist_bins)


def test_vesicles_pool_overflow_and_quanta():
    """A 3-slot pool overflows often: full-pool creations freeze instances (OVERFLOWED, R9/R20)
    identically on both sides, under several quantum sizes."""
    import dataclasses
    md = dataclasses.replace(W.VESICLES, capacity=(("ves", 3),))
    res, *_ = _parity(md, 1200, 60.0, 0.5, 11, hist_bins=256)
    assert res.overflowed > 50
    _parity(md, 1200, 60.0, 0.5, 11, hist_bins=256, quantum_samples=5)


@pytest.mark.parametrize("name", sorted(W.TINY_MODELS))
def test_tiny_models(name):
    _parity(W.TINY_MODELS[name], 257, 6.0, 0.25, 99)


def test_results_outlive_sharded_run():
    """dist.simulate_sharded binds torch-owned buffers; samples read after its run object is
    gone (and after torch reuses freed memory) must still be the simulation's."""
    import gc
    import torch
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    from paper_conf_icdcsw_aldinuccidpmtt14_b200 import dist as cdist
    m = cwc.Model.from_def(W.IMM_DEATH, hist_bins=256)
    cdist.simulate_sharded(m, 500, 100.0, 1.0, 3)
    gc.collect()
    junk = torch.full((64 << 20,), -7, dtype=torch.int32, device="cuda")
    torch.cuda.synchronize()
    raw = m.samples(0, 500)
    del junk
    assert np.array_equal(raw, _oracle(W.IMM_DEATH, 0, 500, 100.0, 1.0, 3).raw)


def test_empty_shard():
    """A rank whose contiguous share is empty (n_total < world): a valid no-op whose statistics
    are all zero and sum neutrally into the all-reduce."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model.from_def(W.LOTKA_VOLTERRA, hist_bins=64)
    m.simulate_range(3, 3, 0, 1.0, 0.1, 9)
    res = m.finalize()
    assert res.finished == 0 and res.reactions == 0
    assert not res.n.any() and not res.sum.any() and not res.hist.any()
    assert np.isnan(res.mean).all()


def test_many_cuts_global_moments():
    """T = 20,001 cuts: the moment accumulators no longer fit in shared memory, so the kernel
    records straight into the global buffer (the other recording path)."""
    _parity(W.IMM_DEATH, 300, 2000.0, 0.1, 77, hist_bins=300)


def test_zero_horizon_and_single_instance():
    _parity(W.LOTKA_VOLTERRA, 1, 0.0, 0.1, 5)
    _parity(W.SCHLOGL, 1, 3.0, 0.1, 5)


# ------------------------------------------------------------------ schedule invariance (R12)
def test_schedule_invariance():
    md = W.SCHLOGL
    base = None
    for opts in ({}, {"quantum_samples": 1}, {"quantum_samples": 7}, {"block_threads": 128},
                 {"fast_cut": 0}, {"fast_cut": 1, "quantum_samples": 3},
                 {"block_threads": 512, "quantum_samples": 2}, {"refill": False}, {"blocks_per_sm": 1},
                 {"refill": False, "quantum_samples": 7},    # per-quantum lockstep launches
                 {"compact": 1}, {"compact": 1, "quantum_samples": 3}, {"compact": 0}):  # compacted launches
        res, raw, flags, reactions, _ = gpu_run(md, 5000, 0, 5000, 4.0, 0.1, 42, hist_bins=512, **opts)
        cur = (res.n, res.sum, res.sqlo, res.sqhi, res.hist, raw, reactions)
        if base is None:
            base = cur
        else:
            for a, b in zip(base, cur):
                assert np.array_equal(a, b), opts


@pytest.mark.parametrize("name,n", [("circadian", 3000), ("vesicles", 3000), ("lv", 2000), ("schlogl", 3000)])
def test_statistics_staging_invariance(name, n):
    """The three per-CTA staging layouts of the cut statistics (global only, sparse u32 limbs with
    zero counts restored at the flush, dense u64) give bit-identical packed statistics, and the
    default one equals the oracle's statistics of its own samples."""
    cfg = W.CONFIGS[name]
    t_end = min(cfg.t_end, 10.0)
    base = None
    for mode in (0, 1, 2, 3):
        res, raw, *_ = gpu_run(cfg.model, n, 0, n, t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins,
                               hist_width=cfg.hist_width, smem_stats=mode)
        cur = (res.n, res.sum, res.sqlo, res.sqhi, res.hist, res.reactions)
        if base is None:
            base = cur
            orun = _oracle(cfg.model, 0, n, t_end, cfg.sample_dt, cfg.seed)
            assert np.array_equal(raw, orun.raw)
            assert_matches_oracle_stats(res, orun.raw, QS)
        else:
            for a, b in zip(base, cur):
                assert np.array_equal(a, b), mode


@pytest.mark.parametrize("opts", [{}, {"quantum_samples": 5}, {"quantum_samples": 13, "block_threads": 256},
                                  {"refill": False, "quantum_samples": 3}, {"compact": 1}, {"fast_cut": 1}])
def test_raw_staging_invariance(opts):
    """Raw cuts staged per lane in shared memory and written as whole 32-byte blocks (option
    raw_stage, the default) equal the direct 4-byte stores and the oracle: blocks cut by quanta
    that are not multiples of 8 cuts, absorbed instances (cuts to K in one go), overflowed ones
    (the staged part of a block, then -1) and a ragged last block (T = 101)."""
    cfg = W.CONFIGS["lv"]
    n, t_end, dt, seed = 600, 50.0, 0.5, cfg.seed + 7
    on, raw_on, fl_on, re_on, _ = gpu_run(cfg.model, n, 0, n, t_end, dt, seed, hist_bins=cfg.hist_bins,
                                          hist_width=cfg.hist_width, **opts)
    off, raw_off, fl_off, re_off, _ = gpu_run(cfg.model, n, 0, n, t_end, dt, seed, hist_bins=cfg.hist_bins,
                                              hist_width=cfg.hist_width, raw_stage=0, **opts)
    assert on.raw_staged == 1 and off.raw_staged == 0
    assert on.absorbed > 0 and on.overflowed > 0
    assert np.array_equal(raw_on, raw_off) and np.array_equal(fl_on, fl_off) and np.array_equal(re_on, re_off)
    orun = _oracle(cfg.model, 0, n, t_end, dt, seed)
    assert np.array_equal(raw_on, orun.raw)
    assert_matches_oracle_stats(on, orun.raw, QS)


def test_bounds_checked_kernel():
    """Every shared-memory and global index of the SSA kernel bounds-checked on the device
    (CWC_CHECKS=1, a violation traps) over raw-cut staging with partial blocks, the three
    statistics layouts, lockstep / compacted launches, pools and a 20,001-cut horizon; results
    equal the oracle's.  Own process: a trap poisons the CUDA context."""
    import os
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, os.path.join(root, "tests", "workers", "bounds_check.py")],
                       capture_output=True, text=True, timeout=900)
    assert r.returncode == 0 and "BOUNDS OK" in r.stdout, r.stdout[-2000:] + r.stderr[-2000:]


@pytest.mark.parametrize("name,defines", [("compartments", ""), ("compartments", "CWC_SPARSE_TICKETS=64"),
                                           ("vesicles", "CWC_COOP_EMIT=1"),
                                           ("vesicles", "CWC_COOP_EMIT=1;CWC_SPARSE_TICKETS=64")])
def test_cooperative_cut_recording(monkeypatch, name, defines):
    """Cuts recorded cooperatively by the warp in the fast step (raw cuts off, sparse statistics:
    lane s records species s of each due lane's cut; compartments by default, vesicles forced),
    including records beyond the sparse admission limit (global path): statistics equal the
    oracle's statistics of its own samples."""
    cfg = W.CONFIGS[name]
    n, t_end = 6000, 30.0
    if defines:
        monkeypatch.setenv("CWC_KERNEL_DEFINES", defines)
    res, *_ = gpu_run(cfg.model, n, 0, n, t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins,
                      hist_width=cfg.hist_width, raw=False, fast_cut=1, quantum_samples=16)
    assert_matches_oracle_stats(res, _oracle(cfg.model, 0, n, t_end, cfg.sample_dt, cfg.seed).raw, QS)


def test_sparse_ticket_overflow_goes_global(monkeypatch):
    """Sparse staging admits at most CWC_SPARSE_TICKETS work items of one quantum per CTA to its
    16-bit limbs; later items record to global memory.  With the limit lowered to 64 most records
    take that path, and the statistics still equal the oracle's (and the default kernel's)."""
    cfg = W.CONFIGS["compartments"]
    n, t_end = 20_000, 10.0
    ref, *_ = gpu_run(cfg.model, n, 0, n, t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins, raw=False)
    monkeypatch.setenv("CWC_KERNEL_DEFINES", "CWC_SPARSE_TICKETS=64")
    res, raw, *_ = gpu_run(cfg.model, n, 0, n, t_end, cfg.sample_dt, cfg.seed, hist_bins=cfg.hist_bins,
                           smem_stats=2)
    for name in ("n", "sum", "sqlo", "sqhi", "hist"):
        assert np.array_equal(getattr(res, name), getattr(ref, name)), name
    assert_matches_oracle_stats(res, _oracle(cfg.model, 0, n, t_end, cfg.sample_dt, cfg.seed).raw, QS)


def test_sharding_invariance():
    """Disjoint ranges summed == one run (what the NCCL all-reduce relies on, §8(e))."""
    md, N, t_end, dt, seed = W.LOTKA_VOLTERRA, 4000, 3.0, 0.1, 7
    full, raw_full, *_ = gpu_run(md, N, 0, N, t_end, dt, seed, hist_bins=64, hist_width=256)
    acc = None
    raws = []
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    for a, b in ((0, 1000), (1000, 2999), (2999, 4000)):
        m = cwc.Model.from_def(md, hist_bins=64, hist_width=256)
        m.simulate_range(N, a, b - a, t_end, dt, seed)
        res = m.finalize()
        raws.append(m.samples(0, b - a))
        cur = [res.n, res.sum, res.sqlo, res.sqhi, res.hist]
        acc = cur if acc is None else [x + y for x, y in zip(acc, cur)]
    for a, b in zip(acc, [full.n, full.sum, full.sqlo, full.sqhi, full.hist]):
        assert np.array_equal(a, b)
    assert np.array_equal(np.concatenate(raws, axis=2), raw_full)


# ------------------------------------------------------------------ bench-size runs
# SURVEY §8(d) "the same sub-ensemble is used for parity": the fixed instances [first, first + N_cpu)
# of the full-size launch (the bench's own launch configuration: every instance of the config in
# one kernel, default options) compared element by element with the oracle.
FULL_SIZE = [  # (config, shards: the last shard of an ensemble sharded over 8 GPUs, N_cpu)
    ("lv", 1, 2_000), ("lv1m", 1, 2_000), ("schlogl", 1, 10_000), ("compartments", 1, 10_000),
    ("circadian", 8, 10_000)]


@pytest.mark.parametrize("cname,shards,n_cpu", FULL_SIZE)
def test_full_size_sub_ensemble_parity(cname, shards, n_cpu):
    """BASELINE sizes in the bench's launch configuration; circadian (10M over 8 GPUs) as the last
    1.25M shard, so instance ids (the Philox key) are global ones far from 0."""
    cfg = W.CONFIGS[cname]
    N = cfg.n_instances
    first = (shards - 1) * N // shards
    count = N - first
    res, _, flags, reactions, m = gpu_run(cfg.model, N, first, count, cfg.t_end, cfg.sample_dt, cfg.seed,
                                          hist_bins=cfg.hist_bins, hist_width=cfg.hist_width, quantiles=QS,
                                          raw=True, copy_raw=False)
    assert res.finished == count and res.reactions == int(reactions.sum())
    # properties of the whole launch that hold at any size
    T, S = res.sum.shape
    assert (res.hist.sum(axis=2) == res.n[:, None]).all() and res.n[0] == count
    assert res.absorbed == int((flags == oracle.FLAG_ABSORBED).sum())
    assert res.overflowed == int((flags == oracle.FLAG_OVERFLOWED).sum())
    # the sub-ensemble [first, first + n_cpu), element by element
    raw = m.samples(0, n_cpu)
    orun = oracle.simulate(flatten_def(cfg.model), first, n_cpu, cfg.t_end, cfg.sample_dt, cfg.seed, nthreads=16)
    same = np.all(raw == orun.raw, axis=(0, 1))
    assert same.all(), f"{(~same).sum()} of {n_cpu} instances differ"
    assert np.array_equal(flags[:n_cpu], orun.flags) and np.array_equal(reactions[:n_cpu], orun.reactions)
    if count * T * S <= 2 * 10 ** 9:    # the raw-vs-stats identity on the whole launch (<= 8 GB of cuts)
        assert_stats_match_raw(res, m.samples(0, count))


def test_device_fast_division_is_ieee():
    """The kernel's branch-free divide (tau = -log(u) / a0) equals IEEE division bit for bit."""
    from paper_conf_icdcsw_aldinuccidpmtt14_b200.api import selftest_div
    rng = np.random.default_rng(4)
    n = 4_000_000
    num = -np.log(rng.random(n))                       # the SSA's numerators: -log(u), u in (0,1)
    num[:1000] = np.exp2(-rng.random(1000) * 53)       # tiny -log(u)
    den = np.exp2(rng.uniform(-60, 60, n)) * rng.uniform(1, 2, n)   # propensity sums over 36 decades
    den[:500] = 1.0
    den[500:1000] = np.round(rng.uniform(1, 1e6, 500))   # exact-quotient / integer cases
    num[500:1000] = den[500:1000] * np.round(rng.uniform(1, 30, 500))
    den[1000:1100] = np.ldexp(1.0, rng.integers(-1020, 1020, 100))  # out of the fast range -> fallback
    got = selftest_div(num, den)
    ref = num / den
    assert np.array_equal(got.view(np.uint64), ref.view(np.uint64))


# ------------------------------------------------------------------ on-line period analysis (R19)
@pytest.mark.parametrize("md,species,lo,hi,t_end,dt,n", [
    (W.CIRCADIAN, "R", 100, 1000, 96.0, 0.5, 1500),
    (W.LOTKA_VOLTERRA, "Y1", 800, 1300, 10.0, 0.05, 1000),
])
def test_period_analysis_matches_oracle(md, species, lo, hi, t_end, dt, n):
    from oracle.period import finalize, period_stats
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    W_ = 24
    m = cwc.Model.from_def(md, hist_bins=64, hist_width=64, period_species=species, period_lo=lo, period_hi=hi,
                           period_window=W_)
    seed = 2024
    m.simulate_range(n, 0, n, t_end, dt, seed)
    m.finalize()
    got = m.period_stats()
    fm = flatten_def(md)
    orun = oracle.simulate(fm, 0, n, t_end, dt, seed, nthreads=16)
    assert np.array_equal(m.samples(0, n), orun.raw)
    ps = period_stats(orun.raw, fm.names.index(species), lo, hi)
    assert got["species"] == fm.names.index(species)
    assert np.array_equal(got["events"], ps.ev) and ps.ev.sum() > n
    assert np.array_equal(got["pc_n"], ps.pc_n) and np.array_equal(got["pc_sum"], ps.pc_sum)
    assert [(int(h) << 32) + int(l) for h, l in zip(got["pc_sqhi"], got["pc_sqlo"])] == list(ps.pc_sq)
    assert np.array_equal(got["lp_n"], ps.lp_n) and np.array_equal(got["lp_sum"], ps.lp_sum)
    assert [(int(h) << 32) + int(l) for h, l in zip(got["lp_sqhi"], got["lp_sqlo"])] == list(ps.lp_sq)
    lp_mean, ma, lp_var = finalize(ps, dt, W_)
    assert np.array_equal(got["lp_mean"], lp_mean, equal_nan=True)
    assert np.array_equal(got["moving_avg"], ma, equal_nan=True)
    assert np.array_equal(got["lp_var"], lp_var, equal_nan=True)
    if md is W.CIRCADIAN:   # Vilar oscillator: local period ~ 20-30 h once every instance has one
        assert 20.0 < np.nanmean(lp_mean[-48:]) < 30.0


def test_neurospora_rate_laws_parity():
    """Functional rate laws (MM / Hill) on the paper's Neurospora model."""
    cfg = W.CONFIGS["neurospora"]
    _parity(cfg.model, 1200, 48.0, cfg.sample_dt, cfg.seed, first=777, hist_bins=cfg.hist_bins)


def test_neurospora_period_analysis_parity():
    from oracle.period import finalize, period_stats
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    pa = W.PERIOD_ANALYSIS["neurospora"]
    md, n, t_end, dt, seed = W.NEUROSPORA, 2000, 96.0, 0.5, 31
    m = cwc.Model.from_def(md, hist_bins=64, period_species=pa["species"], period_lo=pa["lo"], period_hi=pa["hi"],
                           period_window=pa["window"])
    m.simulate_range(n, 0, n, t_end, dt, seed)
    m.finalize()
    got = m.period_stats()
    fm = flatten_def(md)
    orun = oracle.simulate(fm, 0, n, t_end, dt, seed, nthreads=16)
    ps = period_stats(orun.raw, fm.names.index(pa["species"]), pa["lo"], pa["hi"])
    assert np.array_equal(got["events"], ps.ev) and np.array_equal(got["pc_sum"], ps.pc_sum)
    assert np.array_equal(got["lp_n"], ps.lp_n) and np.array_equal(got["lp_sum"], ps.lp_sum)
    lp_mean, ma, lp_var = finalize(ps, dt, pa["window"])
    assert np.array_equal(got["moving_avg"], ma, equal_nan=True)
    assert np.array_equal(got["lp_mean"], lp_mean, equal_nan=True)
    assert 19.0 < ma[-1] < 24.0   # ~21.5 h, the model's published period


# ------------------------------------------------------------------ on-line streaming (§8(f)-2)
def test_streaming_snapshots_are_final_prefixes():
    """Snapshots taken while the kernel runs: the cuts they report final equal the finished run."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS["schlogl"]
    n, t_end = 200_000, 20.0
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, raw_samples=False)
    snaps = [(cf, res) for cf, res in m.stream(n, t_end, cfg.sample_dt, cfg.seed, poll_s=0.005)]
    final = snaps[-1][1]
    T = final.n.size
    assert snaps[-1][0] == T and final.finished == n
    partial = [(cf, r) for cf, r in snaps[:-1] if cf > 0]
    assert len(partial) >= 2, [cf for cf, _ in snaps]          # progress was observed mid-run
    prev = 0
    for cf, r in partial:
        assert prev <= cf < T
        prev = cf
        for name in ("n", "sum", "sqlo", "sqhi", "hist"):
            assert np.array_equal(getattr(r, name)[:cf], getattr(final, name)[:cf]), (cf, name)
        assert np.array_equal(r.mean[:cf], final.mean[:cf], equal_nan=True)
    # and the streamed run equals a normal run
    ref = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, raw_samples=False).simulate(
        n, t_end, cfg.sample_dt, cfg.seed)
    for name in ("n", "sum", "sqlo", "sqhi", "hist"):
        assert np.array_equal(getattr(ref, name), getattr(final, name))


def test_stream_terminate_keeps_final_cuts_exact():
    """Terminating a running simulation (Fig. 2; cwc_cancel via stream(stop=)):
    the kernel stops early, and the cuts reported final are exactly the uninterrupted run's."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS["schlogl"]
    n = cfg.n_instances
    m = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, raw_samples=False)
    out = list(m.stream(n, cfg.t_end, cfg.sample_dt, cfg.seed, poll_s=0.002, stop=lambda cf, res: cf > 0))
    cf, res = out[-1]
    T = res.n.size
    assert 0 < cf < T, [c for c, _ in out]          # stopped after the first final cuts, well before T
    ref = cwc.Model.from_def(cfg.model, hist_bins=cfg.hist_bins, raw_samples=False).simulate(
        n, cfg.t_end, cfg.sample_dt, cfg.seed)
    assert res.reactions < ref.reactions // 2       # most of the work was not done
    for name in ("n", "sum", "sqlo", "sqhi", "hist"):
        assert np.array_equal(getattr(res, name)[:cf], getattr(ref, name)[:cf]), name
    assert (res.n[:cf] == n).all() and (res.n[cf:] < n).any()
    # a new simulation on the same handle is unaffected by the earlier terminate
    again = m.simulate(1000, 5.0, cfg.sample_dt, cfg.seed)
    assert again.finished == 1000


def test_cancel_needs_streaming():
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model.from_def(W.IMM_DEATH, hist_bins=64)
    m.simulate(100, 10.0, 1.0, 1)
    with pytest.raises(cwc.CWCError):
        m.cancel()


def test_checkpoint_resume_bit_identical():
    """Terminate a running simulation, checkpoint it to the host, restore it into a fresh handle
    and resume it: statistics, raw cuts and per-instance records equal the uninterrupted run
    (counter-based RNG); resuming on the same handle gives the same."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    cfg = W.CONFIGS["schlogl"]
    n, t_end = 200_000, 20.0
    kw = dict(hist_bins=cfg.hist_bins, quantiles=QS)
    ref_m = cwc.Model.from_def(cfg.model, **kw)
    ref = ref_m.simulate(n, t_end, cfg.sample_dt, cfg.seed)
    ref_raw = ref_m.samples(0, n)
    ref_flags, ref_react, _ = ref_m.records(0, n)

    m = cwc.Model.from_def(cfg.model, **kw)
    out = list(m.stream(n, t_end, cfg.sample_dt, cfg.seed, poll_s=0.002, stop=lambda cf, r: cf > 0))
    cf, part = out[-1]
    assert 0 < cf < part.n.size and part.reactions < ref.reactions
    ckpt = m.checkpoint()

    m2 = cwc.Model.from_def(cfg.model, **kw)
    m2.restore(ckpt)
    m2.resume()
    for mm in (m2, m):
        if mm is m:
            m.resume()
        res = mm.finalize()
        for name in ("n", "sum", "sqlo", "sqhi", "hist", "quantile"):
            assert np.array_equal(getattr(res, name), getattr(ref, name), equal_nan=True), name
        assert res.reactions == ref.reactions and res.finished == n and res.absorbed == ref.absorbed
        assert np.array_equal(mm.samples(0, n), ref_raw)
        flags, react, _ = mm.records(0, n)
        assert np.array_equal(flags, ref_flags) and np.array_equal(react, ref_react)


def test_checkpoint_rejects_other_model_and_nothing_to_resume():
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model.from_def(W.IMM_DEATH, hist_bins=64)
    m.simulate(100, 10.0, 1.0, 1)
    ckpt = m.checkpoint()
    with pytest.raises(cwc.CWCError):
        m.resume()                                  # a completed run: nothing to resume
    other = cwc.Model.from_def(W.IMM_DEATH, hist_bins=65)
    with pytest.raises(cwc.CWCError):
        other.restore(ckpt)                         # different histogram: different results
    same = cwc.Model.from_def(W.IMM_DEATH, hist_bins=64)
    same.restore(ckpt)                              # a finished run restores and finalises as is
    res = same.finalize()
    assert res.finished == 100 and np.array_equal(res.hist, m.finalize().hist)


def test_checkpoint_resume_with_period_analysis():
    """The on-line period detector's per-instance state travels in the checkpoint: a terminated,
    restored and resumed circadian run gives the uninterrupted run's period statistics."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    pa = W.PERIOD_ANALYSIS["circadian"]
    n, t_end, dt, seed = 40_000, 96.0, 0.5, 17
    kw = dict(hist_bins=64, raw_samples=False, period_species=pa["species"], period_lo=pa["lo"],
              period_hi=pa["hi"], period_window=pa["window"])
    ref_m = cwc.Model.from_def(W.CIRCADIAN, **kw)
    ref = ref_m.simulate(n, t_end, dt, seed)
    ref_p = ref_m.period_stats()
    m = cwc.Model.from_def(W.CIRCADIAN, **kw)
    cf, part = list(m.stream(n, t_end, dt, seed, poll_s=0.001, stop=lambda c, r: c > 0))[-1]
    assert 0 < cf < part.n.size
    m2 = cwc.Model.from_def(W.CIRCADIAN, **kw)
    m2.restore(m.checkpoint())
    m2.resume()
    res = m2.finalize()
    got = m2.period_stats()
    for name in ("n", "sum", "sqlo", "sqhi", "hist"):
        assert np.array_equal(getattr(res, name), getattr(ref, name)), name
    for name in ("events", "pc_n", "pc_sum", "pc_sqlo", "pc_sqhi", "lp_n", "lp_sum", "lp_sqlo", "lp_sqhi"):
        assert np.array_equal(got[name], ref_p[name]), name
    assert np.array_equal(got["moving_avg"], ref_p["moving_avg"], equal_nan=True)


def test_pool_auto_growth_removes_pool_frozen_instances():
    """Reading R20': a run in which a compartment pool was full is repeated with doubled
    capacities; the final result has no pool-frozen instance, and the species outside the pools
    follow exactly the trajectories of an ample pool (the dynamics of a trajectory that never finds
    its pool full do not depend on the capacity)."""
    import dataclasses
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    md = dataclasses.replace(W.VESICLES, capacity=(("ves", 3),))
    n, t_end, dt, seed = 20_000, 60.0, 0.5, 11
    m = cwc.Model.from_def(md, hist_bins=256)
    m.pool_auto = False
    first = m.simulate(n, t_end, dt, seed)
    assert first.pool_full > 50 and first.pool_full <= first.overflowed     # capacity 3 fills often
    m.pool_auto = True
    res = m.simulate(n, t_end, dt, seed)
    assert res.pool_full == 0 and m.pool_capacities()["ves"] >= 6
    big = cwc.Model.from_def(dataclasses.replace(md, capacity=(("ves", 64),)), hist_bins=256).simulate(n, t_end, dt, seed)
    assert big.pool_full == 0
    for sp in ("A", "B", "C"):
        i, j = res.species.index(sp), big.species.index(sp)
        assert np.array_equal(res.sum[:, i], big.sum[:, j]) and np.array_equal(res.hist[:, i], big.hist[:, j]), sp
    assert res.reactions == big.reactions and np.array_equal(res.n, big.n)
