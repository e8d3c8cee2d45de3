// abi.cpp — the extern "C" boundary declared in include/cwc.h.  Argument checking, option
// handling and exception -> status translation; the work is in compiler.cpp / runtime.cpp.
#include <cmath>
#include <cstring>
#include <memory>
#include <new>
#include <string>

#include "cwc.h"
#include "runtime.hpp"

namespace {

thread_local std::string g_err;

template <class F>
cwc_status guard(F&& f) {
    g_err.clear();
    try {
        f();
        return CWC_OK;
    } catch (const cwc::Error& e) {
        g_err = e.what();
        return e.code;
    } catch (const std::bad_alloc&) {
        g_err = "host out of memory";
        return CWC_E_OOM;
    } catch (const std::exception& e) {
        g_err = e.what();
        return CWC_E_INVALID;
    } catch (...) {
        g_err = "unknown error";
        return CWC_E_INVALID;
    }
}

[[noreturn]] void fail(int32_t code, const std::string& msg) { throw cwc::Error(code, msg); }

void need(bool c, const char* msg) {
    if (!c) fail(CWC_E_INVALID, msg);
}

void refresh_info(cwc_model* m) {
    const cwc::FlatModel& fm = m->fm;
    const int S = fm.S(), M = fm.M();
    m->name_ptrs.clear();
    for (auto& n : fm.names) m->name_ptrs.push_back(n.c_str());
    const int R = CWC_MAX_REACTANTS;
    m->info_nreact.assign(M, 0);
    m->info_rspecies.assign((size_t)M * R, 0);
    m->info_rorder.assign((size_t)M * R, 0);
    m->info_delta.assign((size_t)M * S, 0);
    m->info_place_off.assign(1, 0);
    m->info_add_off.assign(1, 0);
    m->info_xfer_off.assign(1, 0);
    m->info_place_alive.clear();
    m->info_add_s.clear();
    m->info_add_n.clear();
    m->info_xfer_src.clear();
    m->info_xfer_dst.clear();
    for (int j = 0; j < M; ++j) {
        m->info_nreact[j] = (int32_t)fm.reactants[j].size();
        for (size_t e = 0; e < fm.reactants[j].size(); ++e) {
            m->info_rspecies[j * R + e] = fm.reactants[j][e].species;
            m->info_rorder[j * R + e] = fm.reactants[j][e].order;
        }
        for (int s = 0; s < S; ++s) m->info_delta[(size_t)j * S + s] = fm.delta[j][s];
        for (const auto& ps : fm.place[j]) {
            m->info_place_alive.push_back(ps.alive);
            for (const auto& a : ps.adds) {
                m->info_add_s.push_back(a.first);
                m->info_add_n.push_back(a.second);
            }
            m->info_add_off.push_back((int32_t)m->info_add_s.size());
        }
        m->info_place_off.push_back((int32_t)m->info_place_alive.size());
        for (const auto& x : fm.transfer[j]) {
            m->info_xfer_src.push_back(x.first);
            m->info_xfer_dst.push_back(x.second);
        }
        m->info_xfer_off.push_back((int32_t)m->info_xfer_src.size());
    }
}

// (Re)flatten the stored load inputs and reset every species-indexed option.
void flatten_into(cwc_model* m) {
    cwc::FlatModel fm = cwc::compile_model(m->in_alphabet, m->in_rules, m->in_rates, m->in_term, m->capacity);
    for (const auto& rl : fm.reactants)
        if ((int)rl.size() > CWC_MAX_REACTANTS)
            fail(CWC_E_UNSUPPORTED, "a flat reaction has more than CWC_MAX_REACTANTS reactant species");
    for (int32_t v : fm.x0)
        if (v > fm.x_cap_max) fail(CWC_E_INVALID, "initial count above the largest exact cap");
    m->fm = std::move(fm);
    m->x_cap = m->fm.x_cap_max;
    m->hist_lo.assign(m->fm.S(), 0);
    m->hist_width.assign(m->fm.S(), 1);
    m->period_species = -1;
    m->compiled_key.clear();
    refresh_info(m);
}

int species_index(const cwc_model* m, const std::string& name) {
    for (int s = 0; s < m->fm.S(); ++s)
        if (m->fm.names[s] == name) return s;
    fail(CWC_E_INVALID, "unknown species '" + name + "'");
}

}  // namespace

extern "C" {

const char* cwc_version(void) { return "cwc-b200 0.1 (sm_100a, NVRTC-specialised SSA)"; }

const char* cwc_last_error(void) { return g_err.c_str(); }

cwc_status cwc_model_load(cwc_model_t* out, int32_t n_species, const char* const* species, int32_t n_rules,
                          const char* const* rules, const double* rates, const char* initial_term) {
    return guard([&] {
        need(out != nullptr, "out is NULL");
        *out = nullptr;
        need(n_species > 0 && species != nullptr, "need at least one species");
        need(n_rules >= 0 && (n_rules == 0 || (rules != nullptr && rates != nullptr)), "bad rule arrays");
        need(initial_term != nullptr, "initial_term is NULL");
        std::vector<std::string> alpha, rs;
        std::vector<double> ks;
        for (int i = 0; i < n_species; ++i) {
            need(species[i] != nullptr, "NULL species name");
            alpha.emplace_back(species[i]);
        }
        for (int i = 0; i < n_rules; ++i) {
            need(rules[i] != nullptr, "NULL rule");
            rs.emplace_back(rules[i]);
            ks.push_back(rates[i]);
        }
        std::unique_ptr<cwc_model> m(new cwc_model());
        m->in_alphabet = alpha;
        m->in_rules = rs;
        m->in_rates = ks;
        m->in_term = initial_term;
        flatten_into(m.get());
        *out = m.release();
    });
}

void cwc_model_free(cwc_model_t m) {
    try {
        delete m;
    } catch (...) {
    }
}

cwc_status cwc_model_info(cwc_model_t m, cwc_model_info_t* out) {
    return guard([&] {
        need(m && out, "NULL argument");
        out->n_species = m->fm.S();
        out->n_reactions = m->fm.M();
        out->n_rules = m->fm.n_rules;
        out->species_names = m->name_ptrs.data();
        out->x0 = m->fm.x0.data();
        out->rates = m->fm.rates.data();
        out->n_reactants = m->info_nreact.data();
        out->reactant_species = m->info_rspecies.data();
        out->reactant_order = m->info_rorder.data();
        out->delta = m->info_delta.data();
        out->rule_of = m->fm.rule_of.data();
        out->x_cap = m->x_cap;
        out->x_cap_max = m->fm.x_cap_max;
        out->hist_bins = m->hist_bins;
        out->hist_lo = m->hist_lo.data();
        out->hist_width = m->hist_width.data();
        out->law = m->fm.law.data();
        out->law_species = m->fm.law_species.data();
        out->law_K = m->fm.law_K.data();
        out->law_n = m->fm.law_n.data();
        out->gate_species = m->fm.gate_species.data();
        out->gate_kind = m->fm.gate_kind.data();
        out->place_off = m->info_place_off.data();
        out->place_alive = m->info_place_alive.data();
        out->add_off = m->info_add_off.data();
        out->add_species = m->info_add_s.data();
        out->add_count = m->info_add_n.data();
        out->xfer_off = m->info_xfer_off.data();
        out->xfer_src = m->info_xfer_src.data();
        out->xfer_dst = m->info_xfer_dst.data();
        out->sentinel = m->fm.sentinel;
        out->flag = m->fm.flag.data();
    });
}

cwc_status cwc_set_option_i64(cwc_model_t m, const char* key, int64_t v) {
    return guard([&] {
        need(m && key, "NULL argument");
        std::string k(key);
        if (k.rfind("capacity.", 0) == 0) {
            need(v >= 1 && v <= 4096, "capacity outside [1, 4096]");
            const std::string label = k.substr(9);
            const auto old = m->capacity;
            m->capacity[label] = v;
            try {
                flatten_into(m);
            } catch (...) {
                m->capacity = old;
                flatten_into(m);
                throw;
            }
        } else if (k == "x_cap") {
            need(v >= 1 && v <= m->fm.x_cap_max, "x_cap outside [1, x_cap_max]");
            for (int32_t x : m->fm.x0) need(x <= v, "x_cap below an initial count");
            m->x_cap = v;
        } else if (k == "raw_samples") {
            need(v == 0 || v == 1, "raw_samples is 0 or 1");
            m->raw_samples = (int)v;
        } else if (k == "hist_bins") {
            need(v >= 1 && v <= (1 << 20), "hist_bins outside [1, 2^20]");
            m->hist_bins = (int)v;
        } else if (k == "hist_width") {
            need(v >= 1 && v <= (int64_t)1 << 40, "hist_width must be >= 1");
            m->hist_width.assign(m->fm.S(), v);
        } else if (k.rfind("hist_width.", 0) == 0) {
            need(v >= 1 && v <= (int64_t)1 << 40, "hist_width must be >= 1");
            m->hist_width[species_index(m, k.substr(11))] = v;
        } else if (k == "hist_lo") {
            need(std::llabs(v) <= (int64_t)1 << 40, "hist_lo out of range");
            m->hist_lo.assign(m->fm.S(), v);
        } else if (k.rfind("hist_lo.", 0) == 0) {
            need(std::llabs(v) <= (int64_t)1 << 40, "hist_lo out of range");
            m->hist_lo[species_index(m, k.substr(8))] = v;
        } else if (k == "quantum_samples") {
            need(v >= 0, "quantum_samples must be >= 0");
            m->quantum_samples = v;
        } else if (k == "block_threads") {
            need(v >= 32 && v <= 1024 && v % 32 == 0, "block_threads: multiple of 32 in [32, 1024]");
            m->block_threads = (int)v;
            m->block_auto = false;
        } else if (k == "period_species") {
            need(v >= -1 && v < m->fm.S(), "period_species: flat species index or -1");
            m->period_species = (int)v;
        } else if (k.rfind("period_species.", 0) == 0) {
            need(v == 0 || v == 1, "period_species.<name> is 0 or 1");
            const int s = species_index(m, k.substr(15));
            if (v) m->period_species = s;
            else if (m->period_species == s) m->period_species = -1;
        } else if (k == "period_lo") {
            need(std::llabs(v) <= (int64_t)1 << 40, "period_lo out of range");
            m->period_lo = v;
        } else if (k == "period_hi") {
            need(std::llabs(v) <= (int64_t)1 << 40, "period_hi out of range");
            m->period_hi = v;
        } else if (k == "period_window") {
            need(v >= 1 && v <= (int64_t)1 << 30, "period_window >= 1");
            m->period_window = (int)v;
        } else if (k == "delta_table") {
            need(v >= -1 && v <= 2, "delta_table is -1 (auto), 0 (select chain), 1 (table) or 2 (telescoped)");
            m->delta_table = (int)v;
        } else if (k == "stream") {
            need(v == 0 || v == 1, "stream is 0 or 1");
            m->stream = (int)v;
        } else if (k == "smem_stats") {
            need(v >= 0 && v <= 3, "smem_stats is 0 (global), 1 (auto), 2 (sparse) or 3 (dense)");
            m->smem_stats = (int)v;
        } else if (k == "draw_batch") {
            need(v == -1 || v == 0 || (v >= 2 && v <= 8), "draw_batch is -1 (auto), 0 or 2..8");
            m->draw_batch = (int)v;
        } else if (k == "raw_stage") {
            need(v == 0 || v == 1, "raw_stage is 0 or 1");
            m->raw_stage = (int)v;
        } else if (k == "ilp") {
            need(v == 1 || v == 2, "ilp is 1 or 2");
            m->ilp = (int)v;
        } else if (k == "fast_cut") {
            need(v >= -1 && v <= 1, "fast_cut is -1 (auto), 0 or 1");
            m->fast_cut = (int)v;
        } else if (k == "seed_jit") {
            need(v == 0 || v == 1, "seed_jit is 0 or 1");
            m->seed_jit = (int)v;
        } else if (k == "min_blocks") {
            need(v >= 0 && v <= 32, "min_blocks in [0, 32]");
            m->min_blocks = (int)v;
        } else if (k == "blocks_per_sm") {
            need(v >= 0 && v <= 64, "blocks_per_sm in [0, 64]");
            m->blocks_per_sm = (int)v;
        } else if (k == "refill") {
            need(v == 0 || v == 1, "refill is 0 or 1");
            m->refill = (int)v;
        } else if (k == "compact") {
            need(v == 0 || v == 1, "compact is 0 or 1");
            m->compact = (int)v;
        } else if (k == "device") {
            need(v >= -1 && v < 1024, "bad device ordinal");
            m->device = (int)v;
        } else {
            fail(CWC_E_INVALID, "unknown option '" + k + "'");
        }
    });
}

cwc_status cwc_set_quantiles(cwc_model_t m, int32_t n, const double* q) {
    return guard([&] {
        need(m && n >= 0 && (n == 0 || q), "bad quantile arguments");
        std::vector<double> v(q, q + n);
        for (double x : v) need(x >= 0 && x <= 1, "quantile levels must be in [0, 1]");
        m->quantiles = v;
    });
}

cwc_status cwc_model_compile(cwc_model_t m, const char** source, const char** log) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::compile(m);
        if (source) *source = m->source.c_str();
        if (log) *log = m->nvrtc_log.c_str();
    });
}

cwc_status cwc_kernel_attributes(cwc_model_t m, int32_t* regs, int32_t* local_bytes, int32_t* max_threads) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        if (m->cubin.empty()) fail(CWC_E_STATE, "kernel not compiled");
        if (regs) *regs = m->regs;
        if (local_bytes) *local_bytes = m->local_bytes;
        if (max_threads) *max_threads = m->max_threads;
    });
}

cwc_status cwc_kernel_image(cwc_model_t m, const void** image, size_t* bytes) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        if (m->cubin.empty()) fail(CWC_E_STATE, "kernel not compiled");
        if (image) *image = m->cubin.data();
        if (bytes) *bytes = m->cubin.size();
    });
}

cwc_status cwc_buffer_sizes(cwc_model_t m, int64_t count, double t_end, double dt, size_t* stats, size_t* raw,
                            size_t* scratch) {
    return guard([&] {
        need(m != nullptr && count >= 0, "bad arguments");
        int64_t K = cwc::grid_K(t_end, dt);
        cwc::buffer_sizes(m, count, K, stats, raw, scratch);
    });
}

cwc_status cwc_bind_device_buffers(cwc_model_t m, int64_t* stats, size_t stats_len, int32_t* raw, size_t raw_len,
                                   void* scratch, size_t scratch_bytes) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::bind_buffers(m, stats, stats_len, raw, raw_len, scratch, scratch_bytes);
    });
}

cwc_status cwc_simulate_range(cwc_model_t m, int64_t n_total, int64_t first, int64_t count, double t_end,
                              double dt, uint64_t seed, void* stream) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::simulate_range(m, n_total, first, count, t_end, dt, seed, (cudaStream_t)stream);
    });
}

cwc_status cwc_simulate(cwc_model_t m, int64_t n, double t_end, double dt, uint64_t seed) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::simulate_range(m, n, 0, n, t_end, dt, seed, nullptr, true);
        cwc::finalize(m, nullptr);
    });
}

cwc_status cwc_stats_device(cwc_model_t m, int64_t** dptr, size_t* n) {
    return guard([&] {
        need(m && dptr && n, "NULL argument");
        if (!m->simulated) fail(CWC_E_STATE, "no simulation yet");
        *dptr = m->d_stats;
        *n = m->last_stats_len;
    });
}

cwc_status cwc_stats_snapshot(cwc_model_t m, int64_t* cuts_final, int64_t* items_done) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::snapshot(m, cuts_final, items_done);
    });
}

cwc_status cwc_stats_host(cwc_model_t m, const int64_t** host_stats, size_t* n_int64) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        if (m->h_stats.empty()) fail(CWC_E_STATE, "no snapshot / finalize yet");
        if (host_stats) *host_stats = m->h_stats.data();
        if (n_int64) *n_int64 = m->h_stats.size();
    });
}

cwc_status cwc_stats_load(cwc_model_t m, const int64_t* host_stats, int64_t cuts_final) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::load_host_stats(m, host_stats, cuts_final);
    });
}

cwc_status cwc_resume(cwc_model_t m, void* cuda_stream) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::resume(m, (cudaStream_t)cuda_stream);
    });
}

cwc_status cwc_checkpoint_bytes(cwc_model_t m, size_t* bytes) {
    return guard([&] {
        need(m != nullptr && bytes != nullptr, "bad arguments");
        *bytes = cwc::checkpoint_bytes(m);
    });
}

cwc_status cwc_checkpoint_save(cwc_model_t m, void* out, size_t bytes) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::checkpoint_save(m, out, bytes);
    });
}

cwc_status cwc_checkpoint_load(cwc_model_t m, const void* in, size_t bytes) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::checkpoint_load(m, in, bytes);
    });
}

cwc_status cwc_cancel(cwc_model_t m) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::cancel(m);
    });
}

cwc_status cwc_stats_finalize(cwc_model_t m, const int64_t* host_stats) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::finalize(m, host_stats);
    });
}

cwc_status cwc_stats(cwc_model_t m, cwc_stats_t* out) {
    return guard([&] {
        need(m && out, "NULL argument");
        if (!m->finalized) fail(CWC_E_STATE, "call cwc_stats_finalize after simulating");
        const int64_t T = m->K + 1;
        const int S = m->fm.S();
        std::memset(out, 0, sizeof *out);
        out->T = (int32_t)T;
        out->S = S;
        out->B = m->hist_bins;
        out->n_q = (int32_t)m->quantiles.size();
        out->times = m->times.data();
        out->n = m->h_n.data();
        out->sum = m->h_sum.data();
        out->sumsq = m->sumsq_d.data();
        out->sqlo = m->h_sqlo.data();
        out->sqhi = m->h_sqhi.data();
        out->mean = m->mean.data();
        out->var = m->var.data();
        out->hist = m->h_hist.data();
        out->hist_lo = m->hist_lo.data();
        out->hist_width = m->hist_width.data();
        out->q = m->quantiles.data();
        out->quantile = m->quant.data();
        const int64_t* ctr = m->h_stats.data() + T * (1 + 3 * (int64_t)S + (int64_t)S * (m->hist_bins + 2));
        out->reactions = ctr[CWC_CTR_REACTIONS];
        out->absorbed = ctr[CWC_CTR_ABSORBED];
        out->overflowed = ctr[CWC_CTR_OVERFLOWED];
        out->finished = ctr[CWC_CTR_FINISHED];
        out->pool_full = ctr[CWC_CTR_POOL_FULL];
        out->launches = m->launches;
        out->raw_staged = m->raw_stage_now;
        out->kernel_ms = m->kernel_ms;
        out->cuts_final = m->cuts_final;
        out->species_names = m->name_ptrs.data();
    });
}

cwc_status cwc_period_stats(cwc_model_t m, cwc_period_stats_t* out) {
    return guard([&] {
        need(m && out, "NULL argument");
        if (!m->finalized) fail(CWC_E_STATE, "call cwc_stats_finalize after simulating");
        if (m->h_period.empty()) fail(CWC_E_STATE, "period analysis was off for the last simulation");
        const int64_t T = m->K + 1;
        const int64_t* q = m->h_period.data();
        std::memset(out, 0, sizeof *out);
        out->T = (int32_t)T;
        out->species = m->period_species;
        out->window = m->period_window;
        out->lo = m->period_lo;
        out->hi = m->period_hi;
        out->events = q;
        out->pc_n = q + T;
        out->pc_sum = q + 2 * T;
        out->pc_sqlo = q + 3 * T;
        out->pc_sqhi = q + 4 * T;
        out->lp_n = q + 5 * T;
        out->lp_sum = q + 6 * T;
        out->lp_sqlo = q + 7 * T;
        out->lp_sqhi = q + 8 * T;
        out->lp_mean = m->lp_mean.data();
        out->lp_var = m->lp_var.data();
        out->moving_avg = m->p_ma.data();
    });
}

cwc_status cwc_samples(cwc_model_t m, int64_t first, int64_t count, int32_t* out) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::copy_samples(m, first, count, out);
    });
}

cwc_status cwc_instance_records(cwc_model_t m, int64_t first, int64_t count, uint8_t* flags, int64_t* reactions,
                                double* t_last) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        cwc::copy_records(m, first, count, flags, reactions, t_last);
    });
}

cwc_status cwc_selftest_philox(int64_t n, const uint32_t* ctr, const uint32_t* key, uint32_t* out) {
    return guard([&] {
        need(n >= 0 && (n == 0 || (ctr && key && out)), "bad arguments");
        cwc::selftest_philox(n, ctr, key, out);
    });
}

cwc_status cwc_selftest_log(int64_t n, const double* x, double* out) {
    return guard([&] {
        need(n >= 0 && (n == 0 || (x && out)), "bad arguments");
        cwc::selftest_log(n, x, out);
    });
}

cwc_status cwc_selftest_div(int64_t n, const double* num, const double* den, double* out) {
    return guard([&] {
        need(n >= 0 && (n == 0 || (num && den && out)), "bad arguments");
        cwc::selftest_div(n, num, den, out);
    });
}

cwc_status cwc_selftest_u01(int64_t n, const uint32_t* w, double* out) {
    return guard([&] {
        need(n >= 0 && (n == 0 || (w && out)), "bad arguments");
        cwc::selftest_u01(n, w, out);
    });
}

cwc_status cwc_selftest_step(cwc_model_t m, int64_t n, int32_t n_draws, const int32_t* x, const double* t,
                             const int64_t* k, double t_end, double sample_dt, const double* u_tau,
                             const double* u_sel, int32_t mode, int32_t* x_out, double* t_out, int64_t* k_out,
                             int32_t* status, int32_t* n_done, int32_t* cuts) {
    return guard([&] {
        need(m != nullptr, "NULL model");
        need(n >= 0 && (n == 0 || (x && t && k && u_tau && u_sel && x_out && t_out && k_out && status && n_done)),
             "bad arguments");
        cwc::selftest_step(m, n, n_draws, x, t, k, t_end, sample_dt, u_tau, u_sel, mode, x_out, t_out, k_out, status,
                           n_done, cuts);
    });
}

}  // extern "C"
