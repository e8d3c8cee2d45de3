// runtime.hpp — the model handle behind cwc_model_t and its device-side runtime.
#pragma once

#include <cuda.h>
#include <cuda_runtime.h>

#include <map>
#include <string>
#include <vector>

#include "codegen.hpp"
#include "compiler.hpp"
#include "device/cwc_params.h"

struct cwc_model {
    cwc::FlatModel fm;
    // load inputs, kept so that "capacity.<label>" can re-flatten (reading R20)
    std::vector<std::string> in_alphabet, in_rules;
    std::vector<double> in_rates;
    std::string in_term;
    std::map<std::string, int64_t> capacity;

    // options (cwc.h)
    int64_t x_cap = 0;
    int raw_samples = 1;
    int hist_bins = 256;
    int seed_jit = 0;
    std::vector<int64_t> hist_lo, hist_width;
    int64_t quantum_samples = 0;
    bool block_auto = true;               // CTA size chosen per launch (until block_threads is set)
    int block_threads = 768;  // one 24-warp CTA per SM (measured best: LV 1.13 vs 1.21 s at 3 x 256)
    int min_blocks = 0;
    int ilp = 1;
    int delta_table = -1;
    int smem_stats = 1;
    int draw_batch = -1;                  // draws per inner-loop trip (0, 2..8; -1 auto)
    int raw_stage = 1;                    // raw-cut staging in shared memory (1 = when it fits)
    int raw_stage_now = 0;                // whether the last launch staged
    // cut recording inside the fast step (1) or on the full-step path (0); -1 = auto: by the
    // reactions per recorded cut of the last simulation on this handle (else a0(x0) * dt)
    int fast_cut = -1;
    double last_reactions_per_cut = 0;
    bool fast_cut_now = true;             // the mode of the kernel being compiled / launched
    // on-line period analysis (reading R19): observable species (-1 = off), Schmitt thresholds,
    // moving-average window in cuts
    int period_species = -1;
    int64_t period_lo = 0, period_hi = 1;
    int period_window = 1;
    int stream = 0;                       // on-line streaming: progress counters + snapshots
    bool cancel_requested = false;        // cwc_cancel on the running simulation
    bool resumable = false;               // terminated (or restored) run that cwc_resume can continue
    cudaStream_t poll_stream = nullptr;   // copy-engine stream for snapshots
    int64_t cuts_final = 0;               // cuts final in the host views (T after finalize)
    int blocks_per_sm = 0;
    int refill = 1;
    // compacted per-quantum launches (0 off, 1 on): one launch per quantum over the instances
    // still running, refill inside the launch, a compaction kernel between launches.  Measured
    // slower than the single persistent launch in the under-filled regime it targets (the launch
    // boundaries cost more than the handed-back lanes gain: LV 100k 1.41e11 -> 1.21e11,
    // profiles/r2_ab_quanta_launch.log), so an ablation mode only
    int compact = 0;
    int launches = 0;                     // SSA + compaction kernels of the last simulate
    int device = -1;
    std::vector<double> quantiles{0.05, 0.25, 0.5, 0.75, 0.95};

    // flat-view storage for cwc_model_info
    std::vector<const char*> name_ptrs;
    std::vector<int32_t> info_nreact, info_rspecies, info_rorder, info_delta;
    std::vector<int32_t> info_place_off, info_place_alive, info_add_off, info_add_s, info_add_n, info_xfer_off,
        info_xfer_src, info_xfer_dst;

    // compiled kernel
    std::string source, nvrtc_log, compiled_key;
    std::vector<char> cubin;
    int regs = -1, local_bytes = -1, max_threads = -1;
    CUmodule module = nullptr;
    CUfunction function = nullptr;
    CUfunction compact_fn = nullptr;
    int module_device = -1;

    // device buffers (owned or bound)
    int64_t* d_stats = nullptr;
    size_t stats_cap = 0;
    int32_t* d_raw = nullptr;
    size_t raw_cap = 0;
    void* d_scratch = nullptr;
    size_t scratch_cap = 0;
    bool bound = false;
    cwc_logtab_entry* d_logtab = nullptr;
    int logtab_device = -1;
    cudaStream_t own_stream = nullptr;
    cudaEvent_t ev0 = nullptr, ev1 = nullptr;

    // last simulated geometry
    bool simulated = false;
    cudaStream_t last_stream = nullptr;
    int64_t n_total = 0, first = 0, count = 0, K = 0;
    double dt = 0, t_end = 0;
    uint64_t seed = 0;
    size_t last_stats_len = 0;
    int64_t items = 0, qs = 0;
    int grid = 0;

    // host results (cwc_stats)
    bool finalized = false;
    std::vector<int64_t> h_stats;
    std::vector<double> times, mean, var, sumsq_d, quant;
    std::vector<int64_t> h_n, h_sum, h_sqlo, h_sqhi, h_hist;
    std::vector<int64_t> h_period;             // CWC_N_PERIOD x T (R19)
    std::vector<double> lp_mean, lp_var, p_ma;  // [T]
    double kernel_ms = 0;

    ~cwc_model();
};

namespace cwc {

size_t stats_len(int64_t T, int S, int B, bool period);
void buffer_sizes(const cwc_model* m, int64_t count, int64_t K, size_t* stats, size_t* raw, size_t* scratch);
void compile(cwc_model* m, const uint64_t* seed = nullptr);  // NVRTC (no GPU needed)
void simulate_range(cwc_model* m, int64_t n_total, int64_t first, int64_t count, double t_end, double dt,
                    uint64_t seed, cudaStream_t stream, bool own_stream = false, bool resume = false);
void resume(cwc_model* m, cudaStream_t stream);
size_t checkpoint_bytes(cwc_model* m);
void checkpoint_save(cwc_model* m, void* out, size_t bytes);
void checkpoint_load(cwc_model* m, const void* in, size_t bytes);
void finalize(cwc_model* m, const int64_t* host_stats);
void snapshot(cwc_model* m, int64_t* cuts_final, int64_t* items_done);
void cancel(cwc_model* m);
void load_host_stats(cwc_model* m, const int64_t* host_stats, int64_t cuts_final);
void bind_buffers(cwc_model* m, int64_t* stats, size_t stats_n, int32_t* raw, size_t raw_n, void* scratch,
                  size_t scratch_bytes);
void copy_samples(cwc_model* m, int64_t first, int64_t count, int32_t* out);
void copy_records(cwc_model* m, int64_t first, int64_t count, uint8_t* flags, int64_t* reactions, double* t_last);
int64_t grid_K(double t_end, double dt);  // R13, throws CWC_E_INVALID

void selftest_philox(int64_t n, const uint32_t* ctr, const uint32_t* key, uint32_t* out);
void selftest_log(int64_t n, const double* x, double* out);
void selftest_u01(int64_t n, const uint32_t* words, double* out);
void selftest_div(int64_t n, const double* num, const double* den, double* out);
void build_log_table(cwc_logtab_entry* tab);
void selftest_step(cwc_model* m, int64_t n, int32_t n_draws, const int32_t* x, const double* t, const int64_t* k,
                   double t_end, double dt, const double* u_tau, const double* u_sel, int32_t mode, int32_t* x_out,
                   double* t_out, int64_t* k_out, int32_t* status, int32_t* n_done, int32_t* cuts);

}  // namespace cwc
