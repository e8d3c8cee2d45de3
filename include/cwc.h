/*
 * cwc.h — C ABI of the B200-native CWC ensemble stochastic simulator.
 *
 * The operation (PAPER.md = Aldinucci et al., ICDCS-W 2014, /root/reference/PAPER.md):
 *   - a CWC model: an alphabet of atoms, multisets of atoms and compartments, labelled
 *     rewrite rules local to a compartment or across compartments           P:L203-215 (§IV)
 *   - Gillespie's stochastic simulation algorithm on CWC terms              P:L216-226 (§IV), ref [1]
 *   - a Monte Carlo ensemble of independent instances ("trajectories")      P:L47-52 (§I)
 *   - cuts of all trajectories at fixed simulation times, analysed on line
 *     by statistical estimators (mean, variance; histograms/quantiles)      P:L244-252 (§IV.A)
 *   - simulation quanta and load re-balancing on the GPU                     P:L300-317 (§IV.C)
 * Readings of what the paper leaves open (R1-R18) are listed in DESIGN.md §3; the numeric
 * contract (Philox stream, CWC-log, evaluation order, sampling convention) is R3-R7.
 *
 * Conventions
 *   - Every function returns a cwc_status; CWC_OK == 0.  On error a thread-local message is
 *     available from cwc_last_error() until the next cwc_* call on that thread.  No function
 *     throws across the ABI.
 *   - "host" pointers are ordinary CPU memory; "device" pointers are CUDA global memory of
 *     the model's device.  All input arrays/strings are borrowed for the duration of the call
 *     and copied; no pointer passed in is retained unless stated ("bound" buffers).
 *   - Handles are not thread safe: one thread at a time per cwc_model_t.
 *   - There is no CPU fallback.  Without a usable CUDA device, simulate calls return
 *     CWC_E_CUDA; model loading, flattening and kernel code generation (NVRTC) work without one.
 */
#ifndef CWC_H_
#define CWC_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef int32_t cwc_status;
#define CWC_OK 0
#define CWC_E_INVALID 1     /* bad argument / value (null, negative, NaN, unknown atom, ...) */
#define CWC_E_PARSE 2       /* syntax error in a term or rule */
#define CWC_E_UNSUPPORTED 3 /* valid CWC outside the hot path: reaction order > 3, closed
                               membrane patterns, moved variables, nested dynamic compartments,
                               more than one compartment created by a rule (reading R20) */
#define CWC_E_CUDA 4        /* CUDA / NVRTC / driver failure, or no device */
#define CWC_E_OOM 5         /* device allocation failed */
#define CWC_E_STATE 6       /* call out of order (e.g. stats before any simulation) */

/* Per-instance flags (reading R8/R9). 0 = reached t_end. */
#define CWC_FLAG_ABSORBED 1   /* a0 == 0: state held to t_end */
#define CWC_FLAG_OVERFLOWED 2 /* a count exceeded x_cap, or a compartment pool was full when a
                                 rule created a compartment (R20): frozen, later samples -1 */

typedef struct cwc_model* cwc_model_t;

/* ------------------------------------------------------------------------------------------
 * Model loading — P:L203-215.
 *   species      [n_species] atom names (the alphabet), [A-Za-z_][A-Za-z0-9_]*; their order is
 *                the species order inside each region of the flat model.
 *   rules        [n_rules] strings "label: lhs -> rhs"; label = "top" or a compartment label.
 *                lhs/rhs: atoms, "n*A", "." (empty), compartments "(wrap $x | content $X)^label".
 *                Rule order is the selection order (R6).
 *   rates        [n_rules] mass-action rate constants, finite and >= 0.
 *   initial_term e.g. "500*L (100*R | (. | 2*G)^nuc)^cell".
 * The static compartment structure is flattened at load (DESIGN.md §3 "flattening"): one flat
 * species per (region, atom), one flat reaction per (rule, context, compartment assignment).
 * Dynamic compartments (reading R20): a rule may create one compartment, written as
 * a ground rhs compartment "(wrap | content)^label" without variables, and may destroy pattern
 * compartments that do not reappear on its rhs; "$x" / "$X" of a destroyed compartment written
 * at rule level on the rhs release its remaining wrap / content into the rule's context, else
 * they vanish.  Compartments of a label some rule creates or destroys ("dynamic" labels) are
 * leaves (atoms only) and live in bounded pools: capacity.<label> slots (default 8) per region
 * that holds them, each slot with an occupancy flag species "#alive@<path>", each pool with a
 * free-slot counter "#free:<label>[@<path>]"; a creation takes the lowest free slot, and a
 * creation at a full pool sets "#full" and freezes the instance as CWC_FLAG_OVERFLOWED.
 * *out receives a library-owned handle (free with cwc_model_free).
 * Errors: CWC_E_INVALID, CWC_E_PARSE, CWC_E_UNSUPPORTED.
 * ---------------------------------------------------------------------------------------- */
cwc_status cwc_model_load(cwc_model_t* out, int32_t n_species, const char* const* species,
                          int32_t n_rules, const char* const* rules, const double* rates,
                          const char* initial_term);

/* Release a handle and every device buffer it owns.  NULL is a no-op. */
void cwc_model_free(cwc_model_t m);

/* Thread-local message of the last failing call ("" if none).  Valid until the next call. */
const char* cwc_last_error(void);

/* Flat view of a loaded model.  All pointers are borrowed views owned by the handle, valid
 * until cwc_model_free (or a cwc_set_option that changes x_cap / histogram layout / capacity).
 *   reactant_species/order: [n_reactions][CWC_MAX_REACTANTS], entries beyond n_reactants[j]
 *                           are 0.
 *   delta: [n_reactions][n_species] dense net change nu_j (row-major).
 * Reading R20 (dynamic compartments; see cwc_model_load), per flat reaction j:
 *   gate_species[j]/gate_kind[j]  -1/0, or a species g with kind 1 (enabled while x_g >= 1: a
 *                                 creation) or 2 (enabled while x_g == 0: its pool is full);
 *                                 the propensity is multiplied by that 0/1 condition.
 *   place_off[j]..place_off[j+1]  candidate slots of a creation, in order: slot p has the
 *                                 occupancy flag place_alive[p] and the additions
 *                                 add_species/add_count[add_off[p]..add_off[p+1]); after
 *                                 x += nu_j the first slot with flag 0 receives its additions.
 *   xfer_off[j]..xfer_off[j+1]    moves of a destruction, after x += nu_j: x[xfer_dst] +=
 *                                 x[xfer_src] (xfer_dst >= 0), then x[xfer_src] = 0.
 *   sentinel                      species "#full" or -1; flag[s] = 1 for occupancy flags. */
#define CWC_MAX_REACTANTS 8
typedef struct {
    int32_t n_species;
    int32_t n_reactions;
    int32_t n_rules;
    const char* const* species_names; /* "A", "R@cell.wrap", "S@cell/nuc", ... */
    const int32_t* x0;
    const double* rates;
    const int32_t* n_reactants;
    const int32_t* reactant_species;
    const int32_t* reactant_order;
    const int32_t* delta;
    const int32_t* rule_of;           /* originating rule index of each flat reaction */
    int64_t x_cap;                    /* current cap (R9) */
    int64_t x_cap_max;                /* largest cap keeping every propensity count < 2^53 */
    int32_t hist_bins;                /* B */
    const int64_t* hist_lo;           /* [n_species] */
    const int64_t* hist_width;        /* [n_species] */
    /* functional rate laws (reading R16'; rule suffix "@ mm(X, K)", "@ hill(X, K, n)",
     * "@ hillr(X, K, n)"): per flat reaction 0 mass action / 1 mm / 2 hill / 3 hillr, the
     * flat species the law reads (-1 for mass action), K and n. */
    const int32_t* law;
    const int32_t* law_species;
    const double* law_K;
    const int32_t* law_n;
    const int32_t* gate_species;      /* [n_reactions] (R20) */
    const int32_t* gate_kind;
    const int32_t* place_off;         /* [n_reactions + 1] */
    const int32_t* place_alive;       /* [place_off[n_reactions]] */
    const int32_t* add_off;           /* [place_off[n_reactions] + 1] */
    const int32_t* add_species;
    const int32_t* add_count;
    const int32_t* xfer_off;          /* [n_reactions + 1] */
    const int32_t* xfer_src;
    const int32_t* xfer_dst;
    int32_t sentinel;
    const uint8_t* flag;              /* [n_species] */
} cwc_model_info_t;
cwc_status cwc_model_info(cwc_model_t m, cwc_model_info_t* out);

/* ------------------------------------------------------------------------------------------
 * Options (cwc_set_option_i64 unless noted).  Keys:
 *   "capacity.<label>"   slots per pool of a dynamic compartment label, [1, 4096] (R20).
 *                        Re-flattens the model: set it first (species-indexed options such as
 *                        hist_width.<name>, period_species and x_cap are reset).   default 8
 *   "x_cap"              1 <= v <= x_cap_max (R9).                       default x_cap_max or model's
 *   "raw_samples"        0/1: keep the raw int32 sample buffer (cwc_samples).       default 1
 *   "hist_bins"          B >= 1 in-range bins per (time, species).               default 256
 *   "hist_width"         bin width >= 1 for every species;  "hist_width.<species name>" for one.
 *   "hist_lo"            left edge of bin 1 for every species; "hist_lo.<species name>" for one.
 *   "quantum_samples"    sample points per simulation quantum (Q/tau); 0 = auto:
 *                        whole trajectories up to one instance per resident lane, else 32
 *                        (up to 4 per lane) or 8 quanta, rounded up to a multiple of 8 cuts.
 *                        Scheduling only: results are bit-identical for every value (R12).
 *   "block_threads"      CUDA block size (multiple of 32, <= 1024).  Default: auto per launch —
 *                        768 (80 registers) from 1.5 instances per resident lane up, else 512
 *                        (113 registers; the instances then exceed the lanes and quanta balance
 *                        the load).
 *   "blocks_per_sm"      persistent CTAs per SM; 0 = occupancy maximum.          default 0
 *   "min_blocks"         register budget: __launch_bounds__ min CTAs per SM; 0 = auto
 *                        (768 / block_threads, i.e. <= 80 registers).
 *   "ilp"                1/2 instances interleaved per thread (ablation knob).      default 1
 *   "stream"             0/1: on-line streaming — progress counters + cwc_stats_snapshot.
 *   "smem_stats"         where the cut statistics accumulate before the flush to the packed
 *                        buffer: 0 global memory only; 2 sparse per-CTA shared counters (u32,
 *                        16-bit limbs, zero counts restored at the flush; T*(1+7S)*4 bytes); 3
 *                        dense per-CTA shared moments (u64, T*(1+3S)*8 bytes); 1 auto = sparse,
 *                        else dense, else global — each only when it fits without lowering
 *                        residency.  Results are bit-identical.                  default 1
 *   "draw_batch"         -1/0/2..8: draws per inner-loop trip — the Philox blocks and CWC-logs of
 *                        the next D steps as D independent chains, then D fast steps (0: the
 *                        next draw inside each fast step); -1 = auto: 4 up to 8 species, 3 up to
 *                        16, else 0.  Performance only: results are bit-identical.   default -1
 *   "raw_stage"          0/1: a lane collects the 8 cuts of one 32-byte block of the raw layout in
 *                        shared memory and writes the block as whole sectors (1: when it fits
 *                        without lowering residency and ilp = 1).  Results are bit-identical.
 *                                                                                   default 1
 *   "fast_cut"           -1/0/1: where cuts are recorded — inside the fast step (1) or on the
 *                        full-step path (0); -1 = auto: 0 when the last simulation on this handle
 *                        (else a0(x0)*sample_dt) had >= 1000 reactions per recorded cut.
 *                        Performance only: results are bit-identical.             default -1
 *   "seed_jit"           0/1: specialise the kernel on the seed (Philox round keys become
 *                        instruction immediates; one NVRTC compile per new seed, cached).
 *   "compact"            0/1: compacted per-quantum launches — one launch per simulation quantum
 *                        over the instances still running (a compaction kernel between launches),
 *                        refill inside each launch (ablation: measured slower than the single
 *                        persistent launch).  Scheduling only: results are bit-identical (R12).
 *                                                                                   default 0
 *   "refill"             0/1: warp-level refill from the global work queue.      default 1
 *                        0 = static assignment: whole trajectories, or with quantum_samples > 0
 *                        the paper's GPU scheme: one launch per simulation quantum,
 *                        every lane running quantum q of its instance, launches as barriers.
 *   "device"             CUDA device ordinal.                                    default current
 * cwc_set_quantiles(m, n, q): quantile levels in [0,1] (R11), default {.05,.25,.5,.75,.95}.
 * Errors: CWC_E_INVALID (unknown key / bad value).
 * ---------------------------------------------------------------------------------------- */
cwc_status cwc_set_option_i64(cwc_model_t m, const char* key, int64_t value);
cwc_status cwc_set_quantiles(cwc_model_t m, int32_t n, const double* q);

/* Generate the model-specialised CUDA translation unit and compile it with NVRTC for sm_100a
 * (cached per process and on disk by source hash).  Works without a GPU.  simulate calls it
 * implicitly.  *source/*log (optional, may be NULL) receive borrowed views of the generated
 * source and the NVRTC log. */
cwc_status cwc_model_compile(cwc_model_t m, const char** source, const char** log);
/* Compiled SASS-level facts of the last compile: registers/thread, local (spill) bytes. */
cwc_status cwc_kernel_attributes(cwc_model_t m, int32_t* regs, int32_t* local_bytes,
                                 int32_t* max_threads);
/* The compiled sm_100a kernel image (cubin) the module is loaded from: a borrowed view, valid
 * until the next compile or cwc_model_free; either pointer may be NULL.  CWC_E_STATE before the
 * first compile. */
cwc_status cwc_kernel_image(cwc_model_t m, const void** image, size_t* bytes);

/* ------------------------------------------------------------------------------------------
 * Device buffers.  By default the handle allocates what it needs.  A caller that owns device
 * memory (PyTorch) may bind its own buffers instead; they must stay valid while bound.
 *   stats   int64[stats_len]   packed ensemble statistics (layout below)
 *   raw     int32[raw_len]     raw samples (only if raw_samples = 1), time-blocked SoA
 *                              [ceil(T/8)][S][count][8]: cut k of species s of local instance i
 *                              at ((k/8*S + s)*count + i)*8 + k%8 (cwc_samples returns [T][S][count])
 *   scratch bytes              per-instance state + work queue
 * cwc_buffer_sizes reports the sizes one cwc_simulate_range(count, t_end, dt) needs.
 * Passing NULL pointers to cwc_bind_device_buffers unbinds (back to library allocation).
 * ---------------------------------------------------------------------------------------- */
cwc_status cwc_buffer_sizes(cwc_model_t m, int64_t count, double t_end, double sample_dt,
                            size_t* stats_len, size_t* raw_len, size_t* scratch_bytes);
cwc_status cwc_bind_device_buffers(cwc_model_t m, int64_t* stats, size_t stats_len, int32_t* raw,
                                   size_t raw_len, void* scratch, size_t scratch_bytes);

/* ------------------------------------------------------------------------------------------
 * Simulation — the hot path.  PAPER.md: "Monte Carlo methods applied to a number of independent
 * instances ... an embarrassingly parallel problem: ... groups of instances can be executed
 * independently" (§I); each instance is a trajectory of "the Gillespie algorithm on CWC
 * terms" (§IV); trajectories are cut "at a given simulation time" and the
 * cuts analysed on line (§IV.A.1-2); simulation quanta with re-scheduling (P:L241-243,
 * §IV.A.1; GPU variant P:L300-317, §IV.C); one ff_mapCUDA per GPU = one shard per device
 * (P:L304-305).  Readings R1-R15 fix what the paper leaves open.
 * cwc_simulate_range simulates the global instances [first, first+count) of an ensemble of
 * n_total instances, from t = 0 to t_end, sampling at t_k = fl(k*sample_dt), k = 0..K,
 * K = llround(t_end/sample_dt) (R7, R13).  Instance i uses the Philox stream keyed by
 * (seed, i) (R3), so any sharding of [0, n_total) gives bit-identical trajectories and
 * statistics.  The packed stats buffer is zeroed and filled by the call.
 * The work is enqueued on cuda_stream (a cudaStream_t; NULL = the legacy default stream) and
 * the call returns without waiting; results are valid once the stream has drained
 * (cwc_stats_finalize / cwc_samples / cwc_instance_records synchronise it).
 * cwc_simulate(m, n, t_end, dt, seed) == cwc_simulate_range(m, n, 0, n, ...) on the handle's
 * own stream followed by cwc_stats_finalize (synchronous).
 * Errors: CWC_E_INVALID (n_total <= 0, count < 0, first+count > n_total, count >= 2^31, t_end < 0,
 *         sample_dt <= 0, |K*dt - t_end| > 1e-9*max(1,t_end), buffers too small);
 *         CWC_E_OOM; CWC_E_CUDA.
 * ---------------------------------------------------------------------------------------- */
cwc_status cwc_simulate(cwc_model_t m, int64_t n_instances, double t_end, double sample_dt,
                        uint64_t seed);
cwc_status cwc_simulate_range(cwc_model_t m, int64_t n_total, int64_t first, int64_t count,
                              double t_end, double sample_dt, uint64_t seed, void* cuda_stream);

/* Packed int64 statistics buffer — the per-cut "statistical estimators (mean, variance ...)"
 * of the analysis pipeline (Fig. 2; on-line estimators P:L689-691; every cut "can be
 * analysed immediately and independently" P:L249-251) and the cut histograms of GPU ensemble
 * tools, accumulated exactly inside the SSA kernel; summed over devices for the
 * multi-GPU combine (one ff_mapCUDA per GPU).  T = K+1 cuts, S species, B bins (all exact integers,
 * order-independent; a sum of buffers = the buffer of the union of instance ranges):
 *   [0, T)                       n[k]            instances present at cut k
 *   [T, T+TS)                    sum[k][s]       sum of x
 *   [T+TS, T+2TS)                sqlo[k][s]      sum of (x^2 mod 2^32)
 *   [T+2TS, T+3TS)               sqhi[k][s]      sum of (x^2 >> 32)       sum x^2 = sqhi*2^32 + sqlo
 *   [T+3TS, T+3TS+TS(B+2))       hist[k][s][b]   b=0 underflow, 1..B bins, B+1 overflow
 *   then 8 counters:             reactions, absorbed, overflowed, finished instances, pool_full, 0...
 *                                (pool_full: the overflowed instances frozen because a compartment pool
 *                                was full, reading R20 — their later cuts are missing; a run with
 *                                pool_full > 0 under-represents compartment-rich trajectories, so the
 *                                Python API re-runs it with doubled capacities, see cwc_stats_t)
 */
#define CWC_CTR_REACTIONS 0
#define CWC_CTR_ABSORBED 1
#define CWC_CTR_OVERFLOWED 2
#define CWC_CTR_FINISHED 3
#define CWC_CTR_POOL_FULL 4
#define CWC_N_CTR 8
/* With period analysis on ("period_species" >= 0), CWC_N_PERIOD arrays of T int64 follow the
 * counters: events, completed periods n / sum / sq_lo / sq_hi, local period n / sum / sq_lo /
 * sq_hi (periods in cuts; sq split like sqlo/sqhi). */
#define CWC_N_PERIOD 9
cwc_status cwc_stats_device(cwc_model_t m, int64_t** dptr, size_t* n_int64);

/* Synchronise, copy the packed stats to the host and derive mean, variance (n-1; int128
 * numerator; NaN if n < 2) and inverted-CDF quantiles (R10, R11) — the "mean, variance" engines
 * of the analysis stage.  If host_stats is non-NULL
 * the packed buffer is taken from it instead (e.g. after an NCCL all-reduce done by the
 * caller into host memory); it must hold stats_len int64 for the last simulated geometry. */
cwc_status cwc_stats_finalize(cwc_model_t m, const int64_t* host_stats);

/* On-line streaming ("once all simulation tasks overcome a
 * given simulation time, an array of results is produced and streamed").  With the
 * option "stream" = 1 the kernel runs in ~16 simulation quanta and counts finished items per
 * quantum; while it is still running, cwc_stats_snapshot copies the progress counters and then
 * the statistics through a copy engine on a separate stream (no synchronisation with the
 * simulation) and derives the cwc_stats views; cuts [0, *cuts_final) of that snapshot are final
 * (identical to the finished run's), later cuts are partial.  *items_done (optional) = finished
 * work items.  Moments then accumulate in global memory (no CTA-local staging).
 * Errors: CWC_E_STATE without a simulation or without "stream". */
cwc_status cwc_stats_snapshot(cwc_model_t m, int64_t* cuts_final, int64_t* items_done);
/* Terminate the running simulation (Fig. 2, "start new simulations, steer and
 * terminate running simulations"; "stream" option only).  The kernel stops handing out work
 * items; items in flight finish their quantum.  Returns without waiting; cwc_stats_finalize then
 * waits for the kernel and reports in cuts_final the prefix of cuts every instance reached (those
 * statistics are exact; later cuts are partial).  Errors: CWC_E_STATE without a streaming
 * simulation. */
cwc_status cwc_cancel(cwc_model_t m);

/* Checkpoint / resume (the paper's tasks are resumable at quantum boundaries,
 * P:L241-243).  Because the RNG is counter-based (R3), the per-instance records (x, t, step, k,
 * flags, period state) and the quanta each instance has done are a complete checkpoint: a resumed
 * run is bit-identical to the uninterrupted one.
 *   cwc_checkpoint_bytes / _save: after the last simulation's kernel has finished (it synchronises)
 *     — statistics, instance records, queue state and raw cuts into a caller-owned host buffer.
 *   cwc_checkpoint_load: into a handle of the same model and result-affecting options (flat
 *     network, histogram, x_cap, raw_samples, period analysis — checked by hash); the run can
 *     then be continued or finalised as it stands.
 *   cwc_resume: continue a run ended by cwc_cancel, or restored, to its horizon on cuda_stream
 *     (NULL = legacy default stream; asynchronous); quanta already done are skipped.
 * Errors: CWC_E_STATE (nothing simulated / nothing to resume), CWC_E_INVALID (buffer too small,
 * not a checkpoint, other model or geometry), CWC_E_CUDA. */
cwc_status cwc_checkpoint_bytes(cwc_model_t m, size_t* bytes);
cwc_status cwc_checkpoint_save(cwc_model_t m, void* out, size_t bytes);
cwc_status cwc_checkpoint_load(cwc_model_t m, const void* in, size_t bytes);
cwc_status cwc_resume(cwc_model_t m, void* cuda_stream);
/* The packed statistics (layout above) behind the current cwc_stats views, as copied by the last
 * snapshot or finalize: a borrowed host view valid until the next snapshot / finalize / load /
 * simulate / free.  CWC_E_STATE before the first snapshot or finalize. */
cwc_status cwc_stats_host(cwc_model_t m, const int64_t** host_stats, size_t* n_int64);
/* Replace the host statistics by a packed buffer of the last simulation's geometry (copied) and
 * re-derive the cwc_stats views with cuts [0, cuts_final) marked final — the multi-GPU on-line
 * path: every rank snapshots its running shard, the packed buffers are summed and the final-cut
 * prefixes min-reduced across ranks (dist.snapshot_sharded), and each rank loads the combined
 * partial result.  No device synchronisation.  Errors: CWC_E_STATE without a simulation;
 * CWC_E_INVALID for a null buffer or cuts_final outside [0, T]. */
cwc_status cwc_stats_load(cwc_model_t m, const int64_t* host_stats, int64_t cuts_final);

/* The finalised statistics of every cut ("an array of results is produced and streamed
 * to the analysis pipeline"; estimators P:L407; readings R10, R11, R14). */
typedef struct {
    int32_t T, S, B, n_q;
    const double* times;      /* [T] t_k = fl(k*dt) */
    const int64_t* n;         /* [T] */
    const int64_t* sum;       /* [T*S] */
    const double* sumsq;      /* [T*S] sum of x^2, rounded to double (exact value via sqlo/sqhi) */
    const int64_t* sqlo;      /* [T*S] */
    const int64_t* sqhi;      /* [T*S] */
    const double* mean;       /* [T*S] */
    const double* var;        /* [T*S] */
    const int64_t* hist;      /* [T*S*(B+2)] */
    const int64_t* hist_lo;   /* [S] */
    const int64_t* hist_width;/* [S] */
    const double* q;          /* [n_q] */
    const double* quantile;   /* [T*S*n_q] (+-inf if in the under/overflow bin, NaN if n = 0) */
    int64_t reactions, absorbed, overflowed, finished;
    double kernel_ms;         /* device time of the last simulate kernel (CUDA events) */
    int64_t cuts_final;       /* cuts [0, cuts_final) are final (T after finalize; see snapshot) */
    const char* const* species_names;
    int64_t pool_full;        /* overflowed instances frozen by a full compartment pool (R20); 0 means
                                 no trajectory was limited by a pool capacity */
    int64_t launches;         /* kernels the last simulate launched (SSA + compaction) */
    int64_t raw_staged;       /* 1: the last simulate staged raw cuts in shared memory (raw_stage) */
} cwc_stats_t;
/* Borrowed views into the handle, valid until the next simulate / finalize / free. */
cwc_status cwc_stats(cwc_model_t m, cwc_stats_t* out);

/* ------------------------------------------------------------------------------------------
 * On-line oscillation-period analysis ("we compute the
 * period of each oscillation and plot the moving average ... of the local period", on sliding
 * windows over the cuts P:L252-258).  Enabled per model with the options
 *   "period_species" (flat index, -1 = off) or "period_species.<name>" = 1,
 *   "period_lo" < "period_hi" (Schmitt-trigger thresholds on the species count),
 *   "period_window" (moving-average window in cuts, default 1).
 * Reading R19: an instance's detector is armed by a cut with x <= lo and fires an
 * event at the first later cut with x >= hi; a period is the number of cuts between consecutive
 * events; the local period of an instance at cut k is its last completed period.  All counts
 * are exact integers accumulated by the SSA kernel (same packed buffer, all-reduce-summable).
 * Views are valid until the next simulate / finalize / free; CWC_E_STATE if the analysis was off. */
typedef struct {
    int32_t T, species, window;
    int64_t lo, hi;
    const int64_t* events;                            /* [T] events at cut k */
    const int64_t *pc_n, *pc_sum, *pc_sqlo, *pc_sqhi; /* [T] periods (in cuts) completing at k */
    const int64_t *lp_n, *lp_sum, *lp_sqlo, *lp_sqhi; /* [T] local periods of instances at k */
    const double* lp_mean;                            /* [T] mean local period, time units */
    const double* lp_var;                             /* [T] its unbiased variance, time^2 */
    const double* moving_avg;                         /* [T] mean of periods completed in the
                                                         `window` cuts ending at k, time units */
} cwc_period_stats_t;
cwc_status cwc_period_stats(cwc_model_t m, cwc_period_stats_t* out);

/* Raw samples of local instances [first, first+count) of the last simulated range, copied to
 * host out[T][S][count] (-1 = missing after an overflow): the trajectory cuts themselves, "an
 * array containing the results of all simulations at a given simulation time", per
 * trajectory "the state of the system at each time step" sampled on the grid (R7).
 * CWC_E_STATE if raw_samples = 0. */
cwc_status cwc_samples(cwc_model_t m, int64_t first, int64_t count, int32_t* out);

/* Per-instance records of the last simulated range (the simulation tasks' final state, P:L238-243;
 * host outputs, any may be NULL):
 * flags (CWC_FLAG_*), reactions applied, final simulation time of the last applied reaction. */
cwc_status cwc_instance_records(cwc_model_t m, int64_t first, int64_t count, uint8_t* flags,
                                int64_t* reactions, double* t_last);

/* ------------------------------------------------------------------------------------------
 * Device self-tests of the hot-path primitives (the same device code the SSA kernel uses):
 * Philox4x32-10 blocks for n (ctr, key) pairs and CWC-log for n doubles, computed on the GPU.
 * Host arrays in, host arrays out.  ctr: [n][4], key: [n][2], out: [n][4]. */
cwc_status cwc_selftest_philox(int64_t n, const uint32_t* ctr, const uint32_t* key, uint32_t* out);
cwc_status cwc_selftest_log(int64_t n, const double* x, double* out);
cwc_status cwc_selftest_u01(int64_t n, const uint32_t* words, double* out); /* words [n][2] */
/* The SSA kernel's branch-free IEEE division (round to nearest) for n pairs, host in/out. */
cwc_status cwc_selftest_div(int64_t n, const double* num, const double* den, double* out);

/* Injected-draw steps of a loaded model (test entry; SURVEY §8(c) "event forced onto a grid
 * point (unit test with crafted u)").  The model's own NVRTC-compiled step code — mode 0: the
 * SSA kernel's fast step followed by the full step when the lane leaves the fast path; mode 1:
 * the full step only — runs n trajectories on the device, trajectory i starting from state
 * x[i][S] at time t[i] with next cut index k[i] (0 <= k <= K+1, K = llround(t_end/sample_dt)),
 * and takes up to n_draws steps with the uniforms u_tau[i][d], u_sel[i][d] in place of the
 * Philox draws (R3), stopping after the first step that is not a jump.  The step is the
 * direct method of P:L216-217 with the cut rule of P:L249-251 (reading R7) and the selection
 * rule R6.  Outputs (host, caller-owned): x_out[i][S], t_out[i] (time of the last jump),
 * k_out[i], status[i] = 0 jump / 2 horizon reached / 3 absorbed / 4 overflowed (the last step's),
 * n_done[i] = steps taken, and (optional) cuts[i][K+1][S]: the cuts these steps emitted, -2 where
 * none, -1 = missing after an overflow.  Errors: CWC_E_INVALID (bad sizes, k outside [0, K+1],
 * mode not 0/1), CWC_E_CUDA (no device). */
cwc_status cwc_selftest_step(cwc_model_t m, int64_t n, int32_t n_draws, const int32_t* x, const double* t,
                             const int64_t* k, double t_end, double sample_dt, const double* u_tau,
                             const double* u_sel, int32_t mode, int32_t* x_out, double* t_out, int64_t* k_out,
                             int32_t* status, int32_t* n_done, int32_t* cuts);

/* Library version string. */
const char* cwc_version(void);

#ifdef __cplusplus
}
#endif
#endif /* CWC_H_ */
