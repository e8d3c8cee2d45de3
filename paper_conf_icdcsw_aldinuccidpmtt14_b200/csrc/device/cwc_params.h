// cwc_params.h — kernel parameter block shared by the host runtime (runtime.cpp) and the
// NVRTC-compiled SSA kernel (cwc_ssa.cuh).  Plain C layout, passed by value as
// __grid_constant__; no includes so NVRTC needs no headers.
#pragma once

struct cwc_round_keys {
    unsigned int k0[10];  // key0 + r * 0x9E3779B9, r = 0..9
    unsigned int k1[10];  // key1 + r * 0xBB67AE85
};

struct cwc_logtab_entry {
    double invc, logc, logclo;
};

struct cwc_params {
    long long first;            // global id of local instance 0
    long long count;            // local instances
    long long K;                // last cut index, T = K + 1
    double dt;                  // sample_dt, t_k = fl(k * dt)
    long long n_items;          // work items = n_quanta * count
    long long qs;               // cuts per quantum (Q/tau)
    int refill;                 // 1 = global atomic work queue with warp-aggregated refill
    int resume;                 // 1: continue a terminated / restored run (skip quanta already done)
    cwc_round_keys rk;          // Philox round keys of the seed
    unsigned long long* stats;  // packed int64 stats (cwc.h layout)
    int* raw;                   // [ceil(T/8)][S][count][8] (time-blocked SoA) or nullptr
    int* st_x;                  // [S][count] saved species counts
    double* st_t;               // [count] saved time
    unsigned long long* st_step;  // [count] saved step (= reactions applied)
    long long* st_k;            // [count] next cut index
    unsigned int* st_flags;     // [count] CWC_FLAG_* | CWC_TERMINAL
    unsigned long long* st_pd;  // [count] period-detector state (R19)
    unsigned int* st_qdone;     // [count] quanta completed (release/acquire)
    unsigned long long* work;   // work-queue counter
    unsigned int* qprog;        // [n_quanta] finished items per quantum (streaming progress) or null
    const unsigned int* cancel; // streaming only: set by the host (cwc_cancel) to stop taking items
    const cwc_logtab_entry* logtab;  // [128]
    long long smem_stats;       // 1: n/sum/sumsq accumulate per CTA in dynamic shared memory
                                //    (T*(1+3S) u64) and are flushed once at the end
    long long q0;               // quantum of work item 0 (per-quantum launches; else 0)
    // compacted per-quantum launches: work item w is quantum q0 of local instance list[w]; the
    // item count is *n_items_dev (written by the previous launch's compaction), else n_items
    const unsigned int* list;
    const unsigned long long* n_items_dev;
    // raw-cut staging (1 = on): each lane collects the 8 cuts of one 32-byte block of the
    // time-blocked raw layout in dynamic shared memory (at byte raw_stage_off: [blockDim][S][8]
    // int32, then one u32 slot mask per lane) and writes the block as whole 32-byte sectors
    int raw_stage;
    int raw_stage_off;
};

#define CWC_TERMINAL 0x80000000u
// raw cuts per 32-byte block of one (species, instance): a lane fills the whole sector while it
// is resident in L2, so the sample stream reaches DRAM as full sectors (no read-for-fill)
#define CWC_RAW_BLOCK 8
