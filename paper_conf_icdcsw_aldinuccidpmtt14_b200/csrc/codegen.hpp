// codegen.hpp — model-specialised CUDA source generation.
#pragma once

#include <string>
#include <vector>

#include "compiler.hpp"

namespace cwc {

struct KernelConfig {
    int block_threads = 256;
    int min_blocks = 0;  // __launch_bounds__ min blocks per SM (0 = let ptxas choose)
    int ilp = 1;         // instances per thread
    int delta_table = -1;  // rewrite: 1 shared-memory delta table, 0 select chain, 2 telescoped predicates, -1 auto
    int hist_bins = 256;
    bool seed_keys = false;  // bake the Philox round keys of `seed` into the kernel (immediates)
    uint64_t seed = 0;
    int period_species = -1;  // on-line period detector on this flat species (-1 = off)
    int64_t period_lo = 0, period_hi = 1;
    int64_t x_cap = 0;
    bool fast_cut = true;  // the fast step records a due cut itself (else it leaves the fast loop)
    bool raw = true;       // raw cuts may be recorded (else every raw-cut path is compiled out)
    int draw_batch = -1;   // draws per inner-loop trip (0 = one per fast step; -1 = auto by species)
    std::vector<int64_t> hist_lo, hist_width;  // [S]
};

// The model section (macros + inline device functions) consumed by device/cwc_ssa.cuh.
std::string generate_model_section(const FlatModel& fm, const KernelConfig& cfg);

// Full NVRTC translation unit: cwc_params.h + cwc_rng.cuh + model section + cwc_ssa.cuh.
std::string generate_kernel_source(const FlatModel& fm, const KernelConfig& cfg);

}  // namespace cwc
