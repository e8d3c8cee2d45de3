// runtime.cpp — NVRTC compilation, device buffers, the simulate launch and host finalisation.
//
// One cwc_simulate_range = two async memsets + ONE launch of the persistent SSA kernel on the
// caller's stream (torch's, when called from Python).  Everything the hot path computes runs in
// that kernel; the host only validates, sizes buffers and, at finalize, turns the exact integer
// accumulators into mean / variance / quantiles (R10, R11).
#include "runtime.hpp"

#include <nvrtc.h>

#include <algorithm>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fstream>
#include <mutex>
#include <dlfcn.h>
#include <nvtx3/nvToolsExt.h>  // header-only NVTX v3: ranges are free unless a profiler injects

// models with at least this many species accumulate cut statistics in the sparse shared layout
// (same-box A/B, profiles/r2_ab_kernel.log, sparse vs dense: vesicles 123 vs 228 ms, compartments
// 625 vs 686, Neurospora 653 vs 684, circadian 1750 vs 1794, Schlogl 1916 vs 1953, LV 1M 1717 vs
// 1725: every model)
#ifndef CWC_SPARSE_MIN_S
#define CWC_SPARSE_MIN_S 1
#endif

// bench.py counts the launch parameter block in its end-to-end H2D bytes (PARAM_BYTES)
static_assert(sizeof(cwc_params) == 280, "cwc_params layout changed: update bench.py PARAM_BYTES");
static_assert(sizeof(cwc_logtab_entry) * 128 == 3072, "log table size");

namespace {
// NVTX range over a host-side phase of the path (visible in nsys / ncu --nvtx timelines)
struct NvtxRange {
    explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
    ~NvtxRange() { nvtxRangePop(); }
    NvtxRange(const NvtxRange&) = delete;
    NvtxRange& operator=(const NvtxRange&) = delete;
};
}  // namespace
#include <sstream>
#include <sys/stat.h>
#include <unistd.h>

#include "cwc.h"

extern const char* const cwc_embedded_params_h;
extern const char* const cwc_embedded_rng_cuh;
extern const char* const cwc_embedded_ssa_cuh;

namespace cwc {

// ------------------------------------------------------------------------------------ errors
[[noreturn]] static void fail(int32_t code, const std::string& msg) { throw Error(code, msg); }

static void ck(cudaError_t e, const char* what) {
    if (e == cudaSuccess) return;
    if (e == cudaErrorMemoryAllocation) fail(CWC_E_OOM, std::string(what) + ": " + cudaGetErrorString(e));
    fail(CWC_E_CUDA, std::string(what) + ": " + cudaGetErrorString(e));
}

// ------------------------------------------------------------------------------------ driver API
// Resolved through the runtime (cudaGetDriverEntryPoint) so the library loads on machines
// without a driver; only simulate needs one.
struct Driver {
    CUresult (*ModuleLoadData)(CUmodule*, const void*) = nullptr;
    CUresult (*ModuleUnload)(CUmodule) = nullptr;
    CUresult (*ModuleGetFunction)(CUfunction*, CUmodule, const char*) = nullptr;
    CUresult (*LaunchKernel)(CUfunction, unsigned, unsigned, unsigned, unsigned, unsigned, unsigned, unsigned,
                             CUstream, void**, void**) = nullptr;
    CUresult (*FuncGetAttribute)(int*, CUfunction_attribute, CUfunction) = nullptr;
    CUresult (*Occupancy)(int*, CUfunction, int, size_t) = nullptr;
    CUresult (*FuncSetAttribute)(CUfunction, CUfunction_attribute, int) = nullptr;
    bool ok = false;
};

static Driver& driver() {
    static Driver d;
    static std::once_flag once;
    std::call_once(once, [] {
        auto get = [](const char* name, void** fn) {
            cudaDriverEntryPointQueryResult q;
            return cudaGetDriverEntryPoint(name, fn, cudaEnableDefault, &q) == cudaSuccess &&
                   q == cudaDriverEntryPointSuccess && *fn;
        };
        d.ok = get("cuModuleLoadData", (void**)&d.ModuleLoadData) &&
               get("cuModuleUnload", (void**)&d.ModuleUnload) &&
               get("cuModuleGetFunction", (void**)&d.ModuleGetFunction) &&
               get("cuLaunchKernel", (void**)&d.LaunchKernel) &&
               get("cuFuncGetAttribute", (void**)&d.FuncGetAttribute) &&
               get("cuOccupancyMaxActiveBlocksPerMultiprocessor", (void**)&d.Occupancy) &&
               get("cuFuncSetAttribute", (void**)&d.FuncSetAttribute);
    });
    if (!d.ok) fail(CWC_E_CUDA, "CUDA driver entry points unavailable (no driver / GPU?)");
    return d;
}

static void ckd(CUresult r, const char* what) {
    if (r != CUDA_SUCCESS) fail(CWC_E_CUDA, std::string(what) + ": CUresult " + std::to_string((int)r));
}

// ------------------------------------------------------------------------------------ sizes
int64_t grid_K(double t_end, double dt) {
    if (!(dt > 0) || !std::isfinite(dt)) fail(CWC_E_INVALID, "sample_dt must be > 0");
    if (!(t_end >= 0) || !std::isfinite(t_end)) fail(CWC_E_INVALID, "t_end must be >= 0");
    double r = std::nearbyint(t_end / dt);
    if (r > 2e9) fail(CWC_E_INVALID, "too many sample points");
    int64_t K = (int64_t)r;
    if (std::fabs((double)K * dt - t_end) > 1e-9 * std::max(1.0, t_end))
        fail(CWC_E_INVALID, "t_end is not a multiple of sample_dt");
    return K;
}

size_t stats_len(int64_t T, int S, int B, bool period) {
    return (size_t)(T * (1 + 3 * (int64_t)S + (int64_t)S * (B + 2)) + CWC_N_CTR + (period ? CWC_N_PERIOD * T : 0));
}

static size_t align256(size_t v) { return (v + 255) & ~(size_t)255; }

struct ScratchLayout {
    size_t x, t, step, k, flags, pd, qdone, work, cancel, qprog, list0, list1, nlive, total;
};

static ScratchLayout scratch_layout(int S, int64_t count, int64_t T) {
    ScratchLayout L{};
    size_t off = 0;
    L.x = off; off = align256(off + (size_t)S * count * 4);
    L.pd = off; off = align256(off + (size_t)count * 8);
    L.t = off; off = align256(off + (size_t)count * 8);
    L.step = off; off = align256(off + (size_t)count * 8);
    L.k = off; off = align256(off + (size_t)count * 8);
    L.flags = off; off = align256(off + (size_t)count * 4);
    L.qdone = off; off += (size_t)count * 4;          // qdone, work and qprog are contiguous:
    off = (off + 7) & ~(size_t)7;                     // one memset clears them
    L.work = off; off += 8;
    L.cancel = off; off += 8;                         // u32 terminate flag (streaming)
    L.qprog = off; off = align256(off + (size_t)T * 4);  // <= T quanta
    L.list0 = off; off = align256(off + (size_t)count * 4);  // compacted launches: running instances
    L.list1 = off; off = align256(off + (size_t)count * 4);
    L.nlive = off; off = align256(off + 16);                 // their counts (two u64)
    L.total = off;
    return L;
}

void buffer_sizes(const cwc_model* m, int64_t count, int64_t K, size_t* stats, size_t* raw, size_t* scratch) {
    const int S = m->fm.S();
    if (stats) *stats = stats_len(K + 1, S, m->hist_bins, m->period_species >= 0);
    if (raw) *raw = m->raw_samples ? (size_t)((K + CWC_RAW_BLOCK) / CWC_RAW_BLOCK) * CWC_RAW_BLOCK * S * (size_t)count : 0;
    if (scratch) *scratch = scratch_layout(S, count, K + 1).total;
}

// ------------------------------------------------------------------------------------ NVRTC
static std::string strip_pragma_once(const char* s) {
    std::string out(s);
    size_t p;
    while ((p = out.find("#pragma once")) != std::string::npos) out.erase(p, 12);
    return out;
}

// Development knob (same-box A/B of kernel revisions): CWC_DEVICE_SRC=<dir> compiles the device
// sources cwc_params.h / cwc_rng.cuh / cwc_ssa.cuh found in <dir> instead of the embedded ones.
static std::string device_source(const char* embedded, const char* file) {
    const char* dir = std::getenv("CWC_DEVICE_SRC");
    if (dir && *dir) {
        std::ifstream f(std::string(dir) + "/" + file);
        if (!f) fail(CWC_E_INVALID, std::string("CWC_DEVICE_SRC: cannot read ") + file);
        return strip_pragma_once(std::string(std::istreambuf_iterator<char>(f), std::istreambuf_iterator<char>()).c_str());
    }
    return strip_pragma_once(embedded);
}

std::string generate_kernel_source(const FlatModel& fm, const KernelConfig& cfg) {
    std::string src = "// CWC ensemble SSA kernel, generated for one model (NVRTC, sm_100a)\n";
    src += device_source(cwc_embedded_params_h, "cwc_params.h");
    src += device_source(cwc_embedded_rng_cuh, "cwc_rng.cuh");
    src += generate_model_section(fm, cfg);
    src += device_source(cwc_embedded_ssa_cuh, "cwc_ssa.cuh");
    return src;
}

static uint64_t fnv1a(const std::string& s) {
    uint64_t h = 1469598103934665603ULL;
    for (unsigned char c : s) { h ^= c; h *= 1099511628211ULL; }
    return h;
}

static std::string cache_dir() {
    const char* e = std::getenv("CWC_CACHE_DIR");
    if (e && *e) return e;
    const char* home = std::getenv("HOME");
    return std::string(home && *home ? home : "/tmp") + "/.cache/cwc_b200";
}

// NVRTC is loaded at run time (dlopen) from the CUDA toolkit of this image rather than linked
// statically (106 MB): the library stays small and loads where NVRTC is absent.
struct Nvrtc {
    decltype(&::nvrtcVersion) Version = nullptr;
    decltype(&::nvrtcCreateProgram) CreateProgram = nullptr;
    decltype(&::nvrtcCompileProgram) CompileProgram = nullptr;
    decltype(&::nvrtcGetProgramLogSize) GetProgramLogSize = nullptr;
    decltype(&::nvrtcGetProgramLog) GetProgramLog = nullptr;
    decltype(&::nvrtcGetCUBINSize) GetCUBINSize = nullptr;
    decltype(&::nvrtcGetCUBIN) GetCUBIN = nullptr;
    decltype(&::nvrtcDestroyProgram) DestroyProgram = nullptr;
    bool ok = false;
    std::string where;
};

static Nvrtc& nvrtc() {
    static Nvrtc n;
    static std::once_flag once;
    std::call_once(once, [] {
        std::vector<std::string> cands;
        if (const char* e = std::getenv("CWC_NVRTC_PATH")) cands.push_back(e);
        const char* home = std::getenv("CUDA_HOME");
        cands.push_back(std::string(home && *home ? home : "/usr/local/cuda") + "/lib64/libnvrtc.so.12");
        cands.push_back("/usr/local/cuda/lib64/libnvrtc.so.12");
        cands.push_back("libnvrtc.so.12");
        void* h = nullptr;
        for (auto& c : cands) {
            h = dlopen(c.c_str(), RTLD_NOW | RTLD_LOCAL);
            if (h) { n.where = c; break; }
        }
        if (!h) return;
        auto sym = [&](const char* s) { return dlsym(h, s); };
        n.Version = (decltype(n.Version))sym("nvrtcVersion");
        n.CreateProgram = (decltype(n.CreateProgram))sym("nvrtcCreateProgram");
        n.CompileProgram = (decltype(n.CompileProgram))sym("nvrtcCompileProgram");
        n.GetProgramLogSize = (decltype(n.GetProgramLogSize))sym("nvrtcGetProgramLogSize");
        n.GetProgramLog = (decltype(n.GetProgramLog))sym("nvrtcGetProgramLog");
        n.GetCUBINSize = (decltype(n.GetCUBINSize))sym("nvrtcGetCUBINSize");
        n.GetCUBIN = (decltype(n.GetCUBIN))sym("nvrtcGetCUBIN");
        n.DestroyProgram = (decltype(n.DestroyProgram))sym("nvrtcDestroyProgram");
        n.ok = n.Version && n.CreateProgram && n.CompileProgram && n.GetProgramLogSize && n.GetProgramLog &&
               n.GetCUBINSize && n.GetCUBIN && n.DestroyProgram;
    });
    if (!n.ok) fail(CWC_E_CUDA, "NVRTC (libnvrtc.so.12) not found; set CWC_NVRTC_PATH");
    return n;
}

static const char* kNvrtcOpts[] = {"--gpu-architecture=sm_100a", "-fmad=false", "-lineinfo", "-std=c++17",
                                   "--ptxas-options=-v", "-DCWC_NVRTC=1"};

// registers / spill stores of the SSA kernel itself (the module also holds the self-test kernel)
static void parse_ptxas(cwc_model* m) {
    m->regs = -1;
    m->local_bytes = 0;
    const std::string& log = m->nvrtc_log;
    size_t start = log.find("entry function 'cwc_ssa_kernel'");
    if (start == std::string::npos) start = 0;
    size_t end = log.find("entry function", start + 1);
    if (end == std::string::npos) end = log.size();
    size_t p = log.find("Used ", start);
    if (p != std::string::npos && p < end) m->regs = std::atoi(log.c_str() + p + 5);
    size_t q = log.find("bytes spill stores", start);
    if (q != std::string::npos && q < end) {
        size_t b = log.rfind(',', q);
        if (b != std::string::npos) m->local_bytes = std::atoi(log.c_str() + b + 1);
    }
}

void compile(cwc_model* m, const uint64_t* seed) {
    NvtxRange nvtx_range("cwc_model_compile");
    KernelConfig cfg;
    cfg.block_threads = m->block_threads;
    // auto register budget: 768 resident threads per SM (<= 80 registers) — measured best for the
    // App. B models (fewer, fatter threads lose more to latency than they gain from registers)
    cfg.min_blocks = m->min_blocks > 0 ? m->min_blocks : std::max(1, 768 / m->block_threads);
    cfg.ilp = m->ilp;
    cfg.delta_table = m->delta_table;
    cfg.period_species = m->period_species;
    cfg.period_lo = m->period_lo;
    cfg.period_hi = m->period_hi;
    cfg.hist_bins = m->hist_bins;
    cfg.x_cap = m->x_cap;
    cfg.fast_cut = m->fast_cut >= 0 ? m->fast_cut != 0 : m->fast_cut_now;  // explicit option wins
    cfg.draw_batch = m->draw_batch;
    cfg.raw = m->raw_samples != 0;
    cfg.hist_lo = m->hist_lo;
    cfg.hist_width = m->hist_width;
    if (seed && m->seed_jit) {
        cfg.seed_keys = true;
        cfg.seed = *seed;
    }
    std::string src = generate_kernel_source(m->fm, cfg);
    // development knob: CWC_KERNEL_DEFINES="A=1;B=2" prepends #defines (kernel variants for A/B
    // timing); part of the source, hence of the cache key
    if (const char* e = std::getenv("CWC_KERNEL_DEFINES")) {
        std::string defs, item;
        for (const char* p = e;; ++p) {
            if (*p == ';' || *p == '\0') {
                size_t eq = item.find('=');
                if (!item.empty())
                    defs += "#define " + (eq == std::string::npos ? item : item.substr(0, eq) + " " + item.substr(eq + 1)) +
                            "\n";
                item.clear();
                if (*p == '\0') break;
            } else {
                item += *p;
            }
        }
        src = defs + src;
    }
    Nvrtc& nv = nvrtc();
    int major = 0, minor = 0;
    nv.Version(&major, &minor);
    std::string key = std::to_string(fnv1a(src)) + "-nvrtc" + std::to_string(major) + "." + std::to_string(minor);
    if (key == m->compiled_key && !m->cubin.empty()) return;

    std::vector<char> cubin;
    std::string log;
    const std::string dir = cache_dir();
    const std::string path = dir + "/" + key + ".cubin", lpath = dir + "/" + key + ".log";
    {
        std::ifstream f(path, std::ios::binary);
        if (f) {
            cubin.assign(std::istreambuf_iterator<char>(f), std::istreambuf_iterator<char>());
            std::ifstream lf(lpath);
            if (lf) log.assign(std::istreambuf_iterator<char>(lf), std::istreambuf_iterator<char>());
        }
    }
    if (cubin.empty()) {
        nvrtcProgram prog;
        if (nv.CreateProgram(&prog, src.c_str(), "cwc_ssa.cu", 0, nullptr, nullptr) != NVRTC_SUCCESS)
            fail(CWC_E_CUDA, "nvrtcCreateProgram failed");
        nvrtcResult r = nv.CompileProgram(prog, (int)(sizeof kNvrtcOpts / sizeof kNvrtcOpts[0]), kNvrtcOpts);
        size_t ls = 0;
        nv.GetProgramLogSize(prog, &ls);
        log.assign(ls, '\0');
        if (ls) nv.GetProgramLog(prog, &log[0]);
        if (!log.empty() && log.back() == '\0') log.pop_back();
        if (r != NVRTC_SUCCESS) {
            nv.DestroyProgram(&prog);
            m->nvrtc_log = log;
            fail(CWC_E_CUDA, "NVRTC compilation failed: " + log.substr(0, 2000));
        }
        size_t cs = 0;
        nv.GetCUBINSize(prog, &cs);
        cubin.resize(cs);
        nv.GetCUBIN(prog, cubin.data());
        nv.DestroyProgram(&prog);
        // best-effort disk cache
        std::string cmd = dir;
        for (size_t i = 1; i <= cmd.size(); ++i)
            if (i == cmd.size() || cmd[i] == '/') mkdir(cmd.substr(0, i).c_str(), 0755);
        std::string tmp = path + ".tmp." + std::to_string((long)getpid());
        {
            std::ofstream f(tmp, std::ios::binary);
            if (f) f.write(cubin.data(), (std::streamsize)cubin.size());
        }
        std::rename(tmp.c_str(), path.c_str());
        std::ofstream lf(lpath);
        if (lf) lf << log;
    }
    if (m->module && driver().ok) driver().ModuleUnload(m->module);
    m->module = nullptr;
    m->function = nullptr;
    m->module_device = -1;
    m->source = src;
    m->nvrtc_log = log;
    m->cubin = std::move(cubin);
    m->compiled_key = key;
    parse_ptxas(m);
}

// ------------------------------------------------------------------------------------ device
static int current_device(cwc_model* m) {
    int dev = m->device;
    if (dev < 0) ck(cudaGetDevice(&dev), "cudaGetDevice");
    ck(cudaSetDevice(dev), "cudaSetDevice");
    ck(cudaFree(nullptr), "CUDA context init");
    return dev;
}

static void ensure_module(cwc_model* m, int dev) {
    if (m->module && m->module_device == dev) return;
    Driver& d = driver();
    if (m->module) d.ModuleUnload(m->module);
    m->module = nullptr;
    ckd(d.ModuleLoadData(&m->module, m->cubin.data()), "cuModuleLoadData");
    ckd(d.ModuleGetFunction(&m->function, m->module, "cwc_ssa_kernel"), "cuModuleGetFunction");
    ckd(d.ModuleGetFunction(&m->compact_fn, m->module, "cwc_compact_kernel"), "cuModuleGetFunction(compact)");
    m->module_device = dev;
    int v = 0;
    if (d.FuncGetAttribute(&v, CU_FUNC_ATTRIBUTE_NUM_REGS, m->function) == CUDA_SUCCESS) m->regs = v;
    if (d.FuncGetAttribute(&v, CU_FUNC_ATTRIBUTE_LOCAL_SIZE_BYTES, m->function) == CUDA_SUCCESS) m->local_bytes = v;
    if (d.FuncGetAttribute(&v, CU_FUNC_ATTRIBUTE_MAX_THREADS_PER_BLOCK, m->function) == CUDA_SUCCESS) m->max_threads = v;
}

static void free_owned(cwc_model* m) {
    if (!m->bound) {
        if (m->d_stats) cudaFree(m->d_stats);
        if (m->d_raw) cudaFree(m->d_raw);
        if (m->d_scratch) cudaFree(m->d_scratch);
    }
    m->d_stats = nullptr; m->d_raw = nullptr; m->d_scratch = nullptr;
    m->stats_cap = m->raw_cap = m->scratch_cap = 0;
}

void bind_buffers(cwc_model* m, int64_t* stats, size_t stats_n, int32_t* raw, size_t raw_n, void* scratch,
                  size_t scratch_bytes) {
    free_owned(m);
    if (!stats && !raw && !scratch) {
        m->bound = false;
        return;
    }
    if (!stats || !scratch) fail(CWC_E_INVALID, "stats and scratch buffers are required when binding");
    m->bound = true;
    m->d_stats = stats;
    m->stats_cap = stats_n * 8;
    m->d_raw = raw;
    m->raw_cap = raw ? raw_n * 4 : 0;
    m->d_scratch = scratch;
    m->scratch_cap = scratch_bytes;
}

template <class T>
static void grow(T*& p, size_t& cap, size_t need_bytes, const char* what) {
    if (cap >= need_bytes && p) return;
    if (p) cudaFree(p);
    p = nullptr;
    cap = 0;
    void* q = nullptr;
    ck(cudaMalloc(&q, std::max<size_t>(need_bytes, 256)), what);
    p = (T*)q;
    cap = need_bytes;
}

// Expected reactions between two cuts from the initial state: a0(x0) * dt (functional laws
// evaluated at x0, gates ignored) — only the first guess of choose_fast_cut.
static double a0_estimate(const FlatModel& fm) {
    double a0 = 0;
    for (int j = 0; j < fm.M(); ++j) {
        double h = 1;
        for (const Reactant& r : fm.reactants[j]) {
            const double x = fm.x0[r.species];
            for (int i = 0; i < r.order; ++i) h *= (x - i) / (i + 1);
            if (h <= 0) { h = 0; break; }
        }
        double a = fm.rates[j] * h;
        if (!fm.law.empty() && fm.law[j] != 0 && fm.law_species[j] >= 0) {
            const double X = fm.x0[fm.law_species[j]], K = fm.law_K[j], n = fm.law.size() ? fm.law_n[j] : 1;
            const double Xn = std::pow(X, n), Kn = std::pow(K, n);
            if (fm.law[j] == 1) a = h > 0 ? fm.rates[j] * X / (K + X) : 0;
            else if (fm.law[j] == 2) a = h > 0 ? fm.rates[j] * Xn / (Kn + Xn) : 0;
            else a = h > 0 ? fm.rates[j] * Kn / (Kn + Xn) : 0;
        }
        a0 += a;
    }
    return a0;
}

// Where the fast step records cuts.  Inline (1) costs the fast loop a call site, which makes
// ptxas rematerialise constants and shuffle registers every step; leaving the fast loop for the
// full step (0) costs a warp-wide exit per recorded cut.  Same-box A/B (profiles/
// r1h_ab_fast_cut.log): leaving wins from ~1,000 reactions per cut (LV 2,800: -2.9 %, circadian
// 1,400: -2.0 %) and loses below (Schlogl 490: +1.2 %, Neurospora 610: +7.6 %, compartments
// 290: +6.3 %).  Auto decides by the last run on this handle, else by a0(x0) * dt.
static bool choose_fast_cut(cwc_model* m, double dt) {
    if (m->fast_cut >= 0) return m->fast_cut != 0;
    const double rpc = m->last_reactions_per_cut > 0 ? m->last_reactions_per_cut : a0_estimate(m->fm) * dt;
    return rpc < 1000.0;
}

void simulate_range(cwc_model* m, int64_t n_total, int64_t first, int64_t count, double t_end, double dt,
                    uint64_t seed, cudaStream_t stream, bool own_stream, bool resume) {
    NvtxRange nvtx_range("cwc_simulate_range");
    if (n_total <= 0) fail(CWC_E_INVALID, "n_total must be > 0");
    if (first < 0 || count < 0 || first + count > n_total) fail(CWC_E_INVALID, "instance range outside [0, n_total)");
    if (count >= ((int64_t)1 << 31)) fail(CWC_E_INVALID, "at most 2^31 - 1 instances per range (shard larger ensembles)");
    const int64_t K = grid_K(t_end, dt);
    if (m->period_species >= 0 && !(m->period_lo < m->period_hi))
        fail(CWC_E_INVALID, "period analysis needs period_lo < period_hi");
    const int64_t T = K + 1;
    const int S = m->fm.S();
    m->fast_cut_now = choose_fast_cut(m, dt);
    // auto CTA size (same-box sweep, profiles/s2r_ab_block_sizes.log, s2s_ab_block_underfilled.log):
    // 768 threads x 80 registers when the instances fill the lanes at least 1.5 times over; below,
    // 512 x 113 registers — the instances then exceed the fewer lanes, so simulation quanta balance
    // the load, and each warp runs a better-scheduled step (LV 100k 969 -> 838 ms, 125k 1065 ->
    // 1034 ms; at 250k-1M and on the 1M configs 768 is best or equal)
    if (m->block_auto && m->ilp == 1) {
        int dv = m->device, sms = 0;
        if (dv < 0 && cudaGetDevice(&dv) != cudaSuccess) dv = -1;
        if (dv >= 0 && cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dv) != cudaSuccess) sms = 0;
        cudaGetLastError();
        if (sms > 0) m->block_threads = count * 2 < (int64_t)sms * 768 * 3 ? 512 : 768;
    }
    compile(m, &seed);
    const int dev = current_device(m);
    ensure_module(m, dev);
    Driver& d = driver();

    size_t need_stats, need_raw, need_scratch;
    buffer_sizes(m, count, K, &need_stats, &need_raw, &need_scratch);
    if (m->bound) {
        if (m->stats_cap < need_stats * 8 || m->scratch_cap < need_scratch || (need_raw && m->raw_cap < need_raw * 4))
            fail(CWC_E_INVALID, "bound device buffers too small (see cwc_buffer_sizes)");
    } else {
        grow(m->d_stats, m->stats_cap, need_stats * 8, "cudaMalloc(stats)");
        if (need_raw) grow(m->d_raw, m->raw_cap, need_raw * 4, "cudaMalloc(raw)");
        grow(m->d_scratch, m->scratch_cap, need_scratch, "cudaMalloc(scratch)");
    }
    if (!m->d_logtab || m->logtab_device != dev) {
        if (m->d_logtab) cudaFree(m->d_logtab);
        m->d_logtab = nullptr;
        cwc_logtab_entry tab[128];
        build_log_table(tab);
        ck(cudaMalloc(&m->d_logtab, sizeof tab), "cudaMalloc(logtab)");
        ck(cudaMemcpy(m->d_logtab, tab, sizeof tab, cudaMemcpyHostToDevice), "upload logtab");
        m->logtab_device = dev;
    }
    if (own_stream) {
        if (!m->own_stream) ck(cudaStreamCreateWithFlags(&m->own_stream, cudaStreamNonBlocking), "cudaStreamCreate");
        stream = m->own_stream;
    }
    if (!m->ev0) {
        ck(cudaEventCreate(&m->ev0), "cudaEventCreate");
        ck(cudaEventCreate(&m->ev1), "cudaEventCreate");
    }

    // launch geometry: persistent grid of (SMs x resident CTAs), no more lanes than instances
    int sms = 0;
    ck(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev), "SM count");
    // per-CTA moment accumulators in dynamic shared memory when they fit without costing residency
    const size_t mom_bytes = (size_t)T * (1 + 3 * (size_t)S) * 8;
    int occ = 0;
    ckd(d.Occupancy(&occ, m->function, m->block_threads, 0), "occupancy");
    if (occ < 1) fail(CWC_E_CUDA, "kernel cannot be resident with block_threads = " + std::to_string(m->block_threads));
    size_t dyn_smem = 0;
    int smem_mode = 0;
    // Per-CTA shared-memory accumulators when they fit without lowering residency: sparse (u32
    // counters and 16-bit limbs with native shared REDs, zero counts skipped and restored at the
    // flush) or dense (u64 n / sum / sum-of-squares halves: 64-bit shared atomics are CAS loops).  Streaming publishes partial
    // statistics while the kernel runs, so it keeps everything in global memory.  (A per-CTA copy
    // of the hottest histogram bin alone was measured slower: vesicles 256 -> 273 ms.)
    const size_t sparse_bytes = (size_t)T * (2 + 7 * (size_t)S) * 4;  // counters + per-quantum admissions
    auto fits = [&](size_t bytes) {
        if (bytes > (size_t)200 * 1024) return false;
        ckd(d.FuncSetAttribute(m->function, CU_FUNC_ATTRIBUTE_MAX_DYNAMIC_SHARED_SIZE_BYTES, (int)bytes),
            "dynamic smem");
        int occ2 = 0;
        ckd(d.Occupancy(&occ2, m->function, m->block_threads, bytes), "occupancy");
        return occ2 >= occ;
    };
    if (m->smem_stats && !m->stream) {
        // (the sparse limbs are exact for any count: a CTA's records beyond 65536 per cut index go to
        // global memory directly)
        const bool want_sparse = m->smem_stats == 2 || (m->smem_stats == 1 && S >= CWC_SPARSE_MIN_S);
        if (want_sparse && fits(sparse_bytes)) smem_mode = 2, dyn_smem = sparse_bytes;
        else if (m->smem_stats != 2 && fits(mom_bytes)) smem_mode = 1, dyn_smem = mom_bytes;
        ckd(d.FuncSetAttribute(m->function, CU_FUNC_ATTRIBUTE_MAX_DYNAMIC_SHARED_SIZE_BYTES, (int)dyn_smem),
            "dynamic smem");
    }
    // raw-cut staging: a lane's 8 cuts of one time block go to DRAM as whole 32-byte sectors
    // instead of eight 4-byte stores that L2 may write back (and re-read for ECC fill) before the
    // sector is complete (LV 1M: 8.3 GB of DRAM traffic per launch for 4.0 GB of raw cuts)
    int raw_stage = 0, raw_stage_off = 0;
    if (need_raw && m->raw_stage && m->ilp == 1) {
        const size_t off = (dyn_smem + 15) / 16 * 16;
        const size_t bytes = off + (size_t)m->block_threads * ((size_t)S * CWC_RAW_BLOCK * 4 + 4);
        if (fits(bytes)) raw_stage = 1, raw_stage_off = (int)off, dyn_smem = bytes;
        ckd(d.FuncSetAttribute(m->function, CU_FUNC_ATTRIBUTE_MAX_DYNAMIC_SHARED_SIZE_BYTES, (int)dyn_smem),
            "dynamic smem");
    }
    m->raw_stage_now = raw_stage;
    int per_sm = m->blocks_per_sm > 0 ? std::min(m->blocks_per_sm, occ) : occ;
    int64_t grid = (int64_t)sms * per_sm;
    // Every resident slot is launched even when there are fewer instances than lanes: warps race
    // for items on the work queue, so the busy warps spread over all SMs instead of packing the
    // first CTAs (391 CTAs of 256 on 148 SMs left 35 % of the SMs with 2 CTAs instead of 3).
    // Only very small ensembles (< 1 warp per CTA) shrink the grid.
    grid = std::min<int64_t>(grid, std::max<int64_t>(sms, (count + 32 * m->ilp - 1) / (32 * m->ilp)));
    const int64_t lanes = grid * m->block_threads * m->ilp;
    int64_t qs;
    // refill off: static assignment of whole trajectories, or — with quantum_samples set — the
    // paper's GPU scheme: one launch per simulation quantum, every lane running its
    // instance's quantum q, the kernel boundary as the barrier between quanta (the T3 ablation)
    // compacted launches (option; ablation of the under-filled regime): a quantum per launch over
    // the instances still running, so the lanes of instances that ended are handed back at every
    // launch instead of idling to the end — measured slower than one persistent launch
    const bool compact = m->refill && !m->stream && !resume && count > 0 && m->compact == 1;
    if (!m->refill) qs = m->quantum_samples > 0 ? std::min<int64_t>(m->quantum_samples, T) : T;
    else if (compact) {
        qs = m->quantum_samples > 0 ? std::min<int64_t>(m->quantum_samples, T) : (T + 7) / 8;
        qs = std::min<int64_t>(T, (qs + CWC_RAW_BLOCK - 1) / CWC_RAW_BLOCK * CWC_RAW_BLOCK);
    } else if (m->quantum_samples > 0) qs = std::min<int64_t>(m->quantum_samples, T);
    else if (m->stream) qs = std::max<int64_t>(1, (T + 15) / 16);  // streaming: progress in ~16 chunks
    // auto (same-box sweeps, profiles/r2_ab_quanta_launch.log): up to one instance per resident lane, whole
    // trajectories (a later quantum could only wait for its predecessor on another lane: LV 100k
    // 1.37e11 whole vs 1.02e11 at 8 quanta); above, quanta let the surplus instances interleave with
    // the first wave instead of forming a second one (LV 125k: 1.05e11 whole, 1.47e11 at 16 quanta,
    // 1.57e11 at 32; LV 250k: 1.32e11 whole, 1.69e11 at 16-32); from 4 per lane the quantum count
    // hardly matters (LV 1M: 1.701 / 1.711 / 1.706e11 at 32 / 16 / 8 quanta) and fewer quanta save
    // state traffic (a save + restore per instance per quantum)
    else if (count <= lanes) qs = T;
    else {
        // 32 quanta up to 4 instances per lane, 8 above; a quantum holds whole 8-cut blocks of the
        // time-blocked raw layout, so each 32-byte sector is written by one lane in one quantum
        // (no partially written sector left in L2 between quanta)
        const int64_t nq_target = count <= 4 * lanes ? 32 : 8;
        qs = (T + nq_target - 1) / nq_target;
        qs = std::min<int64_t>(T, (qs + CWC_RAW_BLOCK - 1) / CWC_RAW_BLOCK * CWC_RAW_BLOCK);
    }
    if (resume) qs = m->qs;  // the work items (quantum, instance) of the run being continued
    const int64_t nq = (T + qs - 1) / qs;

    const ScratchLayout L = scratch_layout(S, count, T);
    char* sc = (char*)m->d_scratch;
    cwc_params P;
    std::memset(&P, 0, sizeof P);
    P.first = first;
    P.count = count;
    P.K = K;
    P.dt = dt;
    P.n_items = nq * count;
    P.qs = qs;
    P.refill = m->refill;
    P.resume = resume ? 1 : 0;
    const uint32_t key0 = (uint32_t)seed, key1 = (uint32_t)(seed >> 32);
    for (int r = 0; r < 10; ++r) {
        P.rk.k0[r] = key0 + (uint32_t)r * 0x9E3779B9u;
        P.rk.k1[r] = key1 + (uint32_t)r * 0xBB67AE85u;
    }
    P.stats = (unsigned long long*)m->d_stats;
    P.raw = need_raw ? m->d_raw : nullptr;
    P.st_x = (int*)(sc + L.x);
    P.st_t = (double*)(sc + L.t);
    P.st_step = (unsigned long long*)(sc + L.step);
    P.st_k = (long long*)(sc + L.k);
    P.st_flags = (unsigned int*)(sc + L.flags);
    P.st_pd = (unsigned long long*)(sc + L.pd);
    P.st_qdone = (unsigned int*)(sc + L.qdone);
    P.work = (unsigned long long*)(sc + L.work);
    P.qprog = m->stream ? (unsigned int*)(sc + L.qprog) : nullptr;
    P.cancel = m->stream ? (const unsigned int*)(sc + L.cancel) : nullptr;
    m->cancel_requested = false;
    P.logtab = m->d_logtab;
    P.smem_stats = smem_mode;
    P.raw_stage = raw_stage;
    P.raw_stage_off = raw_stage_off;

    if (!resume) {
        ck(cudaMemsetAsync(m->d_stats, 0, need_stats * 8, stream), "memset(stats)");
        ck(cudaMemsetAsync(sc + L.qdone, 0, L.qprog + (size_t)T * 4 - L.qdone, stream), "memset(queue)");
    } else {  // keep statistics, instance states, quanta done and progress; restart the hand-out
        ck(cudaMemsetAsync(sc + L.work, 0, L.qprog - L.work, stream), "memset(work, cancel)");
    }
    m->resumable = false;
    ck(cudaEventRecord(m->ev0, stream), "cudaEventRecord");
    const bool lockstep = !m->refill && qs < T;
    const bool per_quantum = (lockstep || compact) && nq > 1;
    unsigned int* lists[2] = {(unsigned int*)(sc + L.list0), (unsigned int*)(sc + L.list1)};
    unsigned long long* nlive = (unsigned long long*)(sc + L.nlive);
    m->launches = 0;
    for (int64_t q = 0; count > 0 && q < (per_quantum ? nq : 1); ++q) {
        if (per_quantum) {  // quantum q only; the previous launch completed every quantum q-1 item
            P.q0 = q;
            P.n_items = count;
        }
        if (compact && q > 0) {  // the instances still running after quantum q-1
            P.list = lists[(q - 1) & 1];
            P.n_items_dev = nlive + ((q - 1) & 1);
            ck(cudaMemsetAsync(P.work, 0, 8, stream), "memset(work)");
        }
        void* args[] = {&P};
        ckd(d.LaunchKernel(m->function, (unsigned)grid, 1, 1, (unsigned)m->block_threads, 1, 1, (unsigned)dyn_smem,
                           (CUstream)stream,
                           args, nullptr),
            "cuLaunchKernel");
        ++m->launches;
        if (compact && q + 1 < nq) {
            unsigned long long* n_out = nlive + (q & 1);
            ck(cudaMemsetAsync(n_out, 0, 8, stream), "memset(nlive)");
            const unsigned int* l_in = q > 0 ? lists[(q - 1) & 1] : nullptr;
            const unsigned long long* n_in_dev = q > 0 ? nlive + ((q - 1) & 1) : nullptr;
            unsigned long long n_in = (unsigned long long)count;
            const unsigned int* flags = (const unsigned int*)P.st_flags;
            unsigned int* l_out = lists[q & 1];
            void* cargs[] = {(void*)&l_in, (void*)&n_in_dev, &n_in, (void*)&flags, &l_out, &n_out};
            const unsigned cgrid = (unsigned)std::min<int64_t>((count + 255) / 256, (int64_t)sms * 8);
            ckd(d.LaunchKernel(m->compact_fn, cgrid, 1, 1, 256, 1, 1, 0, (CUstream)stream, cargs, nullptr),
                "cuLaunchKernel(compact)");
            ++m->launches;
        }
    }
    ck(cudaEventRecord(m->ev1, stream), "cudaEventRecord");
    ck(cudaGetLastError(), "launch");

    m->simulated = true;
    m->finalized = false;
    m->last_stream = stream;
    m->n_total = n_total;
    m->first = first;
    m->count = count;
    m->K = K;
    m->dt = dt;
    m->t_end = t_end;
    m->seed = seed;
    m->last_stats_len = need_stats;
    m->items = nq * count;
    m->qs = qs;
    m->grid = (int)grid;
}

// ------------------------------------------------------------------------------------ finalize
// All quantile levels of one (cut, species) histogram in one scan (R11: the left edge of the
// first bin whose cumulative count reaches max(1, ceil(q n)); under/overflow give -inf/+inf): `order` lists the level indices by increasing level.
static void quantiles_from_hist(const int64_t* h, int B, int64_t n, const std::vector<double>& q,
                                const std::vector<int>& order, int64_t lo, int64_t w, double* out) {
    if (n == 0) {
        for (size_t i = 0; i < q.size(); ++i) out[i] = NAN;
        return;
    }
    size_t next = 0;
    int64_t c = 0;
    for (int b = 0; b < B + 2 && next < order.size(); ++b) {
        c += h[b];
        while (next < order.size()) {
            int64_t need = (int64_t)std::ceil(q[order[next]] * (double)n);
            if (need < 1) need = 1;
            if (c < need) break;
            out[order[next]] = b == 0 ? -INFINITY : (b == B + 1 ? INFINITY : (double)(lo + w * (int64_t)(b - 1)));
            ++next;
        }
    }
    for (; next < order.size(); ++next) out[order[next]] = INFINITY;
}

static void derive(cwc_model* m);
static int64_t final_cuts(cwc_model* m, int64_t* items_done);

void finalize(cwc_model* m, const int64_t* host_stats) {
    NvtxRange nvtx_range("cwc_stats_finalize");
    if (!m->simulated) fail(CWC_E_STATE, "no simulation to finalize");
    const size_t len = m->last_stats_len;
    m->h_stats.resize(len);
    ck(cudaStreamSynchronize(m->last_stream), "simulation");
    float ms = 0;
    if (cudaEventElapsedTime(&ms, m->ev0, m->ev1) == cudaSuccess) m->kernel_ms = ms;
    if (host_stats) std::memcpy(m->h_stats.data(), host_stats, len * 8);
    else ck(cudaMemcpy(m->h_stats.data(), m->d_stats, len * 8, cudaMemcpyDeviceToHost), "copy stats");
    m->cuts_final = m->K + 1;
    if (m->cancel_requested && !host_stats) m->cuts_final = final_cuts(m, nullptr);
    derive(m);
    {   // reactions per recorded cut of this run (choose_fast_cut of the next simulation)
        int64_t recs = 0;
        for (int64_t v : m->h_n) recs += v;
        const int64_t T = m->K + 1, TS = T * m->fm.S(), B = m->hist_bins;
        const int64_t reactions = m->h_stats[T + 3 * TS + TS * (B + 2) + CWC_CTR_REACTIONS];
        if (recs > 0) m->last_reactions_per_cut = (double)reactions / (double)recs;
    }
}

// On-line streaming: while the kernel
// runs, read the per-quantum progress counters and then the statistics through a copy engine on
// a separate stream.  Cuts below (q+1)*qs are final once every item of quanta 0..q has finished
// (an instance that ended early emitted or filled all its later cuts).  The counters are read
// before the statistics, so the snapshot contains every update of the cuts it reports final.
// Cuts [0, result) are final: every item of quanta 0..q-1 has finished (from the progress
// counters; stream option).  *items_done = finished items of all quanta.
static int64_t final_cuts(cwc_model* m, int64_t* items_done) {
    if (!m->poll_stream) ck(cudaStreamCreateWithFlags(&m->poll_stream, cudaStreamNonBlocking), "cudaStreamCreate");
    const int64_t T = m->K + 1, nq = (T + m->qs - 1) / m->qs;
    const ScratchLayout L = scratch_layout(m->fm.S(), m->count, T);
    std::vector<uint32_t> prog((size_t)nq);
    ck(cudaMemcpyAsync(prog.data(), (const char*)m->d_scratch + L.qprog, nq * 4, cudaMemcpyDeviceToHost,
                       m->poll_stream), "copy progress");
    ck(cudaStreamSynchronize(m->poll_stream), "copy progress");
    int64_t q = 0, done = 0;
    while (q < nq && prog[q] >= (uint64_t)m->count) ++q;
    for (uint32_t v : prog) done += v;
    if (items_done) *items_done = done;
    return std::min<int64_t>(q * m->qs, T);
}

// Terminate the running simulation (Fig. 2: "steer and terminate running
// simulations"): the kernel stops handing out work items; items in flight finish their quantum,
// so the cuts the progress counters report final stay exact.  Returns without waiting.
void cancel(cwc_model* m) {
    if (!m->simulated) fail(CWC_E_STATE, "no simulation");
    if (!m->stream) fail(CWC_E_STATE, "cwc_cancel needs the \"stream\" option set before simulating");
    if (!m->poll_stream) ck(cudaStreamCreateWithFlags(&m->poll_stream, cudaStreamNonBlocking), "cudaStreamCreate");
    static const uint32_t one = 1;
    const ScratchLayout L = scratch_layout(m->fm.S(), m->count, m->K + 1);
    // the flag lives in the range simulate_range clears on the launch stream before ev0: order the
    // write after that memset, or a cancel issued while it is still queued would be erased
    ck(cudaStreamWaitEvent(m->poll_stream, m->ev0, 0), "order cancel after the launch's memsets");
    ck(cudaMemcpyAsync((char*)m->d_scratch + L.cancel, &one, 4, cudaMemcpyHostToDevice, m->poll_stream),
       "set cancel flag");
    ck(cudaStreamSynchronize(m->poll_stream), "set cancel flag");
    m->cancel_requested = true;
    m->resumable = true;
}

// Replace the host statistics by a packed buffer of this geometry — e.g. the snapshots of all
// ranks summed while their kernels run — and derive the views; no device synchronisation.
void load_host_stats(cwc_model* m, const int64_t* host_stats, int64_t cuts_final) {
    if (!m->simulated) fail(CWC_E_STATE, "no simulation");
    if (!host_stats) fail(CWC_E_INVALID, "null statistics");
    if (cuts_final < 0 || cuts_final > m->K + 1) fail(CWC_E_INVALID, "cuts_final outside [0, T]");
    m->h_stats.assign(host_stats, host_stats + m->last_stats_len);
    m->cuts_final = cuts_final;
    derive(m);
}

// ------------------------------------------------------------------------ checkpoint / resume
// the counter-based RNG makes the per-instance record (x, t, step, k, flags, period
// state) plus the quanta done a complete checkpoint — a continued run draws exactly the numbers
// the uninterrupted one would have (R3), so resuming is bit-identical.

// What a checkpoint must agree with: the flat model and every option that changes results.
static uint64_t model_identity(const cwc_model* m) {
    std::ostringstream o;
    const FlatModel& f = m->fm;
    char buf[40];
    for (const auto& n : f.names) o << n << ';';
    for (int32_t v : f.x0) o << v << ',';
    for (double r : f.rates) { std::snprintf(buf, sizeof buf, "%a,", r); o << buf; }
    for (const auto& rl : f.reactants) { for (const auto& r : rl) o << r.species << ':' << r.order << ' '; o << '|'; }
    for (const auto& d : f.delta) { for (int32_t v : d) o << v << ','; o << '|'; }
    for (size_t j = 0; j < f.law.size(); ++j) {
        std::snprintf(buf, sizeof buf, "%a", f.law_K[j]);
        o << f.law[j] << ':' << f.law_species[j] << ':' << f.law_n[j] << ':' << buf << ';';
    }
    for (size_t j = 0; j < f.gate_species.size(); ++j) o << f.gate_species[j] << ':' << f.gate_kind[j] << ';';
    for (const auto& pl : f.place)
        for (const auto& sl : pl) { o << sl.alive << '<'; for (const auto& a : sl.adds) o << a.first << '+' << a.second << ' '; }
    for (const auto& tr : f.transfer) for (const auto& t : tr) o << t.first << '>' << t.second << ' ';
    o << '#' << f.sentinel << ';' << m->hist_bins << ';' << m->x_cap << ';' << m->raw_samples << ';'
      << m->period_species << ';' << m->period_lo << ';' << m->period_hi << ';';
    for (size_t s = 0; s < m->hist_lo.size(); ++s) o << m->hist_lo[s] << '/' << m->hist_width[s] << ',';
    return fnv1a(o.str());
}

namespace {
struct CkptHeader {
    char magic[8];
    uint64_t identity;
    int64_t n_total, first, count, K, qs;
    double dt, t_end;
    uint64_t seed;
    uint64_t stats_len, raw_len, scratch_bytes;
};
const char kCkptMagic[8] = {'C', 'W', 'C', 'C', 'K', 'P', 'T', '1'};
}  // namespace

size_t checkpoint_bytes(cwc_model* m) {
    if (!m->simulated) fail(CWC_E_STATE, "no simulation to checkpoint");
    size_t ns, nr, nsc;
    buffer_sizes(m, m->count, m->K, &ns, &nr, &nsc);
    return sizeof(CkptHeader) + ns * 8 + nsc + nr * 4;
}

// After the kernel has finished (a completed or terminated run): header, statistics, instance
// records + queue state, raw cuts.
void checkpoint_save(cwc_model* m, void* out, size_t bytes) {
    const size_t need = checkpoint_bytes(m);
    if (!out || bytes < need) fail(CWC_E_INVALID, "checkpoint buffer too small (see cwc_checkpoint_bytes)");
    ck(cudaStreamSynchronize(m->last_stream), "simulation");
    CkptHeader h{};
    std::memcpy(h.magic, kCkptMagic, 8);
    h.identity = model_identity(m);
    h.n_total = m->n_total; h.first = m->first; h.count = m->count; h.K = m->K; h.qs = m->qs;
    h.dt = m->dt; h.t_end = m->t_end; h.seed = m->seed;
    size_t ns, nr, nsc;
    buffer_sizes(m, m->count, m->K, &ns, &nr, &nsc);
    h.stats_len = ns; h.raw_len = nr; h.scratch_bytes = nsc;
    char* p = (char*)out;
    std::memcpy(p, &h, sizeof h);
    p += sizeof h;
    ck(cudaMemcpy(p, m->d_stats, ns * 8, cudaMemcpyDeviceToHost), "checkpoint stats");
    p += ns * 8;
    ck(cudaMemcpy(p, m->d_scratch, nsc, cudaMemcpyDeviceToHost), "checkpoint scratch");
    p += nsc;
    if (nr) ck(cudaMemcpy(p, m->d_raw, nr * 4, cudaMemcpyDeviceToHost), "checkpoint raw");
}

// Restore a checkpoint into this handle (same model and result-affecting options); the run can
// then be continued with cwc_resume or finalised as it stands.
void checkpoint_load(cwc_model* m, const void* in, size_t bytes) {
    if (!in || bytes < sizeof(CkptHeader)) fail(CWC_E_INVALID, "not a checkpoint");
    CkptHeader h;
    std::memcpy(&h, in, sizeof h);
    if (std::memcmp(h.magic, kCkptMagic, 8) != 0) fail(CWC_E_INVALID, "not a checkpoint");
    if (h.identity != model_identity(m)) fail(CWC_E_INVALID, "checkpoint of a different model or options");
    // the header sizes every buffer and the work-item geometry: validate it before any use
    if (!(h.dt > 0) || !std::isfinite(h.dt) || !(h.t_end >= 0) || !std::isfinite(h.t_end))
        fail(CWC_E_INVALID, "checkpoint header: bad horizon or sample interval");
    int64_t K_hdr = -1;
    try {
        K_hdr = grid_K(h.t_end, h.dt);
    } catch (const Error&) {
        fail(CWC_E_INVALID, "checkpoint header: t_end is not a multiple of sample_dt");
    }
    if (h.K != K_hdr) fail(CWC_E_INVALID, "checkpoint header: K does not match t_end / sample_dt");
    if (h.qs < 1 || h.qs > h.K + 1) fail(CWC_E_INVALID, "checkpoint header: quantum outside [1, K+1]");
    if (h.n_total <= 0 || h.first < 0 || h.count < 0 || h.first > h.n_total || h.count > h.n_total - h.first)
        fail(CWC_E_INVALID, "checkpoint header: instance range outside [0, n_total)");
    size_t ns, nr, nsc;
    buffer_sizes(m, h.count, h.K, &ns, &nr, &nsc);
    if (ns != h.stats_len || nr != h.raw_len || nsc != h.scratch_bytes ||
        bytes < sizeof h + ns * 8 + nsc + nr * 4)
        fail(CWC_E_INVALID, "checkpoint geometry does not match the model's buffers");
    const int dev = current_device(m);
    ck(cudaSetDevice(dev), "cudaSetDevice");
    if (m->bound) {
        if (m->stats_cap < ns * 8 || m->scratch_cap < nsc || (nr && m->raw_cap < nr * 4))
            fail(CWC_E_INVALID, "bound device buffers too small for the checkpoint");
    } else {
        grow(m->d_stats, m->stats_cap, ns * 8, "cudaMalloc(stats)");
        if (nr) grow(m->d_raw, m->raw_cap, nr * 4, "cudaMalloc(raw)");
        grow(m->d_scratch, m->scratch_cap, nsc, "cudaMalloc(scratch)");
    }
    const char* p = (const char*)in + sizeof h;
    ck(cudaMemcpy(m->d_stats, p, ns * 8, cudaMemcpyHostToDevice), "restore stats");
    p += ns * 8;
    ck(cudaMemcpy(m->d_scratch, p, nsc, cudaMemcpyHostToDevice), "restore scratch");
    p += nsc;
    if (nr) ck(cudaMemcpy(m->d_raw, p, nr * 4, cudaMemcpyHostToDevice), "restore raw");
    if (!m->ev0) {
        ck(cudaEventCreate(&m->ev0), "cudaEventCreate");
        ck(cudaEventCreate(&m->ev1), "cudaEventCreate");
    }
    ck(cudaEventRecord(m->ev0, nullptr), "cudaEventRecord");
    ck(cudaEventRecord(m->ev1, nullptr), "cudaEventRecord");
    m->simulated = true;
    m->finalized = false;
    m->last_stream = nullptr;
    m->n_total = h.n_total; m->first = h.first; m->count = h.count; m->K = h.K; m->qs = h.qs;
    m->dt = h.dt; m->t_end = h.t_end; m->seed = h.seed;
    m->last_stats_len = ns;
    m->items = ((h.K + 1 + h.qs - 1) / h.qs) * h.count;
    m->cancel_requested = false;
    m->resumable = true;
}

// Continue a terminated or restored run to its horizon on `stream` (asynchronous, like
// simulate_range): quanta already done are skipped, statistics keep accumulating.
void resume(cwc_model* m, cudaStream_t stream) {
    if (!m->simulated || !m->resumable) fail(CWC_E_STATE, "nothing to resume (terminate or restore a run first)");
    ck(cudaStreamSynchronize(m->last_stream), "terminated simulation");
    simulate_range(m, m->n_total, m->first, m->count, m->t_end, m->dt, m->seed, stream, false, true);
}

void snapshot(cwc_model* m, int64_t* cuts_final, int64_t* items_done) {
    NvtxRange nvtx_range("cwc_stats_snapshot");
    if (!m->simulated) fail(CWC_E_STATE, "no simulation");
    if (!m->stream) fail(CWC_E_STATE, "snapshots need the \"stream\" option set before simulating");
    int64_t done = 0;
    const int64_t cf = final_cuts(m, &done);   // counters first: the stats copy then holds them
    m->h_stats.resize(m->last_stats_len);
    ck(cudaMemcpyAsync(m->h_stats.data(), m->d_stats, m->last_stats_len * 8, cudaMemcpyDeviceToHost, m->poll_stream),
       "copy stats");
    ck(cudaStreamSynchronize(m->poll_stream), "copy stats");
    m->cuts_final = cf;
    derive(m);
    if (cuts_final) *cuts_final = m->cuts_final;
    if (items_done) *items_done = done;
}

static void derive(cwc_model* m) {
    const int64_t T = m->K + 1;
    const int S = m->fm.S(), B = m->hist_bins;
    const int64_t* p = m->h_stats.data();
    const int64_t TS = T * S;
    m->h_n.assign(p, p + T);
    m->h_sum.assign(p + T, p + T + TS);
    m->h_sqlo.assign(p + T + TS, p + T + 2 * TS);
    m->h_sqhi.assign(p + T + 2 * TS, p + T + 3 * TS);
    m->h_hist.assign(p + T + 3 * TS, p + T + 3 * TS + TS * (B + 2));
    // on-line period analysis (R19): per-cut integers -> local-period mean / variance and the
    // moving average of completed periods over the last `window` cuts, in time units
    m->h_period.clear();
    m->lp_mean.assign(T, NAN);
    m->lp_var.assign(T, NAN);
    m->p_ma.assign(T, NAN);
    if (m->period_species >= 0) {
        const int64_t* q = p + T + 3 * TS + TS * (B + 2) + CWC_N_CTR;
        m->h_period.assign(q, q + CWC_N_PERIOD * T);
        const int64_t *pcn = q + T, *pcs = q + 2 * T, *lpn = q + 5 * T, *lps = q + 6 * T;
        const int64_t *lpl = q + 7 * T, *lph = q + 8 * T;
        int64_t wn = 0, ws = 0;
        for (int64_t k = 0; k < T; ++k) {
            const int64_t n = lpn[k];
            if (n > 0) m->lp_mean[k] = (double)lps[k] / (double)n * m->dt;
            if (n > 1) {
                const __int128 sq = ((__int128)(uint64_t)lph[k] << 32) + (__int128)(uint64_t)lpl[k];
                const __int128 s = lps[k];
                const double vc = (double)((__int128)n * sq - s * s) / (double)((__int128)n * (n - 1));
                m->lp_var[k] = vc * m->dt * m->dt;
            }
            wn += pcn[k];
            ws += pcs[k];
            if (k >= m->period_window) {
                wn -= pcn[k - m->period_window];
                ws -= pcs[k - m->period_window];
            }
            if (wn > 0) m->p_ma[k] = (double)ws / (double)wn * m->dt;
        }
    }
    m->times.resize(T);
    m->mean.assign(TS, NAN);
    m->var.assign(TS, NAN);
    m->sumsq_d.resize(TS);
    const int nq = (int)m->quantiles.size();
    m->quant.assign(TS * nq, NAN);
    std::vector<int> qorder(nq);
    for (int qi = 0; qi < nq; ++qi) qorder[qi] = qi;
    std::stable_sort(qorder.begin(), qorder.end(), [&](int a, int b) { return m->quantiles[a] < m->quantiles[b]; });
    for (int64_t k = 0; k < T; ++k) {
        m->times[k] = (double)k * m->dt;
        const int64_t n = m->h_n[k];
        for (int s = 0; s < S; ++s) {
            const int64_t i = k * S + s;
            const __int128 sum = m->h_sum[i];
            const __int128 sq = ((__int128)(uint64_t)m->h_sqhi[i] << 32) + (__int128)(uint64_t)m->h_sqlo[i];
            m->sumsq_d[i] = (double)sq;
            if (n > 0) m->mean[i] = (double)sum / (double)n;
            if (n > 1) m->var[i] = (double)((__int128)n * sq - sum * sum) / (double)((__int128)n * (n - 1));
            quantiles_from_hist(&m->h_hist[i * (B + 2)], B, n, m->quantiles, qorder, m->hist_lo[s],
                                m->hist_width[s], &m->quant[i * nq]);
        }
    }
    m->finalized = true;
}

void copy_samples(cwc_model* m, int64_t first, int64_t count, int32_t* out) {
    NvtxRange nvtx_range("cwc_samples");
    if (!m->simulated) fail(CWC_E_STATE, "no simulation");
    if (!m->raw_samples || !m->d_raw) fail(CWC_E_STATE, "raw samples are disabled");
    if (first < 0 || count < 0 || first + count > m->count) fail(CWC_E_INVALID, "range outside the last simulation");
    if (!out) fail(CWC_E_INVALID, "null output");
    ck(cudaStreamSynchronize(m->last_stream), "simulation");
    if (count == 0) return;
    // device layout [ceil(T/8)][S][m->count][8] (time-blocked) -> out[T][S][count]
    const int64_t S = m->fm.S(), T = m->K + 1, TB = (T + CWC_RAW_BLOCK - 1) / CWC_RAW_BLOCK;
    const size_t row = (size_t)count * CWC_RAW_BLOCK;
    std::vector<int32_t> tmp((size_t)TB * S * row);
    ck(cudaMemcpy2D(tmp.data(), row * 4, m->d_raw + first * CWC_RAW_BLOCK, (size_t)m->count * CWC_RAW_BLOCK * 4,
                    row * 4, (size_t)TB * S, cudaMemcpyDeviceToHost),
       "copy samples");
    for (int64_t k = 0; k < T; ++k)
        for (int64_t s = 0; s < S; ++s) {
            const int32_t* src = tmp.data() + ((size_t)(k / CWC_RAW_BLOCK) * S + s) * row + (k % CWC_RAW_BLOCK);
            int32_t* dst = out + ((size_t)k * S + s) * count;
            for (int64_t j = 0; j < count; ++j) dst[j] = src[(size_t)j * CWC_RAW_BLOCK];
        }
}

void copy_records(cwc_model* m, int64_t first, int64_t count, uint8_t* flags, int64_t* reactions, double* t_last) {
    if (!m->simulated) fail(CWC_E_STATE, "no simulation");
    if (first < 0 || count < 0 || first + count > m->count) fail(CWC_E_INVALID, "range outside the last simulation");
    ck(cudaStreamSynchronize(m->last_stream), "simulation");
    if (count == 0) return;
    const ScratchLayout L = scratch_layout(m->fm.S(), m->count, m->K + 1);
    const char* sc = (const char*)m->d_scratch;
    if (flags) {
        std::vector<uint32_t> f(count);
        ck(cudaMemcpy(f.data(), sc + L.flags + first * 4, count * 4, cudaMemcpyDeviceToHost), "copy flags");
        for (int64_t i = 0; i < count; ++i) flags[i] = (uint8_t)(f[i] & 3u);
    }
    if (reactions)
        ck(cudaMemcpy(reactions, sc + L.step + first * 8, count * 8, cudaMemcpyDeviceToHost), "copy reactions");
    if (t_last) ck(cudaMemcpy(t_last, sc + L.t + first * 8, count * 8, cudaMemcpyDeviceToHost), "copy times");
}


// ------------------------------------------------------------------------ injected-draw self-test
// The SSA kernel's own step code (cwc_step_selftest_kernel in cwc_ssa.cuh, same NVRTC module)
// driven by caller-supplied uniforms from caller-supplied states: one lane per trajectory, up to
// n_draws steps each.  Host arrays in and out; cuts[i][k][s] = -2 where this call emitted no cut.
namespace {
struct SelftestIo {  // mirrors cwc_selftest_io (cwc_ssa.cuh)
    const int* x_in;
    const double* t_in;
    const long long* k_in;
    const double* u_tau;
    const double* u_sel;
    int* x_out;
    double* t_out;
    long long* k_out;
    int* status;
    int* n_done;
    long long n;
    int D;
    int mode;
};
}  // namespace

void selftest_step(cwc_model* m, int64_t n, int32_t n_draws, const int32_t* x, const double* t, const int64_t* k,
                   double t_end, double dt, const double* u_tau, const double* u_sel, int32_t mode, int32_t* x_out,
                   double* t_out, int64_t* k_out, int32_t* status, int32_t* n_done, int32_t* cuts) {
    if (n < 0 || n >= ((int64_t)1 << 31) || n_draws < 1 || (mode != 0 && mode != 1))
        fail(CWC_E_INVALID, "bad self-test arguments");
    const int64_t K = grid_K(t_end, dt), T = K + 1;
    const int S = m->fm.S();
    for (int64_t i = 0; i < n; ++i)
        if (k[i] < 0 || k[i] > T) fail(CWC_E_INVALID, "next cut index outside [0, K+1]");
    if (n == 0) return;
    if (!m->raw_samples) fail(CWC_E_STATE, "the self-test records cuts: raw_samples must be on");
    compile(m, nullptr);
    const int dev = current_device(m);
    ensure_module(m, dev);
    Driver& d = driver();
    CUfunction fn = nullptr;
    ckd(d.ModuleGetFunction(&fn, m->module, "cwc_step_selftest_kernel"), "cuModuleGetFunction(selftest)");
    cwc_logtab_entry tab[128];
    build_log_table(tab);
    const size_t TB = (size_t)((T + CWC_RAW_BLOCK - 1) / CWC_RAW_BLOCK);
    const size_t raw_n = TB * S * (size_t)n * CWC_RAW_BLOCK;
    const size_t st_n = stats_len(T, S, m->hist_bins, m->period_species >= 0);
    const size_t nd = (size_t)n * n_draws;
    // one device block: [logtab | stats | raw | x_in | t | k | u_tau | u_sel | x_out | t_out | k_out | status | n_done]
    size_t off[14], o = 0;
    const size_t sizes[13] = {sizeof tab, st_n * 8, raw_n * 4, (size_t)n * S * 4, (size_t)n * 8, (size_t)n * 8,
                              nd * 8, nd * 8, (size_t)n * S * 4, (size_t)n * 8, (size_t)n * 8, (size_t)n * 4,
                              (size_t)n * 4};
    for (int i = 0; i < 13; ++i) { off[i] = o; o = align256(o + sizes[i]); }
    off[13] = o;
    char* dmem = nullptr;
    ck(cudaMalloc(&dmem, o), "cudaMalloc(self-test)");
    struct Free { char* p; ~Free() { cudaFree(p); } } guard_mem{dmem};
    std::vector<int32_t> raw_init(raw_n, -2);
    std::vector<long long> kk(k, k + n);
    ck(cudaMemcpy(dmem + off[0], tab, sizeof tab, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemset(dmem + off[1], 0, st_n * 8), "memset");
    ck(cudaMemcpy(dmem + off[2], raw_init.data(), raw_n * 4, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemcpy(dmem + off[3], x, (size_t)n * S * 4, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemcpy(dmem + off[4], t, (size_t)n * 8, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemcpy(dmem + off[5], kk.data(), (size_t)n * 8, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemcpy(dmem + off[6], u_tau, nd * 8, cudaMemcpyHostToDevice), "H2D");
    ck(cudaMemcpy(dmem + off[7], u_sel, nd * 8, cudaMemcpyHostToDevice), "H2D");
    cwc_params P;
    std::memset(&P, 0, sizeof P);
    P.first = 0;
    P.count = n;
    P.K = K;
    P.dt = dt;
    P.qs = T;
    P.n_items = n;
    for (int r = 0; r < 10; ++r) {  // seed 0 (the primed Philox draws are overwritten by the injected ones)
        P.rk.k0[r] = (uint32_t)r * 0x9E3779B9u;
        P.rk.k1[r] = (uint32_t)r * 0xBB67AE85u;
    }
    P.stats = (unsigned long long*)(dmem + off[1]);
    P.raw = (int*)(dmem + off[2]);
    P.logtab = (const cwc_logtab_entry*)(dmem + off[0]);
    P.smem_stats = 0;
    SelftestIo io{(const int*)(dmem + off[3]), (const double*)(dmem + off[4]), (const long long*)(dmem + off[5]),
                  (const double*)(dmem + off[6]), (const double*)(dmem + off[7]), (int*)(dmem + off[8]),
                  (double*)(dmem + off[9]), (long long*)(dmem + off[10]), (int*)(dmem + off[11]),
                  (int*)(dmem + off[12]), (long long)n, n_draws, mode};
    void* args[] = {&P, &io};
    const unsigned block = 128;
    ckd(d.LaunchKernel(fn, (unsigned)((n + block - 1) / block), 1, 1, block, 1, 1, 0, nullptr, args, nullptr),
        "cuLaunchKernel(self-test)");
    ck(cudaDeviceSynchronize(), "self-test kernel");
    std::vector<int32_t> raw(raw_n);
    std::vector<long long> ko(n);
    ck(cudaMemcpy(raw.data(), dmem + off[2], raw_n * 4, cudaMemcpyDeviceToHost), "D2H");
    ck(cudaMemcpy(x_out, dmem + off[8], (size_t)n * S * 4, cudaMemcpyDeviceToHost), "D2H");
    ck(cudaMemcpy(t_out, dmem + off[9], (size_t)n * 8, cudaMemcpyDeviceToHost), "D2H");
    ck(cudaMemcpy(ko.data(), dmem + off[10], (size_t)n * 8, cudaMemcpyDeviceToHost), "D2H");
    ck(cudaMemcpy(status, dmem + off[11], (size_t)n * 4, cudaMemcpyDeviceToHost), "D2H");
    ck(cudaMemcpy(n_done, dmem + off[12], (size_t)n * 4, cudaMemcpyDeviceToHost), "D2H");
    for (int64_t i = 0; i < n; ++i) k_out[i] = ko[i];
    if (cuts)  // time-blocked [TB][S][n][8] -> [n][T][S]
        for (int64_t i = 0; i < n; ++i)
            for (int64_t kc = 0; kc < T; ++kc)
                for (int s = 0; s < S; ++s)
                    cuts[(i * T + kc) * S + s] =
                        raw[(((size_t)(kc / CWC_RAW_BLOCK) * S + s) * n + i) * CWC_RAW_BLOCK + kc % CWC_RAW_BLOCK];
}

}  // namespace cwc

cwc_model::~cwc_model() {
    if (module) {
        cwc::Driver& d = cwc::driver();
        d.ModuleUnload(module);
    }
    cwc::free_owned(this);
    if (d_logtab) cudaFree(d_logtab);
    if (own_stream) cudaStreamDestroy(own_stream);
    if (poll_stream) cudaStreamDestroy(poll_stream);
    if (ev0) cudaEventDestroy(ev0);
    if (ev1) cudaEventDestroy(ev1);
}
