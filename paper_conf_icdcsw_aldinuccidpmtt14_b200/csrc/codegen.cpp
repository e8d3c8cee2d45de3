// codegen.cpp — emit the model section of the SSA kernel translation unit.
//
// The flat network from the rule compiler becomes straight-line CUDA: species counts are an
// int array indexed only by compile-time constants (registers), rate constants are exact hex
// literals, propensities are the product of per-species binomial factors (R1) multiplied by
// k_j and summed left to right with explicitly rounded operations (R5), and the rewrite
// x += nu_{j*} is a predicated select chain (no divergent branch on the selected rule).
#include "codegen.hpp"

#include <cstdio>
#include <sstream>

namespace cwc {
namespace {

std::string hexd(double v) {
    char buf[64];
    std::snprintf(buf, sizeof buf, "%a", v);
    return buf;
}

}  // namespace

std::string generate_model_section(const FlatModel& fm, const KernelConfig& cfg) {
    const int S = fm.S(), M = fm.M();
    auto is_flag = [&](int sp) { return fm.flag.size() == (size_t)S && fm.flag[sp]; };
    std::ostringstream o;
    o << "// ---- generated model section: " << S << " species, " << M << " flat reactions\n";
    o << "#define CWC_S " << S << "\n#define CWC_M " << (M > 0 ? M : 1) << "\n#define CWC_B " << cfg.hist_bins
      << "\n#define CWC_BLOCK " << cfg.block_threads << "\n#define CWC_MINB " << cfg.min_blocks << "\n#define CWC_ILP " << cfg.ilp << "\n";
    o << "#define CWC_PERIOD_S " << cfg.period_species << "\n#define CWC_PERIOD_LO " << cfg.period_lo
      << "LL\n#define CWC_PERIOD_HI " << cfg.period_hi << "LL\n";
    o << "#define CWC_RAW " << (cfg.raw ? 1 : 0) << "  // raw cuts recorded (option raw_samples)\n";
    o << "#define CWC_X_CAP " << cfg.x_cap << "\n#define CWC_FAST_CUT " << (cfg.fast_cut ? 1 : 0) << "\n";
    o << "#define CWC_SENTINEL " << fm.sentinel << "  // species \"#full\" of the compartment pools (R20), -1 none\n";
    // branch-free fast commit (cuts on the full-step path) for small models: the select per state
    // word costs less than the divergent branch up to ~4 species (same-box A/B, profiles/
    // r2_ab_kernel.log: LV 1M +2.7 %, 100k +3.3 %; circadian, 9 species, -4 %)
    o << "#ifndef CWC_BRANCHFREE\n#define CWC_BRANCHFREE " << (S <= 4 ? 1 : 0) << "\n#endif\n";
    // draw batch: the next D draws as D independent chains, then D fast steps (same-box sweep,
    // profiles/s2f_ab_draw_batch.log: D = 4 best up to 8 species (LV +3.5-4.1 %, Neurospora +6 %,
    // Schlogl +1 %), 3 for 9-16 (compartments +5.3 %, circadian +7.3 %); larger models keep 0)
    const int db = cfg.draw_batch >= 0 ? cfg.draw_batch : (S <= 8 ? 4 : (S <= 16 ? 3 : 0));
    o << "#ifndef CWC_DRAW_BATCH\n#define CWC_DRAW_BATCH " << (cfg.ilp == 1 ? db : 0) << "\n#endif\n";
    // the batch's draws are committed to the lane state when the warp leaves the loop (LV 1M +6 %,
    // circadian +1.5 %, Neurospora +1 %) — except for one-species models (Schlogl -2.7 %), same box
    o << "#ifndef CWC_DEFER_DRAW\n#define CWC_DEFER_DRAW " << (S > 1 ? 1 : 0) << "\n#endif\n";
    // cooperative cut recording in the fast step (same-box A/B, profiles/s2p_ab_coop_emission.log):
    // it pays when a cut is recorded by few lanes of a warp at a time and its species spread over
    // the lanes — compartments (9 species, a cut every ~290 reactions) +4.4 % — and loses where
    // many lanes record at once (vesicles, 29 species: -40 %) or the cut has 1-3 species
    // (Schlogl, Neurospora: -7 %)
    o << "#ifndef CWC_COOP_EMIT\n#define CWC_COOP_EMIT " << (S >= 8 && S <= 16 ? 1 : 0) << "\n#endif\n\n";
    if (cfg.seed_keys) {
        const uint32_t k0 = (uint32_t)cfg.seed, k1 = (uint32_t)(cfg.seed >> 32);
        o << "#define CWC_STATIC_KEYS 1\nstatic constexpr cwc_round_keys cwc_rk_static = {{";
        for (int r = 0; r < 10; ++r) o << (r ? ", " : "") << (uint32_t)(k0 + (uint32_t)r * 0x9E3779B9u) << "u";
        o << "}, {";
        for (int r = 0; r < 10; ++r) o << (r ? ", " : "") << (uint32_t)(k1 + (uint32_t)r * 0xBB67AE85u) << "u";
        o << "}};\n\n";
    }
    for (int s = 0; s < S; ++s) o << "// species " << s << ": " << fm.names[s] << "\n";

    // x = x0
    o << "__device__ __forceinline__ void cwc_init(int (&x)[CWC_S]) {\n";
    for (int s = 0; s < S; ++s) o << "    x[" << s << "] = " << fm.x0[s] << ";\n";
    o << "}\n\n";

    // propensities: emitted twice, as the running sums (hot) and as "last a_j > 0" (the rare
    // rounding-hole fallback of R6) so only cum[] is live across the step.
    for (int variant = 0; variant < 2; ++variant) {
    if (variant == 0)
        o << "__device__ __forceinline__ double cwc_propensities(const int (&x)[CWC_S], double (&cum)[CWC_M]) {\n"
             "    double a[CWC_M];\n";
    else
        o << "__device__ __forceinline__ int cwc_last_positive(const int (&x)[CWC_S]) {\n    double a[CWC_M];\n";
    // per-(species, order) binomial factors, shared between reactions
    std::vector<std::vector<bool>> need(S, std::vector<bool>(4, false));
    for (int j = 0; j < M; ++j) {
        for (const Reactant& r : fm.reactants[j])
            if (!is_flag(r.species)) need[r.species][r.order] = true;
        if (fm.law[j] != LAW_MASS_ACTION) need[fm.law_species[j]][1] = true;
    }
    for (int s = 0; s < S; ++s) {
        if (need[s][1] || need[s][2]) o << "    const double f" << s << "_1 = (double)x[" << s << "];\n";
        // C(x, 2) = x (x - 1) / 2: x - 1 as an exact DADD (no second conversion); x (x - 1) is an
        // even integer < 2^54, exact in a double, and so is its half (x = 0 gives -0.0, which every
        // use treats as 0: a_j = +-0, cum unchanged, never selected)
        if (need[s][2])
            o << "    const double f" << s << "_2 = __dmul_rn(__dmul_rn(f" << s << "_1, __dsub_rn(f" << s
              << "_1, 1.0)), 0.5);\n";
        if (need[s][3])
            o << "    const double f" << s << "_3 = (double)(((long long)x[" << s << "] * (long long)(x[" << s
              << "] - 1) / 2) * (long long)(x[" << s << "] - 2) / 3);\n";
    }
    if (M == 0) o << "    a[0] = 0.0;\n";
    for (int j = 0; j < M; ++j) {
        std::string h;
        // occupancy flags (R20) are 0/1: k * h * flag == (flag ? k * h : 0.0) exactly, so they
        // select instead of multiplying
        std::string flags;
        for (const Reactant& r : fm.reactants[j])
            if (is_flag(r.species)) flags += std::string(flags.empty() ? "" : " && ") + "x[" + std::to_string(r.species) + "] != 0";
        for (const Reactant& r : fm.reactants[j]) {
            if (is_flag(r.species)) continue;
            std::string f = "f" + std::to_string(r.species) + "_" + std::to_string(r.order);
            h = h.empty() ? f : "__dmul_rn(" + h + ", " + f + ")";
        }
        // reading R20: a gated reaction (creation / pool full) is enabled while x_g >= 1 / x_g == 0
        std::string gate = flags;
        if (!fm.gate_species.empty() && fm.gate_species[j] >= 0)
            gate += std::string(gate.empty() ? "" : " && ") + "x[" + std::to_string(fm.gate_species[j]) +
                    (fm.gate_kind[j] == GATE_POSITIVE ? "] >= 1" : "] == 0");
        if (fm.law[j] == LAW_MASS_ACTION) {
            std::string e = h.empty() ? hexd(fm.rates[j]) : "__dmul_rn(" + hexd(fm.rates[j]) + ", " + h + ")";
            if (!gate.empty()) e = "(" + gate + ") ? " + e + " : 0.0";
            o << "    a[" << j << "] = " << e << ";  // rule " << fm.rule_of[j] << "\n";
            continue;
        }
        if (!gate.empty()) h = h.empty() ? "((" + gate + ") ? 1.0 : 0.0)" : "__dmul_rn(" + h + ", (" + gate + ") ? 1.0 : 0.0)";
        // functional rate law (R16'): k*X/(K+X), k*X^n/(K^n+X^n) or k*K^n/(K^n+X^n), only when the
        // lhs is available; powers are left-to-right products, K^n computed on the host the same way
        const std::string X = "f" + std::to_string(fm.law_species[j]) + "_1";
        std::string Xn = X;
        for (int i = 1; i < fm.law_n[j]; ++i) Xn = "__dmul_rn(" + Xn + ", " + X + ")";
        double Kn = fm.law_K[j];
        for (int i = 1; i < fm.law_n[j]; ++i) Kn = Kn * fm.law_K[j];
        std::string expr;
        if (fm.law[j] == LAW_MM)
            expr = "cwc_div(__dmul_rn(" + hexd(fm.rates[j]) + ", " + X + "), __dadd_rn(" + hexd(fm.law_K[j]) + ", " +
                   X + "))";
        else if (fm.law[j] == LAW_HILL)
            expr = "cwc_div(__dmul_rn(" + hexd(fm.rates[j]) + ", " + Xn + "), __dadd_rn(" + hexd(Kn) + ", " + Xn + "))";
        else
            expr = "cwc_div(__dmul_rn(" + hexd(fm.rates[j]) + ", " + hexd(Kn) + "), __dadd_rn(" + hexd(Kn) + ", " + Xn +
                   "))";
        o << "    a[" << j << "] = " << (h.empty() ? expr : "(" + h + " != 0.0) ? " + expr + " : 0.0")
          << ";  // rule " << fm.rule_of[j] << " (rate law)\n";
    }
    if (variant == 0) {
        o << "    cum[0] = a[0];\n";
        for (int j = 1; j < M; ++j) o << "    cum[" << j << "] = __dadd_rn(cum[" << j - 1 << "], a[" << j << "]);\n";
        o << "    return cum[CWC_M - 1];\n}\n\n";
    } else {
        o << "    int j = 0;\n#pragma unroll\n    for (int i = 0; i < CWC_M; ++i) if (a[i] > 0.0) j = i;\n";
        o << "    return j;\n}\n\n";
    }
    }

    // selection: j* = min{j : cum_j > target} = #{j : cum_j <= target}; rounding hole -> last a_j > 0
    o << "__device__ __forceinline__ int cwc_select(const int (&x)[CWC_S], const double (&cum)[CWC_M], double target) {\n";
    o << "    int j = 0;\n";
    o << "#pragma unroll\n    for (int i = 0; i < CWC_M; ++i) j += (cum[i] <= target) ? 1 : 0;\n";
    o << "    if (j >= CWC_M) j = cwc_last_positive(x);\n";
    o << "    return j;\n}\n\n";

    // rewrite + overflow check on the species some rule increases.  Few (rule, species) pairs:
    // a predicated select chain; many (large networks): the selected rule's row of packed int8
    // deltas from a shared-memory table (one vector load + a sign-extending byte extract per species)
    std::vector<bool> inc(S, false);
    int pairs = 0, maxabs = 0;
    for (int j = 0; j < M; ++j)
        for (int s = 0; s < S; ++s)
            if (fm.delta[j][s]) {
                ++pairs;
                maxabs = std::max(maxabs, std::abs(fm.delta[j][s]));
                if (fm.delta[j][s] > 0) inc[s] = true;
            }
    // reading R20: creations (first free slot of a pool) and destructions (moves of the rest)
    // depend on the state, so they are applied by rule index after the delta
    std::vector<int> special;
    for (int j = 0; j < M; ++j)
        if ((!fm.place.empty() && !fm.place[j].empty()) || (!fm.transfer.empty() && !fm.transfer[j].empty())) {
            special.push_back(j);
            for (const auto& ps : fm.place[j])
                for (const auto& a : ps.adds) inc[a.first] = true;
            for (const auto& x : fm.transfer[j])
                if (x.second >= 0) inc[x.second] = true;
        }
    std::string special_code;
    for (int j : special) {
        std::ostringstream so;
        so << "    if (j == " << j << ") {\n";
        bool first = true;
        for (const auto& ps : fm.place[j]) {
            so << "        " << (first ? "if" : "else if") << " (x[" << ps.alive << "] == 0) {";
            for (const auto& a : ps.adds) so << " x[" << a.first << "] += " << a.second << ";";
            so << " }\n";
            first = false;
        }
        for (const auto& x : fm.transfer[j]) {
            if (x.second >= 0) so << "        x[" << x.second << "] += x[" << x.first << "];\n";
            so << "        x[" << x.first << "] = 0;\n";
        }
        so << "    }\n";
        special_code += so.str();
    }
    const bool table = (cfg.delta_table == 1 || (cfg.delta_table < 0 && pairs > 2 * S)) && maxabs <= 127 && M > 0;
    // fast-path rewrite straight from the selection predicates p_i = (cum_i <= target), which are
    // monotone (cum is non-decreasing), so p_i = [i < j*] and the telescoping sum
    // nu_0 + sum_{i<M-1} (nu_{i+1} - nu_i) p_i = nu_{j*} needs no rule index at all
    const bool telescope = !table && M > 1 && special.empty() && (cfg.delta_table == 2 || cfg.delta_table < 0);
    if (telescope) {
        o << "#define CWC_TELESCOPE 1\n";
        o << "__device__ __forceinline__ bool cwc_apply_p(const bool (&p)[CWC_M], int (&x)[CWC_S]) {\n";
        for (int s = 0; s < S; ++s) {
            const int base = fm.delta[0][s];
            std::vector<std::pair<int, int>> terms;  // (i, nu_{i+1,s} - nu_{i,s})
            for (int i = 0; i + 1 < M; ++i)
                if (fm.delta[i + 1][s] != fm.delta[i][s]) terms.push_back({i, fm.delta[i + 1][s] - fm.delta[i][s]});
            if (terms.empty() && base == 0) continue;
            std::string e;
            for (size_t t = 0; t < terms.size(); ++t) {
                const int d = terms[t].second + (t == 0 ? base : 0), z = (t == 0 ? base : 0);
                e += (t ? " + " : "") + std::string("(p[") + std::to_string(terms[t].first) + "] ? " + std::to_string(d) +
                     " : " + std::to_string(z) + ")";
            }
            if (terms.empty()) e = std::to_string(base);
            o << "    x[" << s << "] += " << e << ";\n";
        }
        o << "    bool over = false;\n";
        for (int s = 0; s < S; ++s)
            if (inc[s]) o << "    over |= x[" << s << "] > CWC_X_CAP;\n";
        o << "    return over;\n}\n\n";
    }
    const int words = (S + 3) / 4, wpad = words <= 1 ? 1 : (words <= 2 ? 2 : (words + 3) / 4 * 4);
    if (table) {
        o << "#define CWC_DELTA_TABLE 1\n#define CWC_DELTA_WORDS " << wpad << "\n";
        o << "__constant__ unsigned int cwc_delta_const[" << M * wpad << "] = {";
        for (int j = 0; j < M; ++j)
            for (int w = 0; w < wpad; ++w) {
                uint32_t word = 0;
                for (int b = 0; b < 4; ++b) {
                    const int s = w * 4 + b;
                    if (s < S) word |= (uint32_t)(uint8_t)(int8_t)fm.delta[j][s] << (8 * b);
                }
                o << (j || w ? ", " : "") << word << "u";
            }
        o << "};\n__shared__ __align__(16) unsigned int cwc_delta_smem[" << M * wpad << "];\n";
        o << "__device__ __forceinline__ void cwc_delta_init() {\n    for (int i = threadIdx.x; i < "
          << M * wpad << "; i += blockDim.x) cwc_delta_smem[i] = cwc_delta_const[i];\n}\n";
        o << "__device__ __forceinline__ bool cwc_apply(int j, int (&x)[CWC_S]) {\n";
        o << "    const unsigned int* row = cwc_delta_smem + j * CWC_DELTA_WORDS;\n";
        o << "    unsigned int w[CWC_DELTA_WORDS];\n";
        if (wpad == 1) o << "    w[0] = row[0];\n";
        else if (wpad == 2) o << "    { const uint2 v = *reinterpret_cast<const uint2*>(row); w[0] = v.x; w[1] = v.y; }\n";
        else
            for (int q = 0; q < wpad / 4; ++q)
                o << "    { const uint4 v = *reinterpret_cast<const uint4*>(row + " << 4 * q << "); w[" << 4 * q
                  << "] = v.x; w[" << 4 * q + 1 << "] = v.y; w[" << 4 * q + 2 << "] = v.z; w[" << 4 * q + 3
                  << "] = v.w; }\n";
        for (int s = 0; s < S; ++s) {
            bool any = false;
            for (int j = 0; j < M; ++j) any |= fm.delta[j][s] != 0;
            if (any)
                o << "    x[" << s << "] += ((int)(w[" << s / 4 << "] << " << 24 - 8 * (s % 4) << ")) >> 24;\n";
        }
    } else {
        o << "__device__ __forceinline__ void cwc_delta_init() {}\n";
        o << "__device__ __forceinline__ bool cwc_apply(int j, int (&x)[CWC_S]) {\n";
        for (int s = 0; s < S; ++s) {
            std::string chain = "0";
            for (int j = M - 1; j >= 0; --j) {
                int d = fm.delta[j][s];
                if (!d) continue;
                chain = "(j == " + std::to_string(j) + " ? " + std::to_string(d) + " : " + chain + ")";
            }
            if (chain != "0") o << "    x[" << s << "] += " << chain << ";\n";
        }
    }
    o << special_code;
    o << "    bool over = false;\n";
    for (int s = 0; s < S; ++s)
        if (inc[s] && !(fm.flag.size() == (size_t)S && fm.flag[s]) && s != fm.sentinel)
            o << "    over |= x[" << s << "] > CWC_X_CAP;\n";
    if (fm.sentinel >= 0) o << "    over |= x[" << fm.sentinel << "] > 0;  // a pool was full (R20)\n";
    o << "    return over;\n}\n\n";

    // histogram bins: 0 underflow, 1..B, B+1 overflow (R11)
    o << "__device__ __forceinline__ int cwc_bin(int s, int v) {\n    long long lo = 0, w = 1;\n    switch (s) {\n";
    for (int s = 0; s < S; ++s)
        o << "        case " << s << ": lo = " << cfg.hist_lo[s] << "LL; w = " << cfg.hist_width[s] << "LL; break;\n";
    o << "        default: break;\n    }\n";
    o << "    const long long d = (long long)v - lo;\n";
    o << "    if (d < 0) return 0;\n    const long long b = d / w;\n    return b >= CWC_B ? CWC_B + 1 : (int)b + 1;\n}\n";
    // the same bins with a run-time species index (cooperative cut recording: lane s records
    // species s), from a shared-memory copy of (lo, width)
    o << "__constant__ long long cwc_hist_c[" << 2 * S << "] = {";
    for (int s = 0; s < S; ++s) o << (s ? ", " : "") << cfg.hist_lo[s] << "LL, " << cfg.hist_width[s] << "LL";
    o << "};\n__shared__ long long cwc_hist_sm[" << 2 * S << "];\n";
    o << "__device__ __forceinline__ void cwc_hist_init() {\n    for (int i = threadIdx.x; i < " << 2 * S
      << "; i += blockDim.x) cwc_hist_sm[i] = cwc_hist_c[i];\n}\n";
    o << "__device__ __forceinline__ int cwc_bin_rt(int s, int v) {\n"
         "    const long long d = (long long)v - cwc_hist_sm[2 * s];\n    if (d < 0) return 0;\n"
         "    const long long b = d / cwc_hist_sm[2 * s + 1];\n    return b >= CWC_B ? CWC_B + 1 : (int)b + 1;\n}\n";
    o << "// ---- end of generated model section\n\n";
    return o.str();
}

}  // namespace cwc
