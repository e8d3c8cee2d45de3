// Rule compiler: CWC terms + rewrite rules -> flat mass-action network.
//
// PAPER.md P:L203-215 (§IV): CWC terms are multisets of atoms and compartments; a compartment
// has a membrane (wrap) multiset, a content term and a label; rules rewrite inside a compartment
// or across nested compartments.  The paper's simulator matches rule patterns against dynamic
// term trees at every step.  For static compartment structure (no creation or
// destruction, R15/R16) every match site is fixed, so this compiler does the tree matching ONCE
// at load and emits one flat reaction per (rule, context, compartment assignment); the GPU then
// never touches a tree.  Compartments that rules create or destroy (reading R20) live in
// bounded pools of slots, each slot a fixed set of regions plus an occupancy flag, so the
// matching is still done once.  DESIGN.md §3 "flattening" is the normative statement.
#pragma once

#include <cstdint>
#include <map>
#include <stdexcept>
#include <string>
#include <vector>

namespace cwc {

struct Error : std::runtime_error {
    int32_t code;  // CWC_E_*
    Error(int32_t c, const std::string& m) : std::runtime_error(m), code(c) {}
};

enum Law : int32_t { LAW_MASS_ACTION = 0, LAW_MM = 1, LAW_HILL = 2, LAW_HILLR = 3 };
enum Gate : int32_t { GATE_NONE = 0, GATE_POSITIVE = 1, GATE_ZERO = 2 };
constexpr int32_t kDefaultCapacity = 8;  // slots per dynamic-compartment pool (reading R20)

struct Reactant {
    int32_t species;
    int32_t order;
    bool operator==(const Reactant& o) const { return species == o.species && order == o.order; }
};

struct FlatModel {
    std::vector<std::string> alphabet;
    std::vector<std::string> names;              // [S]
    std::vector<int32_t> x0;                     // [S]
    std::vector<double> rates;                   // [M]
    std::vector<std::vector<Reactant>> reactants;  // [M], ascending species
    std::vector<std::vector<int32_t>> delta;     // [M][S]
    std::vector<int32_t> rule_of;                // [M]
    // functional rate laws (reading R16'): LAW_* per reaction, the species the law reads (-1
    // for mass action), its constant K and Hill exponent n
    std::vector<int32_t> law, law_species, law_n;  // [M]
    std::vector<double> law_K;                     // [M]
    // dynamic compartments in bounded pools (reading R20): per reaction an optional gate
    // (species, GATE_*), the candidate slots of a creation (the first whose occupancy flag is 0
    // receives its additions), the moves of a destruction (applied after delta: x[dst] += x[src]
    // (dst >= 0), x[src] = 0); per species whether it is a 0/1 occupancy flag; the "#full"
    // species whose increment means a pool overflowed (R9), or -1
    struct PlaceSlot {
        int32_t alive;
        std::vector<std::pair<int32_t, int32_t>> adds;  // (species, count), ascending species
    };
    std::vector<int32_t> gate_species, gate_kind;                  // [M]
    std::vector<std::vector<PlaceSlot>> place;                     // [M]
    std::vector<std::vector<std::pair<int32_t, int32_t>>> transfer;  // [M] (src, dst), ascending src
    std::vector<uint8_t> flag;                                     // [S]
    int32_t sentinel = -1;
    int32_t n_rules = 0;
    int64_t x_cap_max = 0;                       // largest cap with every prod C(cap, r) < 2^53

    int32_t S() const { return (int32_t)names.size(); }
    int32_t M() const { return (int32_t)rates.size(); }
};

// Parse + flatten.  Throws cwc::Error with CWC_E_INVALID / CWC_E_PARSE / CWC_E_UNSUPPORTED.
// capacity: slots per pool of each dynamic compartment label (default kDefaultCapacity).
FlatModel compile_model(const std::vector<std::string>& alphabet,
                        const std::vector<std::string>& rules, const std::vector<double>& rates,
                        const std::string& initial_term,
                        const std::map<std::string, int64_t>& capacity = {});

// Largest cap in [1, limit] such that prod_s C(cap, r_s) < 2^53 for every reaction (R9).
int64_t max_exact_cap(const std::vector<std::vector<Reactant>>& reactants, int64_t limit);

}  // namespace cwc
