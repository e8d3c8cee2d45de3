// Rule compiler implementation — see compiler.hpp and DESIGN.md §3 (input syntax, flattening).
#include "compiler.hpp"

#include <algorithm>
#include <cctype>
#include <cmath>
#include <map>
#include <memory>
#include <set>
#include <unordered_map>

#include "cwc.h"

namespace cwc {
namespace {

// ----------------------------------------------------------------------------------- lexer
enum class Tok { Arrow, Mult, Var, Name, Sym, End };

struct Token {
    Tok kind;
    std::string text;
    int64_t value = 0;
};

bool is_name_start(char c) { return std::isalpha((unsigned char)c) || c == '_'; }
bool is_name_char(char c) { return std::isalnum((unsigned char)c) || c == '_'; }

std::vector<Token> lex(const std::string& s) {
    std::vector<Token> out;
    size_t i = 0, n = s.size();
    while (true) {
        while (i < n && std::isspace((unsigned char)s[i])) ++i;
        if (i >= n) break;
        char c = s[i];
        if (c == '-' && i + 1 < n && s[i + 1] == '>') {
            out.push_back({Tok::Arrow, "->"});
            i += 2;
        } else if (std::isdigit((unsigned char)c)) {
            size_t j = i;
            while (j < n && std::isdigit((unsigned char)s[j])) ++j;
            size_t k = j;
            while (k < n && std::isspace((unsigned char)s[k])) ++k;
            if (k >= n || s[k] != '*')
                throw Error(CWC_E_PARSE, "multiplicity without '*' in '" + s + "'");
            std::string digits = s.substr(i, j - i);
            if (digits.size() > 10) throw Error(CWC_E_INVALID, "multiplicity too large in '" + s + "'");
            Token t{Tok::Mult, digits};
            t.value = std::stoll(digits);
            out.push_back(t);
            i = k + 1;
        } else if (c == '$') {
            size_t j = i + 1;
            if (j >= n || !is_name_start(s[j])) throw Error(CWC_E_PARSE, "bad variable in '" + s + "'");
            while (j < n && is_name_char(s[j])) ++j;
            out.push_back({Tok::Var, s.substr(i, j - i)});
            i = j;
        } else if (is_name_start(c)) {
            size_t j = i;
            while (j < n && is_name_char(s[j])) ++j;
            out.push_back({Tok::Name, s.substr(i, j - i)});
            i = j;
        } else {
            out.push_back({Tok::Sym, std::string(1, c)});
            ++i;
        }
    }
    out.push_back({Tok::End, ""});
    return out;
}

// ----------------------------------------------------------------------------------- trees
using Counts = std::vector<int64_t>;  // indexed by atom

struct Node;  // a term: atoms + compartments
struct Comp {
    std::string label;
    Counts wrap;
    std::unique_ptr<Node> content;
};
struct Node {
    Counts atoms;
    std::vector<Comp> comps;
};

struct PComp {
    std::string label;
    Counts wrap, content;
    std::string wvar, cvar;
};
struct Pattern {
    Counts atoms;
    std::vector<PComp> comps;
};

class Parser {
  public:
    Parser(const std::string& text, const std::unordered_map<std::string, int>& atoms, bool pattern)
        : src_(text), toks_(lex(text)), atoms_(atoms), pattern_(pattern) {}

    const Token& peek() const { return toks_[pos_]; }
    Token take() { return toks_[pos_++]; }
    bool at_end() const { return peek().kind == Tok::End; }

    void expect_sym(char c) {
        Token t = take();
        if (t.kind != Tok::Sym || t.text[0] != c)
            throw Error(CWC_E_PARSE, std::string("expected '") + c + "' in '" + src_ + "'");
    }
    int atom(const std::string& name) {
        auto it = atoms_.find(name);
        if (it == atoms_.end()) throw Error(CWC_E_INVALID, "unknown atom '" + name + "'");
        return it->second;
    }

    // A sequence of atoms / n*A / '.' / variable; compartments only where allowed.
    // Stops at End, Arrow, or one of the stop symbols.
    // comps: 0 = compartment is a parse error, 1 = unsupported, 2 = allowed.
    // vars (a rule's right-hand side at rule level, reading R20): the released variables.
    void sequence(const char* stops, int comps_policy, Counts& atoms, std::string* var,
                  std::vector<Comp>* comps, std::vector<PComp>* pcomps, std::vector<std::string>* vars = nullptr) {
        while (true) {
            const Token& t = peek();
            if (t.kind == Tok::End || t.kind == Tok::Arrow) return;
            if (t.kind == Tok::Sym && std::string(stops).find(t.text[0]) != std::string::npos) return;
            Token tk = take();
            if (tk.kind == Tok::Sym && tk.text == ".") continue;
            if (tk.kind == Tok::Mult) {
                Token nm = take();
                if (nm.kind != Tok::Name) throw Error(CWC_E_PARSE, "expected atom after '*' in '" + src_ + "'");
                atoms[atom(nm.text)] += tk.value;
            } else if (tk.kind == Tok::Name) {
                atoms[atom(tk.text)] += 1;
            } else if (tk.kind == Tok::Var) {
                if (!pattern_) throw Error(CWC_E_PARSE, "variable " + tk.text + " in a term");
                if (vars) {
                    if (std::find(vars->begin(), vars->end(), tk.text) != vars->end())
                        throw Error(CWC_E_UNSUPPORTED, "variable " + tk.text + " released twice: '" + src_ + "'");
                    vars->push_back(tk.text);
                    continue;
                }
                if (!var) throw Error(CWC_E_UNSUPPORTED, "variable at rule level: '" + src_ + "'");
                if (!var->empty()) throw Error(CWC_E_UNSUPPORTED, "two variables in one multiset: '" + src_ + "'");
                *var = tk.text;
            } else if (tk.kind == Tok::Sym && tk.text == "(") {
                if (comps_policy == 0) throw Error(CWC_E_PARSE, "compartment inside a membrane: '" + src_ + "'");
                if (comps_policy == 1)
                    throw Error(CWC_E_UNSUPPORTED, "nested compartment in a pattern compartment: '" + src_ + "'");
                compartment(comps, pcomps);
            } else {
                throw Error(CWC_E_PARSE, "unexpected '" + tk.text + "' in '" + src_ + "'");
            }
        }
    }

    void compartment(std::vector<Comp>* comps, std::vector<PComp>* pcomps) {
        Counts wrap(atoms_.size(), 0), content(atoms_.size(), 0);
        std::string wvar, cvar;
        sequence("|", 0, wrap, pattern_ ? &wvar : nullptr, nullptr, nullptr);
        expect_sym('|');
        std::unique_ptr<Node> inner;
        if (pattern_) {
            sequence(")", 1, content, &cvar, nullptr, nullptr);
        } else {
            inner.reset(new Node{Counts(atoms_.size(), 0), {}});
            sequence(")", 2, inner->atoms, nullptr, &inner->comps, nullptr);
        }
        expect_sym(')');
        expect_sym('^');
        Token lab = take();
        if (lab.kind != Tok::Name) throw Error(CWC_E_PARSE, "expected label after '^' in '" + src_ + "'");
        if (lab.text == "top") throw Error(CWC_E_INVALID, "'top' is reserved for the outermost level");
        if (pattern_) {
            pcomps->push_back(PComp{lab.text, wrap, content, wvar, cvar});
        } else {
            Comp c;
            c.label = lab.text;
            c.wrap = wrap;
            c.content = std::move(inner);
            comps->push_back(std::move(c));
        }
    }

  private:
    std::string src_;
    std::vector<Token> toks_;
    size_t pos_ = 0;
    const std::unordered_map<std::string, int>& atoms_;
    bool pattern_;
};

struct Rule {
    std::string label;
    Pattern lhs, rhs;
    double rate;
    int32_t law = LAW_MASS_ACTION;  // "@ mm(X, K)" / "@ hill(X, K, n)" / "@ hillr(X, K, n)"
    int law_atom = -1;
    double law_K = 0.0;
    int32_t law_n = 1;
    // reading R20: per lhs pattern compartment the rhs compartment it persists as (-1:
    // destroyed), the created rhs compartment (-1: none), the released rule-level variables
    std::vector<int> keep;
    int create = -1;
    std::vector<std::string> release;
};

bool valid_ident(const std::string& s) {
    if (s.empty() || !is_name_start(s[0])) return false;
    for (char c : s)
        if (!is_name_char(c)) return false;
    return true;
}

std::string trim(const std::string& s) {
    size_t a = 0, b = s.size();
    while (a < b && std::isspace((unsigned char)s[a])) ++a;
    while (b > a && std::isspace((unsigned char)s[b - 1])) --b;
    return s.substr(a, b - a);
}

// Rate-law suffix of a rule (reading R16'): "mm(X, K)" | "hill(X, K, n)" | "hillr(X, K, n)".
void parse_law(const std::string& text, const std::unordered_map<std::string, int>& atoms, Rule& r) {
    std::string t = trim(text);
    size_t lp = t.find('('), rp = t.rfind(')');
    if (lp == std::string::npos || rp == std::string::npos || rp < lp || trim(t.substr(rp + 1)) != "")
        throw Error(CWC_E_PARSE, "bad rate law '" + t + "'");
    const std::string name = trim(t.substr(0, lp));
    std::vector<std::string> args;
    std::string cur;
    for (char c : t.substr(lp + 1, rp - lp - 1)) {
        if (c == ',') { args.push_back(trim(cur)); cur.clear(); }
        else cur += c;
    }
    args.push_back(trim(cur));
    if (name == "mm") r.law = LAW_MM;
    else if (name == "hill") r.law = LAW_HILL;
    else if (name == "hillr") r.law = LAW_HILLR;
    else throw Error(CWC_E_PARSE, "unknown rate law '" + name + "'");
    if (args.size() != (r.law == LAW_MM ? 2u : 3u))
        throw Error(CWC_E_PARSE, "wrong number of rate-law arguments in '" + t + "'");
    auto it = atoms.find(args[0]);
    if (it == atoms.end()) throw Error(CWC_E_INVALID, "unknown atom '" + args[0] + "' in rate law");
    r.law_atom = it->second;
    char* end = nullptr;
    r.law_K = std::strtod(args[1].c_str(), &end);
    if (args[1].empty() || *end != '\0') throw Error(CWC_E_PARSE, "bad constant in rate law '" + t + "'");
    if (!std::isfinite(r.law_K) || !(r.law_K > 0))
        throw Error(CWC_E_INVALID, "rate-law constant must be finite and > 0: '" + t + "'");
    if (r.law != LAW_MM) {
        for (char c : args[2])
            if (!std::isdigit((unsigned char)c)) throw Error(CWC_E_PARSE, "bad Hill exponent in '" + t + "'");
        if (args[2].empty() || args[2].size() > 2) throw Error(CWC_E_PARSE, "bad Hill exponent in '" + t + "'");
        r.law_n = std::atoi(args[2].c_str());
        if (r.law_n < 1 || r.law_n > 8) throw Error(CWC_E_INVALID, "Hill exponent must be in [1, 8]: '" + t + "'");
    }
}

Rule parse_rule(const std::string& text, const std::unordered_map<std::string, int>& atoms, double rate) {
    if (!std::isfinite(rate) || rate < 0) throw Error(CWC_E_INVALID, "rate of rule '" + text + "' must be finite and >= 0");
    size_t colon = text.find(':');
    if (colon == std::string::npos) throw Error(CWC_E_PARSE, "rule without label: '" + text + "'");
    Rule r;
    r.label = trim(text.substr(0, colon));
    r.rate = rate;
    if (!valid_ident(r.label)) throw Error(CWC_E_PARSE, "bad rule label '" + r.label + "'");
    std::string body = text.substr(colon + 1);
    const size_t at = body.find('@');
    if (at != std::string::npos) {
        parse_law(body.substr(at + 1), atoms, r);
        body = body.substr(0, at);
    }
    size_t arrow = body.find("->");
    if (arrow == std::string::npos || body.find("->", arrow + 2) != std::string::npos)
        throw Error(CWC_E_PARSE, "rule must contain exactly one '->': '" + text + "'");
    std::string sides[2] = {body.substr(0, arrow), body.substr(arrow + 2)};
    Pattern* pats[2] = {&r.lhs, &r.rhs};
    for (int k = 0; k < 2; ++k) {
        Parser p(sides[k], atoms, true);
        pats[k]->atoms.assign(atoms.size(), 0);
        p.sequence("", 2, pats[k]->atoms, nullptr, nullptr, &pats[k]->comps, k == 1 ? &r.release : nullptr);
        if (!p.at_end()) throw Error(CWC_E_PARSE, "trailing input in '" + sides[k] + "'");
    }
    // Structure (readings R15, R20): an rhs compartment carrying the variables of an lhs pattern
    // compartment is that compartment (same label); an rhs compartment without variables is
    // created (at most one per rule); an lhs compartment that does not reappear is destroyed and
    // its variables may be released at rule level.  Pattern compartments are open (both
    // variables present).
    std::set<std::string> seen;
    for (const PComp& a : r.lhs.comps) {
        if (a.wvar.empty() || a.cvar.empty())
            throw Error(CWC_E_UNSUPPORTED, "pattern compartment without $wrap/$content variables: '" + text + "'");
        for (const std::string* v : {&a.wvar, &a.cvar})
            if (!seen.insert(*v).second) throw Error(CWC_E_UNSUPPORTED, "variable " + *v + " used twice: '" + text + "'");
    }
    r.keep.assign(r.lhs.comps.size(), -1);
    for (size_t bi = 0; bi < r.rhs.comps.size(); ++bi) {
        const PComp& b = r.rhs.comps[bi];
        if (b.wvar.empty() && b.cvar.empty()) {
            if (r.create >= 0) throw Error(CWC_E_UNSUPPORTED, "more than one compartment created: '" + text + "'");
            r.create = (int)bi;
            continue;
        }
        int match = -1;
        for (size_t ai = 0; ai < r.lhs.comps.size(); ++ai)
            if (r.lhs.comps[ai].wvar == b.wvar && r.lhs.comps[ai].cvar == b.cvar) {
                match = (int)ai;
                break;
            }
        if (match < 0 || r.keep[match] >= 0)
            throw Error(CWC_E_UNSUPPORTED, "variables moved between compartments: '" + text + "'");
        if (r.lhs.comps[match].label != b.label) throw Error(CWC_E_UNSUPPORTED, "relabelling a compartment: '" + text + "'");
        r.keep[match] = (int)bi;
    }
    std::set<std::string> gone;
    for (size_t ai = 0; ai < r.lhs.comps.size(); ++ai)
        if (r.keep[ai] < 0) {
            gone.insert(r.lhs.comps[ai].wvar);
            gone.insert(r.lhs.comps[ai].cvar);
        }
    for (const std::string& v : r.release)
        if (!gone.count(v))
            throw Error(CWC_E_UNSUPPORTED, "variable " + v + " released but its compartment is not destroyed: '" + text + "'");
    return r;
}

// ----------------------------------------------------------------------------------- regions
struct Region {
    std::string name;        // "" = top content
    std::string owner;       // owning compartment label ("top")
    bool wrap;
    Counts atoms;
    std::vector<int> child_content, child_wrap;
    int pool = -1, slot = -1;  // the pool slot this region belongs to (reading R20)
};

// Reading R20: the slots for the dynamic compartments of one label in one content region.
struct Pool {
    int parent;
    std::string label;
    std::vector<std::pair<int, int>> slots;  // (wrap region, content region)
    int occupied;                             // slots 0..occupied-1 filled by the initial term
};

struct RegionBuilder {
    std::vector<Region>& regs;
    std::vector<Pool>& pools;
    const std::set<std::string>& dynamic;
    const std::set<std::pair<std::string, std::string>>& creators;  // (context label, created label)
    const std::map<std::string, int64_t>& capacity;

    // Pre-order: the content region, each static child (wrap, content, recursively), then the
    // pools of dynamic children in label order, slot by slot (wrap, content).
    int add_content(const Node& node, const std::string& name, const std::string& owner) {
        int idx = (int)regs.size();
        regs.push_back(Region{name, owner, false, node.atoms, {}, {}});
        std::map<std::string, int> total, seen;
        for (const Comp& c : node.comps)
            if (!dynamic.count(c.label)) total[c.label]++;
        std::map<std::string, std::vector<const Comp*>> dyn;
        for (const Comp& c : node.comps) {
            if (dynamic.count(c.label)) {
                if (!c.content->comps.empty())
                    throw Error(CWC_E_UNSUPPORTED, "dynamic compartment '" + c.label + "' with nested compartments");
                dyn[c.label].push_back(&c);
                continue;
            }
            std::string seg = c.label;
            if (total[c.label] > 1) seg += "#" + std::to_string(seen[c.label]);
            seen[c.label]++;
            std::string path = name.empty() ? seg : name + "/" + seg;
            int w = (int)regs.size();
            regs.push_back(Region{path + ".wrap", c.label, true, c.wrap, {}, {}});
            int ci = add_content(*c.content, path, c.label);
            regs[idx].child_wrap.push_back(w);
            regs[idx].child_content.push_back(ci);
        }
        std::set<std::string> labels;
        for (auto& kv : dyn) labels.insert(kv.first);
        for (auto& cr : creators)
            if (cr.first == owner) labels.insert(cr.second);
        const size_t A = node.atoms.size();
        for (const std::string& l : labels) {
            const std::vector<const Comp*>& init = dyn[l];
            auto it = capacity.find(l);
            const int64_t cap = it == capacity.end() ? kDefaultCapacity : it->second;
            if (cap < 1 || cap > 4096 || (int64_t)init.size() > cap)
                throw Error(CWC_E_INVALID, "capacity of '" + l + "' must be in [1, 4096] and hold the initial compartments");
            const int pid = (int)pools.size();
            pools.push_back(Pool{idx, l, {}, (int)init.size()});
            for (int k = 0; k < (int)cap; ++k) {
                std::string seg = l + "[" + std::to_string(k) + "]";
                std::string path = name.empty() ? seg : name + "/" + seg;
                Counts w(A, 0), ct(A, 0);
                if (k < (int)init.size()) {
                    w = init[k]->wrap;
                    ct = init[k]->content->atoms;
                }
                int wi = (int)regs.size();
                regs.push_back(Region{path + ".wrap", l, true, w, {}, {}, pid, k});
                int ci = (int)regs.size();
                regs.push_back(Region{path, l, false, ct, {}, {}, pid, k});
                regs[idx].child_wrap.push_back(wi);
                regs[idx].child_content.push_back(ci);
                pools[pid].slots.push_back({wi, ci});
            }
        }
        return idx;
    }
};

struct Destroyed {
    int wrap, content;
    bool rel_wrap, rel_content;
};

struct RawReaction {
    int rule;
    double rate;
    int ctx;  // context region (where a rate law's species is read)
    std::map<std::pair<int, int>, int64_t> react;   // (region, atom) -> order
    std::map<std::pair<int, int>, int64_t> delta;   // (region, atom) -> net change (may be 0)
    // reading R20
    std::pair<int, int> gate{-1, -1};
    int gate_kind = GATE_NONE;
    int place_pool = -1;                             // creation into this pool
    const PComp* created = nullptr;
    std::vector<Destroyed> destroyed;
    std::vector<std::pair<std::pair<int, int>, std::pair<int, int>>> xfer;  // src -> dst ((-1,-1) removed)
};

// Enumerate injective, label-matching assignments of pattern compartments to children, in
// lexicographic order of the chosen child indices.
void assignments(const std::vector<Region>& regs, const Region& ctx, const std::vector<PComp>& pc,
                 std::vector<int>& cur, std::vector<bool>& used, std::vector<std::vector<int>>& out) {
    size_t p = cur.size();
    if (p == pc.size()) {
        out.push_back(cur);
        return;
    }
    for (size_t c = 0; c < ctx.child_content.size(); ++c) {
        if (used[c] || regs[ctx.child_content[c]].owner != pc[p].label) continue;
        used[c] = true;
        cur.push_back((int)c);
        assignments(regs, ctx, pc, cur, used, out);
        cur.pop_back();
        used[c] = false;
    }
}

unsigned __int128 binom128(int64_t x, int r) {
    if (x < r) return 0;
    unsigned __int128 c = 1;
    for (int i = 0; i < r; ++i) c = c * (unsigned __int128)(x - i) / (unsigned __int128)(i + 1);
    return c;
}

}  // namespace

int64_t max_exact_cap(const std::vector<std::vector<Reactant>>& reactants, int64_t limit) {
    const unsigned __int128 two53 = (unsigned __int128)1 << 53;
    auto ok = [&](int64_t cap) {
        for (const auto& rl : reactants) {
            unsigned __int128 h = 1;
            for (const Reactant& e : rl) h *= binom128(cap, e.order);
            if (h >= two53) return false;
        }
        return true;
    };
    if (ok(limit)) return limit;
    int64_t lo = 1, hi = limit;
    while (lo < hi) {
        int64_t mid = lo + (hi - lo + 1) / 2;
        if (ok(mid)) lo = mid; else hi = mid - 1;
    }
    return lo;
}

FlatModel compile_model(const std::vector<std::string>& alphabet, const std::vector<std::string>& rules,
                        const std::vector<double>& rates, const std::string& initial_term,
                        const std::map<std::string, int64_t>& capacity) {
    if (alphabet.empty()) throw Error(CWC_E_INVALID, "empty alphabet");
    if (rules.size() != rates.size()) throw Error(CWC_E_INVALID, "one rate per rule");
    std::unordered_map<std::string, int> atoms;
    for (size_t i = 0; i < alphabet.size(); ++i) {
        if (!valid_ident(alphabet[i]) || alphabet[i] == "top") throw Error(CWC_E_INVALID, "bad atom name '" + alphabet[i] + "'");
        if (!atoms.emplace(alphabet[i], (int)i).second) throw Error(CWC_E_INVALID, "duplicate atom '" + alphabet[i] + "'");
    }
    const int A = (int)alphabet.size();

    Node top{Counts(A, 0), {}};
    {
        Parser p(initial_term, atoms, false);
        p.sequence("", 2, top.atoms, nullptr, &top.comps, nullptr);
        if (!p.at_end()) throw Error(CWC_E_PARSE, "trailing input in initial term");
    }
    std::vector<Rule> parsed;
    for (size_t i = 0; i < rules.size(); ++i) parsed.push_back(parse_rule(rules[i], atoms, rates[i]));

    // Reading R20: a label is dynamic when a rule creates or destroys a compartment of it.
    std::set<std::string> dynamic;
    std::set<std::pair<std::string, std::string>> creators;
    for (const Rule& r : parsed) {
        if (r.create >= 0) {
            dynamic.insert(r.rhs.comps[r.create].label);
            creators.insert({r.label, r.rhs.comps[r.create].label});
        }
        for (size_t a = 0; a < r.lhs.comps.size(); ++a)
            if (r.keep[a] < 0) dynamic.insert(r.lhs.comps[a].label);
    }
    for (auto& cr : creators)
        if (dynamic.count(cr.first))
            throw Error(CWC_E_UNSUPPORTED, "compartment '" + cr.second + "' created inside dynamic compartment '" + cr.first + "'");
    for (auto& kv : capacity)
        if (!dynamic.count(kv.first)) throw Error(CWC_E_INVALID, "capacity of '" + kv.first + "': not a dynamic compartment");

    std::vector<Region> regs;
    std::vector<Pool> pools;
    RegionBuilder rb{regs, pools, dynamic, creators, capacity};
    rb.add_content(top, "", "top");
    std::map<std::pair<int, std::string>, int> pool_of;
    for (size_t p = 0; p < pools.size(); ++p) pool_of[{pools[p].parent, pools[p].label}] = (int)p;
    // pseudo-atoms of the flag species (ordered after the alphabet within a region)
    std::vector<std::string> dyn_labels(dynamic.begin(), dynamic.end());  // sorted
    const int ALIVE = A, FULL = A + 1 + (int)dyn_labels.size();
    auto FREE = [&](const std::string& l) {
        return A + 1 + (int)(std::lower_bound(dyn_labels.begin(), dyn_labels.end(), l) - dyn_labels.begin());
    };
    auto alive_of = [&](int region) { return std::make_pair(pools[regs[region].pool].slots[regs[region].slot].second, ALIVE); };

    // Tree matching once: every (rule, context, assignment) is a flat reaction (two for a creation).
    std::vector<RawReaction> raw;
    for (size_t ri = 0; ri < parsed.size(); ++ri) {
        const Rule& rule = parsed[ri];
        for (size_t ci = 0; ci < regs.size(); ++ci) {
            const Region& ctx = regs[ci];
            if (ctx.wrap || ctx.owner != rule.label) continue;
            std::vector<std::vector<int>> found;
            std::vector<int> cur;
            std::vector<bool> used(ctx.child_content.size(), false);
            assignments(regs, ctx, rule.lhs.comps, cur, used, found);
            for (const auto& asg : found) {
                RawReaction rr;
                rr.rule = (int)ri;
                rr.rate = rule.rate;
                rr.ctx = (int)ci;
                std::map<std::pair<int, int>, int64_t> prod;
                auto add = [](std::map<std::pair<int, int>, int64_t>& m, int reg, const Counts& c) {
                    for (size_t a = 0; a < c.size(); ++a)
                        if (c[a]) m[{reg, (int)a}] += c[a];
                };
                add(rr.react, (int)ci, rule.lhs.atoms);
                add(prod, (int)ci, rule.rhs.atoms);
                if (ctx.pool >= 0) {  // inside a pool slot: only while it is occupied
                    rr.react[alive_of((int)ci)] += 1;
                    prod[alive_of((int)ci)] += 1;
                }
                for (size_t p = 0; p < asg.size(); ++p) {
                    int w = ctx.child_wrap[asg[p]], c = ctx.child_content[asg[p]];
                    const PComp& pc = rule.lhs.comps[p];
                    add(rr.react, w, pc.wrap);
                    add(rr.react, c, pc.content);
                    if (regs[c].pool >= 0) rr.react[alive_of(c)] += 1;
                    if (rule.keep[p] >= 0) {
                        const PComp& qc = rule.rhs.comps[rule.keep[p]];
                        add(prod, w, qc.wrap);
                        add(prod, c, qc.content);
                        if (regs[c].pool >= 0) prod[alive_of(c)] += 1;
                    } else {  // destroyed: the slot is freed, the rest moved or removed
                        const Pool& pl = pools[regs[c].pool];
                        prod[{pl.parent, FREE(pl.label)}] += 1;
                        const bool rw = std::find(rule.release.begin(), rule.release.end(), pc.wvar) != rule.release.end();
                        const bool rc = std::find(rule.release.begin(), rule.release.end(), pc.cvar) != rule.release.end();
                        rr.destroyed.push_back(Destroyed{w, c, rw, rc});
                    }
                }
                int64_t order = 0;
                for (auto& kv : rr.react)
                    if (kv.first.second != ALIVE) order += kv.second;
                if (order > 3) throw Error(CWC_E_UNSUPPORTED, "reaction order > 3 in rule " + std::to_string(ri));
                for (auto& kv : prod) rr.delta[kv.first] += kv.second;
                for (auto& kv : rr.react) rr.delta[kv.first] -= kv.second;
                if (rule.create < 0) {
                    raw.push_back(std::move(rr));
                    continue;
                }
                // creation: into the lowest free slot of the pool, else the pool is full
                const PComp& qc = rule.rhs.comps[rule.create];
                const int pid = pool_of.at({(int)ci, qc.label});
                const std::pair<int, int> fkey{(int)ci, FREE(qc.label)};
                RawReaction full = rr;
                rr.gate = fkey;
                rr.gate_kind = GATE_POSITIVE;
                rr.delta[fkey] -= 1;
                rr.place_pool = pid;
                rr.created = &qc;
                full.gate = fkey;
                full.gate_kind = GATE_ZERO;
                full.delta.clear();
                full.delta[{0, FULL}] = 1;
                full.destroyed.clear();
                raw.push_back(std::move(rr));
                raw.push_back(std::move(full));
            }
        }
    }

    // Species: every (region, atom) present initially or touched by a reaction, the flags of
    // every pool, "#full" when a pool can overflow; region pre-order, then alphabet order, then
    // "#alive", "#free:<label>" (label order), "#full".
    std::set<std::pair<int, int>> used;
    for (size_t r = 0; r < regs.size(); ++r)
        for (int a = 0; a < A; ++a)
            if (regs[r].atoms[a] > 0) used.insert({(int)r, a});
    for (const Pool& pl : pools) {
        used.insert({pl.parent, FREE(pl.label)});
        for (auto& sl : pl.slots) used.insert({sl.second, ALIVE});
    }
    bool has_full = false;
    for (const auto& rr : raw) {
        for (auto& kv : rr.react) used.insert(kv.first);
        for (auto& kv : rr.delta) used.insert(kv.first);
        if (rr.gate.first >= 0) used.insert(rr.gate);
        if (rr.gate_kind == GATE_ZERO) has_full = true;
        if (rr.place_pool >= 0)
            for (auto& sl : pools[rr.place_pool].slots)
                for (int a = 0; a < A; ++a) {
                    if (rr.created->wrap[a]) used.insert({sl.first, a});
                    if (rr.created->content[a]) used.insert({sl.second, a});
                }
        if (parsed[rr.rule].law != LAW_MASS_ACTION) used.insert({rr.ctx, parsed[rr.rule].law_atom});
    }
    if (has_full) used.insert({0, FULL});
    for (auto& rr : raw)
        for (const Destroyed& d : rr.destroyed)
            for (int k = 0; k < 2; ++k) {
                const int reg = k == 0 ? d.wrap : d.content;
                const bool rel = k == 0 ? d.rel_wrap : d.rel_content;
                std::vector<std::pair<int, int>> srcs;
                for (auto& ra : used)
                    if (ra.first == reg && ra.second < A) srcs.push_back(ra);
                for (auto& src : srcs) {
                    std::pair<int, int> dst = rel ? std::make_pair(rr.ctx, src.second) : std::make_pair(-1, -1);
                    rr.xfer.push_back({src, dst});
                    if (rel) used.insert(dst);
                }
            }
    if (used.empty()) throw Error(CWC_E_INVALID, "model has no species");

    FlatModel fm;
    fm.alphabet = alphabet;
    fm.n_rules = (int32_t)parsed.size();
    std::map<std::pair<int, int>, int> sidx;
    for (const auto& ra : used) {  // std::set order == (region, atom) lexicographic
        sidx[ra] = (int)fm.names.size();
        const Region& reg = regs[ra.first];
        std::string atom;
        int64_t v = 0;
        if (ra.second < A) {
            atom = alphabet[ra.second];
            v = reg.atoms[ra.second];
        } else if (ra.second == ALIVE) {
            atom = "#alive";
            v = reg.slot < pools[reg.pool].occupied ? 1 : 0;
        } else if (ra.second == FULL) {
            atom = "#full";
        } else {
            const std::string& l = dyn_labels[ra.second - A - 1];
            atom = "#free:" + l;
            const Pool& pl = pools[pool_of.at({ra.first, l})];
            v = (int64_t)pl.slots.size() - pl.occupied;
        }
        fm.names.push_back(reg.name.empty() ? atom : atom + "@" + reg.name);
        if (v > (int64_t)INT32_MAX) throw Error(CWC_E_INVALID, "initial count too large");
        fm.x0.push_back((int32_t)v);
        fm.flag.push_back(ra.second == ALIVE ? 1 : 0);
    }
    fm.sentinel = has_full ? sidx[{0, FULL}] : -1;
    const int S = (int)fm.names.size();
    std::vector<std::vector<Reactant>> cap_lists;
    for (const auto& rr : raw) {
        std::vector<Reactant> rl, rl_cap;
        for (auto& kv : rr.react) rl.push_back(Reactant{sidx[kv.first], (int32_t)kv.second});
        std::sort(rl.begin(), rl.end(), [](const Reactant& a, const Reactant& b) { return a.species < b.species; });
        for (const Reactant& e : rl)
            if (!fm.flag[e.species]) rl_cap.push_back(e);
        cap_lists.push_back(rl_cap);
        std::vector<int32_t> d(S, 0);
        for (auto& kv : rr.delta) d[sidx[kv.first]] += (int32_t)kv.second;
        fm.reactants.push_back(rl);
        fm.delta.push_back(d);
        fm.rates.push_back(rr.rate);
        fm.rule_of.push_back(rr.rule);
        const Rule& rule = parsed[rr.rule];
        fm.law.push_back(rule.law);
        fm.law_species.push_back(rule.law == LAW_MASS_ACTION ? -1 : sidx[{rr.ctx, rule.law_atom}]);
        fm.law_K.push_back(rule.law_K);
        fm.law_n.push_back(rule.law_n);
        fm.gate_species.push_back(rr.gate.first >= 0 ? sidx[rr.gate] : -1);
        fm.gate_kind.push_back(rr.gate_kind);
        std::vector<FlatModel::PlaceSlot> place;
        if (rr.place_pool >= 0)
            for (auto& sl : pools[rr.place_pool].slots) {
                FlatModel::PlaceSlot ps;
                ps.alive = sidx[{sl.second, ALIVE}];
                std::map<int, int32_t> adds;
                adds[ps.alive] += 1;
                for (int a = 0; a < A; ++a) {
                    if (rr.created->wrap[a]) adds[sidx[{sl.first, a}]] += (int32_t)rr.created->wrap[a];
                    if (rr.created->content[a]) adds[sidx[{sl.second, a}]] += (int32_t)rr.created->content[a];
                }
                for (auto& kv : adds) ps.adds.push_back({kv.first, kv.second});
                place.push_back(ps);
            }
        fm.place.push_back(place);
        std::vector<std::pair<int32_t, int32_t>> xf;
        for (auto& e : rr.xfer) xf.push_back({sidx[e.first], e.second.first >= 0 ? sidx[e.second] : -1});
        std::sort(xf.begin(), xf.end());
        fm.transfer.push_back(xf);
    }
    // flags are 0/1 and do not limit the exact propensity range (R9)
    fm.x_cap_max = max_exact_cap(cap_lists, (int64_t)1 << 30);
    return fm;
}

}  // namespace cwc
