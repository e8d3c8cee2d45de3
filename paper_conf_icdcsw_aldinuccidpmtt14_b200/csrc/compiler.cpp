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
    void sequence(const char* stops, int comps_policy, Counts& atoms, std::string* var,
                  std::vector<Comp>* comps, std::vector<PComp>* pcomps) {
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
        p.sequence("", 2, pats[k]->atoms, nullptr, nullptr, &pats[k]->comps);
        if (!p.at_end()) throw Error(CWC_E_PARSE, "trailing input in '" + sides[k] + "'");
    }
    // Static structure: the k-th rhs compartment is the k-th lhs compartment, same label and
    // variables; both variables present (open patterns).
    if (r.lhs.comps.size() != r.rhs.comps.size())
        throw Error(CWC_E_UNSUPPORTED, "compartment creation/destruction: '" + text + "'");
    std::set<std::string> seen;
    for (size_t c = 0; c < r.lhs.comps.size(); ++c) {
        const PComp &a = r.lhs.comps[c], &b = r.rhs.comps[c];
        if (a.label != b.label) throw Error(CWC_E_UNSUPPORTED, "relabelling a compartment: '" + text + "'");
        if (a.wvar.empty() || a.cvar.empty())
            throw Error(CWC_E_UNSUPPORTED, "pattern compartment without $wrap/$content variables: '" + text + "'");
        if (a.wvar != b.wvar || a.cvar != b.cvar)
            throw Error(CWC_E_UNSUPPORTED, "variables moved between compartments: '" + text + "'");
        for (const std::string* v : {&a.wvar, &a.cvar}) {
            if (!seen.insert(*v).second) throw Error(CWC_E_UNSUPPORTED, "variable " + *v + " used twice: '" + text + "'");
        }
    }
    return r;
}

// ----------------------------------------------------------------------------------- regions
struct Region {
    std::string name;        // "" = top content
    std::string owner;       // owning compartment label ("top")
    bool wrap;
    Counts atoms;
    std::vector<int> child_content, child_wrap;
};

int add_content(std::vector<Region>& regs, const Node& node, const std::string& name, const std::string& owner) {
    int idx = (int)regs.size();
    regs.push_back(Region{name, owner, false, node.atoms, {}, {}});
    std::map<std::string, int> total, seen;
    for (const Comp& c : node.comps) total[c.label]++;
    for (const Comp& c : node.comps) {
        std::string seg = c.label;
        if (total[c.label] > 1) seg += "#" + std::to_string(seen[c.label]);
        seen[c.label]++;
        std::string path = name.empty() ? seg : name + "/" + seg;
        int w = (int)regs.size();
        regs.push_back(Region{path + ".wrap", c.label, true, c.wrap, {}, {}});
        int ci = add_content(regs, *c.content, path, c.label);
        regs[idx].child_wrap.push_back(w);
        regs[idx].child_content.push_back(ci);
    }
    return idx;
}

struct RawReaction {
    int rule;
    double rate;
    int ctx;  // context region (where a rate law's species is read)
    std::map<std::pair<int, int>, int64_t> react;   // (region, atom) -> order
    std::map<std::pair<int, int>, int64_t> delta;   // (region, atom) -> net change (may be 0)
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
                        const std::vector<double>& rates, const std::string& initial_term) {
    if (alphabet.empty()) throw Error(CWC_E_INVALID, "empty alphabet");
    if (rules.size() != rates.size()) throw Error(CWC_E_INVALID, "one rate per rule");
    std::unordered_map<std::string, int> atoms;
    for (size_t i = 0; i < alphabet.size(); ++i) {
        if (!valid_ident(alphabet[i]) || alphabet[i] == "top") throw Error(CWC_E_INVALID, "bad atom name '" + alphabet[i] + "'");
        if (!atoms.emplace(alphabet[i], (int)i).second) throw Error(CWC_E_INVALID, "duplicate atom '" + alphabet[i] + "'");
    }
    const size_t A = alphabet.size();

    Node top{Counts(A, 0), {}};
    {
        Parser p(initial_term, atoms, false);
        p.sequence("", 2, top.atoms, nullptr, &top.comps, nullptr);
        if (!p.at_end()) throw Error(CWC_E_PARSE, "trailing input in initial term");
    }
    std::vector<Rule> parsed;
    for (size_t i = 0; i < rules.size(); ++i) parsed.push_back(parse_rule(rules[i], atoms, rates[i]));

    std::vector<Region> regs;
    add_content(regs, top, "", "top");

    // Tree matching once: every (rule, context, assignment) is a flat reaction.
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
                RawReaction rr{(int)ri, rule.rate, (int)ci, {}, {}};
                auto add = [](std::map<std::pair<int, int>, int64_t>& m, int reg, const Counts& c, int64_t sign) {
                    for (size_t a = 0; a < c.size(); ++a)
                        if (c[a]) m[{reg, (int)a}] += sign * c[a];
                };
                add(rr.react, (int)ci, rule.lhs.atoms, 1);
                add(rr.delta, (int)ci, rule.rhs.atoms, 1);
                add(rr.delta, (int)ci, rule.lhs.atoms, -1);
                for (size_t p = 0; p < asg.size(); ++p) {
                    int w = ctx.child_wrap[asg[p]], c = ctx.child_content[asg[p]];
                    add(rr.react, w, rule.lhs.comps[p].wrap, 1);
                    add(rr.react, c, rule.lhs.comps[p].content, 1);
                    add(rr.delta, w, rule.rhs.comps[p].wrap, 1);
                    add(rr.delta, c, rule.rhs.comps[p].content, 1);
                    add(rr.delta, w, rule.lhs.comps[p].wrap, -1);
                    add(rr.delta, c, rule.lhs.comps[p].content, -1);
                }
                int64_t order = 0;
                for (auto& kv : rr.react) order += kv.second;
                if (order > 3) throw Error(CWC_E_UNSUPPORTED, "reaction order > 3 in rule " + std::to_string(ri));
                raw.push_back(std::move(rr));
            }
        }
    }

    // Species: every (region, atom) present initially or touched by a reaction; region
    // pre-order, then alphabet order.
    std::set<std::pair<int, int>> used;
    for (size_t r = 0; r < regs.size(); ++r)
        for (size_t a = 0; a < A; ++a)
            if (regs[r].atoms[a] > 0) used.insert({(int)r, (int)a});
    for (const auto& rr : raw) {
        for (auto& kv : rr.react) used.insert(kv.first);
        for (auto& kv : rr.delta) used.insert(kv.first);
        if (parsed[rr.rule].law != LAW_MASS_ACTION) used.insert({rr.ctx, parsed[rr.rule].law_atom});
    }
    if (used.empty()) throw Error(CWC_E_INVALID, "model has no species");

    FlatModel fm;
    fm.alphabet = alphabet;
    fm.n_rules = (int32_t)parsed.size();
    std::map<std::pair<int, int>, int> sidx;
    for (const auto& ra : used) {  // std::set order == (region, atom) lexicographic
        sidx[ra] = (int)fm.names.size();
        const Region& reg = regs[ra.first];
        fm.names.push_back(reg.name.empty() ? alphabet[ra.second] : alphabet[ra.second] + "@" + reg.name);
        int64_t v = reg.atoms[ra.second];
        if (v > (int64_t)INT32_MAX) throw Error(CWC_E_INVALID, "initial count too large");
        fm.x0.push_back((int32_t)v);
    }
    const int S = (int)fm.names.size();
    for (const auto& rr : raw) {
        std::vector<Reactant> rl;
        for (auto& kv : rr.react) rl.push_back(Reactant{sidx[kv.first], (int32_t)kv.second});
        std::sort(rl.begin(), rl.end(), [](const Reactant& a, const Reactant& b) { return a.species < b.species; });
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
    }
    fm.x_cap_max = max_exact_cap(fm.reactants, (int64_t)1 << 30);
    return fm;
}

}  // namespace cwc
