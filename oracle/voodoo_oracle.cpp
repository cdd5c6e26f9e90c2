// oracle/voodoo_oracle.cpp -- layer 1 of the CPU oracle: a literal,
// single-threaded interpreter of Voodoo programs.
//
// TEST INFRASTRUCTURE ONLY (see oracle.h).  Plain, slow, obviously correct.
//
// Data model (§2.1): a Structured Vector is an ordered
// collection of fixed-size items with one schema.  Here a vector is a map
// from attribute name to a column of slots; every slot is either a value or
// the "empty" value epsilon.  Integers are 128-bit, floats are
// long double.  Every operator materialises its full epsilon-padded output,
// as the paper's interpreter backend does.
//
// Program syntax (SSA, as in Fig 3):
//     name := Op(arg, arg, ...)      // comment
// An argument is a vector name ("v"), an attribute keypath ("v.attr"), or a
// numeric literal.  A bare vector name used where one attribute is needed
// denotes its only attribute.  Ops producing one attribute name it after the
// statement's left-hand side.  Readings of unclear passages are marked with
// their SURVEY.md §8(c) / DESIGN.md id (A1..A27).
#include <algorithm>
#include <cctype>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <map>
#include <memory>
#include <stdexcept>
#include <string>
#include <vector>

#include "oracle.h"

namespace {

typedef __int128 i128;
typedef long double ld;

struct Col {
    bool flt = false;
    std::vector<i128> i;    // used when !flt
    std::vector<ld> f;      // used when flt
    std::vector<uint8_t> e; // 1 = epsilon
    size_t size() const { return e.size(); }
    void resize(size_t n, bool isf) {
        flt = isf;
        e.assign(n, 1);
        if (isf) { f.assign(n, 0); i.clear(); }
        else { i.assign(n, 0); f.clear(); }
    }
    bool eps(size_t k) const { return e[k] != 0; }
    ld asf(size_t k) const { return flt ? f[k] : (ld)i[k]; }
    void set_from(size_t dst, const Col& src, size_t k) {
        e[dst] = src.e[k];
        if (flt) f[dst] = src.asf(k);
        else i[dst] = src.i[k];
    }
};

struct Vec {
    std::map<std::string, Col> attrs;
    size_t n = 0;
    bool scalar = false;  // Constant(c) without a size: broadcasts (Fig 3 line 3)
};

struct Ctx {
    std::map<std::string, Vec> vecs;
};

[[noreturn]] void fail(const std::string& m) { throw std::runtime_error(m); }

// ---- argument handling -------------------------------------------------
struct Arg {
    bool lit = false;
    bool litf = false;
    i128 li = 0;
    ld lf = 0;
    std::string vec, attr;  // attr empty: whole vector / single attribute
};

bool is_number(const std::string& s) {
    if (s.empty()) return false;
    size_t k = (s[0] == '-' || s[0] == '+') ? 1 : 0;
    return k < s.size() && (std::isdigit((unsigned char)s[k]) || s[k] == '.');
}

Arg parse_arg(const std::string& raw) {
    Arg a;
    std::string s = raw;
    if (is_number(s)) {
        a.lit = true;
        if (s.find_first_of(".eE") != std::string::npos) { a.litf = true; a.lf = std::strtold(s.c_str(), nullptr); }
        else a.li = (i128)std::strtoll(s.c_str(), nullptr, 10);
        return a;
    }
    if (!s.empty() && s[0] == '"') { a.vec = s.substr(1, s.size() - 2); return a; }  // Load("name")
    size_t dot = s.find('.');
    if (dot == std::string::npos) a.vec = s;
    else { a.vec = s.substr(0, dot); a.attr = s.substr(dot + 1); }
    return a;
}

const Vec& getvec(Ctx& c, const Arg& a) {
    auto it = c.vecs.find(a.vec);
    if (it == c.vecs.end()) fail("unknown vector '" + a.vec + "'");
    return it->second;
}

// A single attribute operand.  Literals become a broadcast column of length
// `bn` (Constant; Range(c,0) reading A14).
Col getcol(Ctx& c, const Arg& a, size_t bn) {
    if (a.lit) {
        Col k;
        k.resize(bn, a.litf);
        for (size_t j = 0; j < bn; ++j) {
            k.e[j] = 0;
            if (a.litf) k.f[j] = a.lf; else k.i[j] = a.li;
        }
        return k;
    }
    const Vec& v = getvec(c, a);
    if (v.scalar) {
        const Col& s1 = v.attrs.begin()->second;
        Col k;
        k.resize(bn, s1.flt);
        for (size_t j = 0; j < bn; ++j) k.set_from(j, s1, 0);
        return k;
    }
    if (a.attr.empty()) {
        if (v.attrs.size() != 1) fail("vector '" + a.vec + "' has several attributes; use a keypath");
        return v.attrs.begin()->second;
    }
    auto it = v.attrs.find(a.attr);
    if (it == v.attrs.end()) fail("unknown attribute '" + a.vec + "." + a.attr + "'");
    return it->second;
}

size_t arglen(Ctx& c, const Arg& a) {
    if (a.lit) return (size_t)-1;
    const Vec& v = getvec(c, a);
    return v.scalar ? (size_t)-1 : v.n;
}

size_t litint(const Arg& a) {
    if (!a.lit || a.litf) fail("expected an integer literal");
    return (size_t)a.li;
}

// Size argument: an integer literal n or a vector v (|v|)  (Range).
size_t size_arg(Ctx& c, const Arg& a) {
    if (a.lit) return litint(a);
    return getvec(c, a).n;
}

Vec single(const std::string& name, Col col) {
    Vec v;
    v.n = col.size();
    v.attrs[name] = std::move(col);
    return v;
}

// ---- Shape operators (Table 2) ------------------------------
// Range(from, n|v, step): v[i] = from + i*step, i in [0,n) -- 0-based (A1,
// pinned by Fig 9 positions 2,3,7,8,11 and Fig 11 positions 0..9).
Col op_range(ld from_f, i128 from, size_t n, i128 step, bool isf, ld step_f) {
    Col o;
    o.resize(n, isf);
    for (size_t k = 0; k < n; ++k) {
        o.e[k] = 0;
        if (isf) o.f[k] = from_f + (ld)k * step_f;
        else o.i[k] = from + (i128)k * step;
    }
    return o;
}

// Run metadata of a virtual control vector (garbled; reading
// A2): v[i] = (from + floor(i * num / den)) mod cap, cap = 0 meaning "none".
Col op_ctrl(i128 from, i128 num, i128 den, i128 cap, size_t n) {
    if (den <= 0) fail("Ctrl: den must be > 0");
    Col o;
    o.resize(n, false);
    for (size_t k = 0; k < n; ++k) {
        i128 fl = ((i128)k * num) / den;  // k,num >= 0 in every use: truncation == floor
        if ((i128)k * num < 0 && ((i128)k * num) % den != 0) fl -= 1;
        i128 v = from + fl;
        if (cap != 0) v = v % cap;
        o.e[k] = 0;
        o.i[k] = v;
    }
    return o;
}

// ---- Data-parallel operators --------------------
// Output length = the smaller input; an epsilon operand gives
// epsilon (reading A9).
enum BinOp { ADD, SUB, MUL, DIV, MOD, GT, EQ, AND, OR, SHL };

Col op_binary(BinOp op, const Col& a, const Col& b) {
    size_t n = std::min(a.size(), b.size());
    bool cmp = (op == GT || op == EQ || op == AND || op == OR);
    bool isf = !cmp && (a.flt || b.flt);
    if ((op == MOD || op == SHL) && isf) fail("Modulo/BitShift need integers");
    Col o;
    o.resize(n, isf);
    for (size_t k = 0; k < n; ++k) {
        if (a.eps(k) || b.eps(k)) continue;  // stays epsilon
        o.e[k] = 0;
        if (cmp) {
            bool r;
            if (op == GT) r = (a.flt || b.flt) ? (a.asf(k) > b.asf(k)) : (a.i[k] > b.i[k]);
            else if (op == EQ) r = (a.flt || b.flt) ? (a.asf(k) == b.asf(k)) : (a.i[k] == b.i[k]);
            else {
                bool x = a.flt ? a.f[k] != 0 : a.i[k] != 0;
                bool y = b.flt ? b.f[k] != 0 : b.i[k] != 0;
                r = (op == AND) ? (x && y) : (x || y);
            }
            o.i[k] = r ? 1 : 0;  // Greater/Equals yield 1/0 (reading A8)
        } else if (isf) {
            ld x = a.asf(k), y = b.asf(k);
            switch (op) {
            case ADD: o.f[k] = x + y; break;
            case SUB: o.f[k] = x - y; break;
            case MUL: o.f[k] = x * y; break;
            case DIV: o.f[k] = x / y; break;
            default: fail("bad float op");
            }
        } else {
            i128 x = a.i[k], y = b.i[k];
            switch (op) {
            case ADD: o.i[k] = x + y; break;
            case SUB: o.i[k] = x - y; break;
            case MUL: o.i[k] = x * y; break;
            case DIV:  // integer division, C truncation (reading A10)
                if (y == 0) fail("Divide by zero");
                o.i[k] = x / y;
                break;
            case MOD:
                if (y == 0) fail("Modulo by zero");
                o.i[k] = x % y;
                break;
            case SHL: o.i[k] = (y >= 0) ? (x << (int)y) : (x >> (int)(-y)); break;  // BitShift
            default: fail("bad int op");
            }
        }
    }
    return o;
}

// ---- Control-vector runs (reading A3) ------------------------
// A run is a maximal block of ADJACENT slots with equal control values
// (epsilon equals epsilon).  Returns run start offsets plus a final n.
std::vector<size_t> runs_of(const Col& fold, size_t n) {
    std::vector<size_t> starts;
    for (size_t k = 0; k < n; ++k) {
        bool head = (k == 0);
        if (!head) {
            if (fold.e[k] != fold.e[k - 1]) head = true;
            else if (!fold.eps(k)) head = fold.flt ? (fold.f[k] != fold.f[k - 1]) : (fold.i[k] != fold.i[k - 1]);
        }
        if (head) starts.push_back(k);
    }
    starts.push_back(n);
    return starts;
}

// ---- Fold operators (Table 2; Fig 7) ---------------
// FoldSelect: positions of slots whose .s is non-zero (and not epsilon),
// ascending, written from the start of each run; the rest of the run is
// epsilon (order preserving P:L580-582; reading A7, Fig 9).
Col op_fold_select(const Col& fold, const Col& s) {
    size_t n = std::min(fold.size(), s.size());
    Col o;
    o.resize(n, false);
    std::vector<size_t> st = runs_of(fold, n);
    for (size_t r = 0; r + 1 < st.size(); ++r) {
        size_t w = st[r];
        for (size_t k = st[r]; k < st[r + 1]; ++k) {
            if (s.eps(k)) continue;
            bool nz = s.flt ? (s.f[k] != 0) : (s.i[k] != 0);
            if (!nz) continue;
            o.e[w] = 0;
            o.i[w] = (i128)k;
            ++w;
        }
    }
    return o;
}

enum FoldKind { F_SUM, F_COUNT, F_MIN, F_MAX };

// FoldSum/Count/Min/Max: one result per run, written at the run start,
// epsilon elsewhere.  Epsilon inputs are skipped
// (Fig 9: 8+2 = 10).  All-epsilon run: Sum and Count 0, Min/Max epsilon
// (reading A5, parity unpinned by the paper).  FoldCount = FoldSum of 1 over
// non-epsilon slots (reading A6).
Col op_fold(FoldKind kind, const Col& fold, const Col& v) {
    size_t n = std::min(fold.size(), v.size());
    bool isf = (kind == F_COUNT) ? false : v.flt;
    Col o;
    o.resize(n, isf);
    std::vector<size_t> st = runs_of(fold, n);
    for (size_t r = 0; r + 1 < st.size(); ++r) {
        size_t a = st[r], b = st[r + 1];
        i128 si = 0, cnt = 0;
        ld sf = 0;
        bool have = false;
        i128 mi = 0;
        ld mf = 0;
        for (size_t k = a; k < b; ++k) {
            if (v.eps(k)) continue;
            ++cnt;
            if (v.flt) {
                sf += v.f[k];
                if (!have || (kind == F_MIN ? v.f[k] < mf : v.f[k] > mf)) mf = v.f[k];
            } else {
                si += v.i[k];
                if (!have || (kind == F_MIN ? v.i[k] < mi : v.i[k] > mi)) mi = v.i[k];
            }
            have = true;
        }
        switch (kind) {
        case F_SUM:
            o.e[a] = 0;
            if (isf) o.f[a] = sf; else o.i[a] = si;
            break;
        case F_COUNT:
            o.e[a] = 0;
            o.i[a] = cnt;
            break;
        case F_MIN:
        case F_MAX:
            if (have) {
                o.e[a] = 0;
                if (isf) o.f[a] = mf; else o.i[a] = mi;
            }
            break;
        }
    }
    return o;
}

// FoldScan: prefix sum of .s restarting at each run.  Reading A27:
// inclusive; epsilon slots stay epsilon and add nothing.
Col op_fold_scan(const Col& fold, const Col& v) {
    size_t n = std::min(fold.size(), v.size());
    Col o;
    o.resize(n, v.flt);
    std::vector<size_t> st = runs_of(fold, n);
    for (size_t r = 0; r + 1 < st.size(); ++r) {
        i128 si = 0;
        ld sf = 0;
        for (size_t k = st[r]; k < st[r + 1]; ++k) {
            if (v.eps(k)) continue;
            o.e[k] = 0;
            if (v.flt) { sf += v.f[k]; o.f[k] = sf; }
            else { si += v.i[k]; o.i[k] = si; }
        }
    }
    return o;
}

// ---- Gather / Scatter / Partition ---------------
// Gather: output size |pos|; out[k] = V1[pos[k]]; epsilon or out-of-bounds
// positions give epsilon (reading A11).
Col op_gather(const Col& src, const Col& pos) {
    Col o;
    o.resize(pos.size(), src.flt);
    for (size_t k = 0; k < pos.size(); ++k) {
        if (pos.eps(k)) continue;
        if (pos.flt) fail("Gather: positions must be integers");
        i128 p = pos.i[k];
        if (p < 0 || p >= (i128)src.size()) continue;
        o.set_from(k, src, (size_t)p);
    }
    return o;
}

// Scatter: output of the given size, all epsilon; input slots are placed in
// input order, so on conflict the later input wins (reading
// A12: "globally last index wins" is one valid instance of "in order within
// a run, runs unordered").  Out-of-bounds / epsilon positions are dropped.
// An epsilon source value is placed like any value (reading A27b).
Col op_scatter(const Col& src, size_t out_len, const Col& pos) {
    Col o;
    o.resize(out_len, src.flt);
    size_t n = std::min(src.size(), pos.size());
    for (size_t k = 0; k < n; ++k) {
        if (pos.eps(k)) continue;
        i128 p = pos.i[k];
        if (p < 0 || p >= (i128)out_len) continue;
        o.set_from((size_t)p, src, k);
    }
    return o;
}

// Partition(V1.v, pivots): scatter positions that partition V1.v by the
// (ascending) pivots; output size |V1|.  Reading
// A13: stable range partition, bucket = upper_bound(pivots, v) - 1 clamped
// to [0, P-1]; position = (sizes of earlier buckets) + (rank of the slot
// among its bucket's slots in input order) -- pinned by Fig 11.  Epsilon
// values get epsilon positions and occupy no bucket.
Col op_partition(const Col& v, const Col& piv) {
    size_t n = v.size();
    size_t P = piv.size();
    if (P == 0) fail("Partition: empty pivot vector");
    std::vector<ld> pv(P);
    for (size_t j = 0; j < P; ++j) {
        if (piv.eps(j)) fail("Partition: epsilon pivot");
        pv[j] = piv.asf(j);
    }
    for (size_t j = 1; j < P; ++j)
        if (pv[j] < pv[j - 1]) fail("Partition: pivots must be ascending");
    std::vector<size_t> bucket(n, 0);
    std::vector<size_t> count(P, 0);
    for (size_t k = 0; k < n; ++k) {
        if (v.eps(k)) continue;
        ld x = v.asf(k);
        size_t ub = (size_t)(std::upper_bound(pv.begin(), pv.end(), x) - pv.begin());
        size_t b = (ub == 0) ? 0 : ub - 1;
        bucket[k] = b;
        count[b]++;
    }
    std::vector<size_t> next(P, 0);
    size_t acc = 0;
    for (size_t b = 0; b < P; ++b) { next[b] = acc; acc += count[b]; }
    Col o;
    o.resize(n, false);
    for (size_t k = 0; k < n; ++k) {
        if (v.eps(k)) continue;
        o.e[k] = 0;
        o.i[k] = (i128)next[bucket[k]]++;
    }
    return o;
}

// ---- statement dispatch ------------------------------------------------
std::string trim(const std::string& s) {
    size_t a = 0, b = s.size();
    while (a < b && std::isspace((unsigned char)s[a])) ++a;
    while (b > a && std::isspace((unsigned char)s[b - 1])) --b;
    return s.substr(a, b - a);
}

std::vector<std::string> split_args(const std::string& s) {
    std::vector<std::string> out;
    std::string cur;
    int depth = 0;
    bool inq = false;
    for (char ch : s) {
        if (ch == '"') inq = !inq;
        if (!inq && ch == '(') ++depth;
        if (!inq && ch == ')') --depth;
        if (!inq && depth == 0 && ch == ',') { out.push_back(trim(cur)); cur.clear(); continue; }
        cur += ch;
    }
    if (!trim(cur).empty()) out.push_back(trim(cur));
    return out;
}

void exec_stmt(Ctx& c, const std::string& lhs, const std::string& op, const std::vector<Arg>& a) {
    auto need = [&](size_t k) {
        if (a.size() < k) fail(op + ": expected at least " + std::to_string(k) + " arguments");
    };
    auto bin = [&](BinOp b) {
        need(2);
        size_t la = arglen(c, a[0]), lb = arglen(c, a[1]);
        size_t n = std::min(la, lb);
        if (n == (size_t)-1) fail(op + ": two literals");
        c.vecs[lhs] = single(lhs, op_binary(b, getcol(c, a[0], n), getcol(c, a[1], n)));
    };
    // One-run control vector when the fold argument is omitted (Fig 3 line 9).
    auto fold_pair = [&](Col& fold, Col& val) {
        if (a.size() == 1) {
            val = getcol(c, a[0], 0);
            fold = op_range(0, 0, val.size(), 0, false, 0);
        } else {
            need(2);
            size_t la = arglen(c, a[0]), lb = arglen(c, a[1]);
            size_t n = std::min(la, lb);
            fold = getcol(c, a[0], n == (size_t)-1 ? 0 : n);
            val = getcol(c, a[1], n == (size_t)-1 ? fold.size() : n);
        }
    };

    if (op == "Load") {  // Load(.keypath): alias of a bound input vector
        need(1);
        c.vecs[lhs] = getvec(c, a[0]);
    } else if (op == "Range" && a.size() == 1 && !a[0].lit) {  // Range(v): 0..|v|-1 (Fig 3 line 2)
        c.vecs[lhs] = single(lhs, op_range(0, 0, getvec(c, a[0]).n, 1, false, 1));
    } else if (op == "Range") {  // Range(from, n|v, step)
        need(2);
        size_t n = size_arg(c, a[1]);
        i128 step = 1;
        ld stepf = 1;
        bool isf = a[0].litf;
        if (a.size() >= 3) { step = a[2].li; stepf = a[2].litf ? a[2].lf : (ld)a[2].li; isf = isf || a[2].litf; }
        c.vecs[lhs] = single(lhs, op_range(a[0].litf ? a[0].lf : (ld)a[0].li, a[0].li, n, step, isf, stepf));
    } else if (op == "Constant" && a.size() == 1) {  // Constant(c): broadcast scalar (Fig 3 line 3)
        if (!a[0].lit) fail("Constant: literal expected");
        Vec v = single(lhs, op_range(a[0].litf ? a[0].lf : (ld)a[0].li, a[0].li, 1, 0, a[0].litf, 0));
        v.scalar = true;
        c.vecs[lhs] = v;
    } else if (op == "Constant") {  // Constant(c, n|v) == Range(c, n, 0) (A14)
        need(2);
        size_t n = size_arg(c, a[1]);
        c.vecs[lhs] = single(lhs, op_range(a[0].litf ? a[0].lf : (ld)a[0].li, a[0].li, n, 0, a[0].litf, 0));
    } else if (op == "Ctrl") {  // Ctrl(from, num, den, cap, n|v)  (A2)
        need(5);
        c.vecs[lhs] = single(lhs, op_ctrl(a[0].li, a[1].li, a[2].li, a[3].li, size_arg(c, a[4])));
    } else if (op == "Add") bin(ADD);
    else if (op == "Subtract") bin(SUB);
    else if (op == "Multiply") bin(MUL);
    else if (op == "Divide") bin(DIV);
    else if (op == "Modulo") bin(MOD);
    else if (op == "Greater") bin(GT);
    else if (op == "Equals") bin(EQ);
    else if (op == "LogicalAnd") bin(AND);
    else if (op == "LogicalOr") bin(OR);
    else if (op == "BitShift") bin(SHL);
    else if (op == "Zip") {  // Zip: union of the attributes, aligned
        need(2);
        Vec out;
        size_t n = (size_t)-1;
        for (const Arg& x : a) n = std::min(n, arglen(c, x));
        for (const Arg& x : a) {
            if (x.lit) fail("Zip: literal");
            const Vec& v = getvec(c, x);
            for (auto& kv : v.attrs) {
                if (!x.attr.empty() && kv.first != x.attr) continue;
                if (out.attrs.count(kv.first)) fail("Zip: duplicate attribute " + kv.first);
                Col col = kv.second;
                Col cut;
                cut.resize(n, col.flt);
                for (size_t k = 0; k < n; ++k) cut.set_from(k, col, k);
                out.attrs[kv.first] = cut;
            }
        }
        out.n = n;
        c.vecs[lhs] = out;
    } else if (op == "Materialize" || op == "Break") {
        // Materialize(V1, V2.kp) / Break(V1, V2.kp) (Table 2):
        // "materialize V1 in memory ... in chunks of sizes according to runs
        // in V2.kp" / "break up V1 into segments according to the runs in
        // V2.kp (pure tuning hint)".  Both direct HOW a program executes
        // (where the pipeline is cut, how large the buffered chunks are), not
        // what it computes: their value is V1.  The interpreter materialises
        // every intermediate anyway, so it returns V1 unchanged.
        need(2);
        getvec(c, a[1]);  // the control vector must exist
        if (a[0].attr.empty()) c.vecs[lhs] = getvec(c, a[0]);
        else c.vecs[lhs] = single(a[0].attr, getcol(c, a[0], 0));
    } else if (op == "Project") {  // Project(V.kp) -- renamed to lhs
        need(1);
        c.vecs[lhs] = single(lhs, getcol(c, a[0], 0));
    } else if (op == "Rename") {  // Rename(V.kp, name) -- Project(.out, V, .kp)
        need(2);
        c.vecs[lhs] = single(a[1].vec, getcol(c, a[0], 0));
    } else if (op == "FoldSelect") {
        Col f, v;
        fold_pair(f, v);
        c.vecs[lhs] = single(lhs, op_fold_select(f, v));
    } else if (op == "FoldSum" || op == "FoldCount" || op == "FoldMin" || op == "FoldMax") {
        Col f, v;
        fold_pair(f, v);
        FoldKind k = op == "FoldSum" ? F_SUM : op == "FoldCount" ? F_COUNT : op == "FoldMin" ? F_MIN : F_MAX;
        c.vecs[lhs] = single(lhs, op_fold(k, f, v));
    } else if (op == "FoldScan") {
        Col f, v;
        fold_pair(f, v);
        c.vecs[lhs] = single(lhs, op_fold_scan(f, v));
    } else if (op == "Gather") {  // Gather(V1, pos): all attributes of V1 (or V1.kp)
        need(2);
        Col pos = getcol(c, a[1], 0);
        const Vec& src = getvec(c, a[0]);
        Vec out;
        out.n = pos.size();
        for (auto& kv : src.attrs) {
            if (!a[0].attr.empty() && kv.first != a[0].attr) continue;
            out.attrs[a[0].attr.empty() && src.attrs.size() == 1 ? lhs : kv.first] = op_gather(kv.second, pos);
        }
        c.vecs[lhs] = out;
    } else if (op == "Scatter") {  // Scatter(V1, size n|V2, pos)
        need(3);
        size_t out_len = size_arg(c, a[1]);
        Col pos = getcol(c, a[2], 0);
        const Vec& src = getvec(c, a[0]);
        Vec out;
        out.n = out_len;
        for (auto& kv : src.attrs) {
            if (!a[0].attr.empty() && kv.first != a[0].attr) continue;
            out.attrs[kv.first] = op_scatter(kv.second, out_len, pos);
        }
        c.vecs[lhs] = out;
    } else if (op == "Partition" && a.size() == 1) {
        // Partition(V1.v) with no pivot vector (Fig 3 line 5): the pivots are
        // the distinct non-epsilon values of V1.v, ascending (reading A13).
        Col v = getcol(c, a[0], 0);
        std::vector<ld> d;
        for (size_t k = 0; k < v.size(); ++k)
            if (!v.eps(k)) d.push_back(v.asf(k));
        std::sort(d.begin(), d.end());
        d.erase(std::unique(d.begin(), d.end()), d.end());
        Col piv;
        piv.resize(d.size(), true);
        for (size_t k = 0; k < d.size(); ++k) { piv.e[k] = 0; piv.f[k] = d[k]; }
        if (d.empty()) { Col o; o.resize(v.size(), false); c.vecs[lhs] = single(lhs, o); }
        else c.vecs[lhs] = single(lhs, op_partition(v, piv));
    } else if (op == "Partition") {  // Partition(V1.v, pivots)
        need(2);
        c.vecs[lhs] = single(lhs, op_partition(getcol(c, a[0], 0), getcol(c, a[1], 0)));
    } else {
        fail("unknown operator '" + op + "'");
    }
}

void run_program(Ctx& c, const std::string& prog) {
    size_t pos = 0;
    int lineno = 0;
    while (pos <= prog.size()) {
        size_t nl = prog.find('\n', pos);
        if (nl == std::string::npos) nl = prog.size();
        std::string line = prog.substr(pos, nl - pos);
        pos = nl + 1;
        ++lineno;
        size_t cm = line.find("//");
        if (cm != std::string::npos) line = line.substr(0, cm);
        line = trim(line);
        if (line.empty()) continue;
        try {
            size_t as = line.find(":=");
            if (as == std::string::npos) fail("missing ':='");
            std::string lhs = trim(line.substr(0, as));
            std::string rhs = trim(line.substr(as + 2));
            size_t lp = rhs.find('('), rp = rhs.rfind(')');
            if (lp == std::string::npos || rp == std::string::npos || rp < lp) fail("malformed call");
            std::string op = trim(rhs.substr(0, lp));
            std::vector<Arg> args;
            for (auto& s : split_args(rhs.substr(lp + 1, rp - lp - 1))) args.push_back(parse_arg(s));
            exec_stmt(c, lhs, op, args);
        } catch (std::exception& e) {
            throw std::runtime_error("line " + std::to_string(lineno) + ": " + e.what());
        }
        if (nl == prog.size()) break;
    }
}

const Col* find_col(Ctx& c, const char* name) {
    std::string s(name);
    size_t dot = s.find('.');
    std::string v = dot == std::string::npos ? s : s.substr(0, dot);
    auto it = c.vecs.find(v);
    if (it == c.vecs.end()) return nullptr;
    if (dot == std::string::npos) {
        if (it->second.attrs.size() != 1) return nullptr;
        return &it->second.attrs.begin()->second;
    }
    auto jt = it->second.attrs.find(s.substr(dot + 1));
    return jt == it->second.attrs.end() ? nullptr : &jt->second;
}

int set_col(Ctx& c, const char* name, Col col) {
    std::string s(name);
    size_t dot = s.find('.');
    std::string v = dot == std::string::npos ? s : s.substr(0, dot);
    std::string at = dot == std::string::npos ? s : s.substr(dot + 1);
    Vec& vec = c.vecs[v];
    if (!vec.attrs.empty() && vec.n != col.size()) return -1;
    vec.n = col.size();
    vec.attrs[at] = std::move(col);
    return 0;
}

}  // namespace

extern "C" {

void* or_ctx_new(void) { return new Ctx(); }
void or_ctx_free(void* ctx) { delete (Ctx*)ctx; }

int or_ctx_set_i64(void* ctx, const char* name, const int64_t* v, const uint8_t* eps, int64_t n) {
    Col col;
    col.resize((size_t)n, false);
    for (int64_t k = 0; k < n; ++k) { col.i[k] = v[k]; col.e[k] = eps ? (eps[k] != 0) : 0; }
    return set_col(*(Ctx*)ctx, name, std::move(col));
}

int or_ctx_set_f64(void* ctx, const char* name, const double* v, const uint8_t* eps, int64_t n) {
    Col col;
    col.resize((size_t)n, true);
    for (int64_t k = 0; k < n; ++k) { col.f[k] = v[k]; col.e[k] = eps ? (eps[k] != 0) : 0; }
    return set_col(*(Ctx*)ctx, name, std::move(col));
}

int or_ctx_run(void* ctx, const char* program, char* err, int errlen) {
    try {
        run_program(*(Ctx*)ctx, std::string(program));
        if (err && errlen > 0) err[0] = 0;
        return 0;
    } catch (std::exception& e) {
        if (err && errlen > 0) { std::snprintf(err, (size_t)errlen, "%s", e.what()); }
        return 1;
    }
}

int64_t or_ctx_len(void* ctx, const char* name) {
    const Col* c = find_col(*(Ctx*)ctx, name);
    return c ? (int64_t)c->size() : -1;
}

int or_ctx_is_float(void* ctx, const char* name) {
    const Col* c = find_col(*(Ctx*)ctx, name);
    return c ? (c->flt ? 1 : 0) : -1;
}

int or_ctx_get_i128(void* ctx, const char* name, int64_t* lo, int64_t* hi, uint8_t* eps) {
    const Col* c = find_col(*(Ctx*)ctx, name);
    if (!c || c->flt) return -1;
    for (size_t k = 0; k < c->size(); ++k) {
        unsigned __int128 u = (unsigned __int128)c->i[k];
        lo[k] = (int64_t)(uint64_t)u;
        hi[k] = (int64_t)(uint64_t)(u >> 64);
        eps[k] = c->e[k];
    }
    return 0;
}

int or_ctx_get_f64(void* ctx, const char* name, double* v, double* resid, uint8_t* eps) {
    const Col* c = find_col(*(Ctx*)ctx, name);
    if (!c) return -1;
    for (size_t k = 0; k < c->size(); ++k) {
        ld x = c->asf(k);
        v[k] = (double)x;
        if (resid) resid[k] = (double)(x - (ld)v[k]);
        eps[k] = c->e[k];
    }
    return 0;
}

}  // extern "C"
