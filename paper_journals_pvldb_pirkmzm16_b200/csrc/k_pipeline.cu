// k_pipeline.cu -- fused operator chains, vd_run_pipeline (§8(a) a7-a9).
//
// A Voodoo fragment (§3.1) is one fully inlined kernel: scan ->
// predicate -> (FK gather) -> group key -> folds, with materialisation only
// at the seams.  Here the fragments are compiled ahead of time for sm_100a:
//
//   k_pipe_q1      grouped multi-aggregate over <= 8 groups (the Q1 plan of
//                  Fig 10/11): the Partition -> Scatter -> FoldSum/FoldCount
//                  chain stays virtual (§3.1.3) -- each row's
//                  values go straight into its group's register accumulators
//                  (the "scatter position" is the work-item-local key), and
//                  the FoldSelect compaction happens on the host merge.
//   k_pipe_scalar  filtered scalar fold of a product of columns (the Q6 plan
//                  of Fig 8, and the selective aggregation of
//                  Fig 15), branching (late loads) or
//                  predicated (every row loaded, contribution x predicate).
//   k_pipe_generic any vd_pipeline: per-row interpretation of the descriptor
//                  (gathers, key parts, products), per-warp shared-memory
//                  accumulators updated by one leader lane per distinct key.
//
// Hierarchical fold (Fig 3): thread -> warp -> CTA partials in
// the workspace -> the last CTA to finish folds them in CTA order (Fragment 2
// / global barrier) and writes the vd_partials buffer.
#include <float.h>

#include <algorithm>
#include <cmath>
#include <cstdlib>
#include <cstring>
#include <type_traits>

#include "vd_common.cuh"
#include "vd_internal.h"
#include "vd_pred.cuh"

namespace vd {

// ============================================================================
// Output slots
// ============================================================================
// partials: [ngroups][naggs+1] x 16 bytes (include/vd.h vd_partials).
struct Slot16 {
    unsigned long long lo, hi;
};

__device__ __forceinline__ void put_i128(Slot16* s, i128 v) {
    s->lo = (unsigned long long)(u128)v;
    s->hi = (unsigned long long)((u128)v >> 64);
}
__device__ __forceinline__ i128 get_i128(const Slot16& s) { return (i128)(((u128)s.hi << 64) | s.lo); }
__device__ __forceinline__ void put_f64(Slot16* s, double v) {
    s->lo = (unsigned long long)__double_as_longlong(v);
    s->hi = 0;
}
__device__ __forceinline__ double get_f64(const Slot16& s) { return __longlong_as_double((long long)s.lo); }

// The grid level of Fig 3's hierarchical fold, in the last CTA to finish
// (Fragment 2 of Fig 8): slot k = the fold over the CTAs'
// partials parts[b * nslots + k].  One warp per slot, lanes taking blocks
// b = lane, lane + 32, ... -- independent L2 loads, one round trip -- then a
// fixed shuffle tree (deterministic per launch shape).  A thread-per-slot
// loop over the blocks is a chain of gridDim dependent L2 loads (~20 us at
// 148 CTAs: most of a small step, C1).  Every warp of the CTA must call it.
enum FoldKind { FK_I128_SUM = 0, FK_F64_SUM = 1, FK_I128_MIN = 2, FK_I128_MAX = 3, FK_F64_MIN = 4, FK_F64_MAX = 5 };
template <class KindOf>
__device__ __forceinline__ void fold_grid_parts(const Slot16* __restrict__ parts, int nslots, Slot16* dst,
                                                KindOf kind_of) {
    const int lane = threadIdx.x & 31, nw = blockDim.x >> 5;
    const unsigned nb = gridDim.x;
    for (int k = threadIdx.x >> 5; k < nslots; k += nw) {
        const int kd = kind_of(k);
        Slot16 r;
        if (kd == FK_F64_SUM || kd == FK_F64_MIN || kd == FK_F64_MAX) {
            double t = kd == FK_F64_MIN ? DBL_MAX : (kd == FK_F64_MAX ? -DBL_MAX : 0.0);
            for (unsigned b = lane; b < nb; b += 32) {
                const double x = __longlong_as_double((long long)__ldcg(&parts[(size_t)b * nslots + k].lo));
                t = kd == FK_F64_SUM ? t + x : (kd == FK_F64_MIN ? fmin(t, x) : fmax(t, x));
            }
#pragma unroll
            for (int o = 16; o; o >>= 1) {
                const double u = __shfl_xor_sync(VD_FULL, t, o);
                t = kd == FK_F64_SUM ? t + u : (kd == FK_F64_MIN ? fmin(t, u) : fmax(t, u));
            }
            put_f64(&r, t);
        } else {
            i128 t = kd == FK_I128_MIN ? (i128)INT64_MAX : (kd == FK_I128_MAX ? (i128)INT64_MIN : (i128)0);
            for (unsigned b = lane; b < nb; b += 32) {
                Slot16 x;
                x.lo = __ldcg(&parts[(size_t)b * nslots + k].lo);
                x.hi = __ldcg(&parts[(size_t)b * nslots + k].hi);
                const i128 y = get_i128(x);
                t = kd == FK_I128_SUM ? t + y : (kd == FK_I128_MIN ? (y < t ? y : t) : (y > t ? y : t));
            }
#pragma unroll
            for (int o = 16; o; o >>= 1) {
                const i128 u = shfl_xor_i128(t, o);
                t = kd == FK_I128_SUM ? t + u : (kd == FK_I128_MIN ? (u < t ? u : t) : (u > t ? u : t));
            }
            put_i128(&r, t);
        }
        if (lane == 0) dst[k] = r;
    }
}
struct FkI128Sum {
    __device__ __forceinline__ int operator()(int) const { return FK_I128_SUM; }
};

// Maps from a fragment's raw result slots to the plan's [ngroups][naggs+1].
struct Q1Map {
    int32_t naggs, ngroups;
    int32_t src[VD_MAX_AGGS];  // raw slot (0..5) per plan aggregate
};
struct ScalarMap {
    int32_t naggs;
    int32_t src[VD_MAX_AGGS];  // 0 = sum, 1 = count
};
// ============================================================================
// Generic fragment
// ============================================================================
struct GenAgg {
    int32_t kind, nf, isf;
    int32_t col[VD_MAX_FACTORS];
    int64_t a[VD_MAX_FACTORS], b[VD_MAX_FACTORS];
};

struct GenPlan {
    DevPred pred;
    DevCols cols;  // base columns
    // gathers
    int32_t ngathers;
    int32_t g_fk[VD_MAX_GATHERS];
    int64_t g_bias[VD_MAX_GATHERS];
    const void* g_p[VD_MAX_GATHERS];
    int64_t g_len[VD_MAX_GATHERS];
    int32_t g_dt[VD_MAX_GATHERS];
    // key
    int32_t nkey;
    int32_t k_col[VD_MAX_KEYPARTS], k_fn[VD_MAX_KEYPARTS];
    int64_t k_sub[VD_MAX_KEYPARTS], k_mult[VD_MAX_KEYPARTS];
    int64_t ngroups;
    int32_t naggs;
    GenAgg agg[VD_MAX_AGGS];
};

__device__ __forceinline__ Val gen_fetch(const GenPlan& P, int c, int64_t row) {
    if (c < P.cols.ncols) return fetch_typed(P.cols.p[c], P.cols.dt[c], row);
    int g = c - P.cols.ncols;
    Val fk = fetch_typed(P.cols.p[P.g_fk[g]], P.cols.dt[P.g_fk[g]], row);
    Val out;
    out.eps = true;
    out.isf = false;
    out.i = 0;
    out.f = 0;
    if (fk.eps) return out;
    int64_t p = fk.i - P.g_bias[g];
    if (p < 0 || p >= P.g_len[g]) return out;
    return fetch_typed(P.g_p[g], P.g_dt[g], p);
}

__device__ __forceinline__ bool gen_pred(const GenPlan& P, int64_t row) {
    if (P.pred.nconj == 0) return true;
    for (int c = 0; c < P.pred.nconj; ++c) {
        bool ok = true;
        for (int k = 0; k < P.pred.nterms[c] && ok; ++k) {
            const DevTerm& t = P.pred.t[c][k];
            ok = term_true(t, gen_fetch(P, t.col, row));
        }
        if (ok) return true;
    }
    return false;
}

constexpr int GEN_THREADS = 256;
constexpr int GEN_WARPS = GEN_THREADS / 32;

// Row source of the folding loop (vd_materialize): SRC_ROWS evaluates the
// predicate per row (fused); SRC_FLAGS reads the predicate Break
// materialised (one byte per row); SRC_CHUNKS walks the position lists
// Materialize wrote per chunk of C rows (slot c*C + k, k < cnt[c]).
enum { SRC_ROWS = 0, SRC_FLAGS = 1, SRC_CHUNKS = 2 };
struct MatSrc {
    const uint8_t* flags;
    const int32_t* pos;
    const int32_t* cnt;
    int64_t C, nchunks;
};

// slot `it` of the folding loop -> (row, qualifies)
template <int SRC>
__device__ __forceinline__ bool mat_row(const GenPlan& P, const MatSrc& M, int64_t it, int64_t n_iter, int64_t n,
                                        int64_t* row) {
    if (SRC == SRC_ROWS) {
        *row = it;
        return it < n && gen_pred(P, it);
    } else if (SRC == SRC_FLAGS) {
        *row = it;
        return it < n && M.flags[it] != 0;
    } else {
        if (it >= n_iter) { *row = 0; return false; }
        const int64_t c = it / M.C, k = it - c * M.C;
        const bool ok = k < (int64_t)__ldg(M.cnt + c);
        *row = ok ? (int64_t)__ldg(M.pos + it) : 0;
        return ok;
    }
}

// Accumulator slot layout per (group, agg): 16 bytes (i128 or f64/i64 min-max);
// slot [g][naggs] = row count.
template <bool SMEM, int SRC>
__global__ void __launch_bounds__(GEN_THREADS) k_pipe_generic(const __grid_constant__ GenPlan P, int64_t n,
                                                              Slot16* __restrict__ block_parts, int nslots,
                                                              Slot16* __restrict__ gacc,
                                                              unsigned long long* __restrict__ gmask,
                                                              unsigned int* __restrict__ done, Slot16* __restrict__ out,
                                                              unsigned long long* __restrict__ domain_err,
                                                              const MatSrc M, int64_t n_iter) {
    extern __shared__ Slot16 s_mem[];
    // [GEN_WARPS][32][naggs] staging, then (SMEM) [GEN_WARPS][nslots] accumulators
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int NA = P.naggs;
    Slot16* stage = s_mem + (size_t)warp * 32 * (NA + 1);
    Slot16* acc = s_mem + (size_t)GEN_WARPS * 32 * (NA + 1) + (size_t)warp * nslots;
    if (SMEM) {
        for (int k = lane; k < nslots; k += 32) {
            int a = k % (NA + 1);
            Slot16 z{0, 0};
            if (a < NA && (P.agg[a].kind == VD_AGG_MIN || P.agg[a].kind == VD_AGG_MAX)) {
                bool mn = P.agg[a].kind == VD_AGG_MIN;
                if (P.agg[a].isf) put_f64(&z, mn ? DBL_MAX : -DBL_MAX);
                else put_i128(&z, mn ? (i128)INT64_MAX : (i128)INT64_MIN);
            }
            acc[k] = z;
        }
    }
    __syncwarp();
    const int64_t stride = (int64_t)gridDim.x * GEN_THREADS;
    for (int64_t base = (int64_t)blockIdx.x * GEN_THREADS + warp * 32; base < n_iter; base += stride) {
        int64_t row;
        bool ok = mat_row<SRC>(P, M, base + lane, n_iter, n, &row);
        int64_t key = 0;
        if (ok) {
            for (int k = 0; k < P.nkey && ok; ++k) {
                Val v = gen_fetch(P, P.k_col[k], row);
                if (v.eps) { ok = false; break; }
                int64_t x = v.isf ? (int64_t)v.f : v.i;
                if (P.k_fn[k] == 1) x = year_of_day((int32_t)x);
                key += (x - P.k_sub[k]) * P.k_mult[k];
            }
            if (ok && (key < 0 || key >= P.ngroups)) {
                ok = false;
                atomicAdd(domain_err, 1ull);
            }
        }
        if (ok) {
            for (int a = 0; a < NA; ++a) {
                const GenAgg& A = P.agg[a];
                Slot16 v{0, 0};
                if (A.kind == VD_AGG_COUNT) {
                    put_i128(&v, 1);
                } else if (A.isf) {
                    double pr = 1.0;
                    bool e = false;
                    for (int f = 0; f < A.nf; ++f) {
                        double x = 0;
                        if (A.col[f] >= 0) {
                            Val c = gen_fetch(P, A.col[f], row);
                            e |= c.eps;
                            x = c.isf ? c.f : (double)c.i;
                        }
                        pr *= (double)A.a[f] + (double)A.b[f] * x;
                    }
                    if (e) pr = nan("");
                    put_f64(&v, pr);
                } else {
                    i128 pr = 1;
                    bool e = false;
                    for (int f = 0; f < A.nf; ++f) {
                        i128 x = 0;
                        if (A.col[f] >= 0) {
                            Val c = gen_fetch(P, A.col[f], row);
                            e |= c.eps;
                            x = c.i;
                        }
                        pr *= (i128)A.a[f] + (i128)A.b[f] * x;
                    }
                    put_i128(&v, pr);
                    if (e) v.hi = 0x8000000000000000ull;  // epsilon marker (skipped)
                }
                stage[lane * (NA + 1) + a] = v;
            }
        }
        __syncwarp();
        unsigned m = __match_any_sync(VD_FULL, ok ? key : -1ll);
        bool leader = ok && (__ffs(m) - 1 == lane);
        if (leader) {
            for (int a = 0; a <= NA; ++a) {
                const bool cnt = (a == NA);
                const int kind = cnt ? VD_AGG_COUNT : P.agg[a].kind;
                const bool isf = cnt ? false : P.agg[a].isf;
                Slot16 r;
                if (SMEM) r = acc[key * (NA + 1) + a];
                i128 si = 0, mi = 0;
                double sf = 0, mf = 0;
                bool have = false;
                for (unsigned mm = m; mm; mm &= mm - 1) {
                    int l = __ffs(mm) - 1;
                    if (cnt) { si += 1; continue; }
                    Slot16 x = stage[l * (NA + 1) + a];
                    if (!isf && x.hi == 0x8000000000000000ull && kind != VD_AGG_COUNT) continue;
                    if (isf && kind != VD_AGG_COUNT) {
                        double d = get_f64(x);
                        if (d != d) continue;
                        if (kind == VD_AGG_SUM) sf += d;
                        else if (!have || (kind == VD_AGG_MIN ? d < mf : d > mf)) mf = d;
                    } else {
                        i128 y = get_i128(x);
                        if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) si += y;
                        else if (!have || (kind == VD_AGG_MIN ? y < mi : y > mi)) mi = y;
                    }
                    have = true;
                }
                if (SMEM) {
                    if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                        if (isf) put_f64(&r, get_f64(r) + sf);
                        else put_i128(&r, get_i128(r) + si);
                    } else if (have) {
                        if (isf) { double c = get_f64(r); put_f64(&r, kind == VD_AGG_MIN ? fmin(c, mf) : fmax(c, mf)); }
                        else { i128 c = get_i128(r); put_i128(&r, kind == VD_AGG_MIN ? (mi < c ? mi : c) : (mi > c ? mi : c)); }
                    }
                    acc[key * (NA + 1) + a] = r;
                } else {
                    unsigned long long* g = (unsigned long long*)(gacc + key * (NA + 1) + a);
                    if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                        if (isf) atomicAdd((double*)g, sf);
                        else atomic_add_i128(g, si);
                    } else if (have) {
                        if (isf) {
                            // order-preserving integer image of a double
                            long long bits = __double_as_longlong(mf);
                            long long key2 = bits >= 0 ? bits : bits ^ 0x7FFFFFFFFFFFFFFFll;
                            if (kind == VD_AGG_MIN) atomicMin((long long*)g, key2); else atomicMax((long long*)g, key2);
                        } else {
                            if (kind == VD_AGG_MIN) atomicMin((long long*)g, (long long)mi);
                            else atomicMax((long long*)g, (long long)mi);
                        }
                        atomicOr(gmask + key * (NA + 1) + a, 1ull);
                    }
                }
            }
        }
        __syncwarp();
    }
    if (!SMEM) {
        // the last CTA converts min/max images and copies to out
        __syncthreads();
        __shared__ bool s_last;
        if (threadIdx.x == 0) {
            __threadfence();
            s_last = atomicAdd(done, 1u) == gridDim.x - 1;
        }
        __syncthreads();
        if (!s_last) return;
        __threadfence();
        for (int k = threadIdx.x; k < P.ngroups * (NA + 1); k += GEN_THREADS) {
            int a = k % (NA + 1);
            Slot16 v;
            v.lo = __ldcg(&gacc[k].lo);
            v.hi = __ldcg(&gacc[k].hi);
            if (a < NA && (P.agg[a].kind == VD_AGG_MIN || P.agg[a].kind == VD_AGG_MAX)) {
                if (P.agg[a].isf) {
                    long long key2 = (long long)v.lo;
                    long long bits = key2 >= 0 ? key2 : key2 ^ 0x7FFFFFFFFFFFFFFFll;
                    put_f64(&v, __longlong_as_double(bits));
                } else {
                    put_i128(&v, (i128)(long long)v.lo);
                }
            }
            out[k] = v;
        }
        return;
    }
    // fold the warps' accumulators into this CTA's partial, then the grid's
    __syncthreads();
    Slot16* wacc = s_mem + (size_t)GEN_WARPS * 32 * (NA + 1);
    for (int k = threadIdx.x; k < nslots; k += GEN_THREADS) {
        int a = k % (NA + 1);
        const bool cnt = (a == NA);
        const int kind = cnt ? VD_AGG_COUNT : P.agg[a].kind;
        const bool isf = cnt ? false : P.agg[a].isf;
        Slot16 r = wacc[k];
        for (int w = 1; w < GEN_WARPS; ++w) {
            Slot16 x = wacc[(size_t)w * nslots + k];
            if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                if (isf) put_f64(&r, get_f64(r) + get_f64(x)); else put_i128(&r, get_i128(r) + get_i128(x));
            } else if (isf) {
                put_f64(&r, kind == VD_AGG_MIN ? fmin(get_f64(r), get_f64(x)) : fmax(get_f64(r), get_f64(x)));
            } else {
                i128 p = get_i128(r), q = get_i128(x);
                put_i128(&r, kind == VD_AGG_MIN ? (q < p ? q : p) : (q > p ? q : p));
            }
        }
        block_parts[(size_t)blockIdx.x * nslots + k] = r;
    }
    __shared__ bool s_last2;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last2 = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last2) return;
    __threadfence();
    fold_grid_parts(block_parts, nslots, out, [&](int k) {
        const int a = k % (NA + 1);
        const bool cnt = (a == NA);
        const int kind = cnt ? VD_AGG_COUNT : P.agg[a].kind;
        const bool isf = cnt ? false : P.agg[a].isf;
        if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) return isf ? (int)FK_F64_SUM : (int)FK_I128_SUM;
        if (isf) return kind == VD_AGG_MIN ? (int)FK_F64_MIN : (int)FK_F64_MAX;
        return kind == VD_AGG_MIN ? (int)FK_I128_MIN : (int)FK_I128_MAX;
    });
}

// ============================================================================
// Q1-shaped fragment: <= G groups from two u8 key columns, predicate an
// interval on one i32 column, aggregates from four i64 columns V0..V3:
//   S0 = SUM(V0)                          (sum_qty)
//   S1 = SUM(V1)                          (sum_base_price)
//   S2 = SUM(V1*(a1 + b1*V2))             (sum_disc_price)
//   S3 = SUM(V1*(a1 + b1*V2)*(a2 + b2*V3))(sum_charge)
//   S4 = SUM(V2)                          (sum_disc)
//   S5 = COUNT                            (count_order)
// ============================================================================
struct Q1Args {
    const int32_t* d;  // predicate column
    int32_t dlo, dhi;  // lo <= d <= hi
    const uint8_t* k1;
    const uint8_t* k2;
    int32_t m1, m2, koff;  // key = k1*m1 + k2*m2 + koff
    const int64_t* v[4];
    int64_t a1, b1, a2, b2;
    int64_t nquads;  // n / 4 (full quads); the tail is handled by the last CTA
    int64_t n;
};

constexpr int Q1_THREADS = 256;

// packed (disc, count) accumulator: disc in bits 0..39, count in bits 40..63
constexpr int Q1_CSHIFT = 40;

template <int G, bool NARROW>
struct Q1Acc {
    int64_t s0[G], s1[G], s2[G], s3[G], dc[G];
};

// Q1 row values (V0, V1, dp, ch, disc|count word).  EPS (some referenced
// column lacks VD_COL_NOEPS): an epsilon operand makes each product that
// uses it epsilon, and an epsilon value is skipped by its SUM (readings A5,
// A9) -- it contributes 0 while the row still counts (COUNT(*) = the row
// count, as the generic fragment).  Without EPS the metadata has proven
// that no referenced slot is epsilon.
struct Q1Vals {
    int64_t v0, v1, dp, ch, dc;
};
template <bool NARROW, bool EPS>
__device__ __forceinline__ Q1Vals q1_vals(const Q1Args& a, int64_t v0, int64_t v1, int64_t v2, int64_t v3) {
    Q1Vals r;
    if (NARROW) {
        // metadata proves |V1|, |a1+b1*V2|, |dp|, |a2+b2*V3| < 2^31 and the
        // constants fit in 32 bits: the factors are exact in wrapping 32-bit
        // arithmetic and each product is one 32x32->64 IMAD.WIDE
        int32_t f1 = (int32_t)a.a1 + (int32_t)a.b1 * (int32_t)v2;
        r.dp = (int64_t)(int32_t)v1 * (int64_t)f1;
        int32_t f2 = (int32_t)a.a2 + (int32_t)a.b2 * (int32_t)v3;
        r.ch = (int64_t)(int32_t)r.dp * (int64_t)f2;
    } else {
        r.dp = v1 * (a.a1 + a.b1 * v2);
        r.ch = r.dp * (a.a2 + a.b2 * v3);
    }
    if (EPS) {
        const bool e0 = v0 == INT64_MIN, e1 = v1 == INT64_MIN, e2 = v2 == INT64_MIN, e3 = v3 == INT64_MIN;
        r.v0 = e0 ? 0 : v0;
        r.v1 = e1 ? 0 : v1;
        if (e1 | e2) r.dp = 0;
        if (e1 | e2 | e3) r.ch = 0;
        r.dc = (e2 ? 0 : v2) + (1ll << Q1_CSHIFT);
    } else {
        r.v0 = v0;
        r.v1 = v1;
        r.dc = v2 + (1ll << Q1_CSHIFT);
    }
    return r;
}

// key of a row from its two dictionary codes; -1 if either code is epsilon
// (0xFF: the key is epsilon, the row has no group -- Partition drops it, A9)
template <bool EPS>
__device__ __forceinline__ int q1_key(const Q1Args& a, uint32_t c1, uint32_t c2) {
    if (EPS && (c1 == 0xFFu || c2 == 0xFFu)) return -1;
    return (int)c1 * a.m1 + (int)c2 * a.m2 + a.koff;
}

template <int G, bool NARROW, bool EPS>
__device__ __forceinline__ void q1_row(Q1Acc<G, NARROW>& A, const Q1Args& a, bool pass, int key, int64_t v0,
                                       int64_t v1, int64_t v2, int64_t v3) {
    const Q1Vals r = q1_vals<NARROW, EPS>(a, v0, v1, v2, v3);
#pragma unroll
    for (int g = 0; g < G; ++g) {
        if (pass && key == g) {
            A.s0[g] += r.v0;
            A.s1[g] += r.v1;
            A.s2[g] += r.dp;
            A.s3[g] += r.ch;
            A.dc[g] += r.dc;
        }
    }
}

template <int G, bool NARROW, bool EPS>
__global__ void __launch_bounds__(Q1_THREADS, 2) k_pipe_q1(const __grid_constant__ Q1Args a, Slot16* __restrict__ parts,
                                                           unsigned int* __restrict__ done, Slot16* __restrict__ out,
                                                           const Q1Map map) {
    Q1Acc<G, NARROW> A;
#pragma unroll
    for (int g = 0; g < G; ++g) { A.s0[g] = A.s1[g] = A.s2[g] = A.s3[g] = A.dc[g] = 0; }

    const int64_t nthreads = (int64_t)gridDim.x * Q1_THREADS;
    const int64_t tid = (int64_t)blockIdx.x * Q1_THREADS + threadIdx.x;
    // two quads in flight per thread per iteration (q and q + nthreads)
    int64_t q = tid;
    for (; q + nthreads < a.nquads; q += 2 * nthreads) {
        int4 d[2];
        uint32_t k1[2], k2[2];
        longlong2 x[2][4][2];
#pragma unroll
        for (int u = 0; u < 2; ++u) {
            const int64_t qq = q + u * nthreads;
            d[u] = __ldg(reinterpret_cast<const int4*>(a.d) + qq);
            k1[u] = __ldg(reinterpret_cast<const unsigned int*>(a.k1) + qq);
            k2[u] = __ldg(reinterpret_cast<const unsigned int*>(a.k2) + qq);
#pragma unroll
            for (int c = 0; c < 4; ++c) {
                x[u][c][0] = __ldg(reinterpret_cast<const longlong2*>(a.v[c]) + 2 * qq);
                x[u][c][1] = __ldg(reinterpret_cast<const longlong2*>(a.v[c]) + 2 * qq + 1);
            }
        }
#pragma unroll
        for (int u = 0; u < 2; ++u) {
            const int dd[4] = {d[u].x, d[u].y, d[u].z, d[u].w};
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                bool pass = dd[j] >= a.dlo && dd[j] <= a.dhi;
                int key = q1_key<EPS>(a, (k1[u] >> (8 * j)) & 0xFF, (k2[u] >> (8 * j)) & 0xFF);
                int64_t v0 = (j & 1) ? x[u][0][j >> 1].y : x[u][0][j >> 1].x;
                int64_t v1 = (j & 1) ? x[u][1][j >> 1].y : x[u][1][j >> 1].x;
                int64_t v2 = (j & 1) ? x[u][2][j >> 1].y : x[u][2][j >> 1].x;
                int64_t v3 = (j & 1) ? x[u][3][j >> 1].y : x[u][3][j >> 1].x;
                q1_row<G, NARROW, EPS>(A, a, pass, key, v0, v1, v2, v3);
            }
        }
    }
    for (; q < a.nquads; q += nthreads) {
        int4 d = __ldg(reinterpret_cast<const int4*>(a.d) + q);
        uint32_t k1 = __ldg(reinterpret_cast<const unsigned int*>(a.k1) + q);
        uint32_t k2 = __ldg(reinterpret_cast<const unsigned int*>(a.k2) + q);
        longlong2 x[4][2];
#pragma unroll
        for (int c = 0; c < 4; ++c) {
            x[c][0] = __ldg(reinterpret_cast<const longlong2*>(a.v[c]) + 2 * q);
            x[c][1] = __ldg(reinterpret_cast<const longlong2*>(a.v[c]) + 2 * q + 1);
        }
        const int dd[4] = {d.x, d.y, d.z, d.w};
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            bool pass = dd[j] >= a.dlo && dd[j] <= a.dhi;
            int key = q1_key<EPS>(a, (k1 >> (8 * j)) & 0xFF, (k2 >> (8 * j)) & 0xFF);
            int64_t v0 = (j & 1) ? x[0][j >> 1].y : x[0][j >> 1].x;
            int64_t v1 = (j & 1) ? x[1][j >> 1].y : x[1][j >> 1].x;
            int64_t v2 = (j & 1) ? x[2][j >> 1].y : x[2][j >> 1].x;
            int64_t v3 = (j & 1) ? x[3][j >> 1].y : x[3][j >> 1].x;
            q1_row<G, NARROW, EPS>(A, a, pass, key, v0, v1, v2, v3);
        }
    }
    // ragged tail (n % 4 rows): thread 0 of the grid
    if (tid == 0) {
        for (int64_t r = a.nquads * 4; r < a.n; ++r) {
            int dd = a.d[r];
            bool pass = dd >= a.dlo && dd <= a.dhi;
            int key = q1_key<EPS>(a, a.k1[r], a.k2[r]);
            q1_row<G, NARROW, EPS>(A, a, pass, key, a.v[0][r], a.v[1][r], a.v[2][r], a.v[3][r]);
        }
    }

    // ---- hierarchical fold: warp (int64, proven) -> CTA (i128) -> grid ----
    __shared__ i128 s_part[Q1_THREADS / 32][G][6];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
#pragma unroll
    for (int g = 0; g < G; ++g) {
        int64_t v[6] = {A.s0[g], A.s1[g], A.s2[g], A.s3[g], A.dc[g] & ((1ll << Q1_CSHIFT) - 1), A.dc[g] >> Q1_CSHIFT};
#pragma unroll
        for (int k = 0; k < 6; ++k) {
            int64_t w = warp_sum_i64(v[k]);
            if (lane == 0) s_part[warp][g][k] = (i128)w;
        }
    }
    __syncthreads();
    if (threadIdx.x < G * 6) {
        const int g = threadIdx.x / 6, k = threadIdx.x % 6;
        i128 t = 0;
        for (int w = 0; w < Q1_THREADS / 32; ++w) t += s_part[w][g][k];
        put_i128(&parts[(size_t)blockIdx.x * G * 6 + threadIdx.x], t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    __shared__ Slot16 s_raw[G * 6];
    fold_grid_parts(parts, G * 6, s_raw, FkI128Sum());
    __syncthreads();
    // the plan's [ngroups][naggs+1] layout (slot naggs = row count = COUNT)
    for (int k = threadIdx.x; k < map.ngroups * (map.naggs + 1); k += blockDim.x) {
        const int g = k / (map.naggs + 1), ag = k % (map.naggs + 1);
        out[k] = s_raw[g * 6 + ((ag == map.naggs) ? 5 : map.src[ag])];
    }
}

// ---- Q1 fragment, TMA-staged --------------------------------------------------
// The same fragment with its column tiles staged in shared memory by 1D TMA
// bulk copies (cp.async.bulk -> UBLKCP): one producer warp keeps
// Q1T_STAGES tiles of Q1T_TILE rows (7 column slices each) in flight behind
// mbarriers while eight consumer warps fold the previous tiles out of shared
// memory.  Group accumulators live in shared memory, one private set per
// thread laid out [slot][word][thread] (conflict-free: a lane's address
// depends on the slot only through multiples of 32 banks), so a row's
// contribution is one address computation plus load-add-store per word with
// no branch and no per-slot predication; rows failing the predicate land in
// a trash slot G.  This is the virtual scatter of §3.1.3: the group key is a
// work-item-local scatter position that is never materialised.
constexpr int Q1T_CW = 8;                                // consumer warps
constexpr int Q1T_NT = Q1T_CW * 32;                      // consumer threads
constexpr int Q1T_THREADS = Q1T_NT + 32;                 // + 1 producer warp
constexpr int Q1T_TILE = Q1T_CW * 128;                   // rows per stage
constexpr int Q1T_STAGES = 3;
constexpr int Q1T_STAGE_BYTES = Q1T_TILE * (4 + 4 * 8 + 2);
constexpr int Q1T_WORDS = 5;                             // qty, ext, dp, ch, disc|count
__host__ __device__ constexpr size_t q1t_smem(int G) {
    return (size_t)Q1T_STAGES * Q1T_STAGE_BYTES + (size_t)(G + 1) * Q1T_WORDS * Q1T_NT * 8 + 2 * Q1T_STAGES * 8;
}

template <bool NARROW, bool EPS>
__device__ __forceinline__ void q1_row_smem(int64_t* __restrict__ acc_t, const Q1Args& a, int G, int32_t dd,
                                            int key, int64_t v0, int64_t v1, int64_t v2, int64_t v3) {
    // dlo > INT32_MIN (planner), so an epsilon ship date never passes (A9)
    const bool pass = dd >= a.dlo && dd <= a.dhi && (!EPS || key >= 0);
    const int kk = pass ? key : G;  // trash slot for rows that fail the predicate or have no group
    const Q1Vals r = q1_vals<NARROW, EPS>(a, v0, v1, v2, v3);
    int64_t* p = acc_t + (size_t)kk * Q1T_WORDS * Q1T_NT;
    p[0 * Q1T_NT] += r.v0;
    p[1 * Q1T_NT] += r.v1;
    p[2 * Q1T_NT] += r.dp;
    p[3 * Q1T_NT] += r.ch;
    p[4 * Q1T_NT] += r.dc;
}

template <int G, bool NARROW, bool EPS>
__global__ void __launch_bounds__(Q1T_THREADS, 1) k_pipe_q1_tma(const __grid_constant__ Q1Args a, int64_t ntiles,
                                                                Slot16* __restrict__ parts,
                                                                unsigned int* __restrict__ done,
                                                                Slot16* __restrict__ out, const Q1Map map) {
    extern __shared__ __align__(128) uint8_t smem[];
    int64_t* acc = reinterpret_cast<int64_t*>(smem + (size_t)Q1T_STAGES * Q1T_STAGE_BYTES);
    uint64_t* full = reinterpret_cast<uint64_t*>(acc + (size_t)(G + 1) * Q1T_WORDS * Q1T_NT);
    uint64_t* empty = full + Q1T_STAGES;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < Q1T_STAGES; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], Q1T_CW);
        }
        fence_mbar_init();
    }
    for (int k = threadIdx.x; k < (G + 1) * Q1T_WORDS * Q1T_NT; k += Q1T_THREADS) acc[k] = 0;
    __syncthreads();

    if (warp == Q1T_CW) {
        // ---- producer: one elected lane issues the bulk copies ----
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % Q1T_STAGES);
                if (it >= Q1T_STAGES) mbar_wait(&empty[s], (uint32_t)(((it / Q1T_STAGES) - 1) & 1));
                uint8_t* st = smem + (size_t)s * Q1T_STAGE_BYTES;
                const int64_t r0 = tile * Q1T_TILE;
                mbar_expect_tx(&full[s], Q1T_STAGE_BYTES);
                tma_load_1d(st, a.d + r0, Q1T_TILE * 4, &full[s], pol);
#pragma unroll
                for (int c = 0; c < 4; ++c)
                    tma_load_1d(st + Q1T_TILE * 4 + c * Q1T_TILE * 8, a.v[c] + r0, Q1T_TILE * 8, &full[s], pol);
                tma_load_1d(st + Q1T_TILE * 36, a.k1 + r0, Q1T_TILE, &full[s], pol);
                tma_load_1d(st + Q1T_TILE * 37, a.k2 + r0, Q1T_TILE, &full[s], pol);
            }
        }
        __syncwarp();  // reconverge the producer warp before the CTA barrier
    } else {
        // ---- consumers: warp w folds rows w*128 + {2l, 2l+1, 64+2l, 65+2l} ----
        int64_t* acc_t = acc + threadIdx.x;
        const int rb = warp * 128 + 2 * lane;
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % Q1T_STAGES);
            mbar_wait(&full[s], (uint32_t)((it / Q1T_STAGES) & 1));
            const uint8_t* st = smem + (size_t)s * Q1T_STAGE_BYTES;
            int2 dd[2];
            uint32_t kk1[2], kk2[2];
            longlong2 x[2][4];
#pragma unroll
            for (int h = 0; h < 2; ++h) {
                const int r = rb + 64 * h;
                dd[h] = *reinterpret_cast<const int2*>(st + r * 4);
                kk1[h] = *reinterpret_cast<const uint16_t*>(st + Q1T_TILE * 36 + r);
                kk2[h] = *reinterpret_cast<const uint16_t*>(st + Q1T_TILE * 37 + r);
#pragma unroll
                for (int c = 0; c < 4; ++c)
                    x[h][c] = *reinterpret_cast<const longlong2*>(st + Q1T_TILE * 4 + c * Q1T_TILE * 8 + r * 8);
            }
            __syncwarp();  // the warp's reads of the stage are done
            if (lane == 0) mbar_arrive(&empty[s]);
#pragma unroll
            for (int h = 0; h < 2; ++h) {
                const int key0 = q1_key<EPS>(a, kk1[h] & 0xFF, kk2[h] & 0xFF);
                const int key1 = q1_key<EPS>(a, kk1[h] >> 8, kk2[h] >> 8);
                q1_row_smem<NARROW, EPS>(acc_t, a, G, dd[h].x, key0, x[h][0].x, x[h][1].x, x[h][2].x, x[h][3].x);
                q1_row_smem<NARROW, EPS>(acc_t, a, G, dd[h].y, key1, x[h][0].y, x[h][1].y, x[h][2].y, x[h][3].y);
            }
        }
        // ragged tail: rows past the last full tile, CTA 0 only
        if (blockIdx.x == 0) {
            for (int64_t r = ntiles * Q1T_TILE + threadIdx.x; r < a.n; r += Q1T_NT) {
                const int key = q1_key<EPS>(a, a.k1[r], a.k2[r]);
                q1_row_smem<NARROW, EPS>(acc_t, a, G, a.d[r], key, a.v[0][r], a.v[1][r], a.v[2][r], a.v[3][r]);
            }
        }
    }
    __syncthreads();

    // ---- hierarchical fold: thread slots -> warp (int64, proven) -> CTA (i128) -> grid ----
    __shared__ i128 s_part[Q1T_CW][G][6];
    if (warp < Q1T_CW) {
#pragma unroll
        for (int g = 0; g < G; ++g) {
            const int64_t* p = acc + (size_t)g * Q1T_WORDS * Q1T_NT + threadIdx.x;
            const int64_t dcw = p[4 * Q1T_NT];
            int64_t v[6] = {p[0], p[Q1T_NT], p[2 * Q1T_NT], p[3 * Q1T_NT], dcw & ((1ll << Q1_CSHIFT) - 1),
                            dcw >> Q1_CSHIFT};
#pragma unroll
            for (int k = 0; k < 6; ++k) {
                int64_t w = warp_sum_i64(v[k]);
                if (lane == 0) s_part[warp][g][k] = (i128)w;
            }
        }
    }
    __syncthreads();
    if (threadIdx.x < G * 6) {
        const int g = threadIdx.x / 6, k = threadIdx.x % 6;
        i128 t = 0;
        for (int w = 0; w < Q1T_CW; ++w) t += s_part[w][g][k];
        put_i128(&parts[(size_t)blockIdx.x * G * 6 + threadIdx.x], t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    __shared__ Slot16 s_raw[G * 6];
    fold_grid_parts(parts, G * 6, s_raw, FkI128Sum());
    __syncthreads();
    // the plan's [ngroups][naggs+1] layout (slot naggs = row count = COUNT)
    for (int k = threadIdx.x; k < map.ngroups * (map.naggs + 1); k += blockDim.x) {
        const int g = k / (map.naggs + 1), ag = k % (map.naggs + 1);
        out[k] = s_raw[g * 6 + ((ag == map.naggs) ? 5 : map.src[ag])];
    }
}

// Map the Q1 fragment's raw [G][6] sums to the plan's [ngroups][naggs+1].

// ============================================================================
// Scalar fragment (Q6 / selective aggregation):
//   filter: up to 3 columns, ints as inclusive intervals, floats as <= 2 terms
//   value : product of 1 or 2 columns (+ COUNT)
// ============================================================================
template <typename F0, typename F1, typename F2, typename VA, typename VB>
struct ScalarArgs {
    const F0* f0; const F1* f1; const F2* f2;
    int64_t lo[3], hi[3];   // integer intervals
    int32_t fcmp[2];        // float terms on f0 (cmp codes, -1 unused)
    double fc[2];
    const VA* va; const VB* vb;
    int64_t n;
};

struct NoCol {};

template <typename T> struct AccOf { typedef int64_t type; };
template <> struct AccOf<float> { typedef double type; };
template <> struct AccOf<double> { typedef double type; };

template <typename T>
__device__ __forceinline__ bool ftest(T x, int k, const int64_t* lo, const int64_t* hi, const int32_t* fc,
                                      const double* fv) {
    if (IsFloat<T>::value) {
        if (x != x) return false;
        bool ok = true;
        if (fc[0] >= 0) ok = ok && cmp_flt(fc[0], (double)x, fv[0]);
        if (fc[1] >= 0) ok = ok && cmp_flt(fc[1], (double)x, fv[1]);
        return ok;
    }
    return (int64_t)x >= lo[k] && (int64_t)x <= hi[k];
}

constexpr int SC_THREADS = 256;

// MODE 0 branching (late loads: a later column is loaded only for rows whose
// earlier filters passed), MODE 1 predicated (all loads, contribution x p).
// EPS: a value column may hold epsilon (no VD_COL_NOEPS and not a filter
// column, whose interval already excludes it): an epsilon factor makes the
// row's value epsilon, skipped by the SUM (A5) while the row still counts.
template <bool EPS, bool HAS_VB, typename VA, typename VB, typename ACC>
__device__ __forceinline__ ACC scalar_value(VA va, VB vb) {
    ACC v = (ACC)va;
    if (HAS_VB) v *= (ACC)vb;
    if (EPS && (Eps<VA>::is(va) || (HAS_VB && Eps<VB>::is(vb)))) v = (ACC)0;
    return v;
}

template <int MODE, bool EPS, bool HAS_F1, bool HAS_F2, bool HAS_VB, typename F0, typename F1, typename F2,
          typename VA, typename VB>
__global__ void __launch_bounds__(SC_THREADS) k_pipe_scalar(const __grid_constant__ ScalarArgs<F0, F1, F2, VA, VB> a,
                                                            Slot16* __restrict__ parts, unsigned int* __restrict__ done,
                                                            Slot16* __restrict__ out, const ScalarMap map) {
    typedef typename AccOf<VA>::type ACC;
    __shared__ Slot16 s_raw2[2];
    ACC sum = 0;
    int64_t cnt = 0;
    const int64_t nthreads = (int64_t)gridDim.x * SC_THREADS;
    const int64_t tid = (int64_t)blockIdx.x * SC_THREADS + threadIdx.x;
    const int64_t nq = a.n / 4;
    for (int64_t q = tid; q < nq; q += nthreads) {
        F0 x0[4];
        {
            // 4 rows of the first filter column: one 4*sizeof(F0)-byte load
            if (sizeof(F0) == 4) {
                int4 t = __ldg(reinterpret_cast<const int4*>(a.f0) + q);
                memcpy(&x0[0], &t.x, 4); memcpy(&x0[1], &t.y, 4); memcpy(&x0[2], &t.z, 4); memcpy(&x0[3], &t.w, 4);
            } else if (sizeof(F0) == 8) {
                longlong2 t0 = __ldg(reinterpret_cast<const longlong2*>(a.f0) + 2 * q);
                longlong2 t1 = __ldg(reinterpret_cast<const longlong2*>(a.f0) + 2 * q + 1);
                memcpy(&x0[0], &t0.x, 8); memcpy(&x0[1], &t0.y, 8); memcpy(&x0[2], &t1.x, 8); memcpy(&x0[3], &t1.y, 8);
            } else {
#pragma unroll
                for (int j = 0; j < 4; ++j) x0[j] = a.f0[4 * q + j];
            }
        }
        unsigned p = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) p |= (ftest(x0[j], 0, a.lo, a.hi, a.fcmp, a.fc) ? 1u : 0u) << j;
        if (MODE == 0 && p == 0) continue;  // late loads: nothing of this quad survives
        if (HAS_F1) {
            F1 x1[4];
#pragma unroll
            for (int j = 0; j < 4; ++j) x1[j] = (MODE == 1 || ((p >> j) & 1)) ? __ldg(a.f1 + 4 * q + j) : F1(0);
            unsigned p1 = 0;
#pragma unroll
            for (int j = 0; j < 4; ++j) p1 |= (ftest(x1[j], 1, a.lo, a.hi, a.fcmp, a.fc) ? 1u : 0u) << j;
            p &= p1;
            if (MODE == 0 && p == 0) continue;
        }
        if (HAS_F2) {
            F2 x2[4];
#pragma unroll
            for (int j = 0; j < 4; ++j) x2[j] = (MODE == 1 || ((p >> j) & 1)) ? __ldg(a.f2 + 4 * q + j) : F2(0);
            unsigned p2 = 0;
#pragma unroll
            for (int j = 0; j < 4; ++j) p2 |= (ftest(x2[j], 2, a.lo, a.hi, a.fcmp, a.fc) ? 1u : 0u) << j;
            p &= p2;
            if (MODE == 0 && p == 0) continue;
        }
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const bool pj = (p >> j) & 1;
            if (MODE == 0 && !pj) continue;
            VA va = (a.va == (const VA*)a.f0) ? (VA)x0[j] : __ldg(a.va + 4 * q + j);
            const ACC v = scalar_value<EPS, HAS_VB, VA, VB, ACC>(va, HAS_VB ? __ldg(a.vb + 4 * q + j) : VB(1));
            if (MODE == 1) { sum += pj ? v : (ACC)0; cnt += pj; }
            else { sum += v; cnt += 1; }
        }
    }
    if (tid == 0) {
        for (int64_t r = nq * 4; r < a.n; ++r) {
            bool pj = ftest(a.f0[r], 0, a.lo, a.hi, a.fcmp, a.fc);
            if (HAS_F1) pj = pj && ftest(a.f1[r], 1, a.lo, a.hi, a.fcmp, a.fc);
            if (HAS_F2) pj = pj && ftest(a.f2[r], 2, a.lo, a.hi, a.fcmp, a.fc);
            if (!pj) continue;
            sum += scalar_value<EPS, HAS_VB, VA, VB, ACC>(a.va[r], HAS_VB ? a.vb[r] : VB(1));
            cnt += 1;
        }
    }
    // warp -> CTA -> grid
    __shared__ Slot16 s_w[SC_THREADS / 32][2];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    int64_t c = warp_sum_i64(cnt);
    if (IsFloat<VA>::value) {
        double s = warp_sum_f64((double)sum);
        if (lane == 0) put_f64(&s_w[warp][0], s);
    } else {
        i128 s = warp_sum_i128((i128)(int64_t)sum);
        if (lane == 0) put_i128(&s_w[warp][0], s);
    }
    if (lane == 0) put_i128(&s_w[warp][1], (i128)c);
    __syncthreads();
    if (threadIdx.x < 2) {
        Slot16 r = s_w[0][threadIdx.x];
        for (int w = 1; w < SC_THREADS / 32; ++w) {
            if (threadIdx.x == 0 && IsFloat<VA>::value) put_f64(&r, get_f64(r) + get_f64(s_w[w][0]));
            else put_i128(&r, get_i128(r) + get_i128(s_w[w][threadIdx.x]));
        }
        parts[(size_t)blockIdx.x * 2 + threadIdx.x] = r;
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, 2, s_raw2,
                    [](int k) { return (k == 0 && IsFloat<VA>::value) ? (int)FK_F64_SUM : (int)FK_I128_SUM; });
    __syncthreads();
    if (threadIdx.x <= map.naggs) out[threadIdx.x] = s_raw2[(threadIdx.x == map.naggs) ? 1 : map.src[threadIdx.x]];
}

// ---- scalar fragment, TMA-staged -------------------------------------------------
// Up to 5 distinct columns (the filter columns and the value columns, shared
// when a value column is also a filter column, as l_discount in Q6) streamed
// through an SC_STAGES-deep ring of SC_TILE-row slices by one producer warp;
// consumer thread t folds rows t, t+NT, ... of each staged tile.
constexpr int SCT_CW = 8;
constexpr int SCT_NT = SCT_CW * 32;
constexpr int SCT_THREADS = SCT_NT + 32;
constexpr int SCT_TILE = 2048;
constexpr int SCT_MAXSTAGES = 16;

struct ScalarTmaArgs {
    const void* col[5];   // distinct staged columns
    int32_t esz[5];       // element sizes
    int32_t soff[5];      // slice offsets within a stage (bytes)
    int32_t ncol;
    int32_t stage_bytes;
    int32_t nstages;      // ring depth (~180 KB of tiles in flight per SM)
    int32_t role[5];      // staged column of f0, f1, f2, va, vb
    int64_t lo[3], hi[3];
    int32_t fcmp[2];
    double fc[2];
    int64_t n;
};

template <typename T>
__device__ __forceinline__ T role_ld(const uint8_t* st, const ScalarTmaArgs& a, int role, int r) {
    return reinterpret_cast<const T*>(st + a.soff[a.role[role]])[r];
}
template <typename T>
__device__ __forceinline__ T role_ldg(const ScalarTmaArgs& a, int role, int64_t r) {
    return reinterpret_cast<const T*>(a.col[a.role[role]])[r];
}

template <int MODE, bool EPS, int NF, bool HVB, int TILE, typename F0, typename F1, typename F2, typename VA,
          typename VB>
__global__ void __launch_bounds__(SCT_THREADS, 1) k_pipe_scalar_tma(const __grid_constant__ ScalarTmaArgs a,
                                                                    int64_t ntiles, Slot16* __restrict__ parts,
                                                                    unsigned int* __restrict__ done,
                                                                    Slot16* __restrict__ out, const ScalarMap map) {
    typedef typename AccOf<VA>::type ACC;
    __shared__ Slot16 s_raw2[2];
    extern __shared__ __align__(128) uint8_t smem[];
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)a.nstages * a.stage_bytes);
    uint64_t* empty = full + a.nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], SCT_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    ACC sum = 0;
    int64_t cnt = 0;
    auto row = [&](F0 x0, F1 x1, F2 x2, VA va, VB vb) {
        bool p = ftest(x0, 0, a.lo, a.hi, a.fcmp, a.fc);
        if (NF > 1) p = p && ftest(x1, 1, a.lo, a.hi, a.fcmp, a.fc);
        if (NF > 2) p = p && ftest(x2, 2, a.lo, a.hi, a.fcmp, a.fc);
        const ACC v = scalar_value<EPS, HVB, VA, VB, ACC>(va, vb);
        if (MODE == 1) {  // predicated: contribution x predicate
            sum += p ? v : (ACC)0;
            cnt += p;
        } else if (p) {   // branching
            sum += v;
            cnt += 1;
        }
    };
    if (warp == SCT_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % a.nstages);
                if (it >= a.nstages) mbar_wait(&empty[s], (uint32_t)(((it / a.nstages) - 1) & 1));
                uint8_t* st = smem + (size_t)s * a.stage_bytes;
                mbar_expect_tx(&full[s], (uint32_t)a.stage_bytes);
                for (int c = 0; c < a.ncol; ++c)
                    tma_load_1d(st + a.soff[c], (const uint8_t*)a.col[c] + tile * TILE * a.esz[c],
                                (uint32_t)(TILE * a.esz[c]), &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % a.nstages);
            mbar_wait(&full[s], (uint32_t)((it / a.nstages) & 1));
            const uint8_t* st = smem + (size_t)s * a.stage_bytes;
            constexpr int RPT = TILE / SCT_NT;
            F0 x0[RPT]; F1 x1[RPT]; F2 x2[RPT]; VA va[RPT]; VB vb[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) {
                const int r = threadIdx.x + k * SCT_NT;
                x0[k] = role_ld<F0>(st, a, 0, r);
                x1[k] = NF > 1 ? role_ld<F1>(st, a, 1, r) : F1(0);
                x2[k] = NF > 2 ? role_ld<F2>(st, a, 2, r) : F2(0);
                va[k] = role_ld<VA>(st, a, 3, r);
                vb[k] = HVB ? role_ld<VB>(st, a, 4, r) : VB(1);
            }
            __syncwarp();  // the warp's reads of the stage are done
            if (lane == 0) mbar_arrive(&empty[s]);
#pragma unroll
            for (int k = 0; k < RPT; ++k) row(x0[k], x1[k], x2[k], va[k], vb[k]);
        }
        if (blockIdx.x == 0) {
            for (int64_t r = ntiles * TILE + threadIdx.x; r < a.n; r += SCT_NT)
                row(role_ldg<F0>(a, 0, r), NF > 1 ? role_ldg<F1>(a, 1, r) : F1(0),
                    NF > 2 ? role_ldg<F2>(a, 2, r) : F2(0), role_ldg<VA>(a, 3, r), HVB ? role_ldg<VB>(a, 4, r) : VB(1));
        }
    }
    // warp -> CTA -> grid
    __shared__ Slot16 s_w[SCT_THREADS / 32][2];
    int64_t c = warp_sum_i64(cnt);
    if (IsFloat<VA>::value) {
        double sm = warp_sum_f64((double)sum);
        if (lane == 0) put_f64(&s_w[warp][0], sm);
    } else {
        i128 sm = warp_sum_i128((i128)(int64_t)sum);
        if (lane == 0) put_i128(&s_w[warp][0], sm);
    }
    if (lane == 0) put_i128(&s_w[warp][1], (i128)c);
    __syncthreads();
    if (threadIdx.x < 2) {
        Slot16 r = s_w[0][threadIdx.x];
        for (int w = 1; w < SCT_THREADS / 32; ++w) {
            if (threadIdx.x == 0 && IsFloat<VA>::value) put_f64(&r, get_f64(r) + get_f64(s_w[w][0]));
            else put_i128(&r, get_i128(r) + get_i128(s_w[w][threadIdx.x]));
        }
        parts[(size_t)blockIdx.x * 2 + threadIdx.x] = r;
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, 2, s_raw2,
                    [](int k) { return (k == 0 && IsFloat<VA>::value) ? (int)FK_F64_SUM : (int)FK_I128_SUM; });
    __syncthreads();
    if (threadIdx.x <= map.naggs) out[threadIdx.x] = s_raw2[(threadIdx.x == map.naggs) ? 1 : map.src[threadIdx.x]];
}


// ============================================================================
// Gather-fold fragment (FK joins: Q19 / Q9 style, a4 + a7 fused)
// ============================================================================
// Base columns are streamed through a TMA ring (as the scalar fragment);
// per row the predicate's base-column terms are evaluated before any gather
// (late materialisation: the random accesses into the dimension tables --
// identity-hashed FK positions, P:L1054-1056 -- happen only for rows that
// can still qualify), then the gathered terms, the group key (identity or
// calendar year, the latter through a shared-memory lookup table), and
// int64 products (exactness proven from min/max metadata on the host).
// Groups are folded per warp: lanes with equal keys are matched
// (__match_any_sync) and one leader per key adds their staged values into
// the warp's shared-memory slots -- no atomics.
constexpr int GF_CW = 8;
constexpr int GF_NT = GF_CW * 32;
constexpr int GF_THREADS = GF_NT + 32;
constexpr int GF_TILE = 2048;
constexpr int GF_MAXSTAGES = 8;
constexpr int GF_MAXCOLS = 8;
constexpr int GF_MAXYEARDAYS = 8192;

struct GfArgs {
    // staged base columns
    const void* col[GF_MAXCOLS];
    int32_t dt[GF_MAXCOLS], esz[GF_MAXCOLS], soff[GF_MAXCOLS];
    int32_t ncols;
    int32_t stage_bytes, nstages;
    // gathers: reference c = ncols + g
    int32_t ngathers;
    int32_t g_fk[VD_MAX_GATHERS];
    int64_t g_bias[VD_MAX_GATHERS];
    const void* g_p[VD_MAX_GATHERS];
    int64_t g_len[VD_MAX_GATHERS];
    int32_t g_dt[VD_MAX_GATHERS];
    // predicate: per conjunction, base terms first (nbase[c] of them)
    DevPred pred;
    int32_t nbase[VD_MAX_CONJ];
    // base-column terms common to every conjunction, hoisted and tested first
    int32_t ncommon;
    DevTerm common[VD_MAX_TERMS];
    // key
    int32_t nkey;
    int32_t k_col[VD_MAX_KEYPARTS], k_fn[VD_MAX_KEYPARTS];
    int64_t k_sub[VD_MAX_KEYPARTS], k_mult[VD_MAX_KEYPARTS];
    int32_t year_lo, year_days;  // calendar table covers [year_lo, year_lo + year_days)
    int32_t ngroups;
    // aggregates: SUM of prod (a + b*col) (int64), or COUNT
    int32_t naggs;
    int32_t a_kind[VD_MAX_AGGS], a_nf[VD_MAX_AGGS];
    int32_t a_col[VD_MAX_AGGS][VD_MAX_FACTORS];
    int64_t a_a[VD_MAX_AGGS][VD_MAX_FACTORS], a_b[VD_MAX_AGGS][VD_MAX_FACTORS];
    int64_t n;
};

struct GfRow {
    const uint8_t* st;  // stage base (nullptr: read global, tail rows)
    int r;              // row within the tile
    int64_t g;          // global row
};

__device__ __forceinline__ Val gf_base(const GfArgs& a, const GfRow& w, int c) {
    if (w.st) {
        const uint8_t* q = w.st + a.soff[c];
        Val v;
        v.isf = false;
        v.f = 0;
        switch (a.dt[c]) {
        case VD_U8: { uint8_t x = q[w.r]; v.eps = x == 0xFF; v.i = x; break; }
        case VD_I32: { int32_t x = reinterpret_cast<const int32_t*>(q)[w.r]; v.eps = x == INT32_MIN; v.i = x; break; }
        case VD_I64: { int64_t x = reinterpret_cast<const int64_t*>(q)[w.r]; v.eps = x == INT64_MIN; v.i = x; break; }
        case VD_F32: { float x = reinterpret_cast<const float*>(q)[w.r]; v.eps = x != x; v.isf = true; v.f = x; v.i = 0; break; }
        default: { double x = reinterpret_cast<const double*>(q)[w.r]; v.eps = x != x; v.isf = true; v.f = x; v.i = 0; break; }
        }
        return v;
    }
    return fetch_typed(a.col[c], a.dt[c], w.g);
}

// zero_pos: predicated lookups (Fig 16) -- the position is multiplied by the
// 0/1 predicate, so a non-qualifying row reads slot 0.
__device__ __forceinline__ Val gf_fetch(const GfArgs& a, const GfRow& w, int c, bool zero_pos = false) {
    if (c < a.ncols) return gf_base(a, w, c);
    const int g = c - a.ncols;
    Val out;
    out.eps = true;
    out.isf = false;
    out.i = 0;
    out.f = 0;
    int64_t p = 0;
    if (!zero_pos) {
        Val fk = gf_base(a, w, a.g_fk[g]);
        if (fk.eps) return out;
        p = fk.i - a.g_bias[g];
    }
    if (p < 0 || p >= a.g_len[g]) return out;
    return fetch_typed(a.g_p[g], a.g_dt[g], p);
}

__device__ __forceinline__ bool gf_pred(const GfArgs& a, const GfRow& w) {
    for (int k = 0; k < a.ncommon; ++k)
        if (!term_true(a.common[k], gf_base(a, w, a.common[k].col))) return false;
    if (a.pred.nconj == 0) return true;
    // phase 1: base-column terms of every conjunction (no gathers)
    unsigned alive = 0;
    for (int c = 0; c < a.pred.nconj; ++c) {
        bool ok = true;
        for (int k = 0; k < a.nbase[c] && ok; ++k) ok = term_true(a.pred.t[c][k], gf_base(a, w, a.pred.t[c][k].col));
        if (ok) {
            if (a.nbase[c] == a.pred.nterms[c]) return true;
            alive |= 1u << c;
        }
    }
    // phase 2: gathered terms, only for conjunctions still alive
    for (int c = 0; c < a.pred.nconj; ++c) {
        if (!((alive >> c) & 1u)) continue;
        bool ok = true;
        for (int k = a.nbase[c]; k < a.pred.nterms[c] && ok; ++k) {
            const DevTerm& t = a.pred.t[c][k];
            ok = term_true(t, gf_fetch(a, w, t.col));
        }
        if (ok) return true;
    }
    return false;
}

template <int MODE, bool SCALAR>
__global__ void __launch_bounds__(GF_THREADS, 1) k_pipe_gf(const __grid_constant__ GfArgs a, int64_t ntiles,
                                                           Slot16* __restrict__ parts, unsigned int* __restrict__ done,
                                                           Slot16* __restrict__ out) {
    extern __shared__ __align__(128) uint8_t smem[];
    const int NA = a.naggs, NS = a.ngroups * (a.naggs + 1);
    int64_t* acc = reinterpret_cast<int64_t*>(smem + (size_t)a.nstages * a.stage_bytes);  // [GF_CW][NS]
    int64_t* stage_v = acc + (size_t)GF_CW * NS;                                           // [GF_CW][32][NA+1]
    int16_t* ytab = reinterpret_cast<int16_t*>(stage_v + (size_t)GF_CW * 32 * (NA + 1));  // calendar years
    uint64_t* full = reinterpret_cast<uint64_t*>(ytab + ((a.year_days + 7) & ~7));
    uint64_t* empty = full + a.nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], GF_CW);
        }
        fence_mbar_init();
    }
    for (int k = threadIdx.x; k < GF_CW * NS; k += GF_THREADS) acc[k] = 0;
    for (int k = threadIdx.x; k < a.year_days; k += GF_THREADS) ytab[k] = (int16_t)year_of_day(a.year_lo + k);
    __syncthreads();

    int64_t racc[VD_MAX_AGGS + 1];  // SCALAR: per-thread accumulators (one group)
#pragma unroll
    for (int g = 0; g <= VD_MAX_AGGS; ++g) racc[g] = 0;
    auto process = [&](const GfRow& w, bool valid) {
        bool ok = valid && gf_pred(a, w);
        if (SCALAR) {
            // MODE 0 branching: aggregate inputs loaded only for qualifying rows;
            // MODE 1 predicated aggregation: loaded for every row, x predicate;
            // MODE 2 predicated lookups: gathers read position fk*pred (slot 0)
            if (MODE == 0 ? ok : valid) {
                const int64_t pm = ok ? 1 : 0;
#pragma unroll
                for (int g = 0; g < VD_MAX_AGGS; ++g) {
                    if (g >= NA) break;
                    int64_t pr = 1;
                    if (a.a_kind[g] != VD_AGG_COUNT) {
                        bool e = false;
                        for (int f = 0; f < a.a_nf[g]; ++f) {
                            int64_t x = 0;
                            if (a.a_col[g][f] >= 0) {
                                Val v = gf_fetch(a, w, a.a_col[g][f], MODE == 2 && !ok);
                                e |= v.eps;
                                x = v.i;
                            }
                            pr *= a.a_a[g][f] + a.a_b[g][f] * x;
                        }
                        if (e) pr = 0;  // an epsilon input is skipped by the fold (A5)
                    }
                    racc[g] += (MODE == 0) ? pr : pr * pm;
                }
                racc[VD_MAX_AGGS] += pm;
            }
            return;
        }
        if (__ballot_sync(VD_FULL, ok) == 0) return;  // nothing of this 32-row step qualifies
        int64_t key = 0;
        if (ok) {
            for (int k = 0; k < a.nkey && ok; ++k) {
                Val v = gf_fetch(a, w, a.k_col[k]);
                if (v.eps) { ok = false; break; }
                int64_t x = v.i;
                if (a.k_fn[k] == 1) {
                    const int64_t d = x - a.year_lo;
                    x = (d >= 0 && d < a.year_days) ? (int64_t)ytab[d] : (int64_t)year_of_day((int32_t)x);
                }
                key += (x - a.k_sub[k]) * a.k_mult[k];
            }
            if (ok && (key < 0 || key >= a.ngroups)) ok = false;  // excluded by the host's domain proof
        }
        int64_t* sv = stage_v + ((size_t)warp * 32 + lane) * (NA + 1);
        if (ok) {
            for (int g = 0; g < NA; ++g) {
                int64_t pr = 1;
                if (a.a_kind[g] != VD_AGG_COUNT) {
                    bool e = false;
                    for (int f = 0; f < a.a_nf[g]; ++f) {
                        int64_t x = 0;
                        if (a.a_col[g][f] >= 0) {
                            Val v = gf_fetch(a, w, a.a_col[g][f]);
                            e |= v.eps;
                            x = v.i;
                        }
                        pr *= a.a_a[g][f] + a.a_b[g][f] * x;
                    }
                    if (e) pr = 0;  // an epsilon input is skipped by the fold (A5)
                }
                sv[g] = pr;
            }
            sv[NA] = 1;
        }
        __syncwarp();
        const unsigned m = __match_any_sync(VD_FULL, ok ? key : -1ll);
        if (ok && (__ffs(m) - 1) == lane) {
            int64_t* dst = acc + (size_t)warp * NS + key * (NA + 1);
            for (int g = 0; g <= NA; ++g) {
                int64_t t = 0;
                for (unsigned mm = m; mm; mm &= mm - 1)
                    t += stage_v[((size_t)warp * 32 + (__ffs(mm) - 1)) * (NA + 1) + g];
                dst[g] += t;
            }
        }
        __syncwarp();
    };

    if (warp == GF_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % a.nstages);
                if (it >= a.nstages) mbar_wait(&empty[s], (uint32_t)(((it / a.nstages) - 1) & 1));
                uint8_t* st = smem + (size_t)s * a.stage_bytes;
                mbar_expect_tx(&full[s], (uint32_t)a.stage_bytes);
                for (int c = 0; c < a.ncols; ++c)
                    tma_load_1d(st + a.soff[c], (const uint8_t*)a.col[c] + tile * GF_TILE * a.esz[c],
                                (uint32_t)(GF_TILE * a.esz[c]), &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % a.nstages);
            mbar_wait(&full[s], (uint32_t)((it / a.nstages) & 1));
            const uint8_t* st = smem + (size_t)s * a.stage_bytes;
            for (int k = 0; k < GF_TILE / GF_NT; ++k) {
                GfRow w;
                w.st = st;
                w.r = threadIdx.x + k * GF_NT;
                w.g = tile * GF_TILE + w.r;
                process(w, true);
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
        }
        if (blockIdx.x == 0) {
            const int64_t t0 = ntiles * GF_TILE;
            for (int64_t base = t0 + warp * 32; base < a.n; base += GF_NT) {  // warp-uniform trip count
                GfRow w;
                w.st = nullptr;
                w.r = 0;
                w.g = base + lane;
                process(w, w.g < a.n);
            }
        }
    }
    if (SCALAR && warp < GF_CW) {
#pragma unroll
        for (int g = 0; g <= VD_MAX_AGGS; ++g) {
            const int slot = g < NA ? g : (g == VD_MAX_AGGS ? NA : -1);
            const int64_t t = warp_sum_i64(racc[g]);  // per-warp bound proven on the host
            if (lane == 0 && slot >= 0) acc[(size_t)warp * NS + slot] = t;
        }
    }
    __syncthreads();
    // CTA fold of the warps' slots (int128), then the grid's (last CTA)
    for (int k = threadIdx.x; k < NS; k += GF_THREADS) {
        i128 t = 0;
        for (int w = 0; w < GF_CW; ++w) t += (i128)acc[(size_t)w * NS + k];
        put_i128(&parts[(size_t)blockIdx.x * NS + k], t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, NS, out, FkI128Sum());
}

// ============================================================================
// Late-materialisation fragment (branching scalar plans, Fig 15/16 "branching"
// strategy): only the LEAD columns -- the
// columns of predicate terms common to every conjunction whose conjunction
// is an interval (u8: any terms, checked value by value on the host; i32:
// comparisons) -- stream densely (one 128-bit load per 16 rows per u8
// column, four per i32 column).  Rows that pass are compacted per warp
// (popc prefix over the lanes) into a shared-memory queue and folded 32 at a
// time, every lane busy: the rest of the predicate, the FK gathers and the
// aggregate inputs are loaded for those rows only (late loads, reading A31).
// A dense TMA fragment moves every byte of every column; this one moves the
// lead bytes plus the 64-byte blocks that hold a qualifying row.
// ============================================================================
struct LtCons {
    int32_t ref, pad;
    int64_t lo, hi;
    uint64_t in;
};
struct LateLead {
    const uint8_t* c8[2];
    uint32_t lo8[2], hi8[2];  // interval bounds replicated into the 4 bytes
    const int32_t* c32;
    int32_t lo32, hi32;       // lo32 > INT32_MIN: epsilon never passes
    // references (bit c: base column c, bit ncols + g: gather g) read by the
    // rest of the predicate / by the aggregates; FK columns of the gathers
    // included, so that each group of loads is issued at once.  pref1 (a
    // subset of pref): the references of the equality / IN terms, loaded
    // first; the rest of pref only for rows those terms leave undecided
    uint32_t pref, pref1, aref;
    uint32_t grab;  // lead blocks claimed per atomic (dynamic work distribution)
    // the predicate compiled to one constraint per (conjunction, reference):
    // lo <= x <= hi and bit x of `in` (IN sets; ~0 = none), epsilon fails.
    // Row VD_MAX_CONJ holds the common terms.  ncons[0] < 0: a term (NE)
    // has no such form and the term lists of GfArgs are interpreted instead
    int32_t ncons[VD_MAX_CONJ + 1];
    LtCons cons[VD_MAX_CONJ + 1][VD_MAX_TERMS];
    // u8 references (up to LT_MAXTAB): their constraints leave cons[] and
    // become acceptance tables -- tab[k][x] bit c (c < nconj: conjunction c,
    // bit LT_COMMON: the common terms) = value x (255: epsilon) passes every
    // constraint of that conjunction on reference tref[k]; tcm[k] = the
    // conjunctions constraining it.  The predicate becomes an AND of masks.
    int32_t ntab;
    int32_t tref[4];
    uint32_t tcm[4];
    uint8_t tab[4][256];
    // fast first round (PV == 2): the first-round references are one int32
    // FK column and nfg u8 lookups through it whose every constraint is
    // tabulated -- the loads go to registers and the tables decide at once
    // whether any conjunction can still pass (most lead rows: none)
    int32_t fk_col, nfg;
    int32_t fg[VD_MAX_GATHERS];     // gather index of fast lookup j
    int32_t fgtab[VD_MAX_GATHERS];  // its acceptance table
};
constexpr int LT_MAXTAB = 4;
constexpr int LT_COMMON = 4;  // = VD_MAX_CONJ


constexpr int LT_THREADS = 256;
constexpr int LT_QCAP = 32 + 16 * 32;  // < 32 left over + one 16-row step of every lane
// dynamic shared memory of the largest plan (values, accumulators, queues)
constexpr int LT_SMEM_MAX = (GF_MAXCOLS + VD_MAX_GATHERS + VD_MAX_AGGS + 1) * LT_THREADS * 8 + (LT_THREADS / 32) * LT_QCAP * 4;

// Late loads of one row go straight to shared memory (cp.async, no
// registers held while in flight; .L2::64B: each moves one 64-byte block,
// not the default 128-byte line, scripts/ubench_dram_gran.cu): every
// referenced base column at once,
// then the lookups they address.  The thread's values live in its column of
// sv[ref][LT_THREADS] (dynamic reference indices stay in shared memory, not
// in spilled local memory), widened to int64 with epsilon = INT64_MIN.  A u8
// element travels in its aligned 4-byte word (cp.async moves 4, 8 or 16
// bytes), unless that word would run past the column's end.
__device__ __forceinline__ void lt_cp(int64_t* sdst, const void* col, int32_t dt, int64_t i, int64_t len,
                                      uint64_t pol) {
    if (dt == VD_I64) {
        asm volatile("cp.async.ca.shared.global.L2::cache_hint.L2::64B [%0], [%1], 8, %2;" ::"r"(smem_u32(sdst)),
                     "l"((const int64_t*)col + i), "l"(pol)
                     : "memory");
    } else if (dt == VD_I32) {
        asm volatile("cp.async.ca.shared.global.L2::cache_hint.L2::64B [%0], [%1], 4, %2;" ::"r"(smem_u32(sdst)),
                     "l"((const int32_t*)col + i), "l"(pol)
                     : "memory");
    } else if ((i | 3) < len) {
        asm volatile("cp.async.ca.shared.global.L2::cache_hint.L2::64B [%0], [%1], 4, %2;" ::"r"(smem_u32(sdst)),
                     "l"((const uint8_t*)col + (i & ~(int64_t)3)), "l"(pol)
                     : "memory");
    } else {
        *reinterpret_cast<uint32_t*>(sdst) = (uint32_t)__ldg((const uint8_t*)col + i) << (8 * (i & 3));
    }
}
__device__ __forceinline__ int64_t lt_decode(const int64_t* sv, int32_t dt, int64_t i) {
    if (dt == VD_I64) return *sv;
    const uint32_t w = *reinterpret_cast<const uint32_t*>(sv);
    if (dt == VD_I32) return (int32_t)w == INT32_MIN ? INT64_MIN : (int64_t)(int32_t)w;
    const uint32_t x = (w >> (8 * (i & 3))) & 0xFFu;
    return x == 0xFFu ? INT64_MIN : (int64_t)x;
}
__device__ __forceinline__ void cp_async_wait_all() {
    asm volatile("cp.async.commit_group;\n\tcp.async.wait_group 0;" ::: "memory");
}

__device__ __forceinline__ void late_load(const GfArgs& a, uint32_t want, int64_t row, int64_t (*sv)[LT_THREADS],
                                          int tid, uint64_t pol_s, uint64_t pol_d) {
    const uint32_t wb = want & ((1u << a.ncols) - 1);
    for (uint32_t m = wb; m; m &= m - 1) {
        const int c = __ffs(m) - 1;
        lt_cp(&sv[c][tid], a.col[c], a.dt[c], row, a.n, pol_s);
    }
    cp_async_wait_all();
    for (uint32_t m = wb; m; m &= m - 1) {
        const int c = __ffs(m) - 1;
        sv[c][tid] = lt_decode(&sv[c][tid], a.dt[c], row);
    }
    const uint32_t wg = want >> a.ncols;
    if (!wg) return;
    int64_t pidx[VD_MAX_GATHERS];
#pragma unroll
    for (int g = 0; g < VD_MAX_GATHERS; ++g) {
        if (!((wg >> g) & 1u)) continue;
        const int64_t fk = sv[a.g_fk[g]][tid];
        pidx[g] = fk - a.g_bias[g];
        if (fk == INT64_MIN || pidx[g] < 0 || pidx[g] >= a.g_len[g]) {
            pidx[g] = -1;
            sv[a.ncols + g][tid] = INT64_MIN;
        } else {
            lt_cp(&sv[a.ncols + g][tid], a.g_p[g], a.g_dt[g], pidx[g], a.g_len[g], pol_d);
        }
    }
    cp_async_wait_all();
#pragma unroll
    for (int g = 0; g < VD_MAX_GATHERS; ++g)
        if (((wg >> g) & 1u) && pidx[g] >= 0) sv[a.ncols + g][tid] = lt_decode(&sv[a.ncols + g][tid], a.g_dt[g], pidx[g]);
}

// Three-valued predicate over the references loaded so far (`known`): a term
// on a reference not yet loaded is unknown.  Returns 0 (false), 1 (true) or
// 2 (undecided: load the rest and evaluate again).
__device__ __forceinline__ int late_term(const DevTerm& t, const int64_t (*sv)[LT_THREADS], int tid, uint32_t known) {
    if (!((known >> t.col) & 1u)) return 2;
    const int64_t x = sv[t.col][tid];
    return x != INT64_MIN && cmp_int(t.cmp, x, t.iv);  // epsilon is "not selected" (A9)
}

__device__ __forceinline__ int late_pred(const GfArgs& a, const int64_t (*sv)[LT_THREADS], int tid, uint32_t known) {
    int r = 1;
    for (int k = 0; k < a.ncommon; ++k) {
        const int t = late_term(a.common[k], sv, tid, known);
        if (t == 0) return 0;
        r = t == 2 ? 2 : r;
    }
    if (a.pred.nconj == 0) return r;
    int any = 0;  // 0: every conjunction false so far, 2: one undecided
    for (int c = 0; c < a.pred.nconj; ++c) {
        int cj = 1;
        for (int k = 0; k < a.pred.nterms[c] && cj != 0; ++k) {
            const int t = late_term(a.pred.t[c][k], sv, tid, known);
            cj = t == 0 ? 0 : (t == 2 ? 2 : cj);
        }
        if (cj == 1) return r;  // true, unless a common term is undecided
        if (cj == 2) any = 2;
    }
    return any;
}

// The same over the compiled constraints (no per-term comparison switch).
__device__ __forceinline__ int late_cons(const LtCons* cs, int n, const int64_t (*sv)[LT_THREADS], int tid,
                                         uint32_t known) {
    int r = 1;
    for (int k = 0; k < n; ++k) {
        const LtCons& c = cs[k];
        if (!((known >> c.ref) & 1u)) {
            r = 2;
            continue;
        }
        const int64_t x = sv[c.ref][tid];
        if (x == INT64_MIN || x < c.lo || x > c.hi || !((c.in >> (x & 63)) & 1ull)) return 0;
    }
    return r;
}
__device__ __forceinline__ int late_pred_c(const LateLead& ld, int nconj, const int64_t (*sv)[LT_THREADS], int tid,
                                           uint32_t known, const uint8_t (*stab)[256]) {
    const uint32_t conjs = (1u << nconj) - 1;
    uint32_t m = conjs | (1u << LT_COMMON), und = 0;
    for (int k = 0; k < ld.ntab; ++k) {
        const int r = ld.tref[k];
        if (!((known >> r) & 1u)) {
            und |= ld.tcm[k];
            continue;
        }
        const int64_t x = sv[r][tid];
        m &= stab[k][x == INT64_MIN ? 255 : (int)x];
    }
    // the rest, only for the conjunctions (and common terms) still alive
    if (!((m >> LT_COMMON) & 1u) || (nconj > 0 && !(m & conjs))) return 0;
    for (uint32_t live = m; live; live &= live - 1) {
        const int c = __ffs(live) - 1;
        const int t = late_cons(ld.cons[c], ld.ncons[c], sv, tid, known);
        if (t == 0) m &= ~(1u << c);
        if (t == 2) und |= 1u << c;
    }
    if (!((m >> LT_COMMON) & 1u)) return 0;
    if (nconj > 0 && !(m & conjs)) return 0;
    const bool yes = !((und >> LT_COMMON) & 1u) && (nconj == 0 || (m & conjs & ~und));
    return yes ? 1 : 2;
}

__device__ __forceinline__ uint32_t ld64b_hint_u32(const void* p, uint64_t pol) {
    uint32_t v;
    asm volatile("ld.global.nc.L2::cache_hint.L2::64B.u32 %0, [%1], %2;" : "=r"(v) : "l"(p), "l"(pol));
    return v;
}
__device__ __forceinline__ uint32_t ld64b_hint_u8(const void* p, uint64_t pol) {
    uint16_t v;
    asm volatile("ld.global.nc.L2::cache_hint.L2::64B.u8 %0, [%1], %2;" : "=h"(v) : "l"(p), "l"(pol));
    return v;
}
__device__ __forceinline__ uint32_t lt_mask_i32(const int4 (&v)[4], int32_t lo, int32_t hi) {
    uint32_t m = 0;
#pragma unroll
    for (int k = 0; k < 4; ++k) {
        const int32_t x[4] = {v[k].x, v[k].y, v[k].z, v[k].w};
#pragma unroll
        for (int j = 0; j < 4; ++j) m |= (uint32_t)(x[j] >= lo && x[j] <= hi) << (4 * k + j);
    }
    return m;
}
__device__ __forceinline__ int4 lt_ld16(const void* p, uint64_t pol) {
    int4 r;
    asm volatile("ld.global.nc.L1::no_allocate.L2::cache_hint.v4.s32 {%0,%1,%2,%3}, [%4], %5;"
                 : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w)
                 : "l"(p), "l"(pol));
    return r;
}

// PV: the predicate evaluator -- 0: the term lists interpreted; 1: compiled
// to constraints / acceptance tables (ld.ncons[0] >= 0, every plan without
// NE terms); 2: compiled, with the fast first round (ld.nfg > 0).  One
// evaluator per instance keeps the drain's code within the instruction cache
template <int N8, bool I32, int PV>
__global__ void __launch_bounds__(LT_THREADS, 4) k_pipe_late(const __grid_constant__ GfArgs a,
                                                         const __grid_constant__ LateLead ld,
                                                         Slot16* __restrict__ parts, unsigned int* __restrict__ done,
                                                         Slot16* __restrict__ out) {
    // dynamic shared memory: per-thread values [ref][thread], per-thread
    // accumulators [agg][thread] (touched by qualifying rows only, kept out
    // of the register file), per-warp row queues
    extern __shared__ __align__(16) uint8_t lt_smem[];
    // (sized by the plan: ncols + ngathers value rows, naggs + 1 accumulator rows)
    const int NA = a.naggs, nref = a.ncols + a.ngathers;
    int64_t(*s_v)[LT_THREADS] = reinterpret_cast<int64_t(*)[LT_THREADS]>(lt_smem);
    int64_t(*s_a)[LT_THREADS] = reinterpret_cast<int64_t(*)[LT_THREADS]>(lt_smem + nref * LT_THREADS * 8);
    int32_t(*s_q)[LT_QCAP] = reinterpret_cast<int32_t(*)[LT_QCAP]>(lt_smem + (nref + NA + 1) * LT_THREADS * 8);
    __shared__ int64_t s_acc[LT_THREADS / 32][VD_MAX_AGGS + 1];
    __shared__ uint8_t s_tab[LT_MAXTAB][256];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31, tid = threadIdx.x;
    for (int k = 0; k < ld.ntab; ++k) s_tab[k][tid] = ld.tab[k][tid];  // LT_THREADS == 256
    __syncthreads();
    const uint64_t pol_s = policy_evict_first(), pol_d = policy_evict_last();
    int32_t* q_ = s_q[warp];
    int cnt = 0;  // warp-uniform queue depth
    for (int g = 0; g <= NA; ++g) s_a[g][tid] = 0;
    // the rest of the predicate and the aggregate inputs of one lead-qualified row
    constexpr bool CP = PV >= 1;
    // everything after the first round (its references in s_v): the rest of
    // the predicate, the undecided rows' second round, the aggregate inputs
    auto rest_row = [&](int64_t row) {
        int t = CP ? late_pred_c(ld, a.pred.nconj, s_v, tid, ld.pref1, s_tab) : late_pred(a, s_v, tid, ld.pref1);
        if (t == 2) {
            late_load(a, ld.pref & ~ld.pref1, row, s_v, tid, pol_s, pol_d);
            t = CP ? late_pred_c(ld, a.pred.nconj, s_v, tid, ld.pref, s_tab) : late_pred(a, s_v, tid, ld.pref);
        }
        if (t != 1) return;
        late_load(a, ld.aref & ~ld.pref, row, s_v, tid, pol_s, pol_d);
#pragma unroll
        for (int g = 0; g < VD_MAX_AGGS; ++g) {
            if (g >= NA) break;
            int64_t pr = 1;
            if (a.a_kind[g] != VD_AGG_COUNT) {
                bool e = false;
                for (int f = 0; f < a.a_nf[g]; ++f) {
                    int64_t x = 0;
                    if (a.a_col[g][f] >= 0) {
                        x = s_v[a.a_col[g][f]][tid];
                        e |= x == INT64_MIN;
                    }
                    pr *= a.a_a[g][f] + a.a_b[g][f] * x;
                }
                if (e) pr = 0;  // an epsilon input is skipped by the fold (A5)
            }
            s_a[g][tid] += pr;
        }
        s_a[NA][tid] += 1;
    };
    auto fold_row = [&](int64_t row) {
        if (PV == 2) {
            // the FK and the lookups straight to registers (also kept in s_v
            // for the later rounds), the tables ANDed: reject at once unless
            // a conjunction (and the common terms) can still pass (most lead
            // rows: none)
            const int32_t fk = (int32_t)ld64b_hint_u32((const int32_t*)a.col[ld.fk_col] + row, pol_s);
            s_v[ld.fk_col][tid] = fk == INT32_MIN ? INT64_MIN : (int64_t)fk;
            uint32_t m = ((1u << a.pred.nconj) - 1) | (1u << LT_COMMON);
#pragma unroll
            for (int j = 0; j < VD_MAX_GATHERS; ++j) {
                if (j >= ld.nfg) break;
                const int g = ld.fg[j];
                const int64_t pidx = (int64_t)fk - a.g_bias[g];
                uint32_t x = 0xFFu;
                if (fk != INT32_MIN && pidx >= 0 && pidx < a.g_len[g])
                    x = ld64b_hint_u8((const uint8_t*)a.g_p[g] + pidx, pol_d);
                s_v[a.ncols + g][tid] = x == 0xFFu ? INT64_MIN : (int64_t)x;
                m &= s_tab[ld.fgtab[j]][x];
            }
            if (!((m >> LT_COMMON) & 1u) || (a.pred.nconj > 0 && !(m & ((1u << a.pred.nconj) - 1)))) return;
        } else {
            late_load(a, ld.pref1, row, s_v, tid, pol_s, pol_d);
        }
        rest_row(row);
    };
    auto drain = [&](int k) {  // fold the top k (<= 32) queued rows
        __syncwarp();
        if (lane < k) fold_row(q_[cnt - k + lane]);
        cnt -= k;
        __syncwarp();
    };
    const int64_t nq = a.n / 16;
    // lead words of the current step, and of the next one loaded before the
    // current step's drain (the stream stays in flight behind the late loads)
    int4 c8[N8 > 0 ? N8 : 1], c32[4];
    auto load_lead = [&](int64_t q, int4* w8, int4* w32) {
        if (q >= nq) return;
#pragma unroll
        for (int j = 0; j < N8; ++j) w8[j] = lt_ld16(ld.c8[j] + 16 * q, pol_s);
        if (I32) {
#pragma unroll
            for (int k = 0; k < 4; ++k) w32[k] = lt_ld16(ld.c32 + 16 * q + 4 * k, pol_s);
        }
    };
    // dynamic work distribution: a warp claims LT_GRAB consecutive 32-word
    // blocks of the lead at a time from a global counter (done[1]; one
    // same-address atomic per claim, so claims must be coarse), so no warp
    // idles at the end while others still drain
    const unsigned LT_GRAB = ld.grab;
    unsigned rb = 0, re = 0;  // the warp's claimed block range [rb, re)
    auto next_block = [&]() -> int64_t {
        if (rb == re) {
            unsigned b = 0;
            if (lane == 0) b = atomicAdd(done + 1, 1u);
            rb = __shfl_sync(VD_FULL, b, 0) * LT_GRAB;
            re = rb + LT_GRAB;
        }
        return (int64_t)(rb++) * 32;
    };
    int64_t q0 = next_block();
    load_lead(q0 + lane, c8, c32);
    while (q0 < nq) {
        const int64_t q1 = next_block();
        const int64_t q = q0 + lane;
        uint32_t m = 0;
        if (q < nq) {
            m = 0xFFFFu;
            if (N8 > 0) {
                // byte masks of every u8 lead column ANDed word by word, then
                // one byte -> bit extraction
                uint32_t r[4] = {~0u, ~0u, ~0u, ~0u};
#pragma unroll
                for (int j = 0; j < N8; ++j) {
                    const uint32_t w[4] = {(uint32_t)c8[j].x, (uint32_t)c8[j].y, (uint32_t)c8[j].z, (uint32_t)c8[j].w};
                    if (ld.lo8[j] == ld.hi8[j]) {
#pragma unroll
                        for (int i = 0; i < 4; ++i) r[i] &= __vcmpeq4(w[i], ld.lo8[j]);
                    } else {
#pragma unroll
                        for (int i = 0; i < 4; ++i) r[i] &= __vcmpgeu4(w[i], ld.lo8[j]) & __vcmpleu4(w[i], ld.hi8[j]);
                    }
                }
                m = 0;
#pragma unroll
                for (int i = 0; i < 4; ++i) m |= (((r[i] & 0x01010101u) * 0x01020408u) >> 24) << (4 * i);
            }
            if (I32) m &= lt_mask_i32(c32, ld.lo32, ld.hi32);
        }
        load_lead(q1 + lane, c8, c32);
        // compaction: the lanes' qualifying rows, in row order, onto the warp's queue
        const int pc = __popc(m);
        int incl = pc;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const int u = __shfl_up_sync(VD_FULL, incl, o);
            if (lane >= o) incl += u;
        }
        int at = cnt + incl - pc;
        while (m) {
            q_[at++] = (int32_t)(16 * q + (__ffs(m) - 1));
            m &= m - 1;
        }
        cnt += __shfl_sync(VD_FULL, incl, 31);
        while (cnt >= 32) drain(32);
        q0 = q1;
    }
    if (cnt > 0) drain(cnt);
    // ragged tail (< 16 rows): warp 0 of block 0, one row per lane
    if (blockIdx.x == 0 && warp == 0) {
        const int64_t row = nq * 16 + lane;
        if (row < a.n) {
            bool ok = true;
#pragma unroll
            for (int j = 0; j < N8; ++j) {
                const uint32_t x = ld.c8[j][row];
                ok = ok && x >= (ld.lo8[j] & 0xFFu) && x <= (ld.hi8[j] & 0xFFu);
            }
            if (I32) ok = ok && ld.c32[row] >= ld.lo32 && ld.c32[row] <= ld.hi32;
            if (ok) fold_row(row);
        }
    }
    // fold: warp sums (int64, bounded on the host) -> CTA (int128) -> last CTA
    for (int g = 0; g <= NA; ++g) {
        const int64_t t = warp_sum_i64(s_a[g][tid]);
        if (lane == 0) s_acc[warp][g] = t;
    }
    __syncthreads();
    const int NS = NA + 1;
    if (threadIdx.x < NS) {
        const int g = threadIdx.x;  // aggregates, then the row count
        i128 t = 0;
        for (int w = 0; w < LT_THREADS / 32; ++w) t += (i128)s_acc[w][g];
        put_i128(&parts[(size_t)blockIdx.x * NS + threadIdx.x], t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, NS, out, FkI128Sum());
}

// ============================================================================
// FK grouped-fold fragment (Q9 shape): key = (dim[fk - bias] - subA) * mA +
// (f(kb) - subB) * mB with f = calendar year (shared-memory table) or
// identity, value = X * (a + b * Y) (32x32->64 IMAD.WIDE when proven narrow),
// COUNT.  Base columns fk (i32), kb (i32), X, Y (i64) stream through the TMA
// ring (24 B/row); the dimension column (u8) is gathered per row from L2.
// Per-warp shared-memory group slots, filled by one leader lane per distinct
// key of each 32-row step (__match_any_sync) -- the virtual scatter of
// §3.1.3 at warp granularity.
// ============================================================================
constexpr int FKG_TILE = 2048;
constexpr int FKG_CW = 16;  // consumer warps (latency hiding for the L2 gathers)
constexpr int FKG_NT = FKG_CW * 32;
constexpr int FKG_THREADS = FKG_NT + 32;

struct FkgArgs {
    const int32_t* fk;
    const int32_t* kb;
    const int64_t* x;
    const int64_t* y;
    const uint8_t* dim;
    int64_t dim_len, bias;
    int32_t subA, mA, subB, mB;
    int32_t yfn, ylo, ydays;
    int64_t a, b;
    int32_t ngroups;
    int32_t nstages;
    int64_t n;
    int32_t sum_slot, cnt_slot;  // plan aggregate indices (-1: absent)
    int32_t naggs;
};

template <bool NARROW, bool ATOM, bool PIPE>
__global__ void __launch_bounds__(FKG_THREADS, 1) k_pipe_fkg(const __grid_constant__ FkgArgs a, int64_t ntiles,
                                                            Slot16* __restrict__ parts, unsigned int* __restrict__ done,
                                                            Slot16* __restrict__ out) {
    extern __shared__ __align__(128) uint8_t smem[];
    constexpr int SB = FKG_TILE * (4 + 4 + 8 + 8);
    // per-warp group slots as three u32 arrays (sum low word, sum high word,
    // count) so that random keys spread over all 32 banks; + a trash slot
    const int GS = a.ngroups + 1;
    const int GSP = (GS + 31) & ~31;
    uint32_t* acc = reinterpret_cast<uint32_t*>(smem + (size_t)a.nstages * SB);  // [FKG_CW][3][GSP]
    int64_t* sv = reinterpret_cast<int64_t*>(acc + (size_t)FKG_CW * 3 * GSP);   // [FKG_CW][32]
    int16_t* ytab = reinterpret_cast<int16_t*>(sv + FKG_CW * 32);
    uint64_t* full = reinterpret_cast<uint64_t*>(ytab + ((a.ydays + 7) & ~7));
    uint64_t* empty = full + a.nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], FKG_CW);
        }
        fence_mbar_init();
    }
    for (int k = threadIdx.x; k < FKG_CW * 3 * GSP; k += FKG_THREADS) acc[k] = 0;
    for (int k = threadIdx.x; k < a.ydays; k += FKG_THREADS) ytab[k] = (int16_t)year_of_day(a.ylo + k);
    __syncthreads();
    uint32_t* wlo = acc + (size_t)warp * 3 * GSP;
    uint32_t* whi = wlo + GSP;
    uint32_t* wcnt = whi + GSP;
    int64_t* wsv = sv + warp * 32;

    // phase 1 of a 32-row step: the lane's key (-1: no group) and value; the
    // dimension gather is issued here, so the RPT gathers of a tile are in
    // flight together
    // the dimension value of a row (0x100: no dimension row -- epsilon FK or
    // outside the dimension, reading A9/A11); issued early, consumed late
    auto gather = [&](bool valid, int32_t fk) -> int {
        const int64_t p = (int64_t)fk - a.bias;
        return (valid && fk != INT32_MIN && p >= 0 && p < a.dim_len) ? (int)__ldg(a.dim + p) : 0x100;
    };
    // the group key (-1: no group) and value of a row, given its dimension value
    auto keyof = [&](int d, int32_t kb, int64_t x, int64_t y, int64_t& v) {
        int key = -1;
        v = 0;
        if (d != 0x100) {
            int kbv = kb;
            if (a.yfn) {
                const int dd = kb - a.ylo;  // the table covers [min, max] of kb (metadata)
                kbv = (dd >= 0 && dd < a.ydays) ? (int)ytab[dd] : -0x40000000;
            }
            key = (d - a.subA) * a.mA + (kbv - a.subB) * a.mB;
            if (d == 0xFF || kb == INT32_MIN || key < 0 || key >= a.ngroups) key = -1;
            if (NARROW) {
                const int32_t f = (int32_t)((uint32_t)a.a + (uint32_t)a.b * (uint32_t)y);
                v = (int64_t)(int32_t)x * (int64_t)f;
            } else {
                v = x * (a.a + a.b * y);
            }
            if (x == INT64_MIN || y == INT64_MIN) v = 0;  // epsilon factor: skipped by SUM (A5/A9)
        }
        return key;
    };
    // phase 2: fold the step into the warp's group slots -- shared-memory
    // atomics (ATOM) or one leader lane per distinct key (__match_any_sync)
    auto fold = [&](int key, int64_t v) {
        if (ATOM) {
            // native 32-bit shared atomics (a 64-bit one is a CAS loop): the
            // low word returns the old value, the carry goes to the high word
            // -- exact modulo 2^64.  Rows without a group update the trash slot.
            const int g = key >= 0 ? key : a.ngroups;
            const uint64_t uv = (uint64_t)v;
            const uint32_t lo = (uint32_t)uv;
            const uint32_t old = atomicAdd(&wlo[g], lo);
            atomicAdd(&wcnt[g], 1u);  // < 2^32 rows per warp
            const uint32_t hi = (uint32_t)(uv >> 32) + ((uint32_t)(old + lo) < old ? 1u : 0u);
            if (hi) atomicAdd(&whi[g], hi);
            return;
        }
        wsv[lane] = v;
        __syncwarp();
        const unsigned m = __match_any_sync(VD_FULL, key);
        if (key >= 0 && (__ffs(m) - 1) == lane) {
            int64_t t = 0;
            for (unsigned mm = m; mm; mm &= mm - 1) t += wsv[__ffs(mm) - 1];
            const uint64_t cur = ((uint64_t)whi[key] << 32 | wlo[key]) + (uint64_t)t;
            wlo[key] = (uint32_t)cur;
            whi[key] = (uint32_t)(cur >> 32);
            wcnt[key] += __popc(m);
        }
        __syncwarp();
    };
    // RPT rows at once: all low-word atomics are issued before any carry is
    // needed, so their latencies overlap
    constexpr int RPT = FKG_TILE / FKG_NT;
    auto foldn = [&](const int* key, const int64_t* v) {
        if (!ATOM) {
#pragma unroll
            for (int k = 0; k < RPT; ++k) fold(key[k], v[k]);
            return;
        }
        uint32_t old[RPT];
        int g[RPT];
#pragma unroll
        for (int k = 0; k < RPT; ++k) {
            g[k] = key[k] >= 0 ? key[k] : a.ngroups;
            old[k] = atomicAdd(&wlo[g[k]], (uint32_t)(uint64_t)v[k]);
            atomicAdd(&wcnt[g[k]], 1u);
        }
#pragma unroll
        for (int k = 0; k < RPT; ++k) {
            const uint32_t lo = (uint32_t)(uint64_t)v[k];
            const uint32_t hi = (uint32_t)((uint64_t)v[k] >> 32) + ((uint32_t)(old[k] + lo) < old[k] ? 1u : 0u);
            if (hi) atomicAdd(&whi[g[k]], hi);
        }
    };

    if (warp == FKG_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % a.nstages);
                if (it >= a.nstages) mbar_wait(&empty[s], (uint32_t)(((it / a.nstages) - 1) & 1));
                uint8_t* st = smem + (size_t)s * SB;
                const int64_t r0 = tile * FKG_TILE;
                mbar_expect_tx(&full[s], SB);
                tma_load_1d(st, a.fk + r0, FKG_TILE * 4, &full[s], pol);
                tma_load_1d(st + FKG_TILE * 4, a.kb + r0, FKG_TILE * 4, &full[s], pol);
                tma_load_1d(st + FKG_TILE * 8, a.x + r0, FKG_TILE * 8, &full[s], pol);
                tma_load_1d(st + FKG_TILE * 16, a.y + r0, FKG_TILE * 8, &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        // software pipeline: the gathers of tile i are issued, then tile i-1
        // (whose gathers were issued one iteration earlier) is keyed and
        // folded, so each L2 round trip overlaps a whole iteration
        int pd[RPT], pkb[RPT];
        int64_t px[RPT], py[RPT];
        bool have = false;
        auto drain = [&]() {
            int key[RPT];
            int64_t v[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) key[k] = keyof(pd[k], pkb[k], px[k], py[k], v[k]);
            foldn(key, v);
        };
        int s = 0;          // ring stage and its phase, advanced without
        uint32_t ph = 0;    // a division by the runtime stage count
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            mbar_wait(&full[s], ph);
            const uint8_t* st = smem + (size_t)s * SB;
            int32_t f[RPT], kb[RPT];
            int64_t x[RPT], y[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) {
                const int r = threadIdx.x + k * FKG_NT;
                f[k] = reinterpret_cast<const int32_t*>(st)[r];
                kb[k] = reinterpret_cast<const int32_t*>(st + FKG_TILE * 4)[r];
                x[k] = reinterpret_cast<const int64_t*>(st + FKG_TILE * 8)[r];
                y[k] = reinterpret_cast<const int64_t*>(st + FKG_TILE * 16)[r];
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
            if (++s == a.nstages) { s = 0; ph ^= 1u; }
            int d[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) d[k] = gather(true, f[k]);
            if (PIPE && have) drain();
#pragma unroll
            for (int k = 0; k < RPT; ++k) { pd[k] = d[k]; pkb[k] = kb[k]; px[k] = x[k]; py[k] = y[k]; }
            have = true;
            if (!PIPE) { drain(); have = false; }
        }
        if (have) drain();
        if (blockIdx.x == 0) {
            for (int64_t base = ntiles * FKG_TILE + warp * 32; base < a.n; base += FKG_NT) {
                const int64_t r = base + lane;
                const bool ok = r < a.n;
                int64_t v;
                const int key = keyof(gather(ok, ok ? a.fk[r] : 0), ok ? a.kb[r] : 0, ok ? a.x[r] : 0,
                                      ok ? a.y[r] : 0, v);
                fold(key, v);
            }
        }
    }
    __syncthreads();
    const int NS = a.ngroups * (a.naggs + 1);
    // CTA fold (int128) into [ngroups][naggs+1] directly in the plan's layout
    for (int k = threadIdx.x; k < NS; k += FKG_THREADS) {
        const int g = k / (a.naggs + 1), ag = k % (a.naggs + 1);
        const int src = (ag == a.naggs || ag == a.cnt_slot) ? 1 : 0;
        i128 t = 0;
        for (int w = 0; w < FKG_CW; ++w) {
            const uint32_t* b = acc + (size_t)w * 3 * GSP;
            t += src ? (i128)b[2 * GSP + g] : (i128)(int64_t)((uint64_t)b[GSP + g] << 32 | b[g]);
        }
        put_i128(&parts[(size_t)blockIdx.x * NS + k], t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, NS, out, FkI128Sum());
}

// ---- FK grouped fold with per-thread private group slots ----------------------
// The same Q9-shaped fragment when the host proves from min/max metadata that
// every row's value X*(a+bY) lies in [0, 2^31) and the key part B is a
// calendar year inside 1969..2099: each consumer thread owns one packed u64
// slot per group in shared memory, laid out [group][thread] (a warp's 32
// lanes always touch 32 consecutive u64 words: conflict-free whatever the
// keys), holding sum + (count << 48).  A row is one LDS.64 / IADD.64 / STS.64
// -- no atomics, no leader election -- and the group table of the virtual
// scatter (§3.1.3) is private down to the work item, the Fig 3
// hierarchy with one more level.  The host bounds the rows per thread to
// < 2^16 (grid size), so the 16-bit count and 48-bit sum cannot carry.
// CHECKED = false when metadata also proves that every row joins (FK inside
// the dimension, no epsilon) and every key lies in [0, ngroups): then no row
// needs the trash slot and the checks compile away.
// The year comes from (4(d+365)+3) / 1461 + 1969 (exact for 1969-01-01 ..
// 2099-12-31; the host checks the column's range).
constexpr int FKP_TILE = 1024;
constexpr int FKP_CW = 4;
constexpr int FKP_NT = FKP_CW * 32;
constexpr int FKP_THREADS = FKP_NT + 32;
constexpr int FKP_RPT = FKP_TILE / FKP_NT;  // 8 rows per thread per tile, as 4 row pairs
constexpr int FKP_MAXSLOTS = 176;           // ngroups (+ trash) that fit beside a 2-stage ring
constexpr int FKP_STAGES = 2;

template <bool CHECKED, int BATCH>
__global__ void __launch_bounds__(FKP_THREADS, 1) k_pipe_fkg_priv(const __grid_constant__ FkgArgs a, int64_t ntiles,
                                                                  int32_t pf_dist, Slot16* __restrict__ parts,
                                                                  unsigned int* __restrict__ done,
                                                                  Slot16* __restrict__ out) {
    extern __shared__ __align__(128) uint8_t smem[];
    constexpr int SB = FKP_TILE * (4 + 4 + 8 + 8);
    const int GS = a.ngroups + (CHECKED ? 1 : 0);
    uint64_t* tab = reinterpret_cast<uint64_t*>(smem + (size_t)FKP_STAGES * SB);  // [GS][FKP_NT]
    uint64_t* full = tab + (size_t)GS * FKP_NT;
    uint64_t* empty = full + FKP_STAGES;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < FKP_STAGES; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], FKP_CW);
        }
        fence_mbar_init();
    }
    for (int k = threadIdx.x; k < GS * FKP_NT; k += FKP_THREADS) tab[k] = 0;
    __syncthreads();

    constexpr uint64_t ONE = 1ull << 48;
    // key of a row from its dimension value d and base key column value kb
    auto keyof = [&](int d, int32_t kb) -> int {
        const int kbv = a.yfn ? (4 * (kb + 365) + 3) / 1461 + 1969 : kb;
        int key = (d - a.subA) * a.mA + (kbv - a.subB) * a.mB;
        if (CHECKED) {
            if (d == 0x100 || d == 0xFF || kb == INT32_MIN || key < 0 || key >= a.ngroups) key = a.ngroups;
        }
        return key;
    };
    auto gather = [&](int32_t fk) -> int {
        const int64_t p = (int64_t)fk - a.bias;
        if (CHECKED) return (fk != INT32_MIN && p >= 0 && p < a.dim_len) ? (int)__ldg(a.dim + p) : 0x100;
        return (int)__ldg(a.dim + p);
    };
    // an epsilon factor makes the row's value epsilon: skipped by the SUM
    // (reading A5/A9), still counted by COUNT(*)
    auto value = [&](int64_t x, int64_t y) -> uint64_t {
        const int32_t f = (int32_t)((uint32_t)a.a + (uint32_t)a.b * (uint32_t)y);
        const uint64_t v = (uint64_t)((uint32_t)x) * (uint64_t)(uint32_t)f;  // both proven in [0, 2^31)
        if (CHECKED) return (x == INT64_MIN || y == INT64_MIN) ? 0ull : v;
        return v;
    };
    uint64_t* mytab = tab + threadIdx.x;
    auto fold = [&](int key, uint64_t v) {
        uint64_t* p = mytab + (size_t)key * FKP_NT;
        *p += v + ONE;
    };

    if (warp == FKP_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % FKP_STAGES);
                if (pf_dist > 0) {
                    const int64_t pt = tile + (int64_t)pf_dist * gridDim.x;
                    if (pt < ntiles) {
                        const int64_t q0 = pt * FKP_TILE;
                        prefetch_l2_bulk(a.fk + q0, FKP_TILE * 4);
                        prefetch_l2_bulk(a.kb + q0, FKP_TILE * 4);
                        prefetch_l2_bulk(a.x + q0, FKP_TILE * 8);
                        prefetch_l2_bulk(a.y + q0, FKP_TILE * 8);
                    }
                }
                if (it >= FKP_STAGES) mbar_wait(&empty[s], (uint32_t)(((it / FKP_STAGES) - 1) & 1));
                uint8_t* st = smem + (size_t)s * SB;
                const int64_t r0 = tile * FKP_TILE;
                mbar_expect_tx(&full[s], SB);
                tma_load_1d(st, a.fk + r0, FKP_TILE * 4, &full[s], pol);
                tma_load_1d(st + FKP_TILE * 4, a.kb + r0, FKP_TILE * 4, &full[s], pol);
                tma_load_1d(st + FKP_TILE * 8, a.x + r0, FKP_TILE * 8, &full[s], pol);
                tma_load_1d(st + FKP_TILE * 16, a.y + r0, FKP_TILE * 8, &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        // software pipeline: the gathers of tile i are issued before tile i-1
        // (whose gathers flew during the previous iteration) is folded
        // two tiles of gathers in flight: a tile's gathers are issued, then the
        // tile two iterations back is folded (its gathers have had two
        // iterations to return); pd/pkb/pv hold that oldest tile, qd/qkb/qv
        // the one in between
        int pd[FKP_RPT], pkb[FKP_RPT], qd[FKP_RPT], qkb[FKP_RPT];
        uint64_t pv[FKP_RPT], qv[FKP_RPT];
        int have = 0;
        // the RPT read-modify-writes of a batch are independent unless two rows
        // share a key: all loads issue first, a row whose key repeats an
        // earlier row's takes that row's updated value (register selects, no
        // shared-memory round trip), and the stores go out in row order so
        // the last one to an address carries the full sum
        auto drain = [&]() {
#pragma unroll
            for (int b0 = 0; b0 < FKP_RPT; b0 += BATCH) {
                int key[BATCH];
                uint64_t t[BATCH];
#pragma unroll
                for (int k = 0; k < BATCH; ++k) {
                    key[k] = keyof(pd[b0 + k], pkb[b0 + k]);
                    t[k] = mytab[(size_t)key[k] * FKP_NT];
                }
#pragma unroll
                for (int k = 0; k < BATCH; ++k) {
                    uint64_t b = t[k];
#pragma unroll
                    for (int j = 0; j < k; ++j) b = (key[j] == key[k]) ? t[j] : b;
                    t[k] = b + pv[b0 + k] + ONE;
                }
#pragma unroll
                for (int k = 0; k < BATCH; ++k) mytab[(size_t)key[k] * FKP_NT] = t[k];
            }
        };
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % FKP_STAGES);
            mbar_wait(&full[s], (uint32_t)((it / FKP_STAGES) & 1));
            const uint8_t* st = smem + (size_t)s * SB;
            int32_t f[FKP_RPT], kb[FKP_RPT];
            uint64_t v[FKP_RPT];
#pragma unroll
            for (int k = 0; k < FKP_RPT / 2; ++k) {
                const int r = 2 * threadIdx.x + k * 2 * FKP_NT;  // a row pair
                const int2 fk2 = *reinterpret_cast<const int2*>(st + (size_t)r * 4);
                const int2 kb2 = *reinterpret_cast<const int2*>(st + FKP_TILE * 4 + (size_t)r * 4);
                const longlong2 x2 = *reinterpret_cast<const longlong2*>(st + FKP_TILE * 8 + (size_t)r * 8);
                const longlong2 y2 = *reinterpret_cast<const longlong2*>(st + FKP_TILE * 16 + (size_t)r * 8);
                f[2 * k] = fk2.x; f[2 * k + 1] = fk2.y;
                kb[2 * k] = kb2.x; kb[2 * k + 1] = kb2.y;
                v[2 * k] = value(x2.x, y2.x);
                v[2 * k + 1] = value(x2.y, y2.y);
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
            int d[FKP_RPT];
#pragma unroll
            for (int k = 0; k < FKP_RPT; ++k) d[k] = gather(f[k]);
            if (have == 2) drain();
#pragma unroll
            for (int k = 0; k < FKP_RPT; ++k) {
                pd[k] = qd[k]; pkb[k] = qkb[k]; pv[k] = qv[k];
                qd[k] = d[k]; qkb[k] = kb[k]; qv[k] = v[k];
            }
            have = have < 2 ? have + 1 : 2;
        }
        if (have == 2) drain();
        if (have >= 1) {
#pragma unroll
            for (int k = 0; k < FKP_RPT; ++k) { pd[k] = qd[k]; pkb[k] = qkb[k]; pv[k] = qv[k]; }
            drain();
        }
        if (blockIdx.x == 0) {
            // ragged tail (< one tile): direct loads, always checked
            for (int64_t r = ntiles * FKP_TILE + threadIdx.x; r < a.n; r += FKP_NT) {
                const int32_t fk = a.fk[r], kbr = a.kb[r];
                const int64_t p = (int64_t)fk - a.bias;
                const int d = (fk != INT32_MIN && p >= 0 && p < a.dim_len) ? (int)a.dim[p] : 0x100;
                const int kbv = a.yfn ? (4 * (kbr + 365) + 3) / 1461 + 1969 : kbr;
                const int key = (d - a.subA) * a.mA + (kbv - a.subB) * a.mB;
                const bool ok = !(d == 0x100 || d == 0xFF || kbr == INT32_MIN || key < 0 || key >= a.ngroups);
                if (ok) {
                    const int64_t xr = a.x[r], yr = a.y[r];
                    const int32_t f = (int32_t)((uint32_t)a.a + (uint32_t)a.b * (uint32_t)yr);
                    const uint64_t v = (xr == INT64_MIN || yr == INT64_MIN)
                                           ? 0ull : (uint64_t)((uint32_t)xr) * (uint64_t)(uint32_t)f;
                    fold(key, v);
                }
            }
        }
    }
    __syncthreads();
    // CTA fold: per group, the 128 private slots -> (sum, count), int128 into
    // [ngroups][naggs+1] in the plan's layout
    const int NS = a.ngroups * (a.naggs + 1);
    for (int k = threadIdx.x; k < NS; k += FKP_THREADS) {
        const int g = k / (a.naggs + 1), ag = k % (a.naggs + 1);
        const bool cnt = (ag == a.naggs || ag == a.cnt_slot);
        const uint64_t* row = tab + (size_t)g * FKP_NT;
        uint64_t t = 0;
        for (int j = 0; j < FKP_NT; ++j) {
            const uint64_t w = row[(j + threadIdx.x) & (FKP_NT - 1)];  // rotated start: spread banks
            t += cnt ? (w >> 48) : (w & (ONE - 1));
        }
        put_i128(&parts[(size_t)blockIdx.x * NS + k], (i128)t);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, NS, out, FkI128Sum());
}

// ============================================================================
// Star-join scalar fragment (Q19 shape, C5): lineitem x part through a dense
// FK, a disjunction of conjunctions whose terms fall into fixed slots --
//   base  : two u8 set-membership slots (l_shipmode IN, l_shipinstruct IN),
//           one i64 range slot (l_quantity)
//   dim   : two u8 set-membership slots (p_brand, p_container), one i32
//           range slot (p_size), gathered through the FK
// -- and SUM(X * (a + b*Y)) + COUNT over two i64 base columns.  Only the
// filter columns stream through the TMA ring (fk, range column, two u8
// columns: 14 B/row); the union of every conjunction's base slots is tested
// first, the part row is gathered only for the survivors (late
// materialisation), and X / Y are loaded late (branching).
// ============================================================================
__device__ __forceinline__ void scalar2_finish(int64_t sum, int64_t cnt, Slot16* __restrict__ parts,
                                               unsigned int* __restrict__ done, Slot16* __restrict__ out,
                                               int naggs, int cnt_slot);
constexpr int ST_TILE = 4096;
constexpr int ST_MAXCONJ = VD_MAX_CONJ;

struct StarArgs {
    const int32_t* fk;
    const int64_t* rq;        // i64 range column (base)
    const uint8_t* u1;        // u8 columns (base)
    const uint8_t* u2;
    const int64_t* x;         // aggregate columns (late loads)
    const int64_t* y;
    const uint8_t* d1;        // u8 columns (dimension, gathered)
    const uint8_t* d2;
    const int32_t* dr;        // i32 range column (dimension, gathered)
    int64_t dim_len, bias;
    int32_t nconj;
    // lut[k][code]: bit c set <=> code passes conjunction c's terms on u8 slot k
    // (k = 0,1 base, 2,3 dimension); an epsilon code passes only a slot the
    // conjunction does not constrain (reading A9)
    uint8_t lut[4][256];
    int64_t rq_lo[ST_MAXCONJ], rq_hi[ST_MAXCONJ];
    int32_t dr_lo[ST_MAXCONJ], dr_hi[ST_MAXCONJ];
    int64_t a, b;
    int32_t nstages;
    int64_t n;
    int32_t sum_slot, cnt_slot, naggs;
};

template <bool NARROW>
__global__ void __launch_bounds__(FKG_THREADS, 1) k_pipe_star(const __grid_constant__ StarArgs a, int64_t ntiles,
                                                              Slot16* __restrict__ parts,
                                                              unsigned int* __restrict__ done,
                                                              Slot16* __restrict__ out) {
    extern __shared__ __align__(128) uint8_t smem[];
    constexpr int SB = ST_TILE * (4 + 8 + 1 + 1);
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)a.nstages * SB);
    uint64_t* empty = full + a.nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], FKG_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    __shared__ uint32_t s_lut[4][64];  // the four LUTs, byte-addressed
    for (int i = threadIdx.x; i < 256; i += blockDim.x)
        s_lut[i >> 6][i & 63] = reinterpret_cast<const uint32_t*>(&a.lut[0][0])[i];
    __syncthreads();
    const uint8_t* L = reinterpret_cast<const uint8_t*>(&s_lut[0][0]);
    int64_t sum = 0, cnt = 0;
    auto row = [&](int64_t r, int32_t fk, int64_t rq, uint32_t u1, uint32_t u2) {
        uint32_t m = L[u1] & L[256 + u2];
        if (!m) return;  // most rows stop here: two shared-memory byte lookups
#pragma unroll
        for (int c = 0; c < ST_MAXCONJ; ++c)
            if (!(rq >= a.rq_lo[c] && rq <= a.rq_hi[c])) m &= ~(1u << c);
        if (!m) return;
        const int64_t p = (int64_t)fk - a.bias;
        // late gather of the dimension row (only for base-qualified rows); a
        // position outside the dimension gathers epsilon (reading A9)
        uint32_t d1 = 0xFF, d2 = 0xFF;
        int32_t dr = INT32_MIN;
        if (fk != INT32_MIN && p >= 0 && p < a.dim_len) {
            d1 = __ldg(a.d1 + p);
            d2 = __ldg(a.d2 + p);
            dr = __ldg(a.dr + p);
        }
        m &= L[512 + d1] & L[768 + d2];
#pragma unroll
        for (int c = 0; c < ST_MAXCONJ; ++c)
            if (!(dr >= a.dr_lo[c] && dr <= a.dr_hi[c])) m &= ~(1u << c);
        if (!m) return;
        const int64_t x = __ldg(a.x + r), y = __ldg(a.y + r);  // late loads
        cnt += 1;
        if (x == INT64_MIN || y == INT64_MIN) return;  // epsilon factor: contributes nothing
        if (NARROW) sum += (int64_t)(int32_t)x * (int64_t)(int32_t)((uint32_t)a.a + (uint32_t)a.b * (uint32_t)y);
        else sum += x * (a.a + a.b * y);
    };
    if (warp == FKG_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % a.nstages);
                if (it >= a.nstages) mbar_wait(&empty[s], (uint32_t)(((it / a.nstages) - 1) & 1));
                uint8_t* st = smem + (size_t)s * SB;
                const int64_t r0 = tile * ST_TILE;
                mbar_expect_tx(&full[s], SB);
                tma_load_1d(st, a.fk + r0, ST_TILE * 4, &full[s], pol);
                tma_load_1d(st + ST_TILE * 4, a.rq + r0, ST_TILE * 8, &full[s], pol);
                tma_load_1d(st + ST_TILE * 12, a.u1 + r0, ST_TILE, &full[s], pol);
                tma_load_1d(st + ST_TILE * 13, a.u2 + r0, ST_TILE, &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % a.nstages);
            mbar_wait(&full[s], (uint32_t)((it / a.nstages) & 1));
            const uint8_t* st = smem + (size_t)s * SB;
            constexpr int RPT = ST_TILE / FKG_NT;
            int32_t f[RPT];
            int64_t q[RPT];
            uint32_t m1[RPT], m2[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) {
                const int r = threadIdx.x + k * FKG_NT;
                f[k] = reinterpret_cast<const int32_t*>(st)[r];
                q[k] = reinterpret_cast<const int64_t*>(st + ST_TILE * 4)[r];
                m1[k] = st[ST_TILE * 12 + r];
                m2[k] = st[ST_TILE * 13 + r];
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
#pragma unroll
            for (int k = 0; k < RPT; ++k) row(tile * ST_TILE + threadIdx.x + k * FKG_NT, f[k], q[k], m1[k], m2[k]);
        }
        if (blockIdx.x == 0)
            for (int64_t r = ntiles * ST_TILE + threadIdx.x; r < a.n; r += FKG_NT) row(r, a.fk[r], a.rq[r], a.u1[r], a.u2[r]);
    }
    scalar2_finish(sum, cnt, parts, done, out, a.naggs, a.cnt_slot);
}

// ============================================================================
// Selective FK join fragment (Fig 16; NEXT-1):
//   SUM(dim.v[fk - bias]) , COUNT(*)  WHERE lo <= fact.v <= hi
// in the three strategies of Fig 16: MODE 0 branching (gather only for
// qualifying rows), MODE 1 predicated aggregation (gather every row, x pred),
// MODE 2 predicated lookups (gather position (fk - bias) x pred: the
// non-qualifying rows all hit slot 0).  Each thread keeps FJ_R independent
// gathers in flight (memory-level parallelism for the random accesses); the
// sequential columns are read with streaming loads, coalesced per k.
// ============================================================================
constexpr int FJ_THREADS = 256;
constexpr int FJ_R = 8;

struct FkjsArgs {
    const int32_t* fk;
    const void* pv;   // predicate column (i32 / i64)
    const void* dim;  // gathered column (i32 / i64)
    int64_t n, dim_len, bias;
    int64_t lo, hi;   // inclusive predicate interval (lo > epsilon)
    int32_t naggs, sum_slot, cnt_slot;
};

// warp (int64, proven by the planner) -> CTA (int128) -> per-CTA partials ->
// the last CTA sums them in block order and writes the plan's slot layout
// (sum slot, count slot(s)); Fragment 2 of Fig 8 fused into the last CTA.
__device__ __forceinline__ void scalar2_finish(int64_t sum, int64_t cnt, Slot16* __restrict__ parts,
                                               unsigned int* __restrict__ done, Slot16* __restrict__ out,
                                               int naggs, int cnt_slot) {
    __shared__ i128 s_w[32][2];
    __shared__ bool s_last;
    __shared__ Slot16 s_raw2[2];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31, nw = blockDim.x >> 5;
    const int64_t ws_ = warp_sum_i64(sum), wc = warp_sum_i64(cnt);
    if (lane == 0) { s_w[warp][0] = ws_; s_w[warp][1] = wc; }
    __syncthreads();
    if (threadIdx.x < 2) {
        i128 t = 0;
        for (int w = 0; w < nw; ++w) t += s_w[w][threadIdx.x];
        put_i128(&parts[(size_t)blockIdx.x * 2 + threadIdx.x], t);
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, 2, s_raw2, FkI128Sum());
    __syncthreads();
    if (threadIdx.x <= naggs) {
        const int src = (threadIdx.x == naggs || threadIdx.x == cnt_slot) ? 1 : 0;
        out[threadIdx.x] = s_raw2[src];
    }
}

template <int MODE, typename PT, typename DT>
__global__ void __launch_bounds__(FJ_THREADS, 4) k_pipe_fkjs(const __grid_constant__ FkjsArgs a,
                                                             Slot16* __restrict__ parts,
                                                             unsigned int* __restrict__ done,
                                                             Slot16* __restrict__ out) {
    const PT* __restrict__ pv = static_cast<const PT*>(a.pv);
    const DT* __restrict__ dim = static_cast<const DT*>(a.dim);
    const int64_t nthr = (int64_t)gridDim.x * FJ_THREADS;
    const int64_t tid = (int64_t)blockIdx.x * FJ_THREADS + threadIdx.x;
    int64_t sum = 0, cnt = 0;
    // warp-uniform trip count (the __syncwarp below): lanes past n run with in = false
    for (int64_t base = tid; base - (threadIdx.x & 31) < a.n; base += nthr * FJ_R) {
        int64_t p[FJ_R];
        bool q[FJ_R], ok[FJ_R];
#pragma unroll
        for (int k = 0; k < FJ_R; ++k) {
            const int64_t r = base + k * nthr;
            const bool in = r < a.n;
            const int32_t f = in ? __ldcs(a.fk + r) : INT32_MIN;
            const int64_t x = in ? (int64_t)__ldcs(pv + r) : (int64_t)Eps<PT>::value();
            q[k] = in && x >= a.lo && x <= a.hi;
            p[k] = (int64_t)f - a.bias;
            ok[k] = f != INT32_MIN && p[k] >= 0 && p[k] < a.dim_len;  // else the gather gives epsilon
            if (MODE == 2 && !q[k]) { p[k] = 0; ok[k] = a.dim_len > 0; }
        }
        DT g[FJ_R];
        {
            static_assert(FJ_R == 8, "one block of eight gathers");
            const DT* ptr[8];
            bool load[8];
#pragma unroll
            for (int k = 0; k < 8; ++k) {
                load[k] = MODE == 0 ? (q[k] && ok[k]) : ok[k];
                ptr[k] = dim + (load[k] ? p[k] : 0);
            }
            gather8(ptr, load, Eps<DT>::value(), g);
        }
        __syncwarp();  // all eight gathers issued before the first use
#pragma unroll
        for (int k = 0; k < FJ_R; ++k) {
            const int64_t v = Eps<DT>::is(g[k]) ? 0 : (int64_t)g[k];  // an epsilon input adds nothing (A5)
            if (MODE == 0) {
                if (q[k]) { sum += v; cnt += 1; }
            } else {
                const int64_t pm = q[k] ? 1 : 0;
                sum += v * pm;
                cnt += pm;
            }
        }
    }
    scalar2_finish(sum, cnt, parts, done, out, a.naggs, a.cnt_slot);
}

// TMA variant of the Fig 16 fragment: fk and the predicate column stream
// through a bulk-copy ring (producer warp), FJT_CW consumer warps evaluate
// the predicate from shared memory and keep RPT gathers in flight per thread.
constexpr int FJT_CW = 16;  // consumer warps
constexpr int FJT_NT = FJT_CW * 32;
constexpr int FJT_THREADS = FJT_NT + 32;
constexpr int FJT_TILE = FJT_NT * 16;  // 16 gathers in flight per thread

template <int MODE, typename PT, typename DT>
__global__ void __launch_bounds__(FJT_THREADS, 1) k_pipe_fkjs_tma(const __grid_constant__ FkjsArgs a, int nstages,
                                                                  int64_t ntiles, Slot16* __restrict__ parts,
                                                                  unsigned int* __restrict__ done,
                                                                  Slot16* __restrict__ out) {
    extern __shared__ __align__(128) uint8_t smem[];
    constexpr int SB = FJT_TILE * (4 + (int)sizeof(PT));
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)nstages * SB);
    uint64_t* empty = full + nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const PT* __restrict__ pv = static_cast<const PT*>(a.pv);
    const DT* __restrict__ dim = static_cast<const DT*>(a.dim);
    if (threadIdx.x == 0) {
        for (int s = 0; s < nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], FJT_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    int64_t sum = 0, cnt = 0;
    constexpr int RPT = FJT_TILE / FJT_NT;
    // RPT rows of one thread: predicate, then all gathers, then the fold
    auto rows = [&](const int32_t* f, const int64_t* x, const bool* in) {
        int64_t p[RPT];
        bool q[RPT], ok[RPT];
#pragma unroll
        for (int k = 0; k < RPT; ++k) {
            q[k] = in[k] && x[k] >= a.lo && x[k] <= a.hi;
            p[k] = (int64_t)f[k] - a.bias;
            ok[k] = f[k] != INT32_MIN && p[k] >= 0 && p[k] < a.dim_len;
            if (MODE == 2 && !q[k]) { p[k] = 0; ok[k] = a.dim_len > 0; }
        }
        if (MODE == 0) {
            bool any = false;
#pragma unroll
            for (int k = 0; k < RPT; ++k) any |= q[k];
            if (!__any_sync(VD_FULL, any)) return;  // no qualifying row in the warp: no gather, nothing to fold
        }
        DT g[RPT];
        static_assert(RPT % 8 == 0, "gathers are issued in blocks of eight");
#pragma unroll
        for (int k0 = 0; k0 < RPT; k0 += 8) {
            const DT* ptr[8];
            bool load[8];
#pragma unroll
            for (int k = 0; k < 8; ++k) {
                load[k] = MODE == 0 ? (q[k0 + k] && ok[k0 + k]) : (in[k0 + k] && ok[k0 + k]);
                ptr[k] = dim + (load[k] ? p[k0 + k] : 0);
            }
            gather8(ptr, load, Eps<DT>::value(), g + k0);
        }
        __syncwarp();  // loads cannot sink past this point: all RPT are issued before the first use
#pragma unroll
        for (int k = 0; k < RPT; ++k) {
            const int64_t v = Eps<DT>::is(g[k]) ? 0 : (int64_t)g[k];
            if (MODE == 0) {
                if (q[k]) { sum += v; cnt += 1; }
            } else {
                const int64_t pm = q[k] ? 1 : 0;
                sum += v * pm;
                cnt += pm;
            }
        }
    };
    if (warp == FJT_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                const int s = (int)(it % nstages);
                if (it >= nstages) mbar_wait(&empty[s], (uint32_t)(((it / nstages) - 1) & 1));
                uint8_t* st = smem + (size_t)s * SB;
                const int64_t r0 = tile * FJT_TILE;
                mbar_expect_tx(&full[s], SB);
                tma_load_1d(st, a.fk + r0, FJT_TILE * 4, &full[s], pol);
                tma_load_1d(st + FJT_TILE * 4, pv + r0, FJT_TILE * (int)sizeof(PT), &full[s], pol);
            }
        }
        __syncwarp();
    } else {
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            const int s = (int)(it % nstages);
            mbar_wait(&full[s], (uint32_t)((it / nstages) & 1));
            const uint8_t* st = smem + (size_t)s * SB;
            int32_t f[RPT];
            int64_t x[RPT];
            bool in[RPT];
#pragma unroll
            for (int k = 0; k < RPT; ++k) {
                const int r = threadIdx.x + k * FJT_NT;
                f[k] = reinterpret_cast<const int32_t*>(st)[r];
                const PT xv = reinterpret_cast<const PT*>(st + FJT_TILE * 4)[r];
                x[k] = Eps<PT>::is(xv) ? INT64_MIN : (int64_t)xv;  // lo > INT64_MIN: epsilon never qualifies
                in[k] = true;
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
            rows(f, x, in);
        }
        if (blockIdx.x == 0) {  // ragged tail (< one tile)
            for (int64_t base = ntiles * FJT_TILE + threadIdx.x; base - lane < a.n; base += (int64_t)FJT_NT * RPT) {
                int32_t f[RPT];
                int64_t x[RPT];
                bool in[RPT];
#pragma unroll
                for (int k = 0; k < RPT; ++k) {
                    const int64_t r = base + (int64_t)k * FJT_NT;
                    in[k] = r < a.n;
                    f[k] = in[k] ? a.fk[r] : INT32_MIN;
                    const PT xv = in[k] ? pv[r] : Eps<PT>::value();
                    x[k] = Eps<PT>::is(xv) ? INT64_MIN : (int64_t)xv;
                }
                rows(f, x, in);
            }
        }
    }
    __syncthreads();
    scalar2_finish(sum, cnt, parts, done, out, a.naggs, a.cnt_slot);
}

// ============================================================================
// Host planner
// ============================================================================
struct Bound {
    bool known;
    double lo, hi;  // value bounds (doubles: only used for overflow proofs)
};

static Bound col_bound(const vd_pipeline* p, const vd_column* cols, int ncols, const vd_column* dims, int c) {
    const vd_column* col = nullptr;
    if (c < ncols) col = &cols[c];
    else col = &dims[p->gathers[c - ncols].dim_col];
    Bound b;
    b.known = col->has_minmax && col->dtype != VD_F32 && col->dtype != VD_F64;
    b.lo = (double)col->min;
    b.hi = (double)col->max;
    return b;
}

static double factor_absmax(const vd_factor& f, const Bound& b) {
    if (f.col < 0) return std::fabs((double)f.a);
    double x1 = (double)f.a + (double)f.b * b.lo, x2 = (double)f.a + (double)f.b * b.hi;
    return std::max(std::fabs(x1), std::fabs(x2));
}

static int col_dtype(const vd_pipeline* p, const vd_column* cols, int ncols, const vd_column* dims, int c) {
    if (c < ncols) return cols[c].dtype;
    return dims[p->gathers[c - ncols].dim_col].dtype;
}

// Fold the conjunction's integer terms on column c into [lo, hi]; false if a
// term is not an interval (NE / IN) or a float.
static bool term_interval(const vd_term& t, int64_t* lo, int64_t* hi) {
    switch (t.cmp) {
    case VD_CMP_GT: if (t.ival == INT64_MAX) return false; *lo = std::max(*lo, t.ival + 1); return true;
    case VD_CMP_GE: *lo = std::max(*lo, t.ival); return true;
    case VD_CMP_LT: if (t.ival == INT64_MIN) return false; *hi = std::min(*hi, t.ival - 1); return true;
    case VD_CMP_LE: *hi = std::min(*hi, t.ival); return true;
    case VD_CMP_EQ: *lo = std::max(*lo, t.ival); *hi = std::min(*hi, t.ival); return true;
    default: return false;
    }
}

static int grid_persistent(int per_sm) { return num_sms() * per_sm; }

// ---- Q1 matching ---------------------------------------------------------
static bool plain_col(const vd_factor& f) { return f.col >= 0 && f.a == 0 && f.b == 1; }

// Rows one warp of the Q1 fragment folds into its int64 accumulators (the
// bound the overflow proof needs), for the launch shape that runs:
//   TMA: `grid` CTAs x Q1T_CW consumer warps; tile t goes to CTA t % grid and
//        each warp takes 128 rows of it; CTA 0 also folds the ragged tail
//        (< Q1T_TILE rows over Q1T_NT threads: <= 4 rows per thread);
//   LDG: `grid` x Q1_THREADS threads striding over quads (4 rows); thread 0
//        also folds the n % 4 tail rows.
static double q1_rows_per_warp(bool tma, int64_t n, int grid) {
    if (tma) {
        const int64_t ntiles = n / Q1T_TILE;
        const int64_t tiles_per_cta = (ntiles + grid - 1) / grid;
        return (double)tiles_per_cta * 128.0 + 32.0 * 4.0;
    }
    const int64_t threads = (int64_t)grid * Q1_THREADS;
    const int64_t nquads = n / 4;
    return ((double)((nquads + threads - 1) / threads) * 4.0) * 32.0 + 3.0;
}

template <bool NARROW, bool EPS>
static cudaError_t launch_q1(int G, bool use_tma, const Q1Args& qa, int64_t ntiles, int tgrid, int grid,
                             Slot16* parts, unsigned* dn, Slot16* out, const Q1Map& map, cudaStream_t s) {
#define Q1_LAUNCH(GG)                                                                                         \
    if (use_tma) {                                                                                            \
        cudaFuncSetAttribute(k_pipe_q1_tma<GG, NARROW, EPS>, cudaFuncAttributeMaxDynamicSharedMemorySize,      \
                             (int)q1t_smem(GG));                                                              \
        k_pipe_q1_tma<GG, NARROW, EPS><<<tgrid, Q1T_THREADS, q1t_smem(GG), s>>>(qa, ntiles, parts, dn, out, map); \
    } else {                                                                                                  \
        k_pipe_q1<GG, NARROW, EPS><<<grid, Q1_THREADS, 0, s>>>(qa, parts, dn, out, map);                       \
    }
    if (G == 4) { Q1_LAUNCH(4) } else if (G == 6) { Q1_LAUNCH(6) } else { Q1_LAUNCH(8) }
#undef Q1_LAUNCH
    return cudaGetLastError();
}

static vd_status try_q1(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, void* out, void* ws,
                        cudaStream_t s, int* nl, bool* done) {
    *done = false;
    if (p->ngathers != 0 || p->nkeyparts != 2 || p->ngroups > 8 || p->ngroups < 1) return VD_OK;
    for (int k = 0; k < 2; ++k) {
        const vd_keypart& kp = p->key[k];
        if (kp.col >= ncols || kp.fn != 0 || cols[kp.col].dtype != VD_U8) return VD_OK;
        if (kp.mult < -1000 || kp.mult > 1000 || kp.sub < -1000 || kp.sub > 1000) return VD_OK;
        if (!cols[kp.col].has_minmax) return VD_OK;
    }
    // key domain proof from metadata (ctrl/data bit conflict check)
    {
        double klo = 0, khi = 0;
        for (int k = 0; k < 2; ++k) {
            const vd_keypart& kp = p->key[k];
            double a = ((double)cols[kp.col].min - kp.sub) * kp.mult, b = ((double)cols[kp.col].max - kp.sub) * kp.mult;
            klo += std::min(a, b);
            khi += std::max(a, b);
        }
        if (klo < 0 || khi >= (double)p->ngroups) return VD_OK;  // generic path counts violations
    }
    // predicate: one conjunction over a single i32 column, intervals only
    int dcol = -1;
    int64_t lo = INT32_MIN, hi = INT32_MAX;
    if (p->pred.nconj > 1) return VD_OK;
    if (p->pred.nconj == 1) {
        for (int k = 0; k < p->pred.conj[0].nterms; ++k) {
            const vd_term& t = p->pred.conj[0].terms[k];
            if (t.col >= ncols || cols[t.col].dtype != VD_I32) return VD_OK;
            if (dcol >= 0 && t.col != dcol) return VD_OK;
            dcol = t.col;
            if (!term_interval(t, &lo, &hi)) return VD_OK;
        }
    }
    if (dcol < 0) return VD_OK;  // need a predicate column for this fragment
    // INT32_MIN is epsilon: a term over epsilon is false (A9), so the
    // interval never includes it (a one-sided `<=` filter would otherwise)
    lo = std::max<int64_t>(lo, (int64_t)INT32_MIN + 1);
    hi = std::min<int64_t>(hi, INT32_MAX);
    // aggregates -> raw slots; roles V0..V3
    int V[4] = {-1, -1, -1, -1};
    int64_t a1 = 0, b1 = 0, a2 = 0, b2 = 0;
    bool have_lin1 = false, have_lin2 = false;
    Q1Map map;
    map.naggs = p->naggs;
    map.ngroups = (int32_t)p->ngroups;
    auto setrole = [&](int r, int c) {
        if (V[r] >= 0 && V[r] != c) return false;
        V[r] = c;
        return true;
    };
    // first pass: the product aggregates fix V1, V2, V3
    for (int k = 0; k < p->naggs; ++k) {
        const vd_agg& g = p->aggs[k];
        if (g.kind == VD_AGG_COUNT) { map.src[k] = 5; continue; }
        if (g.kind != VD_AGG_SUM) return VD_OK;
        if (g.nfactors < 1 || g.nfactors > 3 || !plain_col(g.f[0])) return VD_OK;
        for (int f = 0; f < g.nfactors; ++f) {
            if (g.f[f].col < 0 || g.f[f].col >= ncols || cols[g.f[f].col].dtype != VD_I64) return VD_OK;
        }
        if (g.nfactors >= 2) {
            if (!setrole(1, g.f[0].col) || !setrole(2, g.f[1].col)) return VD_OK;
            if (have_lin1 && (a1 != g.f[1].a || b1 != g.f[1].b)) return VD_OK;
            a1 = g.f[1].a; b1 = g.f[1].b; have_lin1 = true;
            if (g.nfactors == 3) {
                if (!setrole(3, g.f[2].col)) return VD_OK;
                if (have_lin2 && (a2 != g.f[2].a || b2 != g.f[2].b)) return VD_OK;
                a2 = g.f[2].a; b2 = g.f[2].b; have_lin2 = true;
                map.src[k] = 3;
            } else {
                map.src[k] = 2;
            }
        }
    }
    // second pass: single-column sums take V1 / V2 / V0
    for (int k = 0; k < p->naggs; ++k) {
        const vd_agg& g = p->aggs[k];
        if (g.kind != VD_AGG_SUM || g.nfactors != 1) continue;
        int c = g.f[0].col;
        if (V[1] == c) map.src[k] = 1;
        else if (V[2] == c) map.src[k] = 4;
        else if (V[0] < 0 || V[0] == c) { V[0] = c; map.src[k] = 0; }
        else if (V[1] < 0) { V[1] = c; map.src[k] = 1; }
        else if (V[2] < 0) { V[2] = c; map.src[k] = 4; }
        else return VD_OK;
    }
    // unused roles read some valid column (cheap, keeps one code path)
    int anycol = -1;
    for (int r = 0; r < 4; ++r) if (V[r] >= 0) anycol = V[r];
    if (anycol < 0) anycol = -2;
    // launch shape: the TMA variant (num_sms() CTAs x Q1T_NT consumer
    // threads, 1D bulk copies need every column 16-byte aligned) or the LDG
    // variant (grid_persistent(2) x Q1_THREADS, 4-row vector loads)
    auto al = [](const void* q, size_t a) { return ((uintptr_t)q % a) == 0; };
    const char* var = getenv("VD_Q1_VARIANT");
    const bool al_all = al(cols[dcol].data, 16) && al(cols[p->key[0].col].data, 16) &&
                        al(cols[p->key[1].col].data, 16);
    const bool use_tma = al_all && !(var && strcmp(var, "ldg") == 0);
    const int64_t ntiles = n / Q1T_TILE;
    const int tgrid = num_sms();
    const int grid = grid_persistent(2);
    // overflow proof: each thread folds its rows into int64 slots and the warp
    // sums them in int64 (then int128 above), so the bound is rows per WARP of
    // the variant that launches
    const double rows_per_warp = q1_rows_per_warp(use_tma, n, use_tma ? tgrid : grid);
    Bound bv[4];
    for (int r = 0; r < 4; ++r) {
        int c = V[r] >= 0 ? V[r] : (anycol >= 0 ? anycol : -1);
        if (c < 0) { bv[r].known = true; bv[r].lo = bv[r].hi = 0; continue; }
        bv[r] = col_bound(p, cols, ncols, nullptr, c);
        if (!bv[r].known) return VD_OK;
    }
    auto amax = [](const Bound& b) { return std::max(std::fabs(b.lo), std::fabs(b.hi)); };
    double f1 = std::max(std::fabs((double)a1 + (double)b1 * bv[2].lo), std::fabs((double)a1 + (double)b1 * bv[2].hi));
    double f2 = std::max(std::fabs((double)a2 + (double)b2 * bv[3].lo), std::fabs((double)a2 + (double)b2 * bv[3].hi));
    double dpmax = amax(bv[1]) * f1, chmax = dpmax * f2;
    const double LIM = 9.0e18;
    if (rows_per_warp * std::max({amax(bv[0]), amax(bv[1]), dpmax, chmax}) >= LIM) return VD_OK;
    if (amax(bv[2]) * rows_per_warp >= (double)(1ll << Q1_CSHIFT) || bv[2].lo < 0) return VD_OK;
    if (rows_per_warp >= (double)(1ll << (63 - Q1_CSHIFT))) return VD_OK;
    auto fits32 = [](int64_t x) { return x > INT32_MIN && x < INT32_MAX; };
    bool narrow = amax(bv[1]) < 2147483647.0 && f1 < 2147483647.0 && dpmax < 2147483647.0 && f2 < 2147483647.0 &&
                  amax(bv[2]) < 2147483647.0 && amax(bv[3]) < 2147483647.0 && fits32(a1) && fits32(b1) &&
                  fits32(a2) && fits32(b2);
    // alignment for the vector loads
    if (!al(cols[dcol].data, 16) || !al(cols[p->key[0].col].data, 4) || !al(cols[p->key[1].col].data, 4)) return VD_OK;
    // per-row epsilon checks unless the metadata rules epsilon out of every
    // referenced column (VD_COL_NOEPS)
    bool eps = !(cols[dcol].flags & VD_COL_NOEPS) || !(cols[p->key[0].col].flags & VD_COL_NOEPS) ||
               !(cols[p->key[1].col].flags & VD_COL_NOEPS);
    for (int r = 0; r < 4; ++r)
        if (V[r] >= 0 && !(cols[V[r]].flags & VD_COL_NOEPS)) eps = true;
    Q1Args qa;
    qa.d = (const int32_t*)cols[dcol].data;
    qa.dlo = (int32_t)lo;
    qa.dhi = (int32_t)hi;
    qa.k1 = (const uint8_t*)cols[p->key[0].col].data;
    qa.k2 = (const uint8_t*)cols[p->key[1].col].data;
    qa.m1 = (int32_t)p->key[0].mult;
    qa.m2 = (int32_t)p->key[1].mult;
    qa.koff = (int32_t)(-p->key[0].sub * p->key[0].mult - p->key[1].sub * p->key[1].mult);
    for (int r = 0; r < 4; ++r) {
        int c = V[r] >= 0 ? V[r] : anycol;
        if (c < 0) return VD_OK;
        qa.v[r] = (const int64_t*)cols[c].data;
        if (!al(qa.v[r], 16)) return VD_OK;
    }
    qa.a1 = a1; qa.b1 = b1; qa.a2 = a2; qa.b2 = b2;
    qa.nquads = n / 4;
    qa.n = n;
    // workspace: [done (256B)] [parts grid*G*6*16] [raw G*6*16]
    int G = p->ngroups <= 4 ? 4 : (p->ngroups <= 6 ? 6 : 8);
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    Slot16* raw = parts + (size_t)grid * G * 6;
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    if (narrow) {
        if (eps) e = launch_q1<true, true>(G, use_tma, qa, ntiles, tgrid, grid, parts, dn, (Slot16*)out, map, s);
        else e = launch_q1<true, false>(G, use_tma, qa, ntiles, tgrid, grid, parts, dn, (Slot16*)out, map, s);
    } else {
        if (eps) e = launch_q1<false, true>(G, use_tma, qa, ntiles, tgrid, grid, parts, dn, (Slot16*)out, map, s);
        else e = launch_q1<false, false>(G, use_tma, qa, ntiles, tgrid, grid, parts, dn, (Slot16*)out, map, s);
    }
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    set_fragment(use_tma ? "q1_tma" : "q1_ldg");
    *nl += 1;
    (void)raw;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    *done = true;
    return VD_OK;
}

// ---- scalar matching ----------------------------------------------------------
// ---- selective sum over one f32 column, TMA-staged (Fig 15 / C1) -------------
// select v in [lo, hi] (inclusive f32 bounds; every single-term comparison on
// an f32 value is such an interval: x > c <=> x >= succ(floor32(c))), fold
// the selected values in f64 and count them.  4 rows per LDS.128.
constexpr int SS_TILE = 8192;
constexpr int SS_MAXSTAGES = 6;
// 16 consumer warps (4 per scheduler): with 8 the per-tile instruction
// stream of each warp was exposed (issue active 44%, 5.96 TB/s)
constexpr int SS_CW = 16;
constexpr int SS_NT = SS_CW * 32;
constexpr int SS_THREADS = SS_NT + 32;

struct SelSumArgs {
    const float* v;  // filter column
    const float* w;  // value column (TWO), else the filter column itself
    float lo, hi;
    int64_t n;
    int32_t nstages;
};

// TWO: Fig 15's "select sum(v2) ... where v1 between": the value
// column is a second f32 column staged beside the filter column (both
// tiles in one stage); a NaN (epsilon) value is skipped by the fold while
// its row counts (A5), with EPS set when the value column may hold one.
template <int MODE, bool TWO = false, bool EPS = false>
__global__ void __launch_bounds__(SS_THREADS, 1) k_pipe_selsum_tma(const __grid_constant__ SelSumArgs a,
                                                                    int64_t ntiles, Slot16* __restrict__ parts,
                                                                    unsigned int* __restrict__ done,
                                                                    Slot16* __restrict__ out, const ScalarMap map) {
    extern __shared__ __align__(128) uint8_t smem[];
    __shared__ Slot16 s_raw2[2];
    constexpr int SB = (TWO ? 2 : 1) * SS_TILE * 4;  // stage bytes
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)a.nstages * SB);
    uint64_t* empty = full + a.nstages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], SS_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    double sum = 0;
    int64_t cnt = 0;
    auto row2 = [&](float x, float y) {
        const bool p = x >= a.lo && x <= a.hi;  // NaN (epsilon) fails both
        const double v = (EPS && y != y) ? 0.0 : (double)y;
        if (MODE == 1) {
            sum += p ? v : 0.0;
            cnt += p;
        } else if (p) {
            sum += v;
            cnt += 1;
        }
    };
    auto row = [&](float x) { row2(x, x); };
    if (warp == SS_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int s = 0;
            uint32_t ph = 0;  // parity of the current pass over the ring
            for (int64_t it = 0;; ++it) {
                const int64_t tile = blockIdx.x + it * gridDim.x;
                if (tile >= ntiles) break;
                if (it >= a.nstages) mbar_wait(&empty[s], ph ^ 1u);
                mbar_expect_tx(&full[s], SB);
                tma_load_1d(smem + (size_t)s * SB, a.v + tile * SS_TILE, SS_TILE * 4, &full[s], pol);
                if (TWO)
                    tma_load_1d(smem + (size_t)s * SB + SS_TILE * 4, a.w + tile * SS_TILE, SS_TILE * 4, &full[s], pol);
                if (++s == a.nstages) { s = 0; ph ^= 1u; }
            }
        }
        __syncwarp();
    } else {
        int s = 0;
        uint32_t ph = 0;
        for (int64_t it = 0;; ++it) {
            const int64_t tile = blockIdx.x + it * gridDim.x;
            if (tile >= ntiles) break;
            mbar_wait(&full[s], ph);
            const float4* st = reinterpret_cast<const float4*>(smem + (size_t)s * SB);
            constexpr int K = SS_TILE / 4 / SS_NT;
            float4 x[K], y[K];
#pragma unroll
            for (int k = 0; k < K; ++k) {
                x[k] = st[threadIdx.x + k * SS_NT];
                y[k] = TWO ? st[SS_TILE / 4 + threadIdx.x + k * SS_NT] : x[k];
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
            if (++s == a.nstages) { s = 0; ph ^= 1u; }
#pragma unroll
            for (int k = 0; k < K; ++k) {
                row2(x[k].x, y[k].x);
                row2(x[k].y, y[k].y);
                row2(x[k].z, y[k].z);
                row2(x[k].w, y[k].w);
            }
        }
        if (blockIdx.x == 0)
            for (int64_t r = ntiles * SS_TILE + threadIdx.x; r < a.n; r += SS_NT) row2(a.v[r], TWO ? a.w[r] : a.v[r]);
        (void)row;
    }
    __shared__ Slot16 s_w[SS_THREADS / 32][2];
    const int64_t c = warp_sum_i64(cnt);
    const double sm = warp_sum_f64(sum);
    if (lane == 0) {
        put_f64(&s_w[warp][0], sm);
        put_i128(&s_w[warp][1], (i128)c);
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        double t = 0;
        i128 k = 0;
        for (int w = 0; w < SS_THREADS / 32; ++w) { t += get_f64(s_w[w][0]); k += get_i128(s_w[w][1]); }
        put_f64(&parts[(size_t)blockIdx.x * 2], t);
        put_i128(&parts[(size_t)blockIdx.x * 2 + 1], k);
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, 2, s_raw2, [](int k) { return k == 0 ? (int)FK_F64_SUM : (int)FK_I128_SUM; });
    __syncthreads();
    if (threadIdx.x <= map.naggs) out[threadIdx.x] = s_raw2[(threadIdx.x == map.naggs) ? 1 : map.src[threadIdx.x]];
}

// Inclusive f32 interval [lo, hi] equal to <= 2 comparison terms on an f32
// column: for f32 x and a double constant c, x > c <=> x >= succ(floor32(c)),
// x >= c <=> x >= ceil32(c), x < c <=> x <= pred(ceil32(c)),
// x <= c <=> x <= floor32(c).  NaN (epsilon) fails both comparisons.
static float floor32(double c) {
    float f = (float)c;
    if ((double)f > c) f = nextafterf(f, -INFINITY);
    return f;
}
static float ceil32(double c) {
    float f = (float)c;
    if ((double)f < c) f = nextafterf(f, INFINITY);
    return f;
}
static bool f32_interval(const int32_t fcmp[2], const double fc[2], float* lo, float* hi) {
    float l = -INFINITY, h = INFINITY;
    for (int k = 0; k < 2; ++k) {
        if (fcmp[k] < 0) continue;
        const double c = fc[k];
        switch (fcmp[k]) {
        case VD_CMP_GT: l = fmaxf(l, nextafterf(floor32(c), INFINITY)); break;
        case VD_CMP_GE: l = fmaxf(l, ceil32(c)); break;
        case VD_CMP_LT: h = fminf(h, nextafterf(ceil32(c), -INFINITY)); break;
        case VD_CMP_LE: h = fminf(h, floor32(c)); break;
        case VD_CMP_EQ:
            if ((double)(float)c != c) { l = 1; h = 0; break; }  // no f32 equals c
            l = fmaxf(l, (float)c);
            h = fminf(h, (float)c);
            break;
        default: return false;
        }
    }
    *lo = l;
    *hi = h;
    return true;
}

// Stage layout for the TMA scalar fragment: distinct columns of the 5 roles.
static bool scalar_tma_args(const void* const role_ptr[5], const int role_esz[5], bool present[5], int tile,
                            ScalarTmaArgs* t) {
    t->ncol = 0;
    int off = 0;
    for (int r = 0; r < 5; ++r) {
        t->role[r] = 0;
        if (!present[r]) continue;
        int found = -1;
        for (int c = 0; c < t->ncol; ++c)
            if (t->col[c] == role_ptr[r]) found = c;
        if (found < 0) {
            if (((uintptr_t)role_ptr[r] % 16) != 0) return false;
            found = t->ncol++;
            t->col[found] = role_ptr[r];
            t->esz[found] = role_esz[r];
            t->soff[found] = off;
            off += tile * role_esz[r];
        }
        t->role[r] = found;
    }
    t->stage_bytes = off;
    int ns = (int)((180 * 1024) / (off > 0 ? off : 1));
    t->nstages = ns < 2 ? 2 : (ns > SCT_MAXSTAGES ? SCT_MAXSTAGES : ns);
    return (size_t)off * t->nstages + 2 * t->nstages * 8 <= 220 * 1024;
}

template <int MODE, bool EPS, int NF, bool HVB, int TILE, typename F0, typename F1, typename F2, typename VA,
          typename VB>
static cudaError_t launch_scalar_tma(const ScalarTmaArgs& ta, void* ws, Slot16* out, const ScalarMap& m,
                                     cudaStream_t s, int* nl) {
    int grid = num_sms();
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    Slot16* raw = parts + (size_t)grid * 2;
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) return e;
    size_t smem = (size_t)ta.stage_bytes * ta.nstages + 2 * ta.nstages * 8;
    auto kern = k_pipe_scalar_tma<MODE, EPS, NF, HVB, TILE, F0, F1, F2, VA, VB>;
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    kern<<<grid, SCT_THREADS, smem, s>>>(ta, ta.n / TILE, parts, dn, out, m);
    (void)raw;
    *nl += 1;
    return cudaGetLastError();
}

template <int MODE, bool EPS, bool HF1, bool HF2, bool HVB, typename F0, typename F1, typename F2, typename VA,
          typename VB>
static cudaError_t launch_scalar(const ScalarArgs<F0, F1, F2, VA, VB>& sa, void* ws, Slot16* out, const ScalarMap& m,
                                 cudaStream_t s, int* nl) {
    int grid = grid_persistent(4);
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    Slot16* raw = parts + (size_t)grid * 2;
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) return e;
    k_pipe_scalar<MODE, EPS, HF1, HF2, HVB, F0, F1, F2, VA, VB><<<grid, SC_THREADS, 0, s>>>(sa, parts, dn, out, m);
    (void)raw;
    *nl += 1;
    return cudaGetLastError();
}

// Rows one consumer thread of the scalar fragment folds into its int64 sum,
// the larger over the two launch shapes:
//   TMA: num_sms() CTAs x SCT_NT consumer threads, TILE/SCT_NT rows of each
//        of the CTA's tiles (tile t -> CTA t % grid), + the ragged tail on
//        CTA 0 (< TILE rows: <= TILE/SCT_NT per thread); TILE = 2048 (the
//        i64 value shape);
//   LDG: grid_persistent(4) x SC_THREADS threads striding over quads, + the
//        n % 4 tail on thread 0.
static double scalar_rows_per_thread(int64_t n) {
    const int64_t TILE = 2048, grid = num_sms();
    const int64_t ntiles = n / TILE;
    const double tma = (double)((ntiles + grid - 1) / grid) * (double)(TILE / SCT_NT) + (double)(TILE / SCT_NT);
    const int64_t threads = (int64_t)grid_persistent(4) * SC_THREADS, nq = n / 4;
    const double ldg = (double)((nq + threads - 1) / threads) * 4.0 + 3.0;
    return std::max(tma, ldg);
}

static vd_status try_scalar(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, void* out, void* ws,
                            cudaStream_t s, int* nl, bool* done) {
    *done = false;
    if (p->ngathers != 0 || p->nkeyparts != 0 || p->ngroups != 1) return VD_OK;
    if (p->pred.nconj != 1) return VD_OK;
    // filter columns in order of first appearance
    int fcol[3] = {-1, -1, -1};
    int nf = 0;
    int64_t lo[3] = {INT64_MIN, INT64_MIN, INT64_MIN}, hi[3] = {INT64_MAX, INT64_MAX, INT64_MAX};
    int32_t fcmp[2] = {-1, -1};
    double fc[2] = {0, 0};
    int nfl = 0;
    for (int k = 0; k < p->pred.conj[0].nterms; ++k) {
        const vd_term& t = p->pred.conj[0].terms[k];
        if (t.col >= ncols) return VD_OK;
        int slot = -1;
        for (int j = 0; j < nf; ++j) if (fcol[j] == t.col) slot = j;
        if (slot < 0) {
            if (nf == 3) return VD_OK;
            slot = nf;
            fcol[nf++] = t.col;
        }
        int dt = cols[t.col].dtype;
        if (dt == VD_F32 || dt == VD_F64) {
            if (slot != 0 || nfl == 2 || t.cmp == VD_CMP_IN) return VD_OK;
            fcmp[nfl] = t.cmp;
            fc[nfl] = t.fval;
            ++nfl;
        } else if (!term_interval(t, &lo[slot], &hi[slot])) {
            return VD_OK;
        }
    }
    // aggregates: one SUM of 1-2 plain columns, and/or COUNT
    int va = -1, vb = -1;
    ScalarMap m;
    m.naggs = p->naggs;
    for (int k = 0; k < p->naggs; ++k) {
        const vd_agg& g = p->aggs[k];
        if (g.kind == VD_AGG_COUNT) { m.src[k] = 1; continue; }
        if (g.kind != VD_AGG_SUM || g.nfactors > 2 || va >= 0) return VD_OK;
        for (int f = 0; f < g.nfactors; ++f) if (!plain_col(g.f[f]) || g.f[f].col >= ncols) return VD_OK;
        va = g.f[0].col;
        vb = g.nfactors == 2 ? g.f[1].col : -1;
        m.src[k] = 0;
    }
    if (va < 0) va = fcol[0];
    if (va < 0) return VD_OK;
    // a term over epsilon is false (A9): integer intervals never include the
    // type's epsilon (INT_MIN; a one-sided `<` filter would otherwise)
    for (int j = 0; j < nf; ++j) {
        if (cols[fcol[j]].dtype == VD_I32) lo[j] = std::max<int64_t>(lo[j], (int64_t)INT32_MIN + 1);
        else if (cols[fcol[j]].dtype == VD_I64) lo[j] = std::max<int64_t>(lo[j], INT64_MIN + 1);
        else if (cols[fcol[j]].dtype == VD_U8) hi[j] = std::min<int64_t>(hi[j], 0xFE);
        else if (cols[fcol[j]].dtype != VD_F32 && cols[fcol[j]].dtype != VD_F64) return VD_OK;
    }
    // value columns that may hold epsilon: not proven epsilon-free by the
    // metadata and not a filter column (whose test already rejects epsilon)
    auto may_eps = [&](int c) {
        if (c < 0 || (cols[c].flags & VD_COL_NOEPS)) return false;
        for (int j = 0; j < nf; ++j)
            if (fcol[j] == c) return false;
        return true;
    };
    const bool veps = may_eps(va) || may_eps(vb);
    int t0 = nf > 0 ? cols[fcol[0]].dtype : -1;
    int t1 = nf > 1 ? cols[fcol[1]].dtype : -1;
    int t2 = nf > 2 ? cols[fcol[2]].dtype : -1;
    int tva = cols[va].dtype, tvb = vb >= 0 ? cols[vb].dtype : -1;
    auto al16 = [](const void* q) { return ((uintptr_t)q % 16) == 0; };
    int mode = p->sel_mode == VD_SEL_PREDICATED ? 1 : 0;
    // overflow proof for integer products (per-thread int64, warp in int128)
    if (tva == VD_I64) {
        Bound A = col_bound(p, cols, ncols, nullptr, va);
        Bound B = vb >= 0 ? col_bound(p, cols, ncols, nullptr, vb) : Bound{true, 1, 1};
        if (!A.known || !B.known) return VD_OK;
        double mx = std::max(std::fabs(A.lo), std::fabs(A.hi)) * std::max(std::fabs(B.lo), std::fabs(B.hi));
        // per-thread int64 sum: rows one thread folds in the variant that
        // launches (the larger of the two, the choice is made below)
        if (mx * scalar_rows_per_thread(n) >= 9.0e18) return VD_OK;
    }
    cudaError_t e = cudaSuccess;
    Slot16* o = (Slot16*)out;
    const char* var = getenv("VD_SCALAR_VARIANT");
    const bool use_tma = !(var && strcmp(var, "ldg") == 0);
    float sslo = 0, sshi = 0;
    // Q6 shape: filters (i32, i64, i64), value i64 * i64
    if (nf == 3 && t0 == VD_I32 && t1 == VD_I64 && t2 == VD_I64 && tva == VD_I64 && tvb == VD_I64 &&
        al16(cols[fcol[0]].data)) {
        ScalarArgs<int32_t, int64_t, int64_t, int64_t, int64_t> sa;
        sa.f0 = (const int32_t*)cols[fcol[0]].data;
        sa.f1 = (const int64_t*)cols[fcol[1]].data;
        sa.f2 = (const int64_t*)cols[fcol[2]].data;
        for (int j = 0; j < 3; ++j) { sa.lo[j] = lo[j]; sa.hi[j] = hi[j]; }
        sa.fcmp[0] = sa.fcmp[1] = -1;
        sa.fc[0] = sa.fc[1] = 0;
        sa.va = (const int64_t*)cols[va].data;
        sa.vb = (const int64_t*)cols[vb].data;
        sa.n = n;
        ScalarTmaArgs ta;
        const void* rp[5] = {sa.f0, sa.f1, sa.f2, sa.va, sa.vb};
        const int re[5] = {4, 8, 8, 8, 8};
        bool pr[5] = {true, true, true, true, true};
        if (use_tma && scalar_tma_args(rp, re, pr, 2048, &ta)) {
            for (int j = 0; j < 3; ++j) { ta.lo[j] = lo[j]; ta.hi[j] = hi[j]; }
            ta.fcmp[0] = ta.fcmp[1] = -1;
            ta.fc[0] = ta.fc[1] = 0;
            ta.n = n;
#define SC_Q6_TMA(M, E) launch_scalar_tma<M, E, 3, true, 2048, int32_t, int64_t, int64_t, int64_t, int64_t>(ta, ws, o, m, s, nl)
            if (mode) e = veps ? SC_Q6_TMA(1, true) : SC_Q6_TMA(1, false);
            else e = veps ? SC_Q6_TMA(0, true) : SC_Q6_TMA(0, false);
#undef SC_Q6_TMA
            set_fragment("scalar_tma");
        } else {
            if (mode) e = veps ? launch_scalar<1, true, true, true, true>(sa, ws, o, m, s, nl)
                               : launch_scalar<1, false, true, true, true>(sa, ws, o, m, s, nl);
            else e = veps ? launch_scalar<0, true, true, true, true>(sa, ws, o, m, s, nl)
                          : launch_scalar<0, false, true, true, true>(sa, ws, o, m, s, nl);
            set_fragment("scalar_ldg");
        }
    } else if (nf == 1 && t0 == VD_F32 && tva == VD_F32 && vb < 0 && al16(cols[va].data) &&
               al16(cols[fcol[0]].data) && use_tma && f32_interval(fcmp, fc, &sslo, &sshi)) {
        // selective sum over f32 (Fig 15 / C1): the value column is the filter
        // column or a second one staged beside it
        const bool two = va != fcol[0];
        SelSumArgs ss;
        ss.v = (const float*)cols[fcol[0]].data;
        ss.w = (const float*)cols[va].data;
        ss.lo = sslo;
        ss.hi = sshi;
        ss.n = n;
        ss.nstages = two ? 3 : SS_MAXSTAGES;
        const int grid = num_sms();
        unsigned int* dn = (unsigned int*)ws;
        Slot16* parts = (Slot16*)((char*)ws + 256);
        e = cudaMemsetAsync(dn, 0, 4, s);
        if (e == cudaSuccess) {
            const size_t smem = (size_t)ss.nstages * (two ? 2 : 1) * SS_TILE * 4 + 2 * ss.nstages * 8;
#define SS_GO(M, T, E)                                                                                   \
    {                                                                                                    \
        cudaFuncSetAttribute(k_pipe_selsum_tma<M, T, E>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem); \
        k_pipe_selsum_tma<M, T, E><<<grid, SS_THREADS, smem, s>>>(ss, n / SS_TILE, parts, dn, o, m);     \
    }
            if (!two) { if (mode) SS_GO(1, false, false) else SS_GO(0, false, false) }
            else if (veps) { if (mode) SS_GO(1, true, true) else SS_GO(0, true, true) }
            else { if (mode) SS_GO(1, true, false) else SS_GO(0, true, false) }
#undef SS_GO
            ++*nl;
            e = cudaGetLastError();
        }
        set_fragment("selsum_tma");
    } else if (nf == 1 && t0 == VD_F32 && tva == VD_F32 && vb < 0 && al16(cols[fcol[0]].data)) {
        // selective aggregation over one f32 column (Fig 15 / C1)
        ScalarArgs<float, float, float, float, float> sa;
        sa.f0 = (const float*)cols[fcol[0]].data;
        sa.f1 = sa.f2 = nullptr;
        for (int j = 0; j < 3; ++j) { sa.lo[j] = lo[j]; sa.hi[j] = hi[j]; }
        sa.fcmp[0] = fcmp[0]; sa.fcmp[1] = fcmp[1];
        sa.fc[0] = fc[0]; sa.fc[1] = fc[1];
        sa.va = (const float*)cols[va].data;
        sa.vb = nullptr;
        sa.n = n;
        ScalarTmaArgs ta;
        const void* rp[5] = {sa.f0, nullptr, nullptr, sa.va, nullptr};
        const int re[5] = {4, 4, 4, 4, 4};
        bool pr[5] = {true, false, false, true, false};
        if (use_tma && scalar_tma_args(rp, re, pr, 8192, &ta)) {
            for (int j = 0; j < 3; ++j) { ta.lo[j] = lo[j]; ta.hi[j] = hi[j]; }
            ta.fcmp[0] = fcmp[0]; ta.fcmp[1] = fcmp[1];
            ta.fc[0] = fc[0]; ta.fc[1] = fc[1];
            ta.n = n;
#define SC_F_TMA(M, E) launch_scalar_tma<M, E, 1, false, 8192, float, float, float, float, float>(ta, ws, o, m, s, nl)
            if (mode) e = veps ? SC_F_TMA(1, true) : SC_F_TMA(1, false);
            else e = veps ? SC_F_TMA(0, true) : SC_F_TMA(0, false);
#undef SC_F_TMA
            set_fragment("scalar_tma");
        } else {
            if (mode) e = veps ? launch_scalar<1, true, false, false, false>(sa, ws, o, m, s, nl)
                               : launch_scalar<1, false, false, false, false>(sa, ws, o, m, s, nl);
            else e = veps ? launch_scalar<0, true, false, false, false>(sa, ws, o, m, s, nl)
                          : launch_scalar<0, false, false, false, false>(sa, ws, o, m, s, nl);
            set_fragment("scalar_ldg");
        }
    } else {
        return VD_OK;
    }
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    *done = true;
    return VD_OK;
}

// ---- FK grouped-fold (Q9 shape) matching ---------------------------------------------
static vd_status try_fkg(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, const vd_column* dims,
                         void* out, void* ws, cudaStream_t s, int* nl, bool* done) {
    *done = false;
    const char* var = getenv("VD_FKG_VARIANT");
    if (var && strcmp(var, "off") == 0) return VD_OK;
    if (p->pred.nconj != 0 || p->ngathers != 1 || p->nkeyparts != 2 || p->ngroups > 512) return VD_OK;
    const vd_gatherspec& gs = p->gathers[0];
    const vd_column& dim = dims[gs.dim_col];
    if (cols[gs.fk_col].dtype != VD_I32 || dim.dtype != VD_U8) return VD_OK;
    // key part A: the gathered column (identity); key part B: a base i32 column
    int ia = -1, ib = -1;
    for (int k = 0; k < 2; ++k) {
        if (p->key[k].col == ncols && p->key[k].fn == 0) ia = k;
        else if (p->key[k].col < ncols && cols[p->key[k].col].dtype == VD_I32) ib = k;
    }
    if (ia < 0 || ib < 0) return VD_OK;
    // aggregates: one SUM(X * (a + b*Y)) over i64 base columns, COUNT
    FkgArgs A;
    std::memset(&A, 0, sizeof(A));
    A.sum_slot = A.cnt_slot = -1;
    A.naggs = p->naggs;
    int X = -1, Y = -1;
    for (int g = 0; g < p->naggs; ++g) {
        const vd_agg& ag = p->aggs[g];
        if (ag.kind == VD_AGG_COUNT) { if (A.cnt_slot >= 0) return VD_OK; A.cnt_slot = g; continue; }
        if (ag.kind != VD_AGG_SUM || A.sum_slot >= 0 || ag.nfactors != 2 || !plain_col(ag.f[0])) return VD_OK;
        X = ag.f[0].col;
        Y = ag.f[1].col;
        if (X >= ncols || Y < 0 || Y >= ncols || cols[X].dtype != VD_I64 || cols[Y].dtype != VD_I64) return VD_OK;
        A.a = ag.f[1].a;
        A.b = ag.f[1].b;
        A.sum_slot = g;
    }
    if (A.sum_slot < 0) return VD_OK;
    const int kbcol = p->key[ib].col, fkcol = gs.fk_col;
    for (int c : {fkcol, kbcol, X, Y})
        if (((uintptr_t)cols[c].data % 16) != 0) return VD_OK;
    // exactness: |X*(a+bY)| * rows per warp < 2^63; narrow if everything fits 32 bits
    Bound bx = col_bound(p, cols, ncols, dims, X), by = col_bound(p, cols, ncols, dims, Y);
    if (!bx.known || !by.known) return VD_OK;
    vd_factor fy;
    fy.col = Y; fy.a = A.a; fy.b = A.b;
    const double fmx = factor_absmax(fy, by), xmx = std::max(std::fabs(bx.lo), std::fabs(bx.hi));
    const int grid = num_sms();
    const double rows_per_warp = std::ceil((double)n / ((double)grid * FKG_CW)) + FKG_TILE;
    if (xmx * fmx * rows_per_warp >= 9.0e18) return VD_OK;
    const bool narrow = xmx < 2147483647.0 && fmx < 2147483647.0 && xmx * fmx < 9.0e18 &&
                        std::max(std::fabs(by.lo), std::fabs(by.hi)) < 2147483647.0 && std::fabs((double)A.a) < 2.0e9 &&
                        std::fabs((double)A.b) < 2.0e9;
    A.fk = (const int32_t*)cols[fkcol].data;
    A.kb = (const int32_t*)cols[kbcol].data;
    A.x = (const int64_t*)cols[X].data;
    A.y = (const int64_t*)cols[Y].data;
    A.dim = (const uint8_t*)dim.data;
    A.dim_len = dim.len;
    A.bias = gs.bias;
    A.subA = (int32_t)p->key[ia].sub;
    A.mA = (int32_t)p->key[ia].mult;
    A.subB = (int32_t)p->key[ib].sub;
    A.mB = (int32_t)p->key[ib].mult;
    A.yfn = p->key[ib].fn;
    A.ylo = 0;
    A.ydays = 0;
    if (A.yfn) {
        if (!(cols[kbcol].has_minmax && cols[kbcol].max - cols[kbcol].min < GF_MAXYEARDAYS)) return VD_OK;
        A.ylo = (int32_t)cols[kbcol].min;
        A.ydays = (int32_t)(cols[kbcol].max - cols[kbcol].min + 1);
    }
    A.ngroups = (int32_t)p->ngroups;
    A.n = n;
    // ---- private-slot variant (k_pipe_fkg_priv): values proven in [0, 2^31)
    {
        const double flo = std::min((double)A.a + (double)A.b * by.lo, (double)A.a + (double)A.b * by.hi);
        const vd_column &cfk = cols[fkcol], &ckb = cols[kbcol];
        const bool yr_ok = !A.yfn || (ckb.has_minmax && ckb.min >= -365 && ckb.max <= 47481);
        const bool fits = narrow && bx.lo >= 0 && flo >= 0 && xmx * fmx < 2147483647.0 && yr_ok;
        auto noeps = [](const vd_column& c) { return (c.flags & VD_COL_NOEPS) != 0; };
        bool proven = fits && noeps(cfk) && noeps(ckb) && noeps(cols[X]) && noeps(cols[Y]) && noeps(dim) &&
                      cfk.has_minmax && dim.has_minmax && ckb.has_minmax && cfk.min - gs.bias >= 0 &&
                      cfk.max - gs.bias < dim.len && dim.max < 0xFF;
        if (proven) {
            // key range over the corners of (d, kb') from metadata
            const int64_t k0 = A.yfn ? (4 * (ckb.min + 365) + 3) / 1461 + 1969 : ckb.min;
            const int64_t k1 = A.yfn ? (4 * (ckb.max + 365) + 3) / 1461 + 1969 : ckb.max;
            int64_t kmin = INT64_MAX, kmax = INT64_MIN;
            for (int64_t d : {dim.min, dim.max})
                for (int64_t kk : {k0, k1}) {
                    const int64_t key = (d - A.subA) * (int64_t)A.mA + (kk - A.subB) * (int64_t)A.mB;
                    kmin = std::min(kmin, key);
                    kmax = std::max(kmax, key);
                }
            proven = kmin >= 0 && kmax < A.ngroups;
        }
        const int slots = A.ngroups + (proven ? 0 : 1);
        const int64_t ntiles = n / FKP_TILE;
        // rows per private slot set < 2^16: tiles per CTA * 8 + tail 8
        const int64_t grid = std::max<int64_t>(num_sms(), (ntiles + 8000 - 1) / 8000);
        // opt-in (VD_FKG_VARIANT=priv): one consumer warp per scheduler leaves
        // its dependency chains exposed -- 4.6 ms vs 3.3 ms for the
        // shared-atomic kernel at Q9 SF100 (profiles/round1_q9.md)
        const bool want_priv = var && strcmp(var, "priv") == 0;
        if (want_priv && fits && slots <= FKP_MAXSLOTS && grid <= grid_persistent(4)) {
            const size_t smem = (size_t)FKP_STAGES * FKP_TILE * 24 + (size_t)slots * FKP_NT * 8 + 2 * FKP_STAGES * 8;
            const char* pfv = getenv("VD_FKP_PF");
            const int32_t pf = pfv ? atoi(pfv) : 0;
            unsigned int* dn = (unsigned int*)ws;
            Slot16* parts = (Slot16*)((char*)ws + 256);
            cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
            if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
            auto go = [&](auto kern) {
                cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
                kern<<<(unsigned)grid, FKP_THREADS, smem, s>>>(A, ntiles, pf, parts, dn, (Slot16*)out);
            };
            const char* bv = getenv("VD_FKP_BATCH");
            const int batch = bv ? atoi(bv) : 4;
            if (proven) {
                if (batch == 8) go(k_pipe_fkg_priv<false, 8>);
                else if (batch == 2) go(k_pipe_fkg_priv<false, 2>);
                else go(k_pipe_fkg_priv<false, 4>);
            } else {
                go(k_pipe_fkg_priv<true, 4>);
            }
            ++*nl;
            e = cudaGetLastError();
            if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
            set_fragment(proven ? "fk_group_priv" : "fk_group_priv_checked");
            *done = true;
            return VD_OK;
        }
    }
    constexpr size_t SB = FKG_TILE * 24;
    const size_t fixed = (size_t)FKG_CW * 3 * (((size_t)p->ngroups + 32) & ~(size_t)31) * 4 + FKG_CW * 32 * 8 + (size_t)((A.ydays + 7) & ~7) * 2 +
                         2 * GF_MAXSTAGES * 8;
    const size_t budget = 200 * 1024;
    if (fixed + 2 * SB > budget) return VD_OK;
    // a 2-stage ring (96 KB in flight per SM) is enough to keep HBM busy; the
    // fragment is bound by L2 sector throughput, and deeper rings (4 stages)
    // measured slower: 3.43 vs 3.20 ms at SF100 (streamed sectors queue ahead
    // of the dimension lookups).  VD_FKG_STAGES overrides (2..budget).
    int ns = (int)((budget - fixed) / SB);
    ns = ns > GF_MAXSTAGES ? GF_MAXSTAGES : ns;
    A.nstages = 2;
    if (const char* sv = getenv("VD_FKG_STAGES")) A.nstages = std::max(2, std::min(ns, atoi(sv)));
    const size_t smem = fixed + (size_t)A.nstages * SB;
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    // group-slot update: shared-memory atomics (default) or match_any leaders
    const char* agg = getenv("VD_FKG_AGG");
    const bool atom = !(agg && strcmp(agg, "match") == 0);
    auto go = [&](auto kern) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        kern<<<grid, FKG_THREADS, smem, s>>>(A, n / FKG_TILE, parts, dn, (Slot16*)out);
    };
    const char* pv_ = getenv("VD_FKG_PIPE");
    const bool pipe = pv_ && strcmp(pv_, "1") == 0;
    if (narrow && atom) pipe ? go(k_pipe_fkg<true, true, true>) : go(k_pipe_fkg<true, true, false>);
    else if (narrow) pipe ? go(k_pipe_fkg<true, false, true>) : go(k_pipe_fkg<true, false, false>);
    else if (atom) pipe ? go(k_pipe_fkg<false, true, true>) : go(k_pipe_fkg<false, true, false>);
    else pipe ? go(k_pipe_fkg<false, false, true>) : go(k_pipe_fkg<false, false, false>);
    ++*nl;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    set_fragment("fk_group");
    *done = true;
    return VD_OK;
}

// ---- selective FK join (Fig 16) matching -----------------------------------------------
template <int MODE, typename PT, typename DT>
static void launch_fkjs_tma1(const FkjsArgs& A, int64_t n, Slot16* parts, unsigned* dn, Slot16* out, cudaStream_t s) {
    constexpr size_t SB = FJT_TILE * (4 + sizeof(PT));
    const int nstages = (int)std::min<size_t>(8, (200 * 1024) / SB);
    const size_t smem = (size_t)nstages * SB + 2 * nstages * 8;
    cudaFuncSetAttribute(k_pipe_fkjs_tma<MODE, PT, DT>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    k_pipe_fkjs_tma<MODE, PT, DT><<<num_sms(), FJT_THREADS, smem, s>>>(A, nstages, n / FJT_TILE, parts, dn, out);
}

template <int MODE>
static void launch_fkjs_tma(const FkjsArgs& A, int pdt, int ddt, int64_t n, Slot16* parts, unsigned* dn, Slot16* out,
                            cudaStream_t s) {
    if (pdt == VD_I32 && ddt == VD_I64) launch_fkjs_tma1<MODE, int32_t, int64_t>(A, n, parts, dn, out, s);
    else if (pdt == VD_I32) launch_fkjs_tma1<MODE, int32_t, int32_t>(A, n, parts, dn, out, s);
    else if (ddt == VD_I64) launch_fkjs_tma1<MODE, int64_t, int64_t>(A, n, parts, dn, out, s);
    else launch_fkjs_tma1<MODE, int64_t, int32_t>(A, n, parts, dn, out, s);
}

template <int MODE>
static void launch_fkjs(const FkjsArgs& A, int pdt, int ddt, int grid, Slot16* parts, unsigned* dn, Slot16* out,
                        cudaStream_t s) {
    if (pdt == VD_I32 && ddt == VD_I64) k_pipe_fkjs<MODE, int32_t, int64_t><<<grid, FJ_THREADS, 0, s>>>(A, parts, dn, out);
    else if (pdt == VD_I32) k_pipe_fkjs<MODE, int32_t, int32_t><<<grid, FJ_THREADS, 0, s>>>(A, parts, dn, out);
    else if (ddt == VD_I64) k_pipe_fkjs<MODE, int64_t, int64_t><<<grid, FJ_THREADS, 0, s>>>(A, parts, dn, out);
    else k_pipe_fkjs<MODE, int64_t, int32_t><<<grid, FJ_THREADS, 0, s>>>(A, parts, dn, out);
}

static vd_status try_fkjs(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, const vd_column* dims,
                          void* out, void* ws, cudaStream_t s, int* nl, bool* done) {
    *done = false;
    const char* var = getenv("VD_FKJS_VARIANT");
    if (var && strcmp(var, "off") == 0) return VD_OK;
    if (p->nkeyparts != 0 || p->ngroups != 1 || p->ngathers != 1 || p->pred.nconj != 1) return VD_OK;
    const int fkc = p->gathers[0].fk_col;
    if (fkc >= ncols || cols[fkc].dtype != VD_I32) return VD_OK;
    const vd_column& dim = dims[p->gathers[0].dim_col];
    if (dim.dtype != VD_I32 && dim.dtype != VD_I64) return VD_OK;
    int pc = -1;
    int64_t lo = INT64_MIN + 1, hi = INT64_MAX;
    for (int t = 0; t < p->pred.conj[0].nterms; ++t) {
        const vd_term& tm = p->pred.conj[0].terms[t];
        if (tm.col >= ncols || (pc >= 0 && tm.col != pc)) return VD_OK;
        pc = tm.col;
        if (!term_interval(tm, &lo, &hi)) return VD_OK;
    }
    if (pc < 0 || (cols[pc].dtype != VD_I32 && cols[pc].dtype != VD_I64)) return VD_OK;
    if (cols[pc].dtype == VD_I32) lo = std::max<int64_t>(lo, (int64_t)INT32_MIN + 1);
    FkjsArgs A;
    std::memset(&A, 0, sizeof(A));
    A.sum_slot = A.cnt_slot = -1;
    A.naggs = p->naggs;
    for (int g = 0; g < p->naggs; ++g) {
        const vd_agg& ag = p->aggs[g];
        if (ag.kind == VD_AGG_COUNT) { if (A.cnt_slot >= 0) return VD_OK; A.cnt_slot = g; continue; }
        if (ag.kind != VD_AGG_SUM || A.sum_slot >= 0 || ag.nfactors != 1 || !plain_col(ag.f[0]) ||
            ag.f[0].col != ncols)
            return VD_OK;
        A.sum_slot = g;
    }
    if (A.sum_slot < 0) return VD_OK;
    const Bound bd = col_bound(p, cols, ncols, dims, ncols);
    if (!bd.known) return VD_OK;
    const int grid = num_sms() * 4;
    // both variants: at least num_sms() * FKG_NT threads, plus a ragged tail
    const double rows_per_thread = std::ceil((double)n / ((double)num_sms() * FKG_NT)) + 2.0 * FJT_TILE / FJT_NT;
    if (std::max(std::fabs(bd.lo), std::fabs(bd.hi)) * rows_per_thread * 32.0 >= 9.0e18) return VD_OK;
    A.fk = (const int32_t*)cols[fkc].data;
    A.pv = cols[pc].data;
    A.dim = dim.data;
    A.n = n;
    A.dim_len = dim.len;
    A.bias = p->gathers[0].bias;
    A.lo = lo;
    A.hi = hi;
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    // Branching reads the dimension only for qualifying rows: the TMA ring
    // streams the two columns at full bandwidth (2.5x the plain loads at low
    // selectivity).  The predicated strategies gather every row and are bound
    // by random DRAM accesses, where the plain-load kernel (more warps, fewer
    // LSU stalls) is faster.  VD_FKJS_VARIANT=ldg|tma overrides; TMA needs
    // 16-byte aligned columns.
    bool tma = p->sel_mode == VD_SEL_BRANCH;
    if (var && strcmp(var, "ldg") == 0) tma = false;
    if (var && strcmp(var, "tma") == 0) tma = true;
    tma = tma && ((uintptr_t)A.fk % 16) == 0 && ((uintptr_t)A.pv % 16) == 0;
    const int pdt = cols[pc].dtype, ddt = dim.dtype;
    Slot16* o = (Slot16*)out;
    if (tma) {
        if (p->sel_mode == VD_SEL_BRANCH) launch_fkjs_tma<0>(A, pdt, ddt, n, parts, dn, o, s);
        else if (p->sel_mode == VD_SEL_PREDICATED) launch_fkjs_tma<1>(A, pdt, ddt, n, parts, dn, o, s);
        else launch_fkjs_tma<2>(A, pdt, ddt, n, parts, dn, o, s);
    } else {
        if (p->sel_mode == VD_SEL_BRANCH) launch_fkjs<0>(A, pdt, ddt, grid, parts, dn, o, s);
        else if (p->sel_mode == VD_SEL_PREDICATED) launch_fkjs<1>(A, pdt, ddt, grid, parts, dn, o, s);
        else launch_fkjs<2>(A, pdt, ddt, grid, parts, dn, o, s);
    }
    ++*nl;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    set_fragment("fk_select_sum");
    *done = true;
    return VD_OK;
}

// ---- star-join (Q19 shape) matching -------------------------------------------------
static vd_status try_star(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, const vd_column* dims,
                          void* out, void* ws, cudaStream_t s, int* nl, bool* done) {
    *done = false;
    const char* var = getenv("VD_STAR_VARIANT");
    if (var && strcmp(var, "off") == 0) return VD_OK;
    if (p->nkeyparts != 0 || p->ngroups != 1 || p->pred.nconj < 1 || p->pred.nconj > ST_MAXCONJ) return VD_OK;
    if (p->ngathers < 1 || p->ngathers > 3) return VD_OK;
    const int fkcol = p->gathers[0].fk_col;
    for (int g = 0; g < p->ngathers; ++g)
        if (p->gathers[g].fk_col != fkcol || p->gathers[g].bias != p->gathers[0].bias) return VD_OK;
    if (cols[fkcol].dtype != VD_I32) return VD_OK;
    int64_t dim_len = dims[p->gathers[0].dim_col].len;
    for (int g = 0; g < p->ngathers; ++g)
        if (dims[p->gathers[g].dim_col].len != dim_len) return VD_OK;
    // slot assignment by column: base u8 sets (2), base i64 range (1), dim u8 sets (2), dim i32 range (1)
    int bu[2] = {-1, -1}, br = -1, du[2] = {-1, -1}, dr = -1;
    auto dt_of = [&](int c) { return c < ncols ? cols[c].dtype : dims[p->gathers[c - ncols].dim_col].dtype; };
    auto take = [](int* slot, int nslot, int c) {
        for (int k = 0; k < nslot; ++k) { if (slot[k] == c) return true; if (slot[k] < 0) { slot[k] = c; return true; } }
        return false;
    };
    for (int c = 0; c < p->pred.nconj; ++c)
        for (int t = 0; t < p->pred.conj[c].nterms; ++t) {
            const vd_term& tm = p->pred.conj[c].terms[t];
            const int dt = dt_of(tm.col);
            const bool base = tm.col < ncols;
            bool ok;
            if (dt == VD_U8) ok = base ? take(bu, 2, tm.col) : take(du, 2, tm.col);
            else if (base && dt == VD_I64) ok = take(&br, 1, tm.col);
            else if (!base && dt == VD_I32) ok = take(&dr, 1, tm.col);
            else ok = false;
            if (!ok) return VD_OK;
        }
    StarArgs A;
    std::memset(&A, 0, sizeof(A));
    A.nconj = p->pred.nconj;
    const int uslot[4] = {bu[0], bu[1], du[0], du[1]};
    for (int c = 0; c < ST_MAXCONJ; ++c) {
        int64_t rlo = INT64_MIN, rhi = INT64_MAX, dlo = INT32_MIN, dhi = INT32_MAX;
        if (c >= A.nconj) {  // unused conjunction: never passes
            A.rq_lo[c] = 1; A.rq_hi[c] = 0; A.dr_lo[c] = 1; A.dr_hi[c] = 0;
            continue;
        }
        bool ucon[4] = {false, false, false, false};
        bool pass[4][256];
        for (int k = 0; k < 4; ++k) std::fill(pass[k], pass[k] + 256, true);
        for (int t = 0; t < p->pred.conj[c].nterms; ++t) {
            const vd_term& tm = p->pred.conj[c].terms[t];
            bool ok = true;
            int k = -1;
            for (int q = 0; q < 4; ++q) if (uslot[q] == tm.col) k = q;
            if (k >= 0) {
                ucon[k] = true;
                for (int x = 0; x < 256; ++x) {
                    bool r;
                    switch (tm.cmp) {
                    case VD_CMP_GT: r = x > tm.ival; break;
                    case VD_CMP_LT: r = x < tm.ival; break;
                    case VD_CMP_EQ: r = x == tm.ival; break;
                    case VD_CMP_GE: r = x >= tm.ival; break;
                    case VD_CMP_LE: r = x <= tm.ival; break;
                    case VD_CMP_NE: r = x != tm.ival; break;
                    case VD_CMP_IN: r = x < 64 && (((uint64_t)tm.ival >> x) & 1ull); break;
                    default: return VD_OK;
                    }
                    pass[k][x] = pass[k][x] && r;
                }
            } else if (tm.col == br) {
                ok = term_interval(tm, &rlo, &rhi);
                rlo = std::max<int64_t>(rlo, INT64_MIN + 1);  // epsilon never passes a term
            } else if (tm.col == dr) {
                ok = term_interval(tm, &dlo, &dhi);
                dlo = std::max<int64_t>(dlo, INT32_MIN + 1);
            } else {
                ok = false;
            }
            if (!ok) return VD_OK;
        }
        for (int k = 0; k < 4; ++k) {
            if (ucon[k]) pass[k][255] = false;
            for (int x = 0; x < 256; ++x)
                if (pass[k][x]) A.lut[k][x] |= (uint8_t)(1u << c);
        }
        A.rq_lo[c] = rlo; A.rq_hi[c] = rhi;
        A.dr_lo[c] = (int32_t)std::max<int64_t>(dlo, INT32_MIN);
        A.dr_hi[c] = (int32_t)std::min<int64_t>(dhi, INT32_MAX);
        if (dlo > INT32_MAX || dhi < INT32_MIN) { A.dr_lo[c] = 1; A.dr_hi[c] = 0; }
    }
    // aggregates
    A.sum_slot = A.cnt_slot = -1;
    A.naggs = p->naggs;
    int X = -1, Y = -1;
    for (int g = 0; g < p->naggs; ++g) {
        const vd_agg& ag = p->aggs[g];
        if (ag.kind == VD_AGG_COUNT) { if (A.cnt_slot >= 0) return VD_OK; A.cnt_slot = g; continue; }
        if (ag.kind != VD_AGG_SUM || A.sum_slot >= 0 || ag.nfactors != 2 || !plain_col(ag.f[0])) return VD_OK;
        X = ag.f[0].col;
        Y = ag.f[1].col;
        if (X >= ncols || Y < 0 || Y >= ncols || cols[X].dtype != VD_I64 || cols[Y].dtype != VD_I64) return VD_OK;
        A.a = ag.f[1].a;
        A.b = ag.f[1].b;
        A.sum_slot = g;
    }
    if (A.sum_slot < 0) return VD_OK;
    // slots the predicate does not use read a claimed column through an all-pass LUT
    const int cu1 = bu[0], cu2 = bu[1] >= 0 ? bu[1] : bu[0];
    if (cu1 < 0 || br < 0) return VD_OK;  // the base prefilter needs a u8 and the i64 column
    for (int c : {fkcol, br, cu1, cu2})
        if (((uintptr_t)cols[c].data % 16) != 0) return VD_OK;
    Bound bx = col_bound(p, cols, ncols, dims, X), by = col_bound(p, cols, ncols, dims, Y);
    if (!bx.known || !by.known) return VD_OK;
    vd_factor fy;
    fy.col = Y; fy.a = A.a; fy.b = A.b;
    const double fmx = factor_absmax(fy, by), xmx = std::max(std::fabs(bx.lo), std::fabs(bx.hi));
    const int grid = num_sms();
    const double rows_per_thread = std::ceil((double)n / ((double)grid * FKG_NT)) + ST_TILE;
    if (xmx * fmx * rows_per_thread >= 9.0e18) return VD_OK;
    const bool narrow = xmx < 2147483647.0 && fmx < 2147483647.0 && std::fabs((double)A.a) < 2.0e9 &&
                        std::fabs((double)A.b) < 2.0e9 && std::max(std::fabs(by.lo), std::fabs(by.hi)) < 2147483647.0;
    A.fk = (const int32_t*)cols[fkcol].data;
    A.rq = (const int64_t*)cols[br].data;
    A.u1 = (const uint8_t*)cols[cu1].data;
    A.u2 = (const uint8_t*)cols[cu2].data;
    A.x = (const int64_t*)cols[X].data;
    A.y = (const int64_t*)cols[Y].data;
    auto dimptr = [&](int c) { return dims[p->gathers[c - ncols].dim_col].data; };
    const int cd1 = du[0], cd2 = du[1] >= 0 ? du[1] : du[0];
    if (cd1 < 0 || dr < 0) return VD_OK;
    A.d1 = (const uint8_t*)dimptr(cd1);
    A.d2 = (const uint8_t*)dimptr(cd2);
    A.dr = (const int32_t*)dimptr(dr);
    A.dim_len = dim_len;
    A.bias = p->gathers[0].bias;
    A.n = n;
    constexpr size_t SB = ST_TILE * 14;
    A.nstages = (int)std::min<size_t>(GF_MAXSTAGES, (200 * 1024) / SB);
    const size_t smem = (size_t)A.nstages * SB + 2 * A.nstages * 8;
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    if (narrow) {
        cudaFuncSetAttribute(k_pipe_star<true>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        k_pipe_star<true><<<grid, FKG_THREADS, smem, s>>>(A, n / ST_TILE, parts, dn, (Slot16*)out);
    } else {
        cudaFuncSetAttribute(k_pipe_star<false>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        k_pipe_star<false><<<grid, FKG_THREADS, smem, s>>>(A, n / ST_TILE, parts, dn, (Slot16*)out);
    }
    ++*nl;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    set_fragment("star_join");
    *done = true;
    return VD_OK;
}

// ---- gather-fold matching -------------------------------------------------------
// VD_LATE: "off" disables the late-materialisation fragment, "force" also
// tries it before the dense scalar fragment (plans without gathers: Q6)
static int late_policy() {
    const char* e = getenv("VD_LATE");
    if (e && strcmp(e, "off") == 0) return 0;
    if (e && strcmp(e, "force") == 0) return 2;
    return 1;
}

static bool host_cmp_int(int cmp, int64_t x, int64_t c) {  // = cmp_int (vd_pred.cuh)
    switch (cmp) {
    case VD_CMP_GT: return x > c;
    case VD_CMP_LT: return x < c;
    case VD_CMP_EQ: return x == c;
    case VD_CMP_GE: return x >= c;
    case VD_CMP_LE: return x <= c;
    case VD_CMP_NE: return x != c;
    case VD_CMP_IN: return (uint64_t)x < 64ull && (((uint64_t)c >> (uint64_t)x) & 1ull);
    default: return false;
    }
}

static vd_status try_gf(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, const vd_column* dims,
                        void* out, void* ws, cudaStream_t s, int* nl, bool* done, bool late_only = false) {
    *done = false;
    const char* var = getenv("VD_GF_VARIANT");
    if (var && strcmp(var, "off") == 0) return VD_OK;
    if (ncols > GF_MAXCOLS || p->ngroups > 512) return VD_OK;
    const int nref = ncols + p->ngathers;
    auto dtype_of = [&](int c) { return c < ncols ? cols[c].dtype : dims[p->gathers[c - ncols].dim_col].dtype; };
    auto is_int = [](int dt) { return dt == VD_U8 || dt == VD_I32 || dt == VD_I64; };
    GfArgs A;
    std::memset(&A, 0, sizeof(A));
    // staged columns: all base columns (16B aligned, integer)
    int off = 0;
    for (int c = 0; c < ncols; ++c) {
        if (((uintptr_t)cols[c].data % 16) != 0) return VD_OK;
        A.col[c] = cols[c].data;
        A.dt[c] = cols[c].dtype;
        A.esz[c] = (int)dtype_size(cols[c].dtype);
        A.soff[c] = off;
        off += GF_TILE * A.esz[c];
    }
    A.ncols = ncols;
    A.stage_bytes = off;
    // gathers
    A.ngathers = p->ngathers;
    for (int g = 0; g < p->ngathers; ++g) {
        const vd_column& d = dims[p->gathers[g].dim_col];
        if (!is_int(d.dtype) || !is_int(cols[p->gathers[g].fk_col].dtype)) return VD_OK;
        A.g_fk[g] = p->gathers[g].fk_col;
        A.g_bias[g] = p->gathers[g].bias;
        A.g_p[g] = d.data;
        A.g_len[g] = d.len;
        A.g_dt[g] = d.dtype;
    }
    // predicate: hoist base-column terms shared by every conjunction (AND
    // distributes over OR), then per conjunction base terms first (no gather
    // for a row that already failed), equality / IN terms (usually the most
    // selective) before ranges
    vd_pred pr = p->pred;
    auto same = [](const vd_term& x, const vd_term& y) {
        return x.col == y.col && x.cmp == y.cmp && x.ival == y.ival && x.fval == y.fval;
    };
    A.ncommon = 0;
    if (pr.nconj >= 1) {
        vd_conj& c0 = pr.conj[0];
        for (int t = 0; t < c0.nterms; ++t) {
            const vd_term& cand = c0.terms[t];
            if (cand.col >= ncols) continue;
            bool everywhere = true;
            for (int c = 1; c < pr.nconj && everywhere; ++c) {
                bool found = false;
                for (int u = 0; u < pr.conj[c].nterms; ++u) found = found || same(cand, pr.conj[c].terms[u]);
                everywhere = found;
            }
            if (!everywhere) continue;
            bool dup = false;
            for (int k = 0; k < A.ncommon; ++k)
                dup = dup || (A.common[k].col == cand.col && A.common[k].cmp == cand.cmp && A.common[k].iv == cand.ival &&
                              A.common[k].fv == cand.fval);
            if (!dup && A.ncommon < VD_MAX_TERMS) {
                A.common[A.ncommon].col = cand.col;
                A.common[A.ncommon].cmp = cand.cmp;
                A.common[A.ncommon].iv = cand.ival;
                A.common[A.ncommon].fv = cand.fval;
                ++A.ncommon;
            }
        }
    }
    auto rank = [&](const vd_term& t) {
        const bool base = t.col < ncols;
        const bool eq = t.cmp == VD_CMP_EQ || t.cmp == VD_CMP_IN;
        return (base ? 0 : 2) + (eq ? 0 : 1);
    };
    bool always = false;  // a conjunction reduced to the common terms only
    for (int c = 0; c < pr.nconj; ++c) {
        vd_conj& cj = pr.conj[c];
        vd_term tmp[VD_MAX_TERMS];
        int k = 0;
        for (int r = 0; r < 4; ++r)
            for (int t = 0; t < cj.nterms; ++t) {
                bool hoisted = false;
                for (int h = 0; h < A.ncommon; ++h)
                    hoisted = hoisted || (A.common[h].col == cj.terms[t].col && A.common[h].cmp == cj.terms[t].cmp &&
                                          A.common[h].iv == cj.terms[t].ival && A.common[h].fv == cj.terms[t].fval);
                if (!hoisted && rank(cj.terms[t]) == r) tmp[k++] = cj.terms[t];
            }
        int nb = 0;
        for (int t = 0; t < k; ++t) nb += tmp[t].col < ncols;
        A.nbase[c] = nb;
        cj.nterms = k;
        for (int t = 0; t < k; ++t) cj.terms[t] = tmp[t];
        if (k == 0) always = true;
    }
    if (always) pr.nconj = 0;  // the common terms decide
    make_devpred(&pr, &A.pred);
    // key
    A.nkey = p->nkeyparts;
    int64_t ylo = 0, yhi = -1;
    for (int k = 0; k < p->nkeyparts; ++k) {
        const vd_keypart& kp = p->key[k];
        if (!is_int(dtype_of(kp.col))) return VD_OK;
        A.k_col[k] = kp.col;
        A.k_fn[k] = kp.fn;
        A.k_sub[k] = kp.sub;
        A.k_mult[k] = kp.mult;
        if (kp.fn == 1) {
            const vd_column* kc = kp.col < ncols ? &cols[kp.col] : &dims[p->gathers[kp.col - ncols].dim_col];
            if (kc->has_minmax && kc->max - kc->min < GF_MAXYEARDAYS) { ylo = kc->min; yhi = kc->max; }
        }
    }
    A.year_lo = (int32_t)ylo;
    A.year_days = (int32_t)(yhi - ylo + 1);
    A.ngroups = (int32_t)p->ngroups;
    // aggregates: SUM of int64 products or COUNT; exactness from metadata
    int grid = num_sms();
    double rows_per_warp = std::ceil((double)n / ((double)grid * GF_CW)) + GF_TILE;
    A.naggs = p->naggs;
    for (int g = 0; g < p->naggs; ++g) {
        const vd_agg& ag = p->aggs[g];
        A.a_kind[g] = ag.kind;
        if (ag.kind == VD_AGG_COUNT) continue;
        if (ag.kind != VD_AGG_SUM) return VD_OK;
        A.a_nf[g] = ag.nfactors;
        double mx = 1;
        for (int f = 0; f < ag.nfactors; ++f) {
            A.a_col[g][f] = ag.f[f].col;
            A.a_a[g][f] = ag.f[f].a;
            A.a_b[g][f] = ag.f[f].b;
            if (ag.f[f].col < 0) { mx *= std::fabs((double)ag.f[f].a); continue; }
            if (!is_int(dtype_of(ag.f[f].col))) return VD_OK;
            Bound b = col_bound(p, cols, ncols, dims, ag.f[f].col);
            if (!b.known) return VD_OK;
            mx *= factor_absmax(ag.f[f], b);
        }
        if (mx * rows_per_warp >= 9.0e18) return VD_OK;
    }
    A.n = n;
    if (late_only) {
        // lead columns: base columns of hoisted terms whose conjunction is an
        // interval (u8: checked value by value, epsilon 0xFF never passes;
        // i32: comparisons only, epsilon INT32_MIN never passes)
        const int lmode = p->sel_mode == VD_SEL_BRANCH ? 0 : 1;
        // the warp queues hold int32 row numbers
        if (p->ngroups != 1 || lmode != 0 || p->nkeyparts != 0 || n <= 0 || n >= INT32_MAX) return VD_OK;
        LateLead L;
        std::memset(&L, 0, sizeof(L));
        int n8 = 0;
        bool i32 = false;
        bool lead[GF_MAXCOLS] = {};
        // estimated fraction of rows passing the lead intervals, assuming
        // values spread evenly over each column's [min, max] (metadata)
        double est = 1.0;
        for (int k = 0; k < A.ncommon; ++k) {
            const int c = A.common[k].col;
            if (c >= ncols || lead[c]) continue;
            if (cols[c].dtype == VD_U8 && n8 < 2) {
                bool pass[256];
                int lo = 256, hi = -1;
                for (int x = 0; x < 256; ++x) {
                    bool ok = x != 0xFF;
                    for (int h = 0; h < A.ncommon && ok; ++h)
                        if (A.common[h].col == c) ok = host_cmp_int(A.common[h].cmp, x, A.common[h].iv);
                    pass[x] = ok;
                    if (ok) { lo = std::min(lo, x); hi = std::max(hi, x); }
                }
                bool ivl = true;
                for (int x = lo; x <= hi && ivl; ++x) ivl = pass[x];
                if (!ivl) continue;
                if (hi < lo) { lo = 1; hi = 0; }  // nothing passes
                {
                    const int mn = cols[c].has_minmax ? (int)std::max<int64_t>(0, cols[c].min) : 0;
                    const int mx = cols[c].has_minmax ? (int)std::min<int64_t>(254, cols[c].max) : 254;
                    int np = 0;
                    for (int x = mn; x <= mx; ++x) np += pass[x];
                    est *= mx >= mn ? (double)np / (mx - mn + 1) : 0.0;
                }
                L.c8[n8] = (const uint8_t*)cols[c].data;
                L.lo8[n8] = 0x01010101u * (uint32_t)lo;
                L.hi8[n8] = 0x01010101u * (uint32_t)hi;
                ++n8;
                lead[c] = true;
            } else if (cols[c].dtype == VD_I32 && !i32) {
                int64_t lo = (int64_t)INT32_MIN + 1, hi = INT32_MAX;
                bool ivl = true;
                for (int h = 0; h < A.ncommon && ivl; ++h) {
                    if (A.common[h].col != c) continue;
                    // constants outside the int32 range saturate (no overflow in v +- 1)
                    const int64_t v = std::min<int64_t>(std::max<int64_t>(A.common[h].iv, (int64_t)INT32_MIN - 2),
                                                        (int64_t)INT32_MAX + 2);
                    switch (A.common[h].cmp) {
                    case VD_CMP_GT: lo = std::max(lo, v + 1); break;
                    case VD_CMP_GE: lo = std::max(lo, v); break;
                    case VD_CMP_LT: hi = std::min(hi, v - 1); break;
                    case VD_CMP_LE: hi = std::min(hi, v); break;
                    case VD_CMP_EQ: lo = std::max(lo, v); hi = std::min(hi, v); break;
                    default: ivl = false;
                    }
                }
                if (!ivl) continue;
                if (lo > hi) { lo = 1; hi = 0; }
                if (cols[c].has_minmax && cols[c].max >= cols[c].min) {
                    const double ov = (double)std::min<int64_t>(hi, cols[c].max) - (double)std::max<int64_t>(lo, cols[c].min) + 1;
                    est *= std::max(0.0, ov) / ((double)cols[c].max - (double)cols[c].min + 1);
                }
                L.c32 = (const int32_t*)cols[c].data;
                L.lo32 = (int32_t)lo;
                L.hi32 = (int32_t)hi;
                i32 = true;
                lead[c] = true;
            }
        }
        if (n8 == 0 && !i32) return VD_OK;
        // a late load per surviving row costs more than streaming the row
        // past ~10-20% survivors (Q19 3.6%: 0.69 ms late vs 3.08 ms dense;
        // Fig 16 10%: 0.55 vs 0.57 ms, 20%: 0.91 vs 0.67 ms; Q6 15%: 0.28 vs
        // 0.25 ms): by default only clearly selective leads
        if (late_policy() != 2 && est > 0.12) return VD_OK;
        int nc = 0;  // the lead intervals replace the hoisted terms on their columns
        for (int k = 0; k < A.ncommon; ++k)
            if (!lead[A.common[k].col]) A.common[nc++] = A.common[k];
        A.ncommon = nc;
        // referenced columns (gathers: also their FK column)
        auto ref = [&](uint32_t& m, int c) {
            m |= 1u << c;
            if (c >= ncols) m |= 1u << A.g_fk[c - ncols];
        };
        auto selective = [](int cmp) { return cmp == VD_CMP_EQ || cmp == VD_CMP_IN; };
        for (int k = 0; k < A.ncommon; ++k) {
            ref(L.pref, A.common[k].col);
            if (selective(A.common[k].cmp)) ref(L.pref1, A.common[k].col);
        }
        for (int c = 0; c < A.pred.nconj; ++c)
            for (int k = 0; k < A.pred.nterms[c]; ++k) {
                ref(L.pref, A.pred.t[c][k].col);
                if (selective(A.pred.t[c][k].cmp)) ref(L.pref1, A.pred.t[c][k].col);
            }
        // no equality / IN term: one round over every predicate reference
        if (L.pref1 == 0) L.pref1 = L.pref;
        // compile the terms into per-reference constraints (IN: 0 <= x < 64)
        auto compile = [&](const DevTerm* ts, int nt, LtCons* out) -> int {
            int nc = 0;
            for (int k = 0; k < nt; ++k) {
                const DevTerm& t = ts[k];
                int at = -1;
                for (int h = 0; h < nc; ++h) at = out[h].ref == t.col ? h : at;
                if (at < 0) {
                    at = nc++;
                    out[at].ref = t.col;
                    out[at].pad = 0;
                    out[at].lo = INT64_MIN + 1;
                    out[at].hi = INT64_MAX;
                    out[at].in = ~0ull;
                }
                LtCons& c = out[at];
                const int64_t v = t.iv;
                switch (t.cmp) {
                case VD_CMP_GT: if (v == INT64_MAX) c.hi = c.lo - 1; else c.lo = std::max(c.lo, v + 1); break;
                case VD_CMP_GE: c.lo = std::max(c.lo, v); break;
                case VD_CMP_LT: if (v == INT64_MIN) c.hi = c.lo - 1; else c.hi = std::min(c.hi, v - 1); break;
                case VD_CMP_LE: c.hi = std::min(c.hi, v); break;
                case VD_CMP_EQ: c.lo = std::max(c.lo, v); c.hi = std::min(c.hi, v); break;
                case VD_CMP_IN: c.in &= (uint64_t)v; c.lo = std::max(c.lo, (int64_t)0); c.hi = std::min(c.hi, (int64_t)63); break;
                default: return -1;  // NE
                }
            }
            return nc;
        };
        bool ok = true;
        L.ncons[VD_MAX_CONJ] = compile(A.common, A.ncommon, L.cons[VD_MAX_CONJ]);
        ok = L.ncons[VD_MAX_CONJ] >= 0;
        for (int c = 0; c < A.pred.nconj && ok; ++c) {
            L.ncons[c] = compile(A.pred.t[c], A.pred.nterms[c], L.cons[c]);
            ok = L.ncons[c] >= 0;
        }
        if (!ok) L.ncons[0] = -1;
        else if (A.pred.nconj == 0) L.ncons[0] = 0;
        // u8 references: constraints -> acceptance tables (the common terms
        // sit in row VD_MAX_CONJ = LT_COMMON)
        auto ref_u8 = [&](int r) { return dtype_of(r) == VD_U8; };
        L.ntab = 0;
        if (ok) {
            for (int c = 0; c <= VD_MAX_CONJ; ++c) {
                if (c >= A.pred.nconj && c != VD_MAX_CONJ) continue;
                for (int k = 0; k < L.ncons[c]; ++k) {
                    const int r = L.cons[c][k].ref;
                    if (!ref_u8(r)) continue;
                    int t = -1;
                    for (int h = 0; h < L.ntab; ++h) t = L.tref[h] == r ? h : t;
                    if (t < 0 && L.ntab < LT_MAXTAB) {
                        t = L.ntab++;
                        L.tref[t] = r;
                        L.tcm[t] = 0;
                        std::memset(L.tab[t], 0xFF, 256);
                    }
                    if (t < 0) continue;
                    const LtCons& q = L.cons[c][k];
                    L.tcm[t] |= 1u << c;
                    for (int x = 0; x < 256; ++x) {
                        const bool pass = x != 0xFF && x >= q.lo && x <= q.hi && ((q.in >> (x & 63)) & 1ull);
                        if (!pass) L.tab[t][x] &= (uint8_t)~(1u << c);
                    }
                }
            }
            for (int c = 0; c <= VD_MAX_CONJ; ++c) {  // drop the tabulated constraints
                if (c >= A.pred.nconj && c != VD_MAX_CONJ) continue;
                int nk = 0;
                for (int k = 0; k < L.ncons[c]; ++k) {
                    bool tabbed = false;
                    for (int h = 0; h < L.ntab; ++h) tabbed = tabbed || L.tref[h] == L.cons[c][k].ref;
                    if (!tabbed) L.cons[c][nk++] = L.cons[c][k];
                }
                L.ncons[c] = nk;
            }
        }
        for (int g = 0; g < A.naggs; ++g)
            if (A.a_kind[g] != VD_AGG_COUNT)
                for (int f = 0; f < A.a_nf[g]; ++f)
                    if (A.a_col[g][f] >= 0) ref(L.aref, A.a_col[g][f]);
        // fast first round: pref1 = one int32 FK column + u8 lookups through
        // it whose constraints all became tables
        L.nfg = 0;
        L.fk_col = -1;
        if (ok && A.pred.nconj <= LT_COMMON) {
            const uint32_t base1 = L.pref1 & ((1u << ncols) - 1), gat1 = L.pref1 >> ncols;
            bool fast = base1 != 0 && (base1 & (base1 - 1)) == 0 && gat1 != 0;
            const int fkc = fast ? __builtin_ctz(base1) : -1;
            fast = fast && cols[fkc].dtype == VD_I32;
            for (int g = 0; g < A.ngathers && fast; ++g) {
                if (!((gat1 >> g) & 1u)) continue;
                int k = -1;
                for (int h = 0; h < L.ntab; ++h) k = L.tref[h] == ncols + g ? h : k;
                fast = A.g_fk[g] == fkc && A.g_dt[g] == VD_U8 && k >= 0;
                if (fast) { L.fg[L.nfg] = g; L.fgtab[L.nfg] = k; ++L.nfg; }
            }
            // every constraint on the first-round references is tabulated
            for (int c = 0; c <= VD_MAX_CONJ && fast; ++c) {
                if (c >= A.pred.nconj && c != VD_MAX_CONJ) continue;
                for (int k = 0; k < L.ncons[c] && fast; ++k) fast = !((L.pref1 >> L.cons[c][k].ref) & 1u);
            }
            if (fast) L.fk_col = fkc;
            else L.nfg = 0;
        }
        if (const char* fv = getenv("VD_LATE_FAST"))
            if (strcmp(fv, "0") == 0) L.nfg = 0;
        L.grab = 8;  // measured: 4 and 8 best (0.69 ms at SF100), 64 = static-like (0.76)
        if (const char* gv = getenv("VD_LATE_GRAB")) L.grab = (uint32_t)std::max(1, atoi(gv));
        // the late loads are integer (epsilon = INT64_MIN after widening)
        for (int c = 0; c < ncols; ++c)
            if ((((L.pref | L.aref) >> c) & 1u) && !is_int(cols[c].dtype)) return VD_OK;
        // one wave: as many CTAs per SM as fit (registers allow 4; the
        // pipeline workspace holds 4 x SMs partial slots)
        const size_t lsm = (size_t)(ncols + p->ngathers + p->naggs + 1) * LT_THREADS * 8 +
                           (size_t)(LT_THREADS / 32) * LT_QCAP * 4;
        const int per_sm = std::max(1, std::min(4, (int)((220 * 1024) / (lsm + 1024))));
        const int grid = grid_persistent(per_sm);
        unsigned int* dn = (unsigned int*)ws;
        Slot16* parts = (Slot16*)((char*)ws + 256);
        cudaError_t e = cudaMemsetAsync(dn, 0, 8, s);  // done counter + lead claim counter
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
        // (the attribute is per device context: set on every launch, as for
        // the other dynamic-shared-memory fragments)
#define LT_GO1(N8_, I32_, PV_)                                                                              \
    do {                                                                                                    \
        e = cudaFuncSetAttribute(k_pipe_late<N8_, I32_, PV_>, cudaFuncAttributeMaxDynamicSharedMemorySize, LT_SMEM_MAX); \
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }                     \
        k_pipe_late<N8_, I32_, PV_><<<grid, LT_THREADS, lsm, s>>>(A, L, parts, dn, (Slot16*)out);          \
    } while (0)
#define LT_GO(N8_, I32_)                                                                                    \
    do {                                                                                                    \
        if (L.ncons[0] < 0) LT_GO1(N8_, I32_, 0);                                                           \
        else if (L.nfg > 0) LT_GO1(N8_, I32_, 2);                                                           \
        else LT_GO1(N8_, I32_, 1);                                                                          \
    } while (0)
        if (n8 == 2) { if (i32) LT_GO(2, true); else LT_GO(2, false); }
        else if (n8 == 1) { if (i32) LT_GO(1, true); else LT_GO(1, false); }
        else LT_GO(0, true);
#undef LT_GO
#undef LT_GO1
        ++*nl;
        e = cudaGetLastError();
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
        set_fragment("late");
        *done = true;
        return VD_OK;
    }
    // shared memory: ring + warp slots + staging + calendar + barriers
    const int NS = (int)p->ngroups * (p->naggs + 1);
    size_t fixed = (size_t)GF_CW * NS * 8 + (size_t)GF_CW * 32 * (p->naggs + 1) * 8 +
                   (size_t)((A.year_days + 7) & ~7) * 2 + 2 * GF_MAXSTAGES * 8;
    const size_t budget = 200 * 1024;
    if (fixed + 2 * (size_t)off > budget) return VD_OK;
    int ns = (int)((budget - fixed) / (size_t)off);
    A.nstages = ns < 2 ? 2 : (ns > GF_MAXSTAGES ? GF_MAXSTAGES : ns);
    size_t smem = fixed + (size_t)A.nstages * off;
    unsigned int* dn = (unsigned int*)ws;
    Slot16* parts = (Slot16*)((char*)ws + 256);
    Slot16* rawp = (Slot16*)out;
    cudaError_t e = cudaMemsetAsync(dn, 0, 4, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    const int mode = p->sel_mode == VD_SEL_PREDICATED ? 1 : (p->sel_mode == VD_SEL_PREDICATED_LOOKUP ? 2 : 0);
#define GF_LAUNCH(M, SC)                                                                              \
    cudaFuncSetAttribute(k_pipe_gf<M, SC>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);    \
    k_pipe_gf<M, SC><<<grid, GF_THREADS, smem, s>>>(A, n / GF_TILE, parts, dn, rawp);
    const bool scalar = p->ngroups == 1;
    if (mode == 2) {
        if (scalar) { GF_LAUNCH(2, true) } else { GF_LAUNCH(0, false) }  // grouped: lookups are per qualifying row
    } else if (mode == 1) {
        if (scalar) { GF_LAUNCH(1, true) } else { GF_LAUNCH(1, false) }
    } else {
        if (scalar) { GF_LAUNCH(0, true) } else { GF_LAUNCH(0, false) }
    }
#undef GF_LAUNCH
    ++*nl;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    (void)nref;
    set_fragment("gather_fold");
    *done = true;
    return VD_OK;
}

// ---- generic -------------------------------------------------------------------
static size_t gen_smem(const vd_pipeline* p, bool smem_acc) {
    size_t nslots = (size_t)p->ngroups * (p->naggs + 1);
    size_t b = (size_t)GEN_WARPS * 32 * (p->naggs + 1) * sizeof(Slot16);
    if (smem_acc) b += (size_t)GEN_WARPS * nslots * sizeof(Slot16);
    return b;
}
static const size_t GEN_SMEM_MAX = 200 * 1024;

static size_t fold_ws_bytes_plan(const vd_pipeline* p) {
    size_t nslots = (size_t)p->ngroups * (p->naggs + 1);
    size_t grid = (size_t)grid_persistent(4);
    size_t gen = 256 + grid * nslots * sizeof(Slot16) + 2 * nslots * sizeof(Slot16) + 256;
    size_t q1 = 256 + grid * 8 * 6 * sizeof(Slot16) + 8 * 6 * sizeof(Slot16);
    size_t sc = 256 + grid * 2 * sizeof(Slot16) + 2 * sizeof(Slot16);
    size_t b = std::max(gen, std::max(q1, sc)) + 256;
    return (b + 255) & ~(size_t)255;
}

static int64_t mat_chunk_of(const vd_pipeline* p) { return p->mat_chunk > 0 ? p->mat_chunk : 1024; }

// bytes of the materialised intermediate vector (after the fold workspace)
static size_t mat_bytes(const vd_pipeline* p, int64_t n) {
    if (p->materialize == VD_MAT_BREAK) return ((size_t)n + 255) & ~(size_t)255;
    if (p->materialize == VD_MAT_CHUNKS) {
        const int64_t C = mat_chunk_of(p), nch = (n + C - 1) / C;
        return (((size_t)nch * C * 4 + 255) & ~(size_t)255) + (((size_t)nch * 4 + 255) & ~(size_t)255);
    }
    return 0;
}

size_t pipeline_ws_bytes(const vd_pipeline* p, int64_t n) { return fold_ws_bytes_plan(p) + mat_bytes(p, n); }

static void build_genplan(const vd_pipeline* p, const vd_column* cols, int ncols, const vd_column* dims, GenPlan* out) {
    GenPlan& P = *out;
    std::memset(&P, 0, sizeof(P));
    make_devpred(&p->pred, &P.pred);
    P.cols.ncols = ncols;
    for (int c = 0; c < ncols; ++c) { P.cols.p[c] = cols[c].data; P.cols.dt[c] = cols[c].dtype; }
    P.ngathers = p->ngathers;
    for (int g = 0; g < p->ngathers; ++g) {
        P.g_fk[g] = p->gathers[g].fk_col;
        P.g_bias[g] = p->gathers[g].bias;
        const vd_column& d = dims[p->gathers[g].dim_col];
        P.g_p[g] = d.data;
        P.g_len[g] = d.len;
        P.g_dt[g] = d.dtype;
    }
    P.nkey = p->nkeyparts;
    for (int k = 0; k < p->nkeyparts; ++k) {
        P.k_col[k] = p->key[k].col;
        P.k_fn[k] = p->key[k].fn;
        P.k_sub[k] = p->key[k].sub;
        P.k_mult[k] = p->key[k].mult;
    }
    P.ngroups = p->ngroups;
    P.naggs = p->naggs;
    for (int a = 0; a < p->naggs; ++a) {
        const vd_agg& g = p->aggs[a];
        P.agg[a].kind = g.kind;
        P.agg[a].nf = g.nfactors;
        bool isf = false;
        for (int f = 0; f < g.nfactors; ++f) {
            P.agg[a].col[f] = g.f[f].col;
            P.agg[a].a[f] = g.f[f].a;
            P.agg[a].b[f] = g.f[f].b;
            if (g.kind != VD_AGG_COUNT && g.f[f].col >= 0) {
                int dt = col_dtype(p, cols, ncols, dims, g.f[f].col);
                isf = isf || dt == VD_F32 || dt == VD_F64;
            }
        }
        P.agg[a].isf = isf;
    }
}

template <int SRC>
static vd_status launch_generic(const vd_pipeline* p, const GenPlan& P, int64_t n, int64_t n_iter, const MatSrc& M,
                                void* out, void* ws, cudaStream_t s, int* nl) {
    const int nslots = (int)(p->ngroups * (p->naggs + 1));
    bool smem_acc = gen_smem(p, true) <= GEN_SMEM_MAX;
    size_t smem = gen_smem(p, smem_acc);
    int grid = grid_persistent(smem_acc && smem > 100 * 1024 ? 1 : 2);
    int64_t maxg = (n_iter + GEN_THREADS - 1) / GEN_THREADS;
    if (maxg < 1) maxg = 1;
    if (grid > maxg) grid = (int)maxg;
    unsigned int* dn = (unsigned int*)ws;
    unsigned long long* derr = (unsigned long long*)((char*)ws + 128);
    Slot16* parts = (Slot16*)((char*)ws + 256);
    Slot16* gacc = parts;  // (global-atomic variant) accumulators
    unsigned long long* gmask = (unsigned long long*)(gacc + nslots);
    cudaError_t e = cudaMemsetAsync(ws, 0, 256, s);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    if (smem_acc) {
        if (smem > 48 * 1024)
            cudaFuncSetAttribute(k_pipe_generic<true, SRC>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        k_pipe_generic<true, SRC><<<grid, GEN_THREADS, smem, s>>>(P, n, parts, nslots, gacc, gmask, dn, (Slot16*)out,
                                                                  derr, M, n_iter);
    } else {
        // global accumulators: zero sums, +/- extremes for min/max images
        e = cudaMemsetAsync(gacc, 0, (size_t)nslots * sizeof(Slot16) + (size_t)nslots * 8, s);
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
        bool any_mm = false;
        for (int a = 0; a < p->naggs; ++a) any_mm |= (p->aggs[a].kind == VD_AGG_MIN || p->aggs[a].kind == VD_AGG_MAX);
        if (any_mm) { set_error("MIN/MAX with more groups than fit in shared memory"); return VD_E_UNSUPPORTED; }
        if (smem > 48 * 1024)
            cudaFuncSetAttribute(k_pipe_generic<false, SRC>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        k_pipe_generic<false, SRC><<<grid, GEN_THREADS, smem, s>>>(P, n, parts, nslots, gacc, gmask, dn,
                                                                   (Slot16*)out, derr, M, n_iter);
    }
    ++*nl;
    e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    return VD_OK;
}

static vd_status run_generic(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n, const vd_column* dims,
                             void* out, void* ws, cudaStream_t s, int* nl) {
    GenPlan P;
    build_genplan(p, cols, ncols, dims, &P);
    MatSrc M{};
    vd_status st = launch_generic<SRC_ROWS>(p, P, n, n, M, out, ws, s, nl);
    if (st == VD_OK) set_fragment("generic");
    return st;
}

// ============================================================================
// Materialising plans (vd_materialize): Break and Materialize
// ============================================================================
// First loop.  A single-column interval predicate on an aligned 4-byte
// column (the Fig 15 / C1 shape) is tested with vector loads; any other
// predicate with the generic per-row evaluation.
template <typename T>
struct IvlTerm {
    const T* p;
    T lo, hi;
};

template <typename T, bool FAST>
__device__ __forceinline__ bool mat_pred(const GenPlan& P, const IvlTerm<T>& t, int64_t row) {
    if (FAST) {
        const T v = __ldg(t.p + row);
        return v >= t.lo && v <= t.hi;  // NaN / INT_MIN (epsilon) fail: bounds chosen on the host
    }
    return gen_pred(P, row);
}

// Break (Fig 8): the predicate, fully data parallel, materialised
// as one byte per row; 4 rows per thread per step (one 32-bit store).
template <typename T, bool FAST>
__global__ void __launch_bounds__(256) k_mat_break(const __grid_constant__ GenPlan P, const IvlTerm<T> t, int64_t n,
                                                   uint8_t* __restrict__ flags) {
    const int64_t nq = (n + 3) / 4;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t q = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; q < nq; q += stride) {
        const int64_t r0 = q * 4;
        uint32_t w = 0;
        if (FAST && r0 + 4 <= n) {
            const int4 x = __ldg(reinterpret_cast<const int4*>(t.p) + q);
            T v[4];
            memcpy(&v[0], &x.x, 4); memcpy(&v[1], &x.y, 4); memcpy(&v[2], &x.z, 4); memcpy(&v[3], &x.w, 4);
#pragma unroll
            for (int j = 0; j < 4; ++j) w |= (uint32_t)(v[j] >= t.lo && v[j] <= t.hi) << (8 * j);
        } else {
#pragma unroll
            for (int j = 0; j < 4; ++j)
                if (r0 + j < n) w |= (uint32_t)mat_pred<T, FAST>(P, t, r0 + j) << (8 * j);
        }
        if (r0 + 4 <= n) {
            reinterpret_cast<uint32_t*>(flags)[q] = w;
        } else {
            for (int j = 0; r0 + j < n; ++j) flags[r0 + j] = (uint8_t)(w >> (8 * j));
        }
    }
}

// Materialize (Table 2; Fig 15 "Vectorized" P:L1202-1221): one
// warp per chunk of C rows (a run of Divide(Range, C)) writes the ascending
// positions of its qualifying rows, 32 rows per ballot, to the chunk's slice
// pos[c*C ..] -- the position buffer is filled sequentially within the chunk
// -- and its count to cnt[c].
template <typename T, bool FAST>
__global__ void __launch_bounds__(256) k_mat_chunks(const __grid_constant__ GenPlan P, const IvlTerm<T> t, int64_t n,
                                                    int64_t C, int64_t nchunks, int32_t* __restrict__ pos,
                                                    int32_t* __restrict__ cnt) {
    const int lane = threadIdx.x & 31;
    const unsigned lt = lanemask_lt();
    const int64_t gw = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * blockDim.x) >> 5;
    for (int64_t c = gw; c < nchunks; c += nw) {
        const int64_t r0 = c * C, r1 = min(n, r0 + C);
        int k = 0;
        for (int64_t r = r0 + lane; r - lane < r1; r += 32) {
            const bool f = r < r1 && mat_pred<T, FAST>(P, t, r);
            const unsigned b = __ballot_sync(VD_FULL, f);
            if (f) pos[r0 + k + __popc(b & lt)] = (int32_t)r;
            k += __popc(b);
        }
        if (lane == 0) cnt[c] = k;
    }
}

// Second loop of a scalar plan (one group, SUM/COUNT aggregates): the rows
// the first loop materialised -- flags set, or the positions of each chunk
// -- are resolved (Gather of every factor column at the position) and
// folded per thread (int128 / f64), then warp -> CTA -> grid (the last CTA,
// Fragment 2 of P:L929-931).
constexpr int MF_THREADS = 256;

template <int SRC>
__global__ void __launch_bounds__(MF_THREADS) k_mat_fold(const __grid_constant__ GenPlan P, const MatSrc M, int64_t n,
                                                         Slot16* __restrict__ parts, unsigned int* __restrict__ done,
                                                         Slot16* __restrict__ out) {
    const int NA = P.naggs;
    i128 si[VD_MAX_AGGS];
    double sf[VD_MAX_AGGS];
#pragma unroll
    for (int a = 0; a < VD_MAX_AGGS; ++a) { si[a] = 0; sf[a] = 0; }
    int64_t rows = 0;
    auto fold_row = [&](int64_t row) {
        ++rows;
#pragma unroll
        for (int a = 0; a < VD_MAX_AGGS; ++a) {
            if (a >= NA) break;
            const GenAgg& A = P.agg[a];
            if (A.kind == VD_AGG_COUNT) { si[a] += 1; continue; }
            if (A.isf) {
                double pr = 1.0;
                bool e = false;
                for (int f = 0; f < A.nf; ++f) {
                    double x = 0;
                    if (A.col[f] >= 0) {
                        const Val c = gen_fetch(P, A.col[f], row);
                        e |= c.eps;
                        x = c.isf ? c.f : (double)c.i;
                    }
                    pr *= (double)A.a[f] + (double)A.b[f] * x;
                }
                if (!e) sf[a] += pr;  // an epsilon factor: the value is epsilon, skipped (A5)
            } else {
                i128 pr = 1;
                bool e = false;
                for (int f = 0; f < A.nf; ++f) {
                    i128 x = 0;
                    if (A.col[f] >= 0) {
                        const Val c = gen_fetch(P, A.col[f], row);
                        e |= c.eps;
                        x = c.i;
                    }
                    pr *= (i128)A.a[f] + (i128)A.b[f] * x;
                }
                if (!e) si[a] += pr;
            }
        }
    };
    const int lane = threadIdx.x & 31;
    if (SRC == SRC_FLAGS) {
        const int64_t nq = (n + 3) / 4;
        const int64_t stride = (int64_t)gridDim.x * MF_THREADS;
        for (int64_t q = (int64_t)blockIdx.x * MF_THREADS + threadIdx.x; q < nq; q += stride) {
            const int64_t r0 = q * 4;
            uint32_t w;
            if (r0 + 4 <= n) {
                w = __ldg(reinterpret_cast<const uint32_t*>(M.flags) + q);
            } else {
                w = 0;
                for (int j = 0; r0 + j < n; ++j) w |= (uint32_t)M.flags[r0 + j] << (8 * j);
            }
            for (int j = 0; j < 4; ++j)
                if ((w >> (8 * j)) & 0xFFu) fold_row(r0 + j);
        }
    } else {
        const int64_t gw = ((int64_t)blockIdx.x * MF_THREADS + threadIdx.x) >> 5;
        const int64_t nw = ((int64_t)gridDim.x * MF_THREADS) >> 5;
        for (int64_t c = gw; c < M.nchunks; c += nw) {  // one warp per chunk's position list
            const int k1 = __ldg(M.cnt + c);
            for (int k = lane; k < k1; k += 32) fold_row((int64_t)__ldg(M.pos + c * M.C + k));
        }
    }
    // warp -> CTA -> grid, fixed order
    __shared__ Slot16 s_w[MF_THREADS / 32][VD_MAX_AGGS + 1];
    const int warp = threadIdx.x >> 5;
    for (int a = 0; a <= NA; ++a) {
        Slot16 v;
        if (a < NA && P.agg[a].isf && P.agg[a].kind != VD_AGG_COUNT) {
            put_f64(&v, warp_sum_f64(sf[a]));
        } else {
            put_i128(&v, warp_sum_i128(a < NA ? si[a] : (i128)rows));
        }
        if (lane == 0) s_w[warp][a] = v;
    }
    __syncthreads();
    if (threadIdx.x <= NA) {
        const int a = threadIdx.x;
        const bool fl = a < NA && P.agg[a].isf && P.agg[a].kind != VD_AGG_COUNT;
        Slot16 r = s_w[0][a];
        for (int w = 1; w < MF_THREADS / 32; ++w) {
            if (fl) put_f64(&r, get_f64(r) + get_f64(s_w[w][a]));
            else put_i128(&r, get_i128(r) + get_i128(s_w[w][a]));
        }
        parts[(size_t)blockIdx.x * (NA + 1) + a] = r;
    }
    __shared__ bool s_last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(done, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!s_last) return;
    __threadfence();
    fold_grid_parts(parts, NA + 1, out, [&](int a) {
        return (a < NA && P.agg[a].isf && P.agg[a].kind != VD_AGG_COUNT) ? (int)FK_F64_SUM : (int)FK_I128_SUM;
    });
}

// The predicate's fast form: <= 2 interval terms on ONE 16-byte aligned
// f32 / i32 column (epsilon outside the bounds), else generic evaluation.
template <typename T>
static bool ivl_term(const vd_pipeline* p, const vd_column* cols, int ncols, IvlTerm<T>* t) {
    if (p->ngathers != 0 || p->pred.nconj != 1 || p->pred.conj[0].nterms < 1 || p->pred.conj[0].nterms > 2)
        return false;
    const int c = p->pred.conj[0].terms[0].col;
    for (int k = 0; k < p->pred.conj[0].nterms; ++k)
        if (p->pred.conj[0].terms[k].col != c) return false;
    if (c >= ncols || ((uintptr_t)cols[c].data & 15) != 0) return false;
    const bool isf = std::is_same<T, float>::value;
    if (cols[c].dtype != (isf ? VD_F32 : VD_I32)) return false;
    t->p = (const T*)cols[c].data;
    if (isf) {
        int32_t fcmp[2] = {-1, -1};
        double fc[2] = {0, 0};
        for (int k = 0; k < p->pred.conj[0].nterms; ++k) {
            fcmp[k] = p->pred.conj[0].terms[k].cmp;
            fc[k] = p->pred.conj[0].terms[k].fval;
        }
        float lo, hi;
        if (!f32_interval(fcmp, fc, &lo, &hi)) return false;
        memcpy(&t->lo, &lo, 4);
        memcpy(&t->hi, &hi, 4);
        return true;
    }
    int64_t lo = (int64_t)INT32_MIN + 1, hi = INT32_MAX;  // epsilon never qualifies (A9)
    for (int k = 0; k < p->pred.conj[0].nterms; ++k)
        if (!term_interval(p->pred.conj[0].terms[k], &lo, &hi)) return false;
    if (lo > hi) { lo = 1; hi = 0; }
    int32_t l32 = (int32_t)lo, h32 = (int32_t)hi;
    memcpy(&t->lo, &l32, 4);
    memcpy(&t->hi, &h32, 4);
    return true;
}

template <typename T, bool FAST>
static void launch_mat_first(const vd_pipeline* p, const GenPlan& P, const IvlTerm<T>& t, int64_t n, const MatSrc& M,
                             cudaStream_t s, int* nl) {
    const int64_t grid = grid_persistent(8);
    if (p->materialize == VD_MAT_BREAK)
        k_mat_break<T, FAST><<<(int)std::max<int64_t>(1, std::min<int64_t>(grid, (n + 1023) / 1024)), 256, 0, s>>>(
            P, t, n, const_cast<uint8_t*>(M.flags));
    else
        k_mat_chunks<T, FAST><<<(int)std::max<int64_t>(1, std::min<int64_t>(grid, (M.nchunks + 7) / 8)), 256, 0, s>>>(
            P, t, n, M.C, M.nchunks, const_cast<int32_t*>(M.pos), const_cast<int32_t*>(M.cnt));
    ++*nl;
}

static vd_status run_materialized(const vd_pipeline* p, const vd_column* cols, int ncols, int64_t n,
                                  const vd_column* dims, void* out, void* ws, cudaStream_t s, int* nl) {
    GenPlan P;
    build_genplan(p, cols, ncols, dims, &P);
    char* mat = (char*)ws + fold_ws_bytes_plan(p);
    MatSrc M{};
    int64_t n_iter = n;
    if (p->materialize == VD_MAT_BREAK) {
        M.flags = (const uint8_t*)mat;
    } else {
        M.C = mat_chunk_of(p);
        M.nchunks = (n + M.C - 1) / M.C;
        M.pos = (const int32_t*)mat;
        M.cnt = (const int32_t*)(mat + (((size_t)M.nchunks * M.C * 4 + 255) & ~(size_t)255));
        n_iter = M.nchunks * M.C;
    }
    // first loop: the pipeline breaker writes its vector to memory
    IvlTerm<float> tf{};
    IvlTerm<int32_t> ti{};
    if (ivl_term<float>(p, cols, ncols, &tf)) launch_mat_first<float, true>(p, P, tf, n, M, s, nl);
    else if (ivl_term<int32_t>(p, cols, ncols, &ti)) launch_mat_first<int32_t, true>(p, P, ti, n, M, s, nl);
    else launch_mat_first<float, false>(p, P, tf, n, M, s, nl);
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    // second loop: fold the materialised rows
    const int src = p->materialize == VD_MAT_BREAK ? SRC_FLAGS : SRC_CHUNKS;
    bool simple = p->nkeyparts == 0 && p->ngroups == 1;
    for (int a = 0; a < p->naggs; ++a)
        simple = simple && (p->aggs[a].kind == VD_AGG_SUM || p->aggs[a].kind == VD_AGG_COUNT);
    vd_status st = VD_OK;
    if (simple) {
        unsigned int* dn = (unsigned int*)ws;
        Slot16* parts = (Slot16*)((char*)ws + 256);
        e = cudaMemsetAsync(dn, 0, 4, s);
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
        const int64_t work = src == SRC_FLAGS ? (n + 3) / 4 : M.nchunks * 32;
        const int grid = (int)std::max<int64_t>(
            1, std::min<int64_t>(grid_persistent(4), (work + MF_THREADS - 1) / MF_THREADS));
        if (src == SRC_FLAGS) k_mat_fold<SRC_FLAGS><<<grid, MF_THREADS, 0, s>>>(P, M, n, parts, dn, (Slot16*)out);
        else k_mat_fold<SRC_CHUNKS><<<grid, MF_THREADS, 0, s>>>(P, M, n, parts, dn, (Slot16*)out);
        ++*nl;
        e = cudaGetLastError();
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    } else if (src == SRC_FLAGS) {
        st = launch_generic<SRC_FLAGS>(p, P, n, n_iter, M, out, ws, s, nl);
    } else {
        st = launch_generic<SRC_CHUNKS>(p, P, n, n_iter, M, out, ws, s, nl);
    }
    if (st == VD_OK) set_fragment(p->materialize == VD_MAT_BREAK ? "break" : "mat_chunks");
    return st;
}

vd_status run_pipeline(const vd_pipeline* p, const vd_column* cols, int32_t ncols, int64_t n, const vd_column* dims,
                       int32_t, void* out, void* ws, size_t, cudaStream_t s, int* nl) {
    set_fragment("");
    if (n == 0) {
        set_fragment("empty");
        cudaError_t e = cudaMemsetAsync(out, 0, (size_t)p->ngroups * (p->naggs + 1) * 16, s);
        if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
        return VD_OK;
    }
    if (p->materialize != VD_MAT_NONE) return run_materialized(p, cols, ncols, n, dims, out, ws, s, nl);
    if (!p->force_generic) {
        bool done = false;
        vd_status st = try_q1(p, cols, ncols, n, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
        if (late_policy() == 2) {
            st = try_gf(p, cols, ncols, n, dims, out, ws, s, nl, &done, true);
            if (st != VD_OK || done) return st;
        }
        st = try_scalar(p, cols, ncols, n, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
        st = try_fkg(p, cols, ncols, n, dims, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
        if (late_policy() == 1) {
            // branching scalar FK joins with a selective lead: late loads beat
            // the dense star fragment (Q19) and the per-row selective FK sum
            // (Fig 16 at s <= 10%: 0.22 vs 0.49 ms at 1%)
            st = try_gf(p, cols, ncols, n, dims, out, ws, s, nl, &done, true);
            if (st != VD_OK || done) return st;
        }
        st = try_fkjs(p, cols, ncols, n, dims, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
        st = try_star(p, cols, ncols, n, dims, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
        st = try_gf(p, cols, ncols, n, dims, out, ws, s, nl, &done);
        if (st != VD_OK || done) return st;
    }
    return run_generic(p, cols, ncols, n, dims, out, ws, s, nl);
}

}  // namespace vd
