// k_group.cu -- grouped fold over a large key domain,
// vd_group_fold.  Product code.
//
// The paper's frontend sizes grouping tables from min/max metadata and
// addresses them by identity hashing: group(i) = key[i] -
// key.min in [0, D).  Fig 10/11's chain -- Partition -> Scatter ->
// FoldSum/FoldCount -> FoldSelect compaction -- keeps the
// Partition/Scatter virtual (§3.1.3) exactly as the small-domain
// fragments of k_pipeline.cu do; only the place of the group table changes.
// When D x aggregates no longer fits a shared-memory table (the
// VD_MAX_GROUPS-bounded fragments), the table "spills" to global memory
// (the workspace) and every qualifying row folds into it with global
// reductions (RED.ADD/MIN/MAX.64, resolved in L2).  Then the compaction is
// the FoldSelect of the non-empty slots (row count != 0) with Gathers of the
// slots' aggregates: chunk counts, a look-back scan, and an ordered emit.
//
//   k_grp_init   the table's identity values (sum 0, min +max, max -max)
//   k_grp_fold   scan -> predicate -> key -> values -> global reductions;
//                lanes of a warp holding the same key are combined first
//                (__match_any_sync + one leader), so clustered keys (runs
//                of equal keys, e.g. l_orderkey) cost one reduction per run
//   k_grp_count  non-empty slots per chunk of GRP_CHUNK slots
//   k_grp_emit   ascending keys, 16-byte aggregate slots, row counts
#include <algorithm>
#include <cstdlib>
#include <cstring>

#include "vd_common.cuh"
#include "vd_internal.h"
#include "vd_pred.cuh"

namespace vd {

constexpr int GRP_THREADS = 256;
constexpr int GRP_CHUNK = 4096;  // slots per compaction chunk (256 threads x 16)

// a 16-byte result slot (include/vd.h vd_partials layout)
struct GSlot16 {
    unsigned long long lo, hi;
};

struct GrpArgs {
    DevPred pred;
    DevCols cols;
    int32_t key_col;
    int64_t kmin, D;
    int32_t naggs;
    int32_t kind[VD_MAX_AGGS], nf[VD_MAX_AGGS], isf[VD_MAX_AGGS];
    int32_t fcol[VD_MAX_AGGS][VD_MAX_FACTORS];
    int64_t fa[VD_MAX_AGGS][VD_MAX_FACTORS], fb[VD_MAX_AGGS][VD_MAX_FACTORS];
    unsigned long long* table;  // [D][naggs + 1]
    int64_t n;
};

__global__ void __launch_bounds__(GRP_THREADS) k_grp_init(const __grid_constant__ GrpArgs a) {
    const int W = a.naggs + 1;
    const int64_t total = a.D * W;
    for (int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; k < total; k += (int64_t)gridDim.x * blockDim.x) {
        const int ag = (int)(k % W);
        unsigned long long v = 0;
        if (ag < a.naggs && a.kind[ag] == VD_AGG_MIN) v = (unsigned long long)INT64_MAX;
        if (ag < a.naggs && a.kind[ag] == VD_AGG_MAX) v = (unsigned long long)INT64_MIN;
        a.table[k] = v;
    }
}

// value of aggregate ag at row: product of factors; eps if a factor is epsilon.
// The row is a qualifying row, loaded late: one 64-byte block per factor
// column (fetch_typed_64b), not the default 128-byte line.
__device__ __forceinline__ bool grp_value(const GrpArgs& a, int ag, int64_t row, int64_t* vi, double* vf) {
    bool eps = false;
    if (a.isf[ag]) {
        double p = 1.0;
        for (int f = 0; f < a.nf[ag]; ++f) {
            double x = 0;
            if (a.fcol[ag][f] >= 0) {
                const Val c = fetch_typed_64b(a.cols.p[a.fcol[ag][f]], a.cols.dt[a.fcol[ag][f]], row);
                eps |= c.eps;
                x = c.isf ? c.f : (double)c.i;
            }
            p *= (double)a.fa[ag][f] + (double)a.fb[ag][f] * x;
        }
        *vf = p;
    } else {
        int64_t p = 1;
        for (int f = 0; f < a.nf[ag]; ++f) {
            int64_t x = 0;
            if (a.fcol[ag][f] >= 0) {
                const Val c = fetch_typed_64b(a.cols.p[a.fcol[ag][f]], a.cols.dt[a.fcol[ag][f]], row);
                eps |= c.eps;
                x = c.i;
            }
            p *= a.fa[ag][f] + a.fb[ag][f] * x;  // exact: proven from min/max metadata by the host
        }
        *vi = p;
    }
    return !eps;
}

// one table update: a global reduction that keeps the table's line in L2
// (evict_last) while the scan streams past it (evict_first)
__device__ __forceinline__ void grp_red(unsigned long long* slot, int kind, int isf, int64_t vi, double vf,
                                        uint64_t pol) {
    if (kind == VD_AGG_SUM) {
        if (isf) red_add_f64_hint((double*)slot, vf, pol);
        else red_add_u64_hint(slot, (unsigned long long)vi, pol);
    } else if (kind == VD_AGG_MIN) {
        red_min_s64_hint((long long*)slot, (long long)vi, pol);
    } else if (kind == VD_AGG_MAX) {
        red_max_s64_hint((long long*)slot, (long long)vi, pol);
    } else {
        red_add_u64_hint(slot, (unsigned long long)vi, pol);  // COUNT / row count
    }
}

__global__ void __launch_bounds__(GRP_THREADS) k_grp_fold(const __grid_constant__ GrpArgs a) {
    const uint64_t pol_t = policy_evict_last();
    const int lane = threadIdx.x & 31;
    const int W = a.naggs + 1;
    const int64_t warps = (int64_t)gridDim.x * (GRP_THREADS / 32);
    for (int64_t base = ((int64_t)blockIdx.x * (GRP_THREADS / 32) + (threadIdx.x >> 5)) * 32; base < a.n;
         base += warps * 32) {
        const int64_t row = base + lane;
        bool ok = row < a.n && eval_pred_row(a.pred, a.cols, row);  // branching: later columns only for qualifying rows
        int64_t g = -1;
        if (ok) {
            const Val k = fetch_typed_64b(a.cols.p[a.key_col], a.cols.dt[a.key_col], row);
            if (k.eps) ok = false;  // epsilon key: no group (reading A9)
            else g = k.i - a.kmin;  // in [0, D) by the key's metadata
        }
        if (!__any_sync(VD_FULL, ok)) continue;
        // lanes holding the same group fold through one leader (clustered keys)
        const unsigned m = __match_any_sync(VD_FULL, ok ? g : -1ll);
        if (!ok) continue;  // from here on only lanes of group m shuffle among themselves
        const int leader = __ffs(m) - 1;
        const int nm = __popc(m);
        unsigned long long* slot = a.table + (size_t)g * W;
        for (int ag = 0; ag < a.naggs; ++ag) {
            int64_t vi = 0;
            double vf = 0;
            bool has = false;
            const int kind = a.kind[ag];
            if (kind != VD_AGG_COUNT) has = grp_value(a, ag, row, &vi, &vf);
            if (kind == VD_AGG_COUNT) {
                if (lane == leader) grp_red(&slot[ag], VD_AGG_COUNT, 0, nm, 0, pol_t);
                continue;
            }
            if (nm == 1) {  // the common case for uniform keys: no shuffles
                if (has) grp_red(&slot[ag], kind, a.isf[ag], vi, vf, pol_t);
                continue;
            }
            // combine the group's lanes in lane order (fixed order per warp step)
            int64_t ci = (kind == VD_AGG_MIN) ? INT64_MAX : (kind == VD_AGG_MAX ? INT64_MIN : 0);
            double cf = 0;
            bool any = false;
            for (unsigned mm = m; mm; mm &= mm - 1) {
                const int l = __ffs(mm) - 1;
                const int64_t xi = __shfl_sync(m, vi, l);
                const double xf = __shfl_sync(m, vf, l);
                const bool xh = __shfl_sync(m, has, l);
                if (!xh) continue;
                any = true;
                if (kind == VD_AGG_SUM) { ci += xi; cf += xf; }
                else if (kind == VD_AGG_MIN) ci = xi < ci ? xi : ci;
                else ci = xi > ci ? xi : ci;
            }
            if (lane == leader && any) grp_red(&slot[ag], kind, a.isf[ag], ci, cf, pol_t);
        }
        if (lane == leader) grp_red(&slot[a.naggs], VD_AGG_COUNT, 0, nm, 0, pol_t);  // the group's row count
    }
}

// ---- interval fast path ---------------------------------------------------------
// The predicate is one conjunction of interval terms on at most two integer
// columns (Q15: lo <= l_shipdate <= hi).  Each thread takes 4 consecutive
// rows per step with one 128-bit load of the first filter column (a warp
// reads 512 contiguous bytes), tests the interval (epsilon = INT_MIN lies
// below every lo the host passes), and only qualifying rows touch the second
// filter column, the key and the value columns (branching late loads: for a
// selective filter most sectors of those columns are never read).  Rows fold
// with one global reduction per aggregate, without lane combining.
struct GrpIv {
    const void* c0;
    const void* c1;  // nullptr: no second filter column
    int32_t dt1;
    int64_t lo0, hi0, lo1, hi1;
};

__device__ __forceinline__ void grp_fold_row(const GrpArgs& a, int64_t row, uint64_t pol_t) {
    const Val k = fetch_typed_64b(a.cols.p[a.key_col], a.cols.dt[a.key_col], row);
    if (k.eps) return;
    unsigned long long* slot = a.table + (size_t)(k.i - a.kmin) * (a.naggs + 1);
    for (int ag = 0; ag < a.naggs; ++ag) {
        const int kind = a.kind[ag];
        if (kind == VD_AGG_COUNT) { grp_red(&slot[ag], VD_AGG_COUNT, 0, 1, 0, pol_t); continue; }
        int64_t vi = 0;
        double vf = 0;
        if (!grp_value(a, ag, row, &vi, &vf)) continue;
        grp_red(&slot[ag], kind, a.isf[ag], vi, vf, pol_t);
    }
    grp_red(&slot[a.naggs], VD_AGG_COUNT, 0, 1, 0, pol_t);
}

// Qualifying rows are compacted per warp into a shared-memory stack (ballot
// + popc ranks) and folded 32 at a time with every lane busy, so the
// (branchy, generic) key / value / reduction code runs once per 32
// qualifying rows instead of once per 32-row step that has any.
constexpr int GRP_QCAP = 32 + 4 * 32;  // one drain's worth + one step's worth

template <typename T0>
__global__ void __launch_bounds__(GRP_THREADS) k_grp_fold_iv(const __grid_constant__ GrpArgs a,
                                                            const __grid_constant__ GrpIv iv) {
    __shared__ int64_t s_q[GRP_THREADS / 32][GRP_QCAP];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const uint64_t pol_t = policy_evict_last(), pol_s = policy_evict_first();
    int64_t* q_ = s_q[warp];
    int cnt = 0;  // warp-uniform stack depth
    const unsigned lt = lanemask_lt();
    auto drain = [&](int k) {  // fold the top k (<= 32) stacked rows
        __syncwarp();
        if (lane < k) {
            const int64_t row = q_[cnt - k + lane];
            bool ok = true;
            if (iv.c1) {
                const Val y = fetch_typed_64b(iv.c1, iv.dt1, row);
                ok = !(y.eps || y.i < iv.lo1 || y.i > iv.hi1);
            }
            if (ok) grp_fold_row(a, row, pol_t);
        }
        cnt -= k;
        __syncwarp();
    };
    const int64_t nq = a.n / 4;
    const int64_t wstride = (int64_t)gridDim.x * GRP_THREADS;
    for (int64_t q0 = (int64_t)blockIdx.x * GRP_THREADS + warp * 32; q0 < nq; q0 += wstride) {
        const int64_t q = q0 + lane;
        int64_t x[4] = {INT64_MIN, INT64_MIN, INT64_MIN, INT64_MIN};
        if (q < nq) {
            if (sizeof(T0) == 4) {
                const int4 v = ld_stream16_hint((const int32_t*)iv.c0 + 4 * q, pol_s);
                x[0] = v.x; x[1] = v.y; x[2] = v.z; x[3] = v.w;
            } else {
                const int4 v0 = ld_stream16_hint((const int64_t*)iv.c0 + 4 * q, pol_s);
                const int4 v1 = ld_stream16_hint((const int64_t*)iv.c0 + 4 * q + 2, pol_s);
                x[0] = (int64_t)((uint64_t)(uint32_t)v0.y << 32 | (uint32_t)v0.x);
                x[1] = (int64_t)((uint64_t)(uint32_t)v0.w << 32 | (uint32_t)v0.z);
                x[2] = (int64_t)((uint64_t)(uint32_t)v1.y << 32 | (uint32_t)v1.x);
                x[3] = (int64_t)((uint64_t)(uint32_t)v1.w << 32 | (uint32_t)v1.z);
            }
        }
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const bool pass = x[j] >= iv.lo0 && x[j] <= iv.hi0;
            const unsigned b = __ballot_sync(VD_FULL, pass);
            if (pass) q_[cnt + __popc(b & lt)] = 4 * q + j;
            cnt += __popc(b);
        }
        while (cnt >= 32) drain(32);
    }
    if (cnt > 0) drain(cnt);
    // ragged tail (< 4 rows): one thread
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        for (int64_t row = nq * 4; row < a.n; ++row) {
            const Val x = fetch_typed(iv.c0, sizeof(T0) == 4 ? VD_I32 : VD_I64, row);
            if (x.eps || x.i < iv.lo0 || x.i > iv.hi0) continue;
            if (iv.c1) {
                const Val y = fetch_typed(iv.c1, iv.dt1, row);
                if (y.eps || y.i < iv.lo1 || y.i > iv.hi1) continue;
            }
            grp_fold_row(a, row, pol_t);
        }
    }
}

// non-empty slots per chunk
__global__ void __launch_bounds__(GRP_THREADS) k_grp_count(const unsigned long long* __restrict__ table, int64_t D,
                                                         int W, int32_t* __restrict__ counts) {
    __shared__ int s_w[GRP_THREADS / 32];
    const int64_t c0 = (int64_t)blockIdx.x * GRP_CHUNK;
    int cnt = 0;
    for (int j = threadIdx.x; j < GRP_CHUNK; j += GRP_THREADS) {
        const int64_t g = c0 + j;
        if (g < D && table[(size_t)g * W + (W - 1)] != 0) ++cnt;
    }
    for (int o = 16; o; o >>= 1) cnt += __shfl_xor_sync(VD_FULL, cnt, o);
    if ((threadIdx.x & 31) == 0) s_w[threadIdx.x >> 5] = cnt;
    __syncthreads();
    if (threadIdx.x == 0) {
        int t = 0;
        for (int w = 0; w < GRP_THREADS / 32; ++w) t += s_w[w];
        counts[blockIdx.x] = t;
    }
}

// FoldSelect(row count != 0) + Gathers, in ascending slot order: each
// warp takes 512 consecutive slots (16 per lane-step), ranks by ballot.
__global__ void __launch_bounds__(GRP_THREADS) k_grp_emit(const unsigned long long* __restrict__ table, int64_t D,
                                                        int naggs, const int32_t* __restrict__ isf,
                                                        const int32_t* __restrict__ kinds, int64_t kmin,
                                                        const int32_t* __restrict__ counts,
                                                        const int64_t* __restrict__ offs, int64_t nchunks,
                                                        int64_t* __restrict__ out_keys, GSlot16* __restrict__ out_aggs,
                                                        int64_t* __restrict__ out_rows, int64_t* __restrict__ out_ng) {
    __shared__ int s_w[GRP_THREADS / 32];
    const int W = naggs + 1;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int64_t c0 = (int64_t)blockIdx.x * GRP_CHUNK;
    constexpr int PER_WARP = GRP_CHUNK / (GRP_THREADS / 32);
    // warp prefix within the chunk
    int mine = 0;
    const int64_t w0 = c0 + (int64_t)warp * PER_WARP;
    for (int j = lane; j < PER_WARP; j += 32) {
        const int64_t g = w0 + j;
        if (g < D && table[(size_t)g * W + naggs] != 0) ++mine;
    }
    for (int o = 16; o; o >>= 1) mine += __shfl_xor_sync(VD_FULL, mine, o);
    if (lane == 0) s_w[warp] = mine;
    __syncthreads();
    int64_t pos = offs[blockIdx.x];
    for (int w = 0; w < warp; ++w) pos += s_w[w];
    for (int j0 = 0; j0 < PER_WARP; j0 += 32) {
        const int64_t g = w0 + j0 + lane;
        const unsigned long long rc = g < D ? table[(size_t)g * W + naggs] : 0ull;
        const bool ne = rc != 0;
        const unsigned b = __ballot_sync(VD_FULL, ne);
        if (ne) {
            const int64_t p = pos + __popc(b & lanemask_lt());
            out_keys[p] = g + kmin;
            out_rows[p] = (int64_t)rc;
            for (int ag = 0; ag < naggs; ++ag) {
                unsigned long long v = table[(size_t)g * W + ag];
                // MIN/MAX of a group without a non-epsilon value: still the
                // identity -> epsilon (reading A5; the host proved |values| <
                // INT64_MAX, so the identity is never a real result)
                if (kinds[ag] == VD_AGG_MIN && v == (unsigned long long)INT64_MAX) v = (unsigned long long)INT64_MIN;
                GSlot16 s;
                s.lo = v;
                s.hi = isf[ag] ? 0ull : (((long long)v < 0) ? ~0ull : 0ull);  // i64 -> i128
                out_aggs[(size_t)p * naggs + ag] = s;
            }
        }
        pos += __popc(b);
    }
    if (blockIdx.x == nchunks - 1 && threadIdx.x == 0) *out_ng = offs[blockIdx.x] + counts[blockIdx.x];
}

size_t group_ws_bytes(int64_t D, int naggs) {
    const int64_t nch = (D + GRP_CHUNK - 1) / GRP_CHUNK;
    size_t b = 256;                                                  // isf[] (device copy)
    b += ((size_t)D * (naggs + 1) * 8 + 255) & ~(size_t)255;         // table
    b += ((size_t)nch * 4 + 255) & ~(size_t)255;                     // chunk counts
    b += ((size_t)nch * 8 + 255) & ~(size_t)255;                     // chunk offsets
    b += scan_ws_bytes(nch);
    return b;
}

cudaError_t launch_group_fold(const DevCols& cols, const DevPred& pred, int64_t n, int key_col, int64_t kmin,
                              int64_t D, const vd_agg* aggs, const int32_t* isf, int naggs, int64_t* out_keys,
                              void* out_aggs, int64_t* out_rows, int64_t* out_ng, void* ws, cudaStream_t s,
                              int* nl) {
    GrpArgs A;
    std::memset(&A, 0, sizeof(A));
    A.pred = pred;
    A.cols = cols;
    A.key_col = key_col;
    A.kmin = kmin;
    A.D = D;
    A.naggs = naggs;
    A.n = n;
    for (int g = 0; g < naggs; ++g) {
        A.kind[g] = aggs[g].kind;
        A.nf[g] = aggs[g].kind == VD_AGG_COUNT ? 0 : aggs[g].nfactors;
        A.isf[g] = isf[g];
        for (int f = 0; f < A.nf[g]; ++f) {
            A.fcol[g][f] = aggs[g].f[f].col;
            A.fa[g][f] = aggs[g].f[f].a;
            A.fb[g][f] = aggs[g].f[f].b;
        }
    }
    const int64_t nch = (D + GRP_CHUNK - 1) / GRP_CHUNK;
    char* w = (char*)ws;
    int32_t* d_isf = (int32_t*)w;
    w += 256;
    A.table = (unsigned long long*)w;
    w += ((size_t)D * (naggs + 1) * 8 + 255) & ~(size_t)255;
    int32_t* counts = (int32_t*)w;
    w += ((size_t)nch * 4 + 255) & ~(size_t)255;
    int64_t* offs = (int64_t*)w;
    w += ((size_t)nch * 8 + 255) & ~(size_t)255;
    void* scan_ws = w;

    int32_t hdr[2 * VD_MAX_AGGS];
    for (int g = 0; g < VD_MAX_AGGS; ++g) {
        hdr[g] = g < naggs ? isf[g] : 0;
        hdr[VD_MAX_AGGS + g] = g < naggs ? aggs[g].kind : 0;
    }
    cudaError_t e = cudaMemcpyAsync(d_isf, hdr, sizeof(hdr), cudaMemcpyHostToDevice, s);
    if (e != cudaSuccess) return e;
    const int sms = num_sms();
    k_grp_init<<<sms * 8, GRP_THREADS, 0, s>>>(A);
    ++*nl;
    // interval fast path: one conjunction of integer interval terms on at
    // most two columns, the first one i32/i64 and 16-byte aligned
    GrpIv iv;
    std::memset(&iv, 0, sizeof(iv));
    bool fast = !getenv("VD_GRP_GENERIC") && pred.nconj == 1 && pred.nterms[0] >= 1;
    int fc[2] = {-1, -1};
    int64_t lo[2] = {INT64_MIN + 1, INT64_MIN + 1}, hi[2] = {INT64_MAX, INT64_MAX};
    for (int k = 0; fast && k < pred.nterms[0]; ++k) {
        const DevTerm& t = pred.t[0][k];
        int slot = t.col == fc[0] ? 0 : (t.col == fc[1] ? 1 : (fc[0] < 0 ? 0 : (fc[1] < 0 ? 1 : -1)));
        if (slot < 0 || cols.dt[t.col] == VD_F32 || cols.dt[t.col] == VD_F64) { fast = false; break; }
        fc[slot] = t.col;
        switch (t.cmp) {
        case VD_CMP_GT: if (t.iv == INT64_MAX) fast = false; else lo[slot] = std::max(lo[slot], t.iv + 1); break;
        case VD_CMP_GE: lo[slot] = std::max(lo[slot], t.iv); break;
        case VD_CMP_LT: if (t.iv == INT64_MIN) fast = false; else hi[slot] = std::min(hi[slot], t.iv - 1); break;
        case VD_CMP_LE: hi[slot] = std::min(hi[slot], t.iv); break;
        case VD_CMP_EQ: lo[slot] = std::max(lo[slot], t.iv); hi[slot] = std::min(hi[slot], t.iv); break;
        default: fast = false;
        }
    }
    if (fast) {
        // epsilon (the type's minimum) must fall outside the interval
        for (int j = 0; j < 2; ++j) {
            if (fc[j] < 0) continue;
            const int32_t dt = cols.dt[fc[j]];
            const int64_t eps = dt == VD_I32 ? (int64_t)INT32_MIN : (dt == VD_I64 ? INT64_MIN : 0xFF);
            if (dt == VD_U8) { if (hi[j] >= eps) hi[j] = eps - 1; }
            else if (lo[j] <= eps) lo[j] = eps + 1;
        }
        fast = (cols.dt[fc[0]] == VD_I32 || cols.dt[fc[0]] == VD_I64) && ((uintptr_t)cols.p[fc[0]] % 16) == 0;
    }
    if (fast && n > 0) {
        iv.c0 = cols.p[fc[0]];
        iv.lo0 = lo[0];
        iv.hi0 = hi[0];
        if (fc[1] >= 0) {
            iv.c1 = cols.p[fc[1]];
            iv.dt1 = cols.dt[fc[1]];
            iv.lo1 = lo[1];
            iv.hi1 = hi[1];
        }
        const int64_t nq = n / 4;
        const int grid = (int)std::max<int64_t>(1, std::min<int64_t>((nq + GRP_THREADS - 1) / GRP_THREADS,
                                                                     (int64_t)sms * 8));
        if (cols.dt[fc[0]] == VD_I32) k_grp_fold_iv<int32_t><<<grid, GRP_THREADS, 0, s>>>(A, iv);
        else k_grp_fold_iv<int64_t><<<grid, GRP_THREADS, 0, s>>>(A, iv);
        ++*nl;
    } else if (n > 0) {
        const int64_t warps_needed = (n + 31) / 32;
        const int64_t blocks = (warps_needed + GRP_THREADS / 32 - 1) / (GRP_THREADS / 32);
        const int grid = (int)std::min<int64_t>(blocks, (int64_t)sms * 8);
        k_grp_fold<<<grid, GRP_THREADS, 0, s>>>(A);
        ++*nl;
    }
    k_grp_count<<<(unsigned)nch, GRP_THREADS, 0, s>>>(A.table, D, naggs + 1, counts);
    ++*nl;
    e = launch_scan_i32(counts, nch, offs, scan_ws, s, nl);
    if (e != cudaSuccess) return e;
    k_grp_emit<<<(unsigned)nch, GRP_THREADS, 0, s>>>(A.table, D, naggs, d_isf, d_isf + VD_MAX_AGGS, kmin, counts, offs, nch, out_keys,
                                                    (GSlot16*)out_aggs, out_rows, out_ng);
    ++*nl;
    return cudaGetLastError();
}

}  // namespace vd
