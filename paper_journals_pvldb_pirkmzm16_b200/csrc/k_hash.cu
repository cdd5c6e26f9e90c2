// k_hash.cu -- grouped fold over SPARSE keys with open-addressing hash tables
// (SURVEY §8(f) NEXT-4), vd_hash_group_fold / vd_merge_groups.  Product code.
//
// The paper's frontend groups through "identity hashing on open hashtables"
// sized "from the input domain (using only min and max)" --
// vd_group_fold.  That stops working when the domain max - min + 1 is far
// larger than the number of distinct keys (64-bit surrogate keys, hashed
// strings, keys of a filtered sub-population): the table would not fit.
// Here the table is sized from a distinct-key estimate instead and keys are
// placed by a 64-bit mixing hash with linear probing:
//
//   level 1, shared memory : each CTA folds its rows into a private table of
//       HG_SLOTS entries (key + one 64-bit word per aggregate + row count);
//       a key that finds no free slot within HG_PROBES probes SPILLS --
//   level 2, global memory : the workspace table of `capacity` entries,
//       keys claimed with atomicCAS, aggregates folded with global
//       reductions (RED.ADD / MIN / MAX.64, resolved in L2).  At the end of
//       its rows a CTA flushes its shared table into the global one, one
//       reduction per (key, aggregate).
//   compaction: the FoldSelect of the occupied slots with Gathers of their
//       keys and aggregates (Fig 11's compaction), in TABLE order
//       (a hash table has no key order; vd_group_fold keeps ascending order).
//
// Lanes of a warp holding the same key are combined first (__match_any_sync
// + one leader), so clustered keys cost one table update per run.  The
// Partition / Scatter of Fig 10/11 stay virtual: a row's slot is the
// scatter position, never materialised (§3.1.3).
//
// vd_merge_groups is the cross-GPU step for compacted groups: every rank's
// (keys, aggregates, rows) lists, concatenated, are re-inserted into one
// table with 128-bit / f64 / min / max combination and compacted again.
#include <algorithm>
#include <cstdlib>
#include <cstring>

#include "vd_common.cuh"
#include "vd_internal.h"
#include "vd_pred.cuh"

namespace vd {

constexpr int HG_THREADS = 256;
constexpr int HG_SLOTS = 1024;  // shared-memory table entries per CTA
constexpr int HG_PROBES = 8;    // probes in the shared table before spilling
constexpr int HG_CHUNK = 4096;  // slots per compaction chunk
constexpr int64_t HG_EMPTY = INT64_MIN;  // epsilon keys never enter a table (A9)

__device__ __forceinline__ uint64_t hg_mix(int64_t k) {  // splitmix64 finaliser
    uint64_t x = (uint64_t)k;
    x ^= x >> 30;
    x *= 0xBF58476D1CE4E5B9ull;
    x ^= x >> 27;
    x *= 0x94D049BB133111EBull;
    x ^= x >> 31;
    return x;
}

struct HgArgs {
    DevPred pred;
    DevCols cols;
    int32_t key_col;
    int32_t naggs;
    int32_t kind[VD_MAX_AGGS], nf[VD_MAX_AGGS], isf[VD_MAX_AGGS];
    int32_t fcol[VD_MAX_AGGS][VD_MAX_FACTORS];
    int64_t fa[VD_MAX_AGGS][VD_MAX_FACTORS], fb[VD_MAX_AGGS][VD_MAX_FACTORS];
    int64_t n;
    uint64_t mask;                // capacity - 1 (power of two)
    int64_t* keys;                // [capacity]
    unsigned long long* vals;     // [capacity][naggs + 1]
    unsigned long long* overflow; // set when the global table is full
};

__device__ __forceinline__ unsigned long long hg_identity(int kind) {
    if (kind == VD_AGG_MIN) return (unsigned long long)INT64_MAX;
    if (kind == VD_AGG_MAX) return (unsigned long long)INT64_MIN;
    return 0ull;
}

__global__ void __launch_bounds__(HG_THREADS) k_hg_init(const __grid_constant__ HgArgs a) {
    const int W = a.naggs + 1;
    const int64_t cap = (int64_t)a.mask + 1;
    for (int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; k < cap * W; k += (int64_t)gridDim.x * blockDim.x) {
        const int ag = (int)(k % W);
        a.vals[k] = ag < a.naggs ? hg_identity(a.kind[ag]) : 0ull;
        if (ag == 0) a.keys[k / W] = HG_EMPTY;
    }
}

// value of aggregate ag at `row`: the product of its factors; false if a
// factor is epsilon (the value is epsilon, skipped by the fold: A5)
__device__ __forceinline__ bool hg_value(const HgArgs& a, int ag, int64_t row, unsigned long long* v) {
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
        *v = (unsigned long long)__double_as_longlong(p);
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
        *v = (unsigned long long)p;
    }
    return !eps;
}

// combine two 64-bit aggregate words (SUM/COUNT add, MIN/MAX)
__device__ __forceinline__ unsigned long long hg_comb(int kind, int isf, unsigned long long x, unsigned long long y) {
    if (kind == VD_AGG_SUM && isf)
        return (unsigned long long)__double_as_longlong(__longlong_as_double((long long)x) +
                                                        __longlong_as_double((long long)y));
    if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) return x + y;
    const long long a = (long long)x, b = (long long)y;
    return (unsigned long long)(kind == VD_AGG_MIN ? (a < b ? a : b) : (a > b ? a : b));
}

// fold one word into a table slot with the matching atomic (shared or global)
__device__ __forceinline__ void hg_atomic(unsigned long long* p, int kind, int isf, unsigned long long v) {
    if (kind == VD_AGG_SUM && isf) atomicAdd((double*)p, __longlong_as_double((long long)v));
    else if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) atomicAdd(p, v);
    else if (kind == VD_AGG_MIN) atomicMin((long long*)p, (long long)v);
    else atomicMax((long long*)p, (long long)v);
}

// global insert-or-find: the slot index of `key`, -1 if the table is full
__device__ __forceinline__ int64_t hg_global_slot(const HgArgs& a, int64_t key) {
    uint64_t h = hg_mix(key) & a.mask;
    for (uint64_t probe = 0; probe <= a.mask; ++probe) {
        const int64_t cur = ((volatile int64_t*)a.keys)[h];
        if (cur == key) return (int64_t)h;
        if (cur == HG_EMPTY) {
            const long long prev = atomicCAS((unsigned long long*)&a.keys[h], (unsigned long long)HG_EMPTY,
                                             (unsigned long long)key);
            if (prev == (long long)HG_EMPTY || prev == key) return (int64_t)h;
        }
        h = (h + 1) & a.mask;
    }
    atomicOr(a.overflow, 1ull);
    return -1;
}

// Fold one row's words (v[ag], has[ag]; the row count is word naggs) into
// the CTA's shared table, or spill to the global one.  Once the shared table
// is 3/4 full a new key gets only 2 probes there: with uniform keys over a
// large domain a CTA sees few repeats, and probing a full table only adds
// latency.
__device__ __forceinline__ void hg_insert(const HgArgs& a, long long* s_key, unsigned long long* s_val,
                                          int* s_used, int64_t key, const unsigned long long* v, const bool* has,
                                          uint64_t pol_t) {
    const int W = a.naggs + 1;
    uint32_t h = (uint32_t)(hg_mix(key) & (HG_SLOTS - 1));
    const int probes = *((volatile int*)s_used) < HG_SLOTS * 3 / 4 ? HG_PROBES : 2;
    int slot = -1;
    for (int p = 0; p < probes; ++p) {
        const long long cur = s_key[h];
        if (cur == key) { slot = (int)h; break; }
        if (cur == HG_EMPTY) {
            const long long prev = (long long)atomicCAS((unsigned long long*)&s_key[h], (unsigned long long)HG_EMPTY,
                                                        (unsigned long long)key);
            if (prev == HG_EMPTY) { atomicAdd(s_used, 1); slot = (int)h; break; }
            if (prev == key) { slot = (int)h; break; }
        }
        h = (h + 1) & (HG_SLOTS - 1);
    }
    if (slot >= 0) {
        unsigned long long* dst = s_val + (size_t)slot * W;
        for (int ag = 0; ag <= a.naggs; ++ag)
            if (has[ag]) hg_atomic(dst + ag, ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT, ag < a.naggs ? a.isf[ag] : 0, v[ag]);
        return;
    }
    const int64_t g = hg_global_slot(a, key);  // level 2: spill to the global table
    if (g < 0) return;
    unsigned long long* dst = a.vals + (size_t)g * W;
    for (int ag = 0; ag <= a.naggs; ++ag) {
        if (!has[ag]) continue;
        const int kind = ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT;
        const int fl = ag < a.naggs ? a.isf[ag] : 0;
        if (kind == VD_AGG_SUM && fl) red_add_f64_hint((double*)(dst + ag), __longlong_as_double((long long)v[ag]), pol_t);
        else if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) red_add_u64_hint(dst + ag, v[ag], pol_t);
        else if (kind == VD_AGG_MIN) red_min_s64_hint((long long*)(dst + ag), (long long)v[ag], pol_t);
        else red_max_s64_hint((long long*)(dst + ag), (long long)v[ag], pol_t);
    }
}

// flush the CTA's shared table into the global one
__device__ __forceinline__ void hg_flush(const HgArgs& a, const long long* s_key, const unsigned long long* s_val) {
    const int W = a.naggs + 1;
    for (int k = threadIdx.x; k < HG_SLOTS; k += HG_THREADS) {
        const long long key = s_key[k];
        if (key == HG_EMPTY) continue;
        const int64_t g = hg_global_slot(a, key);
        if (g < 0) continue;
        for (int ag = 0; ag <= a.naggs; ++ag) {
            const int kind = ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT;
            const unsigned long long x = s_val[(size_t)k * W + ag];
            if (x == hg_identity(kind) && kind != VD_AGG_SUM && kind != VD_AGG_COUNT) continue;
            hg_atomic(a.vals + (size_t)g * W + ag, kind, ag < a.naggs ? a.isf[ag] : 0, x);
        }
    }
}

// Interval fast path (the predicate is one conjunction of integer interval
// terms on at most two columns, the first 16-byte aligned -- Q15's
// l_shipdate window): 4 rows per thread per 128-bit evict-first load of the
// filter column, qualifying rows compacted per warp into a shared-memory
// queue and folded 32 at a time with every lane busy (key, values and the
// second filter column loaded late, 64-byte blocks).
struct HgIv {
    const void* c0;
    const void* c1;  // nullptr: no second filter column
    int32_t dt0, dt1;
    int64_t lo0, hi0, lo1, hi1;
};
constexpr int HG_QCAP = 32 + 4 * 32;

__global__ void __launch_bounds__(HG_THREADS) k_hg_fold_iv(const __grid_constant__ HgArgs a,
                                                          const __grid_constant__ HgIv iv) {
    extern __shared__ __align__(16) unsigned long long s_tab[];
    __shared__ int64_t s_q[HG_THREADS / 32][HG_QCAP];
    __shared__ int s_used;
    const int W = a.naggs + 1;
    long long* s_key = (long long*)s_tab;
    unsigned long long* s_val = s_tab + HG_SLOTS;
    for (int k = threadIdx.x; k < HG_SLOTS; k += HG_THREADS) s_key[k] = HG_EMPTY;
    for (int k = threadIdx.x; k < HG_SLOTS * W; k += HG_THREADS) {
        const int ag = k % W;
        s_val[k] = ag < a.naggs ? hg_identity(a.kind[ag]) : 0ull;
    }
    if (threadIdx.x == 0) s_used = 0;
    __syncthreads();
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const uint64_t pol_t = policy_evict_last(), pol_s = policy_evict_first();
    int64_t* q_ = s_q[warp];
    int cnt = 0;
    const unsigned lt = lanemask_lt();
    auto fold_row = [&](int64_t row) {
        if (iv.c1) {
            const Val y = fetch_typed_64b(iv.c1, iv.dt1, row);
            if (y.eps || y.i < iv.lo1 || y.i > iv.hi1) return;
        }
        const Val k = fetch_typed_64b(a.cols.p[a.key_col], a.cols.dt[a.key_col], row);
        if (k.eps) return;  // epsilon key: no group (A9)
        unsigned long long v[VD_MAX_AGGS + 1];
        bool has[VD_MAX_AGGS + 1];
        for (int ag = 0; ag < a.naggs; ++ag) {
            if (a.kind[ag] == VD_AGG_COUNT) { v[ag] = 1; has[ag] = true; }
            else has[ag] = hg_value(a, ag, row, &v[ag]);
        }
        v[a.naggs] = 1;
        has[a.naggs] = true;
        hg_insert(a, s_key, s_val, &s_used, k.i, v, has, pol_t);
    };
    auto drain = [&](int k) {  // fold the top k (<= 32) queued rows
        __syncwarp();
        if (lane < k) fold_row(q_[cnt - k + lane]);
        cnt -= k;
        __syncwarp();
    };
    const int64_t nq = a.n / 4;
    const int64_t wstride = (int64_t)gridDim.x * HG_THREADS;
    for (int64_t q0 = (int64_t)blockIdx.x * HG_THREADS + warp * 32; q0 < nq; q0 += wstride) {
        const int64_t q = q0 + lane;
        int64_t x[4] = {INT64_MIN, INT64_MIN, INT64_MIN, INT64_MIN};
        if (q < nq) {
            if (iv.dt0 == VD_I32) {
                const int4 w = ld_stream16_hint((const int32_t*)iv.c0 + 4 * q, pol_s);
                x[0] = w.x; x[1] = w.y; x[2] = w.z; x[3] = w.w;
            } else {
                const int4 w0 = ld_stream16_hint((const int64_t*)iv.c0 + 4 * q, pol_s);
                const int4 w1 = ld_stream16_hint((const int64_t*)iv.c0 + 4 * q + 2, pol_s);
                x[0] = (int64_t)((uint64_t)(uint32_t)w0.y << 32 | (uint32_t)w0.x);
                x[1] = (int64_t)((uint64_t)(uint32_t)w0.w << 32 | (uint32_t)w0.z);
                x[2] = (int64_t)((uint64_t)(uint32_t)w1.y << 32 | (uint32_t)w1.x);
                x[3] = (int64_t)((uint64_t)(uint32_t)w1.w << 32 | (uint32_t)w1.z);
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
    if (blockIdx.x == 0 && threadIdx.x == 0) {  // ragged tail (< 4 rows)
        for (int64_t row = nq * 4; row < a.n; ++row) {
            const Val x = fetch_typed(iv.c0, iv.dt0, row);
            if (!(x.eps || x.i < iv.lo0 || x.i > iv.hi0)) fold_row(row);
        }
    }
    __syncthreads();
    hg_flush(a, s_key, s_val);
}

__global__ void __launch_bounds__(HG_THREADS) k_hg_fold(const __grid_constant__ HgArgs a) {
    extern __shared__ __align__(16) unsigned long long s_tab[];  // [HG_SLOTS] keys, then [HG_SLOTS][W] words
    const int W = a.naggs + 1;
    long long* s_key = (long long*)s_tab;
    unsigned long long* s_val = s_tab + HG_SLOTS;
    for (int k = threadIdx.x; k < HG_SLOTS; k += HG_THREADS) s_key[k] = HG_EMPTY;
    for (int k = threadIdx.x; k < HG_SLOTS * W; k += HG_THREADS) {
        const int ag = k % W;
        s_val[k] = ag < a.naggs ? hg_identity(a.kind[ag]) : 0ull;
    }
    __syncthreads();
    const int lane = threadIdx.x & 31;
    const int64_t warps = (int64_t)gridDim.x * (HG_THREADS / 32);
    for (int64_t base = ((int64_t)blockIdx.x * (HG_THREADS / 32) + (threadIdx.x >> 5)) * 32; base < a.n;
         base += warps * 32) {
        const int64_t row = base + lane;
        bool ok = row < a.n && eval_pred_row(a.pred, a.cols, row);
        int64_t key = HG_EMPTY;
        if (ok) {
            const Val k = fetch_typed_64b(a.cols.p[a.key_col], a.cols.dt[a.key_col], row);
            if (k.eps) ok = false;  // epsilon key: no group (A9)
            else key = k.i;
        }
        if (!__any_sync(VD_FULL, ok)) continue;
        // this row's aggregate words (the row count is word naggs)
        unsigned long long v[VD_MAX_AGGS + 1];
        bool has[VD_MAX_AGGS + 1];
#pragma unroll
        for (int ag = 0; ag <= VD_MAX_AGGS; ++ag) { v[ag] = 0; has[ag] = false; }
        if (ok) {
            for (int ag = 0; ag < a.naggs; ++ag) {
                if (a.kind[ag] == VD_AGG_COUNT) { v[ag] = 1; has[ag] = true; }
                else has[ag] = hg_value(a, ag, row, &v[ag]);
            }
            v[a.naggs] = 1;
            has[a.naggs] = true;
        }
        // lanes with the same key: one leader carries the combined words
        const unsigned m = __match_any_sync(VD_FULL, ok ? key : HG_EMPTY);
        if (!ok) continue;
        const int leader = __ffs(m) - 1;
        for (int ag = 0; ag <= a.naggs; ++ag) {
            const int kind = ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT;
            const int fl = ag < a.naggs ? a.isf[ag] : 0;
            unsigned long long c = hg_identity(kind);
            bool any = false;
            for (unsigned mm = m; mm; mm &= mm - 1) {  // lane order: fixed per warp step
                const int l = __ffs(mm) - 1;
                const unsigned long long x = __shfl_sync(m, v[ag], l);
                const bool xh = __shfl_sync(m, has[ag], l);
                if (xh) { c = any ? hg_comb(kind, fl, c, x) : x; any = true; }
            }
            v[ag] = c;
            has[ag] = any;
        }
        if (lane != leader) continue;
        // level 1: the CTA's shared table
        uint32_t h = (uint32_t)(hg_mix(key) & (HG_SLOTS - 1));
        int slot = -1;
        for (int p = 0; p < HG_PROBES; ++p) {
            const long long cur = s_key[h];
            if (cur == key) { slot = (int)h; break; }
            if (cur == HG_EMPTY) {
                const long long prev = (long long)atomicCAS((unsigned long long*)&s_key[h],
                                                            (unsigned long long)HG_EMPTY, (unsigned long long)key);
                if (prev == HG_EMPTY || prev == key) { slot = (int)h; break; }
            }
            h = (h + 1) & (HG_SLOTS - 1);
        }
        unsigned long long* dst;
        if (slot >= 0) {
            dst = s_val + (size_t)slot * W;
        } else {  // level 2: spill to the global table
            const int64_t g = hg_global_slot(a, key);
            if (g < 0) continue;
            dst = a.vals + (size_t)g * W;
        }
        for (int ag = 0; ag <= a.naggs; ++ag)
            if (has[ag]) hg_atomic(dst + ag, ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT, ag < a.naggs ? a.isf[ag] : 0, v[ag]);
    }
    // flush the shared table into the global one
    __syncthreads();
    for (int k = threadIdx.x; k < HG_SLOTS; k += HG_THREADS) {
        const long long key = s_key[k];
        if (key == HG_EMPTY) continue;
        const int64_t g = hg_global_slot(a, key);
        if (g < 0) continue;
        for (int ag = 0; ag <= a.naggs; ++ag) {
            const int kind = ag < a.naggs ? a.kind[ag] : VD_AGG_COUNT;
            const unsigned long long x = s_val[(size_t)k * W + ag];
            if (x == hg_identity(kind) && kind != VD_AGG_SUM && kind != VD_AGG_COUNT) continue;
            hg_atomic(a.vals + (size_t)g * W + ag, kind, ag < a.naggs ? a.isf[ag] : 0, x);
        }
    }
}

// occupied slots per chunk (the FoldSelect counts)
__global__ void __launch_bounds__(HG_THREADS) k_hg_count(const int64_t* __restrict__ keys, int64_t cap,
                                                       int32_t* __restrict__ counts) {
    __shared__ int s_w[HG_THREADS / 32];
    const int64_t c0 = (int64_t)blockIdx.x * HG_CHUNK;
    int cnt = 0;
    for (int j = threadIdx.x; j < HG_CHUNK; j += HG_THREADS) {
        const int64_t g = c0 + j;
        if (g < cap && keys[g] != HG_EMPTY) ++cnt;
    }
    for (int o = 16; o; o >>= 1) cnt += __shfl_xor_sync(VD_FULL, cnt, o);
    if ((threadIdx.x & 31) == 0) s_w[threadIdx.x >> 5] = cnt;
    __syncthreads();
    if (threadIdx.x == 0) {
        int t = 0;
        for (int w = 0; w < HG_THREADS / 32; ++w) t += s_w[w];
        counts[blockIdx.x] = t;
    }
}

struct HgEmit {
    int32_t naggs;
    int32_t kind[VD_MAX_AGGS], isf[VD_MAX_AGGS];
    int32_t wide;  // 1: the table holds 16-byte aggregate slots (merge), 0: 8-byte words (fold)
};

// FoldSelect(occupied) + Gathers in table order; aggregates as 16-byte slots
__global__ void __launch_bounds__(HG_THREADS) k_hg_emit(const int64_t* __restrict__ keys,
                                                      const unsigned long long* __restrict__ vals, int64_t cap,
                                                      const HgEmit e, const int32_t* __restrict__ counts,
                                                      const int64_t* __restrict__ offs, int64_t nchunks,
                                                      int64_t* __restrict__ out_keys,
                                                      unsigned long long* __restrict__ out_aggs,
                                                      int64_t* __restrict__ out_rows, int64_t* __restrict__ out_ng,
                                                      const unsigned long long* __restrict__ overflow) {
    __shared__ int s_w[HG_THREADS / 32];
    const int NA = e.naggs;
    const int W = e.wide ? 2 * NA + 1 : NA + 1;  // words per slot; the row count is the last word
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    constexpr int PER_WARP = HG_CHUNK / (HG_THREADS / 32);
    const int64_t w0 = (int64_t)blockIdx.x * HG_CHUNK + (int64_t)warp * PER_WARP;
    int mine = 0;
    for (int j = lane; j < PER_WARP; j += 32) {
        const int64_t g = w0 + j;
        if (g < cap && keys[g] != HG_EMPTY) ++mine;
    }
    for (int o = 16; o; o >>= 1) mine += __shfl_xor_sync(VD_FULL, mine, o);
    if (lane == 0) s_w[warp] = mine;
    __syncthreads();
    int64_t pos = offs[blockIdx.x];
    for (int w = 0; w < warp; ++w) pos += s_w[w];
    for (int j0 = 0; j0 < PER_WARP; j0 += 32) {
        const int64_t g = w0 + j0 + lane;
        const bool occ = g < cap && keys[g] != HG_EMPTY;
        const unsigned b = __ballot_sync(VD_FULL, occ);
        if (occ) {
            const int64_t p = pos + __popc(b & lanemask_lt());
            const unsigned long long* src = vals + (size_t)g * W;
            out_keys[p] = keys[g];
            out_rows[p] = (int64_t)src[W - 1];
            for (int ag = 0; ag < NA; ++ag) {
                unsigned long long lo, hi;
                if (e.wide) {
                    lo = src[2 * ag];
                    hi = src[2 * ag + 1];
                    if (e.kind[ag] == VD_AGG_MIN || e.kind[ag] == VD_AGG_MAX || e.isf[ag]) hi = e.isf[ag] ? 0ull : (((long long)lo < 0) ? ~0ull : 0ull);
                } else {
                    lo = src[ag];
                    hi = e.isf[ag] ? 0ull : (((long long)lo < 0) ? ~0ull : 0ull);  // i64 -> i128
                }
                // MIN/MAX with no non-epsilon value: still the identity -> epsilon (A5)
                if (e.kind[ag] == VD_AGG_MIN && lo == (unsigned long long)INT64_MAX) { lo = (unsigned long long)INT64_MIN; hi = ~0ull; }
                out_aggs[2 * ((size_t)p * NA + ag)] = lo;
                out_aggs[2 * ((size_t)p * NA + ag) + 1] = hi;
            }
        }
        pos += __popc(b);
    }
    // a full table (more distinct keys than the capacity allows) reports -1
    if (blockIdx.x == nchunks - 1 && threadIdx.x == 0)
        *out_ng = *overflow ? -1 : offs[blockIdx.x] + counts[blockIdx.x];
}

// ---- cross-GPU merge of compacted groups ------------------------------------------
struct HmArgs {
    const int64_t* in_keys;
    const unsigned long long* in_aggs;  // [nparts * stride][naggs] 16-byte slots
    const int64_t* in_rows;
    const int64_t* in_counts;           // [nparts] valid groups per part
    int64_t stride;                     // groups per part block
    int64_t m;                          // nparts * stride
    int32_t naggs;
    int32_t kind[VD_MAX_AGGS], isf[VD_MAX_AGGS];
    uint64_t mask;
    int64_t* keys;
    unsigned long long* vals;  // [capacity][2 * naggs + 1]
    unsigned long long* overflow;
};

__global__ void __launch_bounds__(HG_THREADS) k_hm_init(const __grid_constant__ HmArgs a) {
    const int W = 2 * a.naggs + 1;
    const int64_t cap = (int64_t)a.mask + 1;
    for (int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; k < cap * W; k += (int64_t)gridDim.x * blockDim.x) {
        const int w = (int)(k % W);
        unsigned long long v = 0;
        if (w < 2 * a.naggs && (w & 1) == 0) {
            const int ag = w >> 1;
            if (a.kind[ag] == VD_AGG_MIN || a.kind[ag] == VD_AGG_MAX) v = hg_identity(a.kind[ag]);
        }
        a.vals[k] = v;
        if (w == 0) a.keys[k / W] = HG_EMPTY;
    }
}

__global__ void __launch_bounds__(HG_THREADS) k_hm_insert(const __grid_constant__ HmArgs a) {
    const int W = 2 * a.naggs + 1;
    HgArgs g;  // the probe loop of the fold
    g.mask = a.mask;
    g.keys = a.keys;
    g.overflow = a.overflow;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < a.m; i += (int64_t)gridDim.x * blockDim.x) {
        const int64_t part = i / a.stride;
        if (i - part * a.stride >= __ldg(a.in_counts + part)) continue;  // padding past the part's groups
        const int64_t key = a.in_keys[i];
        const int64_t s = hg_global_slot(g, key);
        if (s < 0) continue;
        unsigned long long* dst = a.vals + (size_t)s * W;
        for (int ag = 0; ag < a.naggs; ++ag) {
            const unsigned long long lo = a.in_aggs[2 * ((size_t)i * a.naggs + ag)];
            const unsigned long long hi = a.in_aggs[2 * ((size_t)i * a.naggs + ag) + 1];
            const int kind = a.kind[ag];
            if (kind == VD_AGG_SUM && a.isf[ag]) {
                atomicAdd((double*)&dst[2 * ag], __longlong_as_double((long long)lo));
            } else if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                atomic_add_i128(&dst[2 * ag], (i128)(((u128)hi << 64) | lo));  // exact, order independent
            } else if ((long long)lo != INT64_MIN) {  // an epsilon MIN/MAX (no value) contributes nothing
                if (kind == VD_AGG_MIN) atomicMin((long long*)&dst[2 * ag], (long long)lo);
                else atomicMax((long long*)&dst[2 * ag], (long long)lo);
            }
        }
        atomicAdd(&dst[W - 1], (unsigned long long)a.in_rows[i]);
    }
}

// ---- host launchers ---------------------------------------------------------------
static size_t al256(size_t b) { return (b + 255) & ~(size_t)255; }

static int64_t hg_capacity(int64_t est) {
    int64_t c = 1024;
    while (c < 2 * est) c <<= 1;  // load factor <= 1/2
    return c;
}

size_t hash_group_ws_bytes(int64_t est, int naggs, bool wide) {
    const int64_t cap = hg_capacity(est);
    const int64_t nch = (cap + HG_CHUNK - 1) / HG_CHUNK;
    const int W = wide ? 2 * naggs + 1 : naggs + 1;
    return 256 + al256((size_t)cap * 8) + al256((size_t)cap * W * 8) + al256((size_t)nch * 4) + al256((size_t)nch * 8) +
           scan_ws_bytes(nch);
}

struct HgLayout {
    unsigned long long* overflow;
    int64_t* keys;
    unsigned long long* vals;
    int32_t* counts;
    int64_t* offs;
    void* scan_ws;
    int64_t cap, nch;
};
static HgLayout hg_layout(void* ws, int64_t est, int W) {
    HgLayout L;
    L.cap = hg_capacity(est);
    L.nch = (L.cap + HG_CHUNK - 1) / HG_CHUNK;
    char* w = (char*)ws;
    L.overflow = (unsigned long long*)w;
    w += 256;
    L.keys = (int64_t*)w;
    w += al256((size_t)L.cap * 8);
    L.vals = (unsigned long long*)w;
    w += al256((size_t)L.cap * W * 8);
    L.counts = (int32_t*)w;
    w += al256((size_t)L.nch * 4);
    L.offs = (int64_t*)w;
    w += al256((size_t)L.nch * 8);
    L.scan_ws = w;
    return L;
}

static cudaError_t hg_compact(const HgLayout& L, const HgEmit& e, int64_t* out_keys, void* out_aggs,
                              int64_t* out_rows, int64_t* out_ng, cudaStream_t s, int* nl) {
    k_hg_count<<<(unsigned)L.nch, HG_THREADS, 0, s>>>(L.keys, L.cap, L.counts);
    ++*nl;
    cudaError_t err = launch_scan_i32(L.counts, L.nch, L.offs, L.scan_ws, s, nl);
    if (err != cudaSuccess) return err;
    k_hg_emit<<<(unsigned)L.nch, HG_THREADS, 0, s>>>(L.keys, L.vals, L.cap, e, L.counts, L.offs, L.nch, out_keys,
                                                     (unsigned long long*)out_aggs, out_rows, out_ng, L.overflow);
    ++*nl;
    return cudaGetLastError();
}

cudaError_t launch_hash_group_fold(const DevCols& cols, const DevPred& pred, int64_t n, int key_col,
                                   const vd_agg* aggs, const int32_t* isf, int naggs, int64_t est, int64_t* out_keys,
                                   void* out_aggs, int64_t* out_rows, int64_t* out_ng, void* ws, cudaStream_t s,
                                   int* nl) {
    HgArgs A;
    std::memset(&A, 0, sizeof(A));
    A.pred = pred;
    A.cols = cols;
    A.key_col = key_col;
    A.naggs = naggs;
    A.n = n;
    HgEmit e;
    std::memset(&e, 0, sizeof(e));
    e.naggs = naggs;
    for (int g = 0; g < naggs; ++g) {
        A.kind[g] = e.kind[g] = aggs[g].kind;
        A.isf[g] = e.isf[g] = isf[g];
        A.nf[g] = aggs[g].kind == VD_AGG_COUNT ? 0 : aggs[g].nfactors;
        for (int f = 0; f < A.nf[g]; ++f) {
            A.fcol[g][f] = aggs[g].f[f].col;
            A.fa[g][f] = aggs[g].f[f].a;
            A.fb[g][f] = aggs[g].f[f].b;
        }
    }
    const HgLayout L = hg_layout(ws, est, naggs + 1);
    A.mask = (uint64_t)(L.cap - 1);
    A.keys = L.keys;
    A.vals = L.vals;
    A.overflow = L.overflow;
    cudaError_t err = cudaMemsetAsync(L.overflow, 0, 8, s);
    if (err != cudaSuccess) return err;
    const int sms = num_sms();
    k_hg_init<<<sms * 8, HG_THREADS, 0, s>>>(A);
    ++*nl;
    // interval fast path: one conjunction of integer interval terms on at most
    // two columns, the first i32/i64 and 16-byte aligned
    HgIv iv;
    std::memset(&iv, 0, sizeof(iv));
    bool fast = pred.nconj == 1 && pred.nterms[0] >= 1;
    int fc[2] = {-1, -1};
    int64_t lo[2] = {INT64_MIN + 1, INT64_MIN + 1}, hi[2] = {INT64_MAX, INT64_MAX};
    for (int k = 0; fast && k < pred.nterms[0]; ++k) {
        const DevTerm& t = pred.t[0][k];
        const int slot = t.col == fc[0] ? 0 : (t.col == fc[1] ? 1 : (fc[0] < 0 ? 0 : (fc[1] < 0 ? 1 : -1)));
        if (slot < 0 || (cols.dt[t.col] != VD_I32 && cols.dt[t.col] != VD_I64)) { fast = false; break; }
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
        for (int j = 0; j < 2; ++j) {  // epsilon (the type's minimum) outside the interval (A9)
            if (fc[j] < 0) continue;
            const int64_t eps = cols.dt[fc[j]] == VD_I32 ? (int64_t)INT32_MIN : INT64_MIN;
            if (lo[j] <= eps) lo[j] = eps + 1;
        }
        fast = ((uintptr_t)cols.p[fc[0]] % 16) == 0 && !getenv("VD_HASH_GENERIC");
    }
    if (n > 0 && fast) {
        iv.c0 = cols.p[fc[0]];
        iv.dt0 = cols.dt[fc[0]];
        iv.lo0 = lo[0];
        iv.hi0 = hi[0];
        if (fc[1] >= 0) {
            iv.c1 = cols.p[fc[1]];
            iv.dt1 = cols.dt[fc[1]];
            iv.lo1 = lo[1];
            iv.hi1 = hi[1];
        }
        const size_t smem = (size_t)HG_SLOTS * 8 * (naggs + 2);
        cudaFuncSetAttribute(k_hg_fold_iv, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        int per_sm = 0;
        if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_hg_fold_iv, HG_THREADS, smem) != cudaSuccess ||
            per_sm < 1)
            per_sm = 1;
        const int64_t nq = n / 4;
        const int grid = (int)std::max<int64_t>(
            1, std::min<int64_t>((nq + HG_THREADS - 1) / HG_THREADS, (int64_t)sms * per_sm));
        k_hg_fold_iv<<<grid, HG_THREADS, smem, s>>>(A, iv);
        ++*nl;
    } else if (n > 0) {
        const size_t smem = (size_t)HG_SLOTS * 8 * (naggs + 2);
        cudaFuncSetAttribute(k_hg_fold, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        int per_sm = 0;
        if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_hg_fold, HG_THREADS, smem) != cudaSuccess ||
            per_sm < 1)
            per_sm = 1;
        const int64_t blocks = ((n + 31) / 32 + HG_THREADS / 32 - 1) / (HG_THREADS / 32);
        const int grid = (int)std::max<int64_t>(1, std::min<int64_t>(blocks, (int64_t)sms * per_sm));
        k_hg_fold<<<grid, HG_THREADS, smem, s>>>(A);
        ++*nl;
    }
    return hg_compact(L, e, out_keys, out_aggs, out_rows, out_ng, s, nl);
}

cudaError_t launch_merge_groups(const int64_t* keys, const void* aggs, const int64_t* rows, const int64_t* counts,
                                int nparts, int64_t stride, const int32_t* kinds, const int32_t* isf, int naggs,
                                int64_t est, int64_t* out_keys, void* out_aggs, int64_t* out_rows, int64_t* out_ng,
                                void* ws, cudaStream_t s, int* nl) {
    HmArgs A;
    std::memset(&A, 0, sizeof(A));
    A.in_keys = keys;
    A.in_aggs = (const unsigned long long*)aggs;
    A.in_rows = rows;
    A.in_counts = counts;
    A.stride = stride;
    const int64_t m = (int64_t)nparts * stride;
    A.m = m;
    A.naggs = naggs;
    HgEmit e;
    std::memset(&e, 0, sizeof(e));
    e.naggs = naggs;
    e.wide = 1;
    for (int g = 0; g < naggs; ++g) {
        A.kind[g] = e.kind[g] = kinds[g];
        A.isf[g] = e.isf[g] = isf[g];
    }
    const HgLayout L = hg_layout(ws, est, 2 * naggs + 1);
    A.mask = (uint64_t)(L.cap - 1);
    A.keys = L.keys;
    A.vals = L.vals;
    A.overflow = L.overflow;
    cudaError_t err = cudaMemsetAsync(L.overflow, 0, 8, s);
    if (err != cudaSuccess) return err;
    const int sms = num_sms();
    k_hm_init<<<sms * 8, HG_THREADS, 0, s>>>(A);
    ++*nl;
    if (m > 0) {
        const int grid = (int)std::max<int64_t>(1, std::min<int64_t>((m + HG_THREADS - 1) / HG_THREADS, (int64_t)sms * 8));
        k_hm_insert<<<grid, HG_THREADS, 0, s>>>(A);
        ++*nl;
    }
    return hg_compact(L, e, out_keys, out_aggs, out_rows, out_ng, s, nl);
}

}  // namespace vd
