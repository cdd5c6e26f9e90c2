// k_fold.cu -- controlled folds FoldSum/Count/Min/Max (§8(a) a6).
//
// Table 2 and §2.2: one aggregate per run of
// adjacent equal control values, epsilon inputs skipped (Fig 9), results in
// the empty-slot-suppressed form of §3.1.2: slot r = run r.
//
// Fold placement decides the kernel:
//   one run (constant ctrl)   -> k_fold_one: grid-stride partials per
//       thread -> CTA -> grid, the last CTA folding the CTA partials in a
//       fixed order (the "global barrier" Fragment 2 of Fig 8, P:L929-931,
//       without a second launch).
//   runs of any other shape    -> k_fold_seg: tiles of FOLD_TILE rows; each
//       thread folds 16 consecutive rows into segments, a CTA-wide
//       segmented scan joins segments across threads, runs that start and
//       end inside a tile are written directly, and the first / last run of
//       each tile leaves a partial record that k_fold_fixup joins across
//       tiles (in tile order, so results do not depend on scheduling).
// Integer sums are exact 128-bit, float sums f64.
#include <float.h>

#include <cstring>

#include "vd_common.cuh"
#include "vd_internal.h"

namespace vd {

constexpr int FOLD_THREADS = 256;
constexpr int FOLD_ITEMS = 16;
constexpr int FOLD_TILE = FOLD_THREADS * FOLD_ITEMS;

template <typename T, int OP>
struct FAgg {
    i128 vi;
    double vf;
    int64_t c;
    __device__ __forceinline__ void init() {
        c = 0;
        vi = 0;
        vf = 0;
        if (OP == FOLD_MIN) { vi = (i128)INT64_MAX; vf = DBL_MAX; }
        if (OP == FOLD_MAX) { vi = (i128)INT64_MIN; vf = -DBL_MAX; }
    }
    __device__ __forceinline__ void add(T x) {
        if (Eps<T>::is(x)) return;
        ++c;
        if (IsFloat<T>::value) {
            double d = (double)x;
            if (OP == FOLD_SUM) vf += d;
            else if (OP == FOLD_MIN) vf = d < vf ? d : vf;
            else if (OP == FOLD_MAX) vf = d > vf ? d : vf;
        } else {
            i128 v = (i128)(int64_t)x;
            if (OP == FOLD_SUM) vi += v;
            else if (OP == FOLD_MIN) vi = v < vi ? v : vi;
            else if (OP == FOLD_MAX) vi = v > vi ? v : vi;
        }
    }
    __device__ __forceinline__ void merge(const FAgg& o) {
        c += o.c;
        if (OP == FOLD_SUM) { vi += o.vi; vf += o.vf; }
        else if (OP == FOLD_MIN) { vi = o.vi < vi ? o.vi : vi; vf = o.vf < vf ? o.vf : vf; }
        else if (OP == FOLD_MAX) { vi = o.vi > vi ? o.vi : vi; vf = o.vf > vf ? o.vf : vf; }
    }
};

// Store run r's result in the suppressed output (include/vd.h vd_fold_*).
template <typename T, int OP>
__device__ __forceinline__ void store_result(void* out, int64_t* counts, int64_t r, const FAgg<T, OP>& a) {
    if (counts) counts[r] = a.c;
    if (OP == FOLD_COUNT) {
        ((int64_t*)out)[r] = a.c;
    } else if (OP == FOLD_SUM) {
        if (IsFloat<T>::value) ((double*)out)[r] = a.vf;
        else st_i128((char*)out + 16 * r, a.vi);
    } else {
        T v;
        if (a.c == 0) v = Eps<T>::value();  // all-epsilon run (reading A5)
        else v = IsFloat<T>::value ? (T)a.vf : (T)(int64_t)a.vi;
        ((T*)out)[r] = v;
    }
}

template <typename T, int OP>
__device__ __forceinline__ FAgg<T, OP> shfl_agg(const FAgg<T, OP>& a, int o) {
    FAgg<T, OP> b;
    b.vi = shfl_xor_i128(a.vi, o);
    b.vf = __shfl_xor_sync(VD_FULL, a.vf, o);
    b.c = __shfl_xor_sync(VD_FULL, a.c, o);
    return b;
}

// ---- one run ---------------------------------------------------------------
template <typename T, int OP>
__global__ void __launch_bounds__(FOLD_THREADS) k_fold_one(const T* __restrict__ v, int64_t n, void* out,
                                                           int64_t* counts, int64_t* nruns_out,
                                                           FAgg<T, OP>* __restrict__ partials,
                                                           unsigned int* __restrict__ done) {
    FAgg<T, OP> a;
    a.init();
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) a.add(__ldg(v + i));
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) a.merge(shfl_agg(a, o));
    __shared__ FAgg<T, OP> s_w[FOLD_THREADS / 32];
    __shared__ bool s_last;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (lane == 0) s_w[warp] = a;
    __syncthreads();
    if (threadIdx.x == 0) {
        FAgg<T, OP> b = s_w[0];
        for (int w = 1; w < FOLD_THREADS / 32; ++w) b.merge(s_w[w]);
        partials[blockIdx.x] = b;
        __threadfence();
        s_last = (atomicAdd(done, 1u) == gridDim.x - 1);
    }
    __syncthreads();
    if (s_last && threadIdx.x == 0) {
        __threadfence();
        FAgg<T, OP> b;
        b.init();
        for (unsigned k = 0; k < gridDim.x; ++k) {
            // L2 loads: the partials were written by other CTAs
            FAgg<T, OP> p;
            const unsigned long long* q = (const unsigned long long*)(partials + k);
            p.vi = (i128)(((u128)__ldcg(q + 1) << 64) | __ldcg(q));
            p.vf = __longlong_as_double((long long)__ldcg(q + 2));
            p.c = (int64_t)__ldcg(q + 3);
            b.merge(p);
        }
        store_result<T, OP>(out, counts, 0, b);
        if (nruns_out) *nruns_out = 1;
    }
}

// ---- runs of arbitrary shape -----------------------------------------------
struct RidSrc {
    int cls;          // RUNS_FIXED or RUNS_GENERAL
    int64_t R;        // fixed run length
    const void* mat;  // GENERAL: control values (materialized) or NULL (virtual)
    int32_t dt;
    int64_t from, num, den, cap;
    const int32_t* starts;    // GENERAL: run starts (ascending)
    const int64_t* nstarts;   // GENERAL: number of runs (device)
    __device__ __forceinline__ int64_t value(int64_t i) const {
        if (mat) return dt == VD_I32 ? (int64_t)__ldg((const int32_t*)mat + i) : (int64_t)__ldg((const long long*)mat + i);
        i128 q = ((i128)i * num) / den;
        i128 v = (i128)from + q;
        if (cap != 0) v %= cap;
        return (int64_t)v;
    }
};

template <typename T, int OP>
struct SegElem {
    int64_t rid;
    int cont;  // this span's tail segment extends to the span's left edge
    FAgg<T, OP> a;
};

template <typename T, int OP>
__device__ __forceinline__ SegElem<T, OP> seg_combine(const SegElem<T, OP>& L, const SegElem<T, OP>& Rt) {
    SegElem<T, OP> o;
    o.rid = Rt.rid;
    bool join = Rt.cont && (L.rid == Rt.rid);
    o.a = Rt.a;
    if (join) o.a.merge(L.a);
    o.cont = join && L.cont;
    return o;
}

template <typename T, int OP>
struct SegRec {
    int64_t rid;
    int32_t valid;     // record present
    int32_t starts;    // the run starts inside this tile
    int32_t single;    // the tile holds one run only (first == last)
    FAgg<T, OP> a;
};

template <typename T, int OP>
__global__ void __launch_bounds__(FOLD_THREADS) k_fold_seg(const T* __restrict__ v, int64_t n, RidSrc rs,
                                                           void* out, int64_t* counts,
                                                           SegRec<T, OP>* __restrict__ rec_first,
                                                           SegRec<T, OP>* __restrict__ rec_last) {
    __shared__ SegElem<T, OP> s_scan[2][FOLD_THREADS];
    __shared__ int64_t s_first_rid;
    __shared__ int s_first_head;
    __shared__ int s_heads[FOLD_THREADS];
    __shared__ int64_t s_hrid[FOLD_THREADS];
    const int t = threadIdx.x;
    const int64_t tile = blockIdx.x;
    const int64_t a0 = tile * FOLD_TILE;
    const int64_t row0 = a0 + (int64_t)t * FOLD_ITEMS;

    // run ids of this thread's rows; rows >= n continue the last run
    int64_t rid[FOLD_ITEMS];
    if (rs.cls == RUNS_FIXED) {
        int64_t first = row0 < n ? row0 : n - 1;
        int64_t r = first / rs.R, rem = first - r * rs.R;
#pragma unroll
        for (int j = 0; j < FOLD_ITEMS; ++j) {
            rid[j] = r;
            if (row0 + j + 1 < n) {
                if (++rem == rs.R) { ++r; rem = 0; }
            }
        }
        if (t == 0) { s_first_rid = a0 / rs.R; s_first_head = (a0 % rs.R) == 0; }
    } else {
        int hc = 0;
        unsigned hm = 0;
#pragma unroll
        for (int j = 0; j < FOLD_ITEMS; ++j) {
            int64_t i = row0 + j;
            bool h = (i < n) && (i > a0) && (rs.value(i) != rs.value(i - 1));
            hm |= (h ? 1u : 0u) << j;
            hc += h;
        }
        s_heads[t] = hc;
        if (t == 0) {
            // run containing row a0 = (number of run starts <= a0) - 1
            int64_t lo = 0, hi = *rs.nstarts;
            while (lo < hi) {
                int64_t mid = (lo + hi) >> 1;
                if ((int64_t)rs.starts[mid] <= a0) lo = mid + 1; else hi = mid;
            }
            s_first_rid = lo - 1;
            s_first_head = (a0 == 0) || (rs.value(a0) != rs.value(a0 - 1));
        }
        __syncthreads();
        // exclusive scan of head counts (simple, FOLD_THREADS entries)
        for (int o = 1; o < FOLD_THREADS; o <<= 1) {
            int x = (t >= o) ? s_heads[t - o] : 0;
            __syncthreads();
            s_heads[t] += x;
            __syncthreads();
        }
        int64_t r = s_first_rid + (s_heads[t] - hc);
#pragma unroll
        for (int j = 0; j < FOLD_ITEMS; ++j) {
            if ((hm >> j) & 1u) ++r;
            rid[j] = r;
        }
    }
    __syncthreads();
    const int64_t first_rid = s_first_rid;
    const bool first_head = s_first_head != 0;

    // thread-level segments
    T x[FOLD_ITEMS];
#pragma unroll
    for (int j = 0; j < FOLD_ITEMS; ++j) x[j] = (row0 + j < n) ? __ldg(v + row0 + j) : Eps<T>::value();
    FAgg<T, OP> head, cur;
    head.init();
    cur.init();
    int64_t head_rid = rid[0], cur_rid = rid[0];
    bool single = true;
#pragma unroll
    for (int j = 0; j < FOLD_ITEMS; ++j) {
        if (rid[j] != cur_rid) {
            if (single) {
                head = cur;
                single = false;
            } else if (cur_rid != first_rid) {
                store_result<T, OP>(out, counts, cur_rid, cur);  // complete, interior
            }
            cur.init();
            cur_rid = rid[j];
        }
        cur.add(x[j]);
    }
    s_hrid[t] = head_rid;
    // CTA segmented scan of (tail rid, tail agg, cont)
    SegElem<T, OP> me;
    me.rid = cur_rid;
    me.cont = single ? 1 : 0;
    me.a = cur;
    int pb = 0;
    s_scan[0][t] = me;
    __syncthreads();
    for (int o = 1; o < FOLD_THREADS; o <<= 1) {
        SegElem<T, OP> y = s_scan[pb][t];
        if (t >= o) y = seg_combine(s_scan[pb][t - o], y);
        s_scan[pb ^ 1][t] = y;
        pb ^= 1;
        __syncthreads();
    }
    // exclusive carry for thread t
    SegElem<T, OP> carry;
    bool have_carry = t > 0;
    if (have_carry) carry = s_scan[pb][t - 1];

    if (!single) {
        // head segment ends inside this thread
        FAgg<T, OP> h = head;
        if (have_carry && carry.rid == head_rid) h.merge(carry.a);
        if (head_rid == first_rid) {
            SegRec<T, OP> r;
            r.rid = head_rid; r.valid = 1; r.starts = first_head; r.single = 0; r.a = h;
            rec_first[tile] = r;
        } else {
            store_result<T, OP>(out, counts, head_rid, h);
        }
    }
    if (t < FOLD_THREADS - 1 && s_hrid[t + 1] != cur_rid) {
        // this thread's tail run ends exactly at the thread boundary
        SegElem<T, OP> tot = s_scan[pb][t];  // inclusive: the run's in-tile aggregate
        if (cur_rid == first_rid) {
            SegRec<T, OP> r;
            r.rid = cur_rid; r.valid = 1; r.starts = first_head; r.single = 0; r.a = tot.a;
            rec_first[tile] = r;
        } else {
            store_result<T, OP>(out, counts, cur_rid, tot.a);
        }
    }
    if (t == FOLD_THREADS - 1) {
        SegElem<T, OP> tot = s_scan[pb][t];  // inclusive: the tile's last run in-tile aggregate
        SegRec<T, OP> r;
        r.rid = tot.rid; r.valid = 1; r.a = tot.a;
        if (tot.rid == first_rid) {
            r.starts = first_head; r.single = 1;
            rec_first[tile] = r;
            SegRec<T, OP> z;
            z.valid = 0; z.rid = -1; z.starts = 0; z.single = 0; z.a.init();
            rec_last[tile] = z;
        } else {
            r.starts = 1; r.single = 0;
            rec_last[tile] = r;
        }
    }
}

// Join the partial records of runs that cross tile boundaries, in tile order.
template <typename T, int OP>
__global__ void k_fold_fixup(const SegRec<T, OP>* __restrict__ rec_first, const SegRec<T, OP>* __restrict__ rec_last,
                             int64_t ntiles, void* out, int64_t* counts) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t t = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; t < ntiles; t += stride) {
        // run owned through rec_first (starts at this tile's first row)
        SegRec<T, OP> f = rec_first[t];
        if (f.valid && f.starts) {
            FAgg<T, OP> a = f.a;
            if (f.single)
                for (int64_t u = t + 1; u < ntiles && rec_first[u].rid == f.rid && !rec_first[u].starts; ++u) {
                    a.merge(rec_first[u].a);
                    if (!rec_first[u].single) break;
                }
            store_result<T, OP>(out, counts, f.rid, a);
        }
        SegRec<T, OP> l = rec_last[t];
        if (l.valid) {
            FAgg<T, OP> a = l.a;
            for (int64_t u = t + 1; u < ntiles && rec_first[u].rid == l.rid && !rec_first[u].starts; ++u) {
                a.merge(rec_first[u].a);
                if (!rec_first[u].single) break;
            }
            store_result<T, OP>(out, counts, l.rid, a);
        }
    }
}

__global__ void k_store_i64(int64_t* p, int64_t v) { *p = v; }
__global__ void k_copy_i64(int64_t* dst, const int64_t* src) { *dst = *src; }

size_t fold_ws_bytes(int64_t n) {
    int64_t ntiles = (n + FOLD_TILE - 1) / FOLD_TILE;
    size_t rec = sizeof(SegRec<int64_t, FOLD_SUM>);  // all instantiations have the same layout size
    size_t seg = 2 * (size_t)ntiles * rec + 256;
    size_t one = (size_t)num_sms() * 8 * 64 + 256;
    size_t b = seg > one ? seg : one;
    return (b + 255) & ~(size_t)255;
}

template <typename T, int OP>
static cudaError_t fold_typed(const vd_column& vals, const CtrlInfo& ci, const int32_t* starts,
                              const int64_t* nstarts, void* out, int64_t* counts, int64_t* nruns_out, void* ws,
                              cudaStream_t s, int* nl) {
    const int64_t n = vals.len;
    const T* v = (const T*)vals.data;
    if (ci.cls == RUNS_ONE) {
        if (n == 0) {
            if (nruns_out) { k_store_i64<<<1, 1, 0, s>>>(nruns_out, 0); ++*nl; }
            return cudaGetLastError();
        }
        int64_t blocks = (n + FOLD_THREADS * 4 - 1) / (FOLD_THREADS * 4);
        int64_t cap = (int64_t)num_sms() * 4;
        if (blocks > cap) blocks = cap;
        unsigned int* done = (unsigned int*)ws;
        FAgg<T, OP>* partials = (FAgg<T, OP>*)((char*)ws + 256);
        cudaError_t e = cudaMemsetAsync(done, 0, 4, s);
        if (e != cudaSuccess) return e;
        k_fold_one<T, OP><<<(int)blocks, FOLD_THREADS, 0, s>>>(v, n, out, counts, nruns_out, partials, done);
        ++*nl;
        return cudaGetLastError();
    }
    int64_t ntiles = (n + FOLD_TILE - 1) / FOLD_TILE;
    if (ntiles > 0) {
        RidSrc rs;
        rs.cls = ci.cls; rs.R = ci.R; rs.mat = ci.mat; rs.dt = ci.mat_dtype;
        rs.from = ci.from; rs.num = ci.num; rs.den = ci.den; rs.cap = ci.cap;
        rs.starts = starts; rs.nstarts = nstarts;
        SegRec<T, OP>* rf = (SegRec<T, OP>*)((char*)ws + 256);
        SegRec<T, OP>* rl = rf + ntiles;
        k_fold_seg<T, OP><<<(int)ntiles, FOLD_THREADS, 0, s>>>(v, n, rs, out, counts, rf, rl);
        ++*nl;
        int64_t fb = (ntiles + 255) / 256;
        k_fold_fixup<T, OP><<<(int)fb, 256, 0, s>>>(rf, rl, ntiles, out, counts);
        ++*nl;
    }
    if (nruns_out) {
        if (ci.cls == RUNS_GENERAL) k_copy_i64<<<1, 1, 0, s>>>(nruns_out, nstarts);
        else k_store_i64<<<1, 1, 0, s>>>(nruns_out, ci.nruns);
        ++*nl;
    }
    return cudaGetLastError();
}

template <int OP>
static cudaError_t fold_op(const vd_column& vals, const CtrlInfo& ci, const int32_t* starts, const int64_t* nstarts,
                           void* out, int64_t* counts, int64_t* nruns_out, void* ws, cudaStream_t s, int* nl) {
    switch (vals.dtype) {
    case VD_U8: return fold_typed<uint8_t, OP>(vals, ci, starts, nstarts, out, counts, nruns_out, ws, s, nl);
    case VD_I32: return fold_typed<int32_t, OP>(vals, ci, starts, nstarts, out, counts, nruns_out, ws, s, nl);
    case VD_I64: return fold_typed<int64_t, OP>(vals, ci, starts, nstarts, out, counts, nruns_out, ws, s, nl);
    case VD_F32: return fold_typed<float, OP>(vals, ci, starts, nstarts, out, counts, nruns_out, ws, s, nl);
    default: return fold_typed<double, OP>(vals, ci, starts, nstarts, out, counts, nruns_out, ws, s, nl);
    }
}

// ws layout for GENERAL controls: [select ws | starts (n int32) | nstarts | fold ws]
cudaError_t launch_fold(FoldOp op, const vd_column& vals, const CtrlInfo& ci, void* out, int64_t* out_counts,
                        int64_t* out_nruns, void* ws, size_t, cudaStream_t s, int* nl) {
    const int32_t* starts = nullptr;
    const int64_t* nstarts = nullptr;
    char* fws = (char*)ws;
    if (ci.cls == RUNS_GENERAL) {
        size_t sel = select_ws_bytes(vals.len);
        int32_t* st = (int32_t*)(fws + sel);
        size_t stb = (((size_t)vals.len * 4 + 255) & ~(size_t)255);
        int64_t* ns = (int64_t*)(fws + sel + stb);
        cudaError_t e = launch_select_heads(ci, vals.len, st, ns, fws, sel, s, nl);
        if (e != cudaSuccess) return e;
        starts = st;
        nstarts = ns;
        fws = fws + sel + stb + 256;
    }
    switch (op) {
    case FOLD_SUM: return fold_op<FOLD_SUM>(vals, ci, starts, nstarts, out, out_counts, out_nruns, fws, s, nl);
    case FOLD_COUNT: return fold_op<FOLD_COUNT>(vals, ci, starts, nstarts, out, out_counts, out_nruns, fws, s, nl);
    case FOLD_MIN: return fold_op<FOLD_MIN>(vals, ci, starts, nstarts, out, out_counts, out_nruns, fws, s, nl);
    default: return fold_op<FOLD_MAX>(vals, ci, starts, nstarts, out, out_counts, out_nruns, fws, s, nl);
    }
}

// ============================================================================
// FoldScan(.out, V1, .fold, .s) (Table 2): prefix sum of the values,
// a new run of the control vector starting a new sum; inclusive, epsilon
// slots stay epsilon and add nothing (reading A27).  One pass: tiles of
// SCAN_T rows taken in order from an atomic counter; each thread scans 16
// rows in registers, a CTA segmented scan (flag = "a run starts here")
// joins threads, and a decoupled look-back over per-tile (flag, value) words
// supplies the carry into the tile's first run.  A tile that contains a run
// start publishes its inclusive prefix at once (the sum of its last run
// does not depend on earlier tiles), so look-back chains stop there.
// Integer input -> int64 (exactness proven on the host), float -> f64.
// ============================================================================
constexpr int FSC_THREADS = 256;
constexpr int FSC_ITEMS = 16;
constexpr int FSC_TILE = FSC_THREADS * FSC_ITEMS;

struct FscStatus {
    unsigned long long flag;  // 0 not ready, 1 aggregate ready, 2 inclusive prefix ready
    unsigned long long agg;   // int64 or f64 bits; written once
    unsigned long long pfx;   // written once, before flag = 2
};

template <typename A> __device__ __forceinline__ unsigned long long fsc_bits(A v);
template <> __device__ __forceinline__ unsigned long long fsc_bits<int64_t>(int64_t v) { return (unsigned long long)v; }
template <> __device__ __forceinline__ unsigned long long fsc_bits<double>(double v) {
    return (unsigned long long)__double_as_longlong(v);
}
template <typename A> __device__ __forceinline__ A fsc_val(unsigned long long b);
template <> __device__ __forceinline__ int64_t fsc_val<int64_t>(unsigned long long b) { return (int64_t)b; }
template <> __device__ __forceinline__ double fsc_val<double>(unsigned long long b) {
    return __longlong_as_double((long long)b);
}

__device__ __forceinline__ void fsc_publish(FscStatus* st, unsigned long long flag, unsigned long long val) {
    if (flag == 2ull) st->pfx = val;
    else st->agg = val;
    __threadfence();
    asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(&st->flag), "l"(flag) : "memory");
}

template <typename T, typename A>
__global__ void __launch_bounds__(FSC_THREADS) k_fold_scan(const T* __restrict__ v, int64_t n, RidSrc rs,
                                                           A* __restrict__ out, FscStatus* __restrict__ status,
                                                           unsigned long long* __restrict__ tile_ctr) {
    __shared__ int64_t s_tile;
    __shared__ int s_wf[FSC_THREADS / 32];
    __shared__ A s_ws[FSC_THREADS / 32];
    __shared__ A s_carry;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    if (t == 0) s_tile = (int64_t)atomicAdd(tile_ctr, 1ull);
    __syncthreads();
    const int64_t tile = s_tile;
    const int64_t row0 = tile * FSC_TILE + (int64_t)t * FSC_ITEMS;

    // thread-local inclusive segmented scan
    A y[FSC_ITEMS];
    unsigned hm = 0, em = 0;
    A run = 0;
#pragma unroll
    for (int j = 0; j < FSC_ITEMS; ++j) {
        const int64_t i = row0 + j;
        bool h = false;
        if (i < n) {
            if (rs.cls == RUNS_ONE) h = (i == 0);
            else if (rs.cls == RUNS_FIXED) h = (i % rs.R) == 0;
            else h = (i == 0) || (rs.value(i) != rs.value(i - 1));
        }
        if (h) run = 0;
        T x = i < n ? __ldg(v + i) : Eps<T>::value();
        const bool e = Eps<T>::is(x);
        if (!e) run += (A)x;
        y[j] = run;
        hm |= (h ? 1u : 0u) << j;
        em |= (e ? 1u : 0u) << j;
    }
    // CTA segmented inclusive scan of (flag, sum) over threads
    int f = hm != 0;
    A sum = run;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        const int fp = __shfl_up_sync(VD_FULL, f, o);
        const A sp = __shfl_up_sync(VD_FULL, sum, o);
        if (lane >= o) {
            if (!f) sum += sp;
            f |= fp;
        }
    }
    if (lane == 31) { s_wf[warp] = f; s_ws[warp] = sum; }
    __syncthreads();
    if (warp == 0) {
        int wf = lane < FSC_THREADS / 32 ? s_wf[lane] : 0;
        A wsum = lane < FSC_THREADS / 32 ? s_ws[lane] : (A)0;
#pragma unroll
        for (int o = 1; o < FSC_THREADS / 32; o <<= 1) {
            const int fp = __shfl_up_sync(VD_FULL, wf, o);
            const A sp = __shfl_up_sync(VD_FULL, wsum, o);
            if (lane >= o) {
                if (!wf) wsum += sp;
                wf |= fp;
            }
        }
        // tile aggregate = inclusive value of the last warp
        const int tf = __shfl_sync(VD_FULL, wf, FSC_THREADS / 32 - 1);
        const A tsum = __shfl_sync(VD_FULL, wsum, FSC_THREADS / 32 - 1);
        if (lane < FSC_THREADS / 32) { s_wf[lane] = wf; s_ws[lane] = wsum; }  // inclusive per warp
        // look-back: the carry into this tile's first run
        A carry = 0;
        if (tile > 0) {
            if (lane == 0 && tf) fsc_publish(&status[tile], 2ull, fsc_bits<A>(tsum));
            else if (lane == 0) fsc_publish(&status[tile], 1ull, fsc_bits<A>(tsum));
            int64_t end = tile - 1;
            for (;;) {
                const int64_t idx = end - lane;
                unsigned long long fl = 2ull, vb = fsc_bits<A>((A)0);
                if (idx >= 0) {
                    do {
                        asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(fl) : "l"(&status[idx].flag) : "memory");
                    } while (fl == 0);
                    vb = fl == 2ull ? __ldcg(&status[idx].pfx) : __ldcg(&status[idx].agg);
                }
                const unsigned pm = __ballot_sync(VD_FULL, fl == 2ull);
                const int stop = pm ? (__ffs(pm) - 1) : 31;
                A c = lane <= stop ? fsc_val<A>(vb) : (A)0;
                // fixed-order reduction (deterministic for floats)
#pragma unroll
                for (int o = 16; o > 0; o >>= 1) c += __shfl_xor_sync(VD_FULL, c, o);
                carry += c;
                if (pm) break;
                end -= 32;
            }
            if (lane == 0 && !tf) fsc_publish(&status[tile], 2ull, fsc_bits<A>(carry + tsum));
        } else if (lane == 0) {
            fsc_publish(&status[0], 2ull, fsc_bits<A>(tsum));
        }
        if (lane == 0) s_carry = carry;
    }
    __syncthreads();
    // exclusive (flag, sum) before this thread, then the tile carry
    int pf = 0;
    A ps = 0;
    {
        const int fp = __shfl_up_sync(VD_FULL, f, 1);
        const A sp = __shfl_up_sync(VD_FULL, sum, 1);
        if (lane > 0) { pf = fp; ps = sp; }
        if (warp > 0) {
            // prepend the previous warps' inclusive value
            const int wf = s_wf[warp - 1];
            const A wsv = s_ws[warp - 1];
            if (!pf) { ps += wsv; pf = wf; }
        }
        if (!pf) ps += s_carry;
    }
#pragma unroll
    for (int j = 0; j < FSC_ITEMS; ++j) {
        const int64_t i = row0 + j;
        if (i >= n) break;
        const bool before_head = (hm & ((2u << j) - 1u)) == 0;  // no run start in rows 0..j of this thread
        A r = y[j] + (before_head ? ps : (A)0);
        if ((em >> j) & 1u) {
            out[i] = fsc_val<A>(sizeof(A) == 8 && !IsFloat<A>::value ? 0x8000000000000000ull : 0x7ff8000000000000ull);
        } else {
            out[i] = r;
        }
    }
}

size_t fold_scan_ws_bytes(int64_t n) {
    const int64_t ntiles = (n + FSC_TILE - 1) / FSC_TILE;
    return 256 + (((size_t)ntiles * sizeof(FscStatus) + 255) & ~(size_t)255);
}

template <typename T, typename A>
static cudaError_t fold_scan_typed(const vd_column& vals, const CtrlInfo& ci, void* out, void* ws, cudaStream_t s,
                                   int* nl) {
    const int64_t n = vals.len;
    const int64_t ntiles = (n + FSC_TILE - 1) / FSC_TILE;
    if (ntiles == 0) return cudaSuccess;
    cudaError_t e = cudaMemsetAsync(ws, 0, fold_scan_ws_bytes(n), s);
    if (e != cudaSuccess) return e;
    RidSrc rs;
    std::memset(&rs, 0, sizeof(rs));
    rs.cls = ci.cls; rs.R = ci.R; rs.mat = ci.mat; rs.dt = ci.mat_dtype;
    rs.from = ci.from; rs.num = ci.num; rs.den = ci.den; rs.cap = ci.cap;
    k_fold_scan<T, A><<<(unsigned)ntiles, FSC_THREADS, 0, s>>>((const T*)vals.data, n, rs, (A*)out,
                                                               (FscStatus*)((char*)ws + 256),
                                                               (unsigned long long*)ws);
    ++*nl;
    return cudaGetLastError();
}

cudaError_t launch_fold_scan(const vd_column& vals, const CtrlInfo& ci, void* out, void* ws, cudaStream_t s, int* nl) {
    switch (vals.dtype) {
    case VD_U8: return fold_scan_typed<uint8_t, int64_t>(vals, ci, out, ws, s, nl);
    case VD_I32: return fold_scan_typed<int32_t, int64_t>(vals, ci, out, ws, s, nl);
    case VD_I64: return fold_scan_typed<int64_t, int64_t>(vals, ci, out, ws, s, nl);
    case VD_F32: return fold_scan_typed<float, double>(vals, ci, out, ws, s, nl);
    default: return fold_scan_typed<double, double>(vals, ci, out, ws, s, nl);
    }
}

}  // namespace vd
