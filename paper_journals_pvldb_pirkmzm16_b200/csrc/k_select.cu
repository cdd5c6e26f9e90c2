// k_select.cu -- order-preserving selection -> position list (§8(a) a2+a3).
//
// FoldSelect (Table 2) is order preserving: the
// output position of a qualifying row depends on how many qualifying rows
// precede it.  One pass over the input: every tile of SEL_TILE rows
// evaluates the predicate, ranks its qualifying rows with warp ballots /
// popc, and learns how many rows all earlier tiles selected through a
// single-pass decoupled look-back over per-tile status words.  Tiles are
// handed out by an atomic counter, so every predecessor of a tile is
// already running or done (forward progress).
//
// Two write strategies (Fig 1):
//   MODE 0, branching  : only qualifying lanes store their position, directly
//                        to global memory at cursor + rank.
//   MODE 1, predicated : cursor arithmetic (Ross) -- every row is written at
//                        the warp's cursor into a shared-memory stage, the
//                        cursor advancing by the predicate; rows that do not
//                        qualify land past the cursor and are overwritten by
//                        the next step.  The valid prefix is then streamed
//                        out with coalesced stores.  No lane of one store
//                        instruction shares an address with another.
#include "vd_common.cuh"
#include "vd_internal.h"
#include "vd_lookback.cuh"
#include "vd_pred.cuh"

namespace vd {

constexpr int SEL_THREADS = 256;
constexpr int SEL_WARPS = SEL_THREADS / 32;
constexpr int SEL_CH = 4;                          // chunks of 128 rows per warp
constexpr int SEL_WROWS = SEL_CH * 128;            // rows per warp per tile
constexpr int SEL_TILE = SEL_WARPS * SEL_WROWS;    // 4096 rows per tile

// ---- flag providers: flags of 4 consecutive rows starting at row0 ----------
struct GenericFlags {
    DevPred P;
    DevCols C;
    __device__ __forceinline__ void flags4(int64_t row0, int64_t n, bool f[4]) const {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            int64_t r = row0 + j;
            f[j] = (r < n) && eval_pred_row(P, C, r);
        }
    }
};

template <typename T> struct Vec4Load;
template <> struct Vec4Load<float> {
    static __device__ __forceinline__ void ld(const float* p, float v[4]) {
        float4 x = __ldg(reinterpret_cast<const float4*>(p));
        v[0] = x.x; v[1] = x.y; v[2] = x.z; v[3] = x.w;
    }
};
template <> struct Vec4Load<int32_t> {
    static __device__ __forceinline__ void ld(const int32_t* p, int32_t v[4]) {
        int4 x = __ldg(reinterpret_cast<const int4*>(p));
        v[0] = x.x; v[1] = x.y; v[2] = x.z; v[3] = x.w;
    }
};
template <> struct Vec4Load<int64_t> {
    static __device__ __forceinline__ void ld(const int64_t* p, int64_t v[4]) {
        longlong2 a = __ldg(reinterpret_cast<const longlong2*>(p));
        longlong2 b = __ldg(reinterpret_cast<const longlong2*>(p) + 1);
        v[0] = a.x; v[1] = a.y; v[2] = b.x; v[3] = b.y;
    }
};
template <> struct Vec4Load<double> {
    static __device__ __forceinline__ void ld(const double* p, double v[4]) {
        double2 a = __ldg(reinterpret_cast<const double2*>(p));
        double2 b = __ldg(reinterpret_cast<const double2*>(p) + 1);
        v[0] = a.x; v[1] = a.y; v[2] = b.x; v[3] = b.y;
    }
};
template <> struct Vec4Load<uint8_t> {
    static __device__ __forceinline__ void ld(const uint8_t* p, uint8_t v[4]) {
        uint32_t x = __ldg(reinterpret_cast<const unsigned int*>(p));
        v[0] = x & 0xFF; v[1] = (x >> 8) & 0xFF; v[2] = (x >> 16) & 0xFF; v[3] = x >> 24;
    }
};

// One term over one column; 4 rows per vector load when the column base is
// aligned to the vector width (checked on the host).
template <typename T, bool ALIGNED>
struct TermFlags {
    const T* p;
    int cmp;
    int64_t iv;
    double fv;
    __device__ __forceinline__ bool test(T x) const {
        if (Eps<T>::is(x)) return false;
        if (IsFloat<T>::value) return cmp_flt(cmp, (double)x, fv);
        return cmp_int(cmp, (int64_t)x, iv);
    }
    __device__ __forceinline__ void flags4(int64_t row0, int64_t n, bool f[4]) const {
        T v[4];
        if (ALIGNED && row0 + 4 <= n) {
            Vec4Load<T>::ld(p + row0, v);
#pragma unroll
            for (int j = 0; j < 4; ++j) f[j] = test(v[j]);
        } else {
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                int64_t r = row0 + j;
                f[j] = (r < n) && test(__ldg(p + r));
            }
        }
    }
};

// Run heads of a control vector: row 0 and every row whose control value
// differs from its predecessor's (adjacent runs, reading A3).
struct HeadFlags {
    const void* mat;
    int32_t dt;
    int64_t from, num, den, cap;
    __device__ __forceinline__ int64_t value(int64_t i) const {
        if (mat) return dt == VD_I32 ? (int64_t)__ldg((const int32_t*)mat + i) : (int64_t)__ldg((const long long*)mat + i);
        i128 q = ((i128)i * num) / den;
        i128 v = (i128)from + q;
        if (cap != 0) v %= cap;
        return (int64_t)v;
    }
    __device__ __forceinline__ void flags4(int64_t row0, int64_t n, bool f[4]) const {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            int64_t r = row0 + j;
            f[j] = (r < n) && (r == 0 || value(r) != value(r - 1));
        }
    }
};

template <int MODE, class F>
__global__ void __launch_bounds__(SEL_THREADS) k_select(F fl, int64_t n, int32_t* __restrict__ out,
                                                        int64_t* __restrict__ out_count, uint64_t* __restrict__ status,
                                                        unsigned long long* __restrict__ tile_ctr, int64_t ntiles) {
    __shared__ int64_t s_tile;
    __shared__ int64_t s_base;
    __shared__ int s_wtot[SEL_WARPS];
    __shared__ int s_woff[SEL_WARPS];
    __shared__ int32_t s_stage[MODE == 1 ? SEL_WARPS * SEL_WROWS : 1];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const unsigned lt = lanemask_lt();

    for (;;) {
        if (threadIdx.x == 0) s_tile = (int64_t)atomicAdd(tile_ctr, 1ull);
        __syncthreads();
        const int64_t tile = s_tile;
        if (tile >= ntiles) break;
        const int64_t row_w = tile * SEL_TILE + (int64_t)warp * SEL_WROWS;

        unsigned fm = 0;  // bit k*4+j: row row_w + k*128 + lane*4 + j qualifies
#pragma unroll
        for (int k = 0; k < SEL_CH; ++k) {
            bool f[4];
            fl.flags4(row_w + k * 128 + lane * 4, n, f);
#pragma unroll
            for (int j = 0; j < 4; ++j) fm |= (f[j] ? 1u : 0u) << (k * 4 + j);
        }
        unsigned b[SEL_CH][4];
        int ck[SEL_CH];
        int wtot = 0;
#pragma unroll
        for (int k = 0; k < SEL_CH; ++k) {
            ck[k] = 0;
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                b[k][j] = __ballot_sync(VD_FULL, (fm >> (k * 4 + j)) & 1u);
                ck[k] += __popc(b[k][j]);
            }
            wtot += ck[k];
        }
        if (lane == 0) s_wtot[warp] = wtot;
        __syncthreads();
        if (warp == 0) {
            int v = lane < SEL_WARPS ? s_wtot[lane] : 0;
            int incl = v;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                int u = __shfl_up_sync(VD_FULL, incl, o);
                if (lane >= o) incl += u;
            }
            if (lane < SEL_WARPS) s_woff[lane] = incl - v;
            int64_t agg = __shfl_sync(VD_FULL, incl, SEL_WARPS - 1);
            int64_t base = lookback_exclusive(status, tile, agg, lane);
            if (lane == 0) {
                s_base = base;
                if (tile == ntiles - 1) *out_count = base + agg;
            }
        }
        __syncthreads();
        const int64_t base = s_base + s_woff[warp];

        if (MODE == 0) {
            int cur = 0;
#pragma unroll
            for (int k = 0; k < SEL_CH; ++k) {
                int before = 0;
#pragma unroll
                for (int j = 0; j < 4; ++j) before += __popc(b[k][j] & lt);
#pragma unroll
                for (int j = 0; j < 4; ++j) {
                    if ((fm >> (k * 4 + j)) & 1u) {
                        out[base + cur + before] = (int32_t)(row_w + k * 128 + lane * 4 + j);
                        ++before;
                    }
                }
                cur += ck[k];
            }
        } else {
            int32_t* st = s_stage + warp * SEL_WROWS;
            int cur = 0;
#pragma unroll
            for (int k = 0; k < SEL_CH; ++k) {
                int sel_before = 0;
#pragma unroll
                for (int j = 0; j < 4; ++j) sel_before += __popc(b[k][j] & lt);
                int item_before = lane * 4;
#pragma unroll
                for (int j = 0; j < 4; ++j) {
                    int f = (fm >> (k * 4 + j)) & 1u;
                    int addr = cur + (f ? sel_before : ck[k] + (item_before - sel_before));
                    st[addr] = (int32_t)(row_w + k * 128 + lane * 4 + j);  // unconditional write
                    sel_before += f;                                         // cursor += predicate
                    ++item_before;
                }
                cur += ck[k];
                __syncwarp();
            }
            for (int i = lane; i < wtot; i += 32) out[base + i] = st[i];
            __syncwarp();
        }
        __syncthreads();
    }
}

size_t select_ws_bytes(int64_t n) {
    int64_t ntiles = (n + SEL_TILE - 1) / SEL_TILE;
    size_t b = 256 + (size_t)ntiles * 8;
    return (b + 255) & ~(size_t)255;
}

static int select_grid(int64_t ntiles) {
    int64_t g = (int64_t)num_sms() * 8;
    if (ntiles < g) g = ntiles;
    return (int)(g < 1 ? 1 : g);
}

template <int MODE, class F>
static cudaError_t run_select(const F& fl, int64_t n, int32_t* out_pos, int64_t* out_count, void* ws,
                              cudaStream_t s, int* nl) {
    int64_t ntiles = (n + SEL_TILE - 1) / SEL_TILE;
    if (ntiles == 0) return cudaMemsetAsync(out_count, 0, sizeof(int64_t), s);
    unsigned long long* ctr = (unsigned long long*)ws;
    uint64_t* status = (uint64_t*)((char*)ws + 256);
    cudaError_t e = cudaMemsetAsync(ws, 0, 256 + (size_t)ntiles * 8, s);
    if (e != cudaSuccess) return e;
    k_select<MODE, F><<<select_grid(ntiles), SEL_THREADS, 0, s>>>(fl, n, out_pos, out_count, status, ctr, ntiles);
    ++*nl;
    return cudaGetLastError();
}

template <int MODE, typename T>
static cudaError_t dispatch_term(const void* p, const DevTerm& t, int64_t n, int32_t* out_pos, int64_t* out_count,
                                 void* ws, cudaStream_t s, int* nl) {
    size_t vecbytes = sizeof(T) * 4 > 16 ? 16 : sizeof(T) * 4;
    bool aligned = ((uintptr_t)p % vecbytes) == 0;
    if (aligned) {
        TermFlags<T, true> f{(const T*)p, t.cmp, t.iv, t.fv};
        return run_select<MODE>(f, n, out_pos, out_count, ws, s, nl);
    }
    TermFlags<T, false> f{(const T*)p, t.cmp, t.iv, t.fv};
    return run_select<MODE>(f, n, out_pos, out_count, ws, s, nl);
}

template <int MODE>
static cudaError_t select_mode(const DevCols& cols, const DevPred& pred, int64_t n, int32_t* out_pos,
                               int64_t* out_count, void* ws, cudaStream_t s, int* nl) {
    if (pred.nconj == 1 && pred.nterms[0] == 1) {
        const DevTerm& t = pred.t[0][0];
        const void* p = cols.p[t.col];
        switch (cols.dt[t.col]) {
        case VD_U8: return dispatch_term<MODE, uint8_t>(p, t, n, out_pos, out_count, ws, s, nl);
        case VD_I32: return dispatch_term<MODE, int32_t>(p, t, n, out_pos, out_count, ws, s, nl);
        case VD_I64: return dispatch_term<MODE, int64_t>(p, t, n, out_pos, out_count, ws, s, nl);
        case VD_F32: return dispatch_term<MODE, float>(p, t, n, out_pos, out_count, ws, s, nl);
        default: return dispatch_term<MODE, double>(p, t, n, out_pos, out_count, ws, s, nl);
        }
    }
    GenericFlags g{pred, cols};
    return run_select<MODE>(g, n, out_pos, out_count, ws, s, nl);
}

cudaError_t launch_select(int mode, const DevCols& cols, const DevPred& pred, int64_t n, int32_t* out_pos,
                          int64_t* out_count, void* ws, size_t, cudaStream_t s, int* nl) {
    if (mode == VD_SEL_PREDICATED) return select_mode<1>(cols, pred, n, out_pos, out_count, ws, s, nl);
    return select_mode<0>(cols, pred, n, out_pos, out_count, ws, s, nl);
}

cudaError_t launch_select_heads(const CtrlInfo& ci, int64_t n, int32_t* out_pos, int64_t* out_count, void* ws,
                                size_t, cudaStream_t s, int* nl) {
    HeadFlags h{ci.mat, ci.mat_dtype, ci.from, ci.num, ci.den, ci.cap};
    return run_select<0>(h, n, out_pos, out_count, ws, s, nl);
}

// out_run_off[r] = number of selected positions before run r's first row
// (lower_bound of the run start in the ascending position list); the last
// entry is the total count.
__global__ void k_run_offsets(int cls, int64_t R, int64_t nruns_host, const int32_t* __restrict__ pos,
                              const int64_t* __restrict__ count, const int32_t* __restrict__ starts,
                              const int64_t* __restrict__ nruns_dev, int64_t* __restrict__ out,
                              int64_t* __restrict__ out_nruns) {
    const int64_t nr = (cls == RUNS_GENERAL) ? *nruns_dev : nruns_host;
    const int64_t cnt = *count;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t r = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; r <= nr; r += stride) {
        if (r == nr) {
            if (out) out[r] = cnt;
            continue;
        }
        int64_t st = (cls == RUNS_FIXED) ? r * R : (cls == RUNS_ONE ? 0 : (int64_t)starts[r]);
        int64_t lo = 0, hi = cnt;
        while (lo < hi) {
            int64_t mid = (lo + hi) >> 1;
            if ((int64_t)pos[mid] < st) lo = mid + 1; else hi = mid;
        }
        if (out) out[r] = lo;
    }
    if (blockIdx.x == 0 && threadIdx.x == 0 && out_nruns) *out_nruns = nr;
}

cudaError_t launch_run_offsets(const CtrlInfo& ci, int64_t n, const int32_t* pos, const int64_t* count,
                               const int32_t* run_starts, const int64_t* nruns_dev, int64_t* out_run_off,
                               int64_t* out_nruns, cudaStream_t s, int* nl) {
    int64_t work = (ci.cls == RUNS_GENERAL) ? n + 1 : ci.nruns + 1;
    int64_t blocks = (work + 255) / 256;
    int64_t cap = (int64_t)num_sms() * 8;
    if (blocks > cap) blocks = cap;
    if (blocks < 1) blocks = 1;
    k_run_offsets<<<(int)blocks, 256, 0, s>>>((int)ci.cls, ci.R, ci.nruns, pos, count, run_starts, nruns_dev,
                                               out_run_off, out_nruns);
    ++*nl;
    return cudaGetLastError();
}

}  // namespace vd
