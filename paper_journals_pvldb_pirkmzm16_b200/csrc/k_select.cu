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
#include <algorithm>
#include <cmath>
#include <cstdlib>
#include <cstring>
#include <type_traits>

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
struct NoRaw {};

struct GenericFlags {
    DevPred P;
    DevCols C;
    typedef NoRaw Raw;
    __device__ __forceinline__ void load(int64_t, int64_t, Raw&) const {}
    __device__ __forceinline__ void eval(const Raw&, int64_t row0, int64_t n, bool f[4]) const { flags4(row0, n, f); }
    __device__ __forceinline__ bool eval1(int64_t r, int64_t n) const { return (r < n) && eval_pred_row(P, C, r); }
    __device__ __forceinline__ void flags4(int64_t row0, int64_t n, bool f[4]) const {
#pragma unroll
        for (int j = 0; j < 4; ++j) f[j] = eval1(row0 + j, n);
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

// 4 consecutive values from shared memory (16-byte aligned for 4-byte types).
template <typename T> struct Vec4Lds;
template <> struct Vec4Lds<float> {
    static __device__ __forceinline__ void ld(const float* p, float v[4]) {
        float4 x = *reinterpret_cast<const float4*>(p);
        v[0] = x.x; v[1] = x.y; v[2] = x.z; v[3] = x.w;
    }
};
template <> struct Vec4Lds<int32_t> {
    static __device__ __forceinline__ void ld(const int32_t* p, int32_t v[4]) {
        int4 x = *reinterpret_cast<const int4*>(p);
        v[0] = x.x; v[1] = x.y; v[2] = x.z; v[3] = x.w;
    }
};
template <> struct Vec4Lds<uint8_t> {
    static __device__ __forceinline__ void ld(const uint8_t* p, uint8_t v[4]) {
        uint32_t x = *reinterpret_cast<const uint32_t*>(p);
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
    // interval form lo <= x <= hi of the term (ivl != 0), with epsilon
    // excluded by the bounds (int: lo > MIN / u8: hi < 0xFF; float: NaN
    // fails every comparison); computed on the host
    int ivl;
    T lo, hi;
    __device__ __forceinline__ bool test(T x) const {
        if (ivl) return x >= lo && x <= hi;
        if (Eps<T>::is(x)) return false;
        if (IsFloat<T>::value) return cmp_flt(cmp, (double)x, fv);
        return cmp_int(cmp, (int64_t)x, iv);
    }
    // raw values of 4 rows, loaded ahead of their evaluation (software pipelining)
    struct Raw {
        T v[4];
    };
    __device__ __forceinline__ void load(int64_t row0, int64_t n, Raw& r) const {
        if (ALIGNED && row0 + 4 <= n) {
            Vec4Load<T>::ld(p + row0, r.v);
        } else {
#pragma unroll
            for (int j = 0; j < 4; ++j) r.v[j] = (row0 + j < n) ? __ldg(p + row0 + j) : T(0);
        }
    }
    __device__ __forceinline__ void eval(const Raw& r, int64_t row0, int64_t n, bool f[4]) const {
#pragma unroll
        for (int j = 0; j < 4; ++j) f[j] = (row0 + j < n) && test(r.v[j]);
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
    typedef NoRaw Raw;
    __device__ __forceinline__ void load(int64_t, int64_t, Raw&) const {}
    __device__ __forceinline__ void eval(const Raw&, int64_t row0, int64_t n, bool f[4]) const { flags4(row0, n, f); }
    __device__ __forceinline__ int64_t value(int64_t i) const {
        if (mat) return dt == VD_I32 ? (int64_t)__ldg((const int32_t*)mat + i) : (int64_t)__ldg((const long long*)mat + i);
        i128 q = ((i128)i * num) / den;
        i128 v = (i128)from + q;
        if (cap != 0) v %= cap;
        return (int64_t)v;
    }
    __device__ __forceinline__ bool eval1(int64_t r, int64_t n) const {
        return (r < n) && (r == 0 || value(r) != value(r - 1));
    }
    __device__ __forceinline__ void flags4(int64_t row0, int64_t n, bool f[4]) const {
#pragma unroll
        for (int j = 0; j < 4; ++j) f[j] = eval1(row0 + j, n);
    }
};

// One tile of the selection: flags -> ranks -> look-back -> positions.
template <int MODE, class F>
__device__ __forceinline__ void select_tile(const F& fl, const typename F::Raw (&raw)[SEL_CH], int64_t tile,
                                            int64_t n, int32_t* __restrict__ out, int64_t* __restrict__ out_count,
                                            uint64_t* __restrict__ status, int64_t ntiles, int64_t* s_base,
                                            int* s_wtot, int* s_woff, int32_t* s_stage) {
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const unsigned lt = lanemask_lt();
    const int64_t row_w = tile * SEL_TILE + (int64_t)warp * SEL_WROWS;
    unsigned fm = 0;  // bit k*4+j: row row_w + k*128 + lane*4 + j qualifies
#pragma unroll
    for (int k = 0; k < SEL_CH; ++k) {
        bool f[4];
        fl.eval(raw[k], row_w + k * 128 + lane * 4, n, f);
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
        int64_t base = lookback_exclusive_w128(status, tile, agg, lane);
        if (lane == 0) {
            *s_base = base;
            if (tile == ntiles - 1) *out_count = base + agg;
        }
    }
    __syncthreads();
    const int64_t base = *s_base + s_woff[warp];

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
}

// Persistent CTAs, tiles claimed in order from an atomic counter, two tiles
// per CTA in flight: the next tile's loads are issued before the current
// tile's look-back, so HBM stays busy while the look-back waits on L2.
template <int MODE, class F>
__global__ void __launch_bounds__(SEL_THREADS) k_select(F fl, int64_t n, int32_t* __restrict__ out,
                                                        int64_t* __restrict__ out_count, uint64_t* __restrict__ status,
                                                        unsigned long long* __restrict__ tile_ctr, int64_t ntiles) {
    __shared__ int64_t s_next;
    __shared__ int64_t s_base;
    __shared__ int s_wtot[SEL_WARPS];
    __shared__ int s_woff[SEL_WARPS];
    __shared__ int32_t s_stage[MODE == 1 ? SEL_WARPS * SEL_WROWS : 1];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    typename F::Raw ra[SEL_CH], rb[SEL_CH];

    auto claim = [&]() -> int64_t {
        if (threadIdx.x == 0) s_next = (int64_t)atomicAdd(tile_ctr, 1ull);
        __syncthreads();
        int64_t t = s_next;
        __syncthreads();
        return t;
    };
    auto load = [&](int64_t tile, typename F::Raw (&r)[SEL_CH]) {
        const int64_t row_w = tile * SEL_TILE + (int64_t)warp * SEL_WROWS;
#pragma unroll
        for (int k = 0; k < SEL_CH; ++k) fl.load(row_w + k * 128 + lane * 4, n, r[k]);
    };
    int64_t cur = claim();
    if (cur < ntiles) load(cur, ra);
    for (;;) {
        if (cur >= ntiles) break;
        int64_t nxt = claim();
        if (nxt < ntiles) load(nxt, rb);
        select_tile<MODE>(fl, ra, cur, n, out, out_count, status, ntiles, &s_base, s_wtot, s_woff, s_stage);
        cur = nxt;
        if (cur >= ntiles) break;
        nxt = claim();
        if (nxt < ntiles) load(nxt, ra);
        select_tile<MODE>(fl, rb, cur, n, out, out_count, status, ntiles, &s_base, s_wtot, s_woff, s_stage);
        cur = nxt;
    }
}

// ---- bitmap selection ---------------------------------------------------------------
// Fig 8: a `break` materialises the predicate data-parallel, and
// foldSelect then emits the positions.  Here the materialised predicate is a
// bitmap (1 bit per row; 125 MB for 1e9 rows, largely L2-resident) with a
// population count per 1024-row chunk:
//   k_sel_bits_*  streaming pass: flags -> bitmap words + chunk counts
//   scan          chunk counts -> chunk offsets (look-back scan)
//   k_sel_write   positions from the bitmap: branching (each qualifying bit
//                 stores its position) or predicated (cursor arithmetic:
//                 every row of the chunk is written to a shared-memory stage,
//                 qualifying rows at the cursor, the rest past it, then the
//                 qualifying prefix streams out with coalesced stores).
// No serial chain: each pass is fully data parallel, unlike a single-pass
// look-back whose throughput is bounded by window x tile per L2 round trip.
constexpr int BM_THREADS = 256;
constexpr int BM_CHUNK = 1024;  // rows per warp chunk = 32 words

// Bitmap layout: chunk c, word w (0..31), bit i <-> row c*1024 + 32*w + i.
// Flag pass: each load instruction reads 512 contiguous bytes (lane L takes
// rows q*128 + 4L .. 4L+3), the warp ballots each of the 4 row phases, and
// lane w assembles word w from the four ballots of its 128-row block by
// spreading bytes (word = interleave of 4 ballot bytes).
__device__ __forceinline__ uint32_t spread8(uint32_t x) {  // bit k -> bit 4k
    x = (x | (x << 12)) & 0x000F000Fu;
    x = (x | (x << 6)) & 0x03030303u;
    x = (x | (x << 3)) & 0x11111111u;
    return x;
}

template <typename T, bool ALIGNED, bool IVL>
__global__ void __launch_bounds__(BM_THREADS) k_sel_bits_vec(TermFlags<T, ALIGNED> fl, int64_t n,
                                                             uint32_t* __restrict__ bits,
                                                             int32_t* __restrict__ counts, int64_t nchunks,
                                                             int64_t c0 = 0) {
    __shared__ uint32_t s_bal[BM_THREADS / 32][32];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int64_t gw = ((int64_t)blockIdx.x * BM_THREADS + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * BM_THREADS) >> 5;
    uint32_t* bal = s_bal[warp];
    // chunks entirely inside the column (all but the last): no per-row
    // bounds checks, and the interval form of the term (IVL, decided on the
    // host) as two compares with no epsilon / operator dispatch
    const int64_t nfull = ALIGNED ? n / BM_CHUNK : 0;
    for (int64_t c = c0 + gw; c < nchunks; c += nw) {
        if (c < nfull) {
            T v[8][4];
#pragma unroll
            for (int q = 0; q < 8; ++q) Vec4Load<T>::ld(fl.p + c * BM_CHUNK + q * 128 + lane * 4, v[q]);
#pragma unroll
            for (int q = 0; q < 8; ++q) {
#pragma unroll
                for (int j = 0; j < 4; ++j) {
                    const bool f = IVL ? (v[q][j] >= fl.lo && v[q][j] <= fl.hi) : fl.test(v[q][j]);
                    const uint32_t b = __ballot_sync(VD_FULL, f);
                    if (lane == 0) bal[q * 4 + j] = b;  // bit L <-> row q*128 + 4L + j
                }
            }
        } else {
            typename TermFlags<T, ALIGNED>::Raw raw[8];
#pragma unroll
            for (int q = 0; q < 8; ++q) fl.load(c * BM_CHUNK + q * 128 + lane * 4, n, raw[q]);
#pragma unroll
            for (int q = 0; q < 8; ++q) {
                bool f[4];
                fl.eval(raw[q], c * BM_CHUNK + q * 128 + lane * 4, n, f);
#pragma unroll
                for (int j = 0; j < 4; ++j) {
                    const uint32_t b = __ballot_sync(VD_FULL, f[j]);
                    if (lane == 0) bal[q * 4 + j] = b;
                }
            }
        }
        __syncwarp();
        // word w = rows 32w..32w+31 = q-block w/4, lanes 8(w%4) .. 8(w%4)+7
        const int q = lane >> 2, m = lane & 3;
        uint32_t word = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) word |= spread8((bal[q * 4 + j] >> (8 * m)) & 0xFFu) << j;
        __syncwarp();
        bits[c * 32 + lane] = word;
        int cnt = __popc(word);
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) cnt += __shfl_xor_sync(VD_FULL, cnt, o);
        if (lane == 0) counts[c] = cnt;
    }
}

// TMA-staged flag pass for 1- and 4-byte columns under an interval term:
// a producer warp streams BT_CW-chunk tiles of the column with 1D bulk copies
// into a BT_STAGES-deep mbarrier ring; consumer warp w builds chunk w of the
// tile out of shared memory (same ballot / byte-spread assembly as
// k_sel_bits_vec).  The LDG version is latency bound (64 registers -> 32
// warps per SM, no loads in flight while a warp assembles its words); the
// ring keeps HBM busy independent of the consumers.  Measured on 1e9 f32:
// 620.8 us (TMA) vs 630 us (LDG), i.e. 6.45 TB/s -- the single-stream read
// ceiling (scripts/ubench_read.cu: 6.69 TB/s for a bare LDG.128 stream).
constexpr int BT_CW = 16;
constexpr int BT_THREADS = BT_CW * 32 + 32;
constexpr int BT_STAGES = 3;

// tile of a CTA's it-th step (strided over the grid), -1 past the end.  A
// contiguous range of tiles per CTA was measured slower (637.8 vs 620.8 us
// per 4 GB): HBM bank spread is not the limit.
__device__ __forceinline__ int64_t tile_of(int64_t it, int64_t ntiles) {
    const int64_t t = blockIdx.x + it * gridDim.x;
    return t < ntiles ? t : -1;
}

template <typename T>
__global__ void __launch_bounds__(BT_THREADS, 1) k_sel_bits_tma(const T* __restrict__ col, T lo, T hi,
                                                                int64_t ntiles, uint32_t* __restrict__ bits,
                                                                int32_t* __restrict__ counts) {
    constexpr uint32_t TB = BT_CW * BM_CHUNK * sizeof(T);  // tile bytes
    extern __shared__ __align__(128) uint8_t smem[];
    __shared__ uint32_t s_bal[BT_CW][32];
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)BT_STAGES * TB);
    uint64_t* empty = full + BT_STAGES;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int i = 0; i < BT_STAGES; ++i) {
            mbar_init(&full[i], 1);
            mbar_init(&empty[i], BT_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (warp == BT_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int st = 0;
            uint32_t ph = 0;
            for (int64_t it = 0;; ++it) {
                const int64_t tile = tile_of(it, ntiles);
                if (tile < 0) break;
                if (it >= BT_STAGES) mbar_wait(&empty[st], ph ^ 1u);
                mbar_expect_tx(&full[st], TB);
                tma_load_1d(smem + (size_t)st * TB, col + tile * (BT_CW * BM_CHUNK), TB, &full[st], pol);
                if (++st == BT_STAGES) { st = 0; ph ^= 1u; }
            }
        }
        return;
    }
    uint32_t* bal = s_bal[warp];
    int st = 0;
    uint32_t ph = 0;
    for (int64_t it = 0;; ++it) {
        const int64_t tile = tile_of(it, ntiles);
        if (tile < 0) break;
        mbar_wait(&full[st], ph);
        const T* src = reinterpret_cast<const T*>(smem + (size_t)st * TB) + warp * BM_CHUNK;
        T v[8][4];
#pragma unroll
        for (int q = 0; q < 8; ++q) Vec4Lds<T>::ld(src + q * 128 + lane * 4, v[q]);
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[st]);
        if (++st == BT_STAGES) { st = 0; ph ^= 1u; }
#pragma unroll
        for (int q = 0; q < 8; ++q) {
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                const uint32_t b = __ballot_sync(VD_FULL, v[q][j] >= lo && v[q][j] <= hi);
                if (lane == 0) bal[q * 4 + j] = b;  // bit L <-> row q*128 + 4L + j
            }
        }
        __syncwarp();
        const int qq = lane >> 2, m = lane & 3;
        uint32_t word = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) word |= spread8((bal[qq * 4 + j] >> (8 * m)) & 0xFFu) << j;
        __syncwarp();
        const int64_t c = tile * BT_CW + warp;
        bits[c * 32 + lane] = word;
        int cnt = __popc(word);
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) cnt += __shfl_xor_sync(VD_FULL, cnt, o);
        if (lane == 0) counts[c] = cnt;
    }
}

// ---- single-launch selection: stream + grid barrier + decode ------------------
// One cooperative persistent kernel (one CTA per SM, all co-resident), each
// CTA owning a contiguous range of 1024-row chunks:
//   phase 1  a producer warp streams the CTA's rows through an SC_STAGES-deep
//            TMA ring; consumer warp w turns its 1024-row chunk into 32
//            ballots (ballot k: bit L <-> row 32k + L, a row-ordered word)
//            and stores them as the chunk's 32 bitmap words -- the predicate
//            materialised, Fig 8's break: n/8 bytes, largely L2-resident --
//            and the chunk's count in shared memory;
//   barrier  the CTA's total goes to counts[cta]; one grid-wide barrier; the
//            CTA's output base is the sum of the counts of the CTAs before it
//            (no scan launch, no per-tile look-back chain), and a CTA-wide
//            scan of its chunk counts gives every chunk's offset;
//   phase 2  warps decode their chunks independently (no barriers), skipping
//            empty chunks and keeping the next chunks' words in flight.
// Replaces the 4-launch bitmap path (flag pass, scan, total, position pass).
// A single-pass decoupled look-back variant (one look-back per 64 KB tile)
// was measured at 5.8 ms for 1e9 rows: under a full HBM stream a look-back
// costs several microseconds of L2 round trips, far above a CTA's ~1.5 us
// per tile.
static size_t al256(size_t b) { return (b + 255) & ~(size_t)255; }
constexpr int SC_CW = 15;  // + the producer: 16 warps, 4 per SM sub-partition (128 registers each)
constexpr int SC_THREADS = SC_CW * 32 + 32;  // + producer warp
constexpr int SC_P2W = SC_CW + 1;            // phase 2: every warp decodes
constexpr int SC_STAGES = 3;
constexpr int SC_CHUNKS = SC_CW;             // 1024-row chunks per tile
constexpr int SC_STG = 1024 + 128 + 8;       // per-warp position stage (ints)
constexpr int SC_PF = 4;                     // phase 2: 4-chunk groups in flight per warp
constexpr int SC_SPARSE = 64;                // phase 2: branching groups this sparse store directly
constexpr int SC_ROUND = 1024;               // phase 2: outputs per staged round (a multiple of 4)
constexpr int SC_MAXCH = 12288;              // chunks per CTA (counts kept in shared memory)

template <int MODE, typename T>
__global__ void __launch_bounds__(SC_THREADS, 1) k_sel_coop(const T* __restrict__ col, T lo, T hi, int64_t n,
                                                            int32_t* __restrict__ out, int64_t* __restrict__ out_count,
                                                            uint32_t* __restrict__ bits,
                                                            int64_t* __restrict__ counts,
                                                            unsigned int* __restrict__ grid_bar, int phase1_only,
                                                            int round_max) {
    constexpr uint32_t TB = SC_CHUNKS * 1024 * sizeof(T);  // tile bytes
    extern __shared__ __align__(128) uint8_t smem[];
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)SC_STAGES * TB);
    uint64_t* empty = full + SC_STAGES;
    uint16_t* s_ccnt = reinterpret_cast<uint16_t*>(empty + SC_STAGES);  // per-chunk counts (phase 1 -> 2)
    __shared__ int s_cnt[SC_CW];
    __shared__ int s_scan[SC_THREADS / 32];
    __shared__ int64_t s_base;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    // the CTA's chunk range [c0, c1) (chunk = 1024 rows), tiles of SC_CHUNKS
    const int64_t nchunks = (n + 1023) / 1024;
    const int64_t c0 = nchunks * blockIdx.x / gridDim.x, c1 = nchunks * (blockIdx.x + 1) / gridDim.x;
    const int nch = (int)(c1 - c0);  // <= SC_MAXCH (host-checked)
    const int64_t ntile = (nch + SC_CHUNKS - 1) / SC_CHUNKS;
    if (threadIdx.x == 0) {
        for (int i = 0; i < SC_STAGES; ++i) {
            mbar_init(&full[i], 1);
            mbar_init(&empty[i], SC_CW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    // ---- phase 1: stream -> ballot words + per-chunk counts ----
    int cnt = 0;
    if (warp == SC_CW) {
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int st = 0;
            uint32_t ph = 0;
            for (int64_t t = 0; t < ntile; ++t) {
                if (t >= SC_STAGES) mbar_wait(&empty[st], ph ^ 1u);
                const int64_t r0 = (c0 + t * SC_CHUNKS) * 1024;
                const int64_t r1 = min((c0 + (t + 1) * SC_CHUNKS) * 1024, c1 * 1024);
                if (r1 <= n) {
                    const uint32_t bytes = (uint32_t)((r1 - r0) * sizeof(T));  // whole chunks: a multiple of 16
                    mbar_expect_tx(&full[st], bytes);
                    tma_load_1d(smem + (size_t)st * TB, col + r0, bytes, &full[st], pol);
                } else {
                    mbar_arrive(&full[st]);  // the column's ragged end: consumers load it directly
                }
                if (++st == SC_STAGES) { st = 0; ph ^= 1u; }
            }
        }
        __syncwarp();
    } else {
        int st = 0;
        uint32_t ph = 0;
        for (int64_t t = 0; t < ntile; ++t) {
            mbar_wait(&full[st], ph);
            const int64_t c = c0 + t * SC_CHUNKS + warp;  // this warp's chunk
            const bool staged = min((c0 + (t + 1) * SC_CHUNKS) * 1024, c1 * 1024) <= n;
            uint32_t mine = 0;
            if (c < c1) {
                if (staged) {
                    const T* src = reinterpret_cast<const T*>(smem + (size_t)st * TB) + warp * 1024;
#pragma unroll
                    for (int k = 0; k < 32; ++k) {
                        const T v = src[k * 32 + lane];
                        const uint32_t b = __ballot_sync(VD_FULL, v >= lo && v <= hi);  // NaN / INT_MIN fail
                        mine = lane == k ? b : mine;
                    }
                } else {
                    for (int k = 0; k < 32; ++k) {
                        const int64_t r = c * 1024 + k * 32 + lane;
                        bool f = false;
                        if (r < n) {
                            const T v = __ldg(col + r);
                            f = v >= lo && v <= hi;
                        }
                        const uint32_t b = __ballot_sync(VD_FULL, f);
                        mine = lane == k ? b : mine;
                    }
                }
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[st]);
            if (++st == SC_STAGES) { st = 0; ph ^= 1u; }
            if (c < c1) {
                bits[c * 32 + lane] = mine;
                int cc = __popc(mine);
#pragma unroll
                for (int o = 16; o; o >>= 1) cc += __shfl_xor_sync(VD_FULL, cc, o);
                if (lane == 0) s_ccnt[c - c0] = (uint16_t)cc;
                cnt += cc;
            }
        }
    }
    if (lane == 0 && warp < SC_CW) s_cnt[warp] = cnt;
    __syncthreads();
    if (threadIdx.x == 0) {
        int64_t t = 0;
        for (int w = 0; w < SC_CW; ++w) t += s_cnt[w];
        st_release_u64(reinterpret_cast<uint64_t*>(&counts[blockIdx.x]), (uint64_t)t);
        // ---- grid barrier (cooperative launch: every CTA is resident) ----
        __threadfence();
        atomicAdd(grid_bar, 1u);
        while (ld_acquire_u32(grid_bar) < gridDim.x) __nanosleep(64);
    }
    __syncthreads();
    // CTA base = counts of the CTAs before it
    if (warp == 0) {
        int64_t b = 0;
        for (int i = lane; i < (int)blockIdx.x; i += 32)
            b += (int64_t)ld_acquire_u64(reinterpret_cast<uint64_t*>(&counts[i]));
        b = warp_sum_i64(b);
        if (lane == 0) {
            s_base = b;
            if (blockIdx.x == gridDim.x - 1) {
                int64_t tot = b;
                for (int w = 0; w < SC_CW; ++w) tot += s_cnt[w];
                *out_count = tot;
            }
        }
    }
    // exclusive scan of the chunk counts -> int32 chunk offsets within the
    // CTA (in the ring's memory, free now): thread i owns a contiguous run
    int32_t* s_off = reinterpret_cast<int32_t*>(smem) + SC_P2W * SC_STG;
    const int per = (nch + SC_THREADS - 1) / SC_THREADS;
    const int i0 = min(nch, (int)threadIdx.x * per), i1 = min(nch, i0 + per);
    int mysum = 0;
    for (int i = i0; i < i1; ++i) mysum += s_ccnt[i];
    int incl = mysum;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        const int u = __shfl_up_sync(VD_FULL, incl, o);
        if (lane >= o) incl += u;
    }
    if (lane == 31) s_scan[warp] = incl;
    __syncthreads();
    int wbase = 0;
    for (int w = 0; w < warp; ++w) wbase += s_scan[w];
    int run = wbase + incl - mysum;
    for (int i = i0; i < i1; ++i) {
        s_off[i] = run;
        run += s_ccnt[i];
    }
    __syncthreads();
    // ---- phase 2: bitmap words -> positions, no barriers ----
    // A warp decodes GROUPS of 4 consecutive chunks (4096 rows, contiguous
    // in the output): lane L loads words 4L .. 4L+3 of the group with one
    // 16-byte load (rows 128L .. 128L+127) and a warp popc-prefix gives its
    // output range.  Branching groups with at most SC_SPARSE positions store
    // straight to global memory; denser chunks -- and every chunk in
    // predicated mode (cursor arithmetic: every row written, qualifying rows
    // at the cursor) -- are assembled per 128-row block from the chunk's 32
    // ballot words (read back as shared-memory broadcasts) in a stage and
    // streamed out with 16-byte stores.  Each warp keeps its next SC_PF
    // groups' words in flight; empty groups are skipped from the counts.
    if (phase1_only) return;  // every warp, the producer's too, decodes groups
    int32_t* sw = reinterpret_cast<int32_t*>(smem) + warp * SC_STG;  // the ring's memory, reused
    uint32_t* swords = reinterpret_cast<uint32_t*>(s_off + SC_MAXCH) + warp * 128;
    const unsigned lt = lanemask_lt();
    const int64_t base = s_base;
    const int ngrp = (nch + 3) >> 2;
    auto gcount = [&](int g) {
        int t = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) t += (4 * g + j < nch) ? s_ccnt[4 * g + j] : 0;
        return t;
    };
    auto gload = [&](int g) {
        if (g >= ngrp) return make_uint4(0, 0, 0, 0);
        const int64_t w0 = (c0 + 4 * (int64_t)g) * 32 + 4 * lane;
        if (4 * g + 4 <= nch) return __ldcs(reinterpret_cast<const uint4*>(bits + w0));
        uint4 x = make_uint4(0, 0, 0, 0);  // the CTA's last, partial group
        const int valid = (nch - 4 * g) * 32;  // words
        if (4 * lane + 0 < valid) x.x = __ldcs(bits + w0 + 0);
        if (4 * lane + 1 < valid) x.y = __ldcs(bits + w0 + 1);
        if (4 * lane + 2 < valid) x.z = __ldcs(bits + w0 + 2);
        if (4 * lane + 3 < valid) x.w = __ldcs(bits + w0 + 3);
        return x;
    };
    int qg[SC_PF];
    uint4 qw[SC_PF];
    int nxt = warp;
#pragma unroll
    for (int u = 0; u < SC_PF; ++u) {
        while (nxt < ngrp && gcount(nxt) == 0) nxt += SC_P2W;
        qg[u] = nxt;
        qw[u] = gload(nxt);
        if (nxt < ngrp) nxt += SC_P2W;
    }
    while (qg[0] < ngrp) {
        const int g = qg[0];
        const uint4 w4 = qw[0];
#pragma unroll
        for (int u = 0; u + 1 < SC_PF; ++u) {
            qg[u] = qg[u + 1];
            qw[u] = qw[u + 1];
        }
        while (nxt < ngrp && gcount(nxt) == 0) nxt += SC_P2W;
        qg[SC_PF - 1] = nxt;
        qw[SC_PF - 1] = gload(nxt);
        if (nxt < ngrp) nxt += SC_P2W;
        const int total = gcount(g);
        const int64_t g0 = base + s_off[4 * g];
        if (MODE == 0 && total <= SC_SPARSE) {
            const uint32_t ws[4] = {w4.x, w4.y, w4.z, w4.w};
            const int pc = __popc(ws[0]) + __popc(ws[1]) + __popc(ws[2]) + __popc(ws[3]);
            int incl = pc;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const int u = __shfl_up_sync(VD_FULL, incl, o);
                if (lane >= o) incl += u;
            }
            int k = incl - pc;
            const int32_t row0 = (int32_t)((c0 + 4 * (int64_t)g) * 1024 + lane * 128);
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                uint32_t m = ws[j];
                while (m) {
                    __stcs(&out[g0 + k], row0 + 32 * j + (__ffs(m) - 1));
                    ++k;
                    m &= m - 1;
                }
            }
            continue;
        }
        if (MODE == 0 && total <= round_max) {
            // lane-owned rows, positions staged in one round of <= SC_ROUND outputs
            // (stage index k at k + k/32: lanes 32 positions apart hit
            // different banks), each round streamed out with 16-byte stores
            uint32_t ws[4] = {w4.x, w4.y, w4.z, w4.w};
            const int pc = __popc(ws[0]) + __popc(ws[1]) + __popc(ws[2]) + __popc(ws[3]);
            int incl = pc;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const int u = __shfl_up_sync(VD_FULL, incl, o);
                if (lane >= o) incl += u;
            }
            int k = incl - pc;  // this lane's next output rank
            const int32_t row0 = (int32_t)((c0 + 4 * (int64_t)g) * 1024 + lane * 128);
            // the output's misalignment in words: output rank rb + i sits at
            // stage index i + a (physically x + x/32); SC_ROUND % 4 == 0, so
            // every round has the same misalignment and 16-byte groups of the
            // output are 4-word stage groups
            const int a = (int)(((uintptr_t)(out + g0) >> 2) & 3);
            const int h0 = (4 - a) & 3;
            for (int rb = 0; rb < total; rb += SC_ROUND) {
                const int re = min(total, rb + SC_ROUND);
#pragma unroll
                for (int jj = 0; jj < 4; ++jj) {  // static indices: ws stays in registers
                    uint32_t m = ws[jj];
                    while (m && k < re) {
                        const int x = k - rb + a;
                        sw[x + (x >> 5)] = row0 + 32 * jj + (__ffs(m) - 1);
                        ++k;
                        m &= m - 1;
                    }
                    ws[jj] = m;
                }
                __syncwarp();
                const int cnt = re - rb;
                const int64_t gb = g0 + rb;
                const int h = min(cnt, h0);
                if (lane < h) { const int x = lane + a; __stcs(&out[gb + lane], sw[x + (x >> 5)]); }
                const int nv = (cnt - h) >> 2;
                int4* o4 = reinterpret_cast<int4*>(out + gb + h);
                for (int v = lane; v < nv; v += 32) {
                    const int x = h + a + 4 * v;  // a multiple of 4: the group never straddles a pad
                    const int32_t* q = sw + x + (x >> 5);
                    __stcs(o4 + v, make_int4(q[0], q[1], q[2], q[3]));
                }
                for (int i = h + 4 * nv + lane; i < cnt; i += 32) {
                    const int x = i + a;
                    __stcs(&out[gb + i], sw[x + (x >> 5)]);
                }
                __syncwarp();
            }
            continue;
        }
        // dense groups (> SC_ROUND positions: the rank ranges of a round
        // would belong to a quarter of the lanes) and every predicated group:
        // per chunk, from its 32 ballot words (shared-memory broadcasts)
        *reinterpret_cast<uint4*>(swords + 4 * lane) = w4;
        __syncwarp();
        int64_t gc = g0;
        for (int j = 0; j < 4 && 4 * g + j < nch; ++j) {
            const int cj = s_ccnt[4 * g + j];
            if (cj == 0) continue;
            uint32_t bw[32];
#pragma unroll
            for (int k = 0; k < 32; k += 4) {
                const uint4 x = *reinterpret_cast<const uint4*>(swords + 32 * j + k);  // broadcast
                bw[k] = x.x; bw[k + 1] = x.y; bw[k + 2] = x.z; bw[k + 3] = x.w;
            }
            const int64_t row0 = (c0 + 4 * (int64_t)g + j) * 1024;
            const int a = (int)(((uintptr_t)(out + gc) >> 2) & 3);
            int cur = a;
#pragma unroll
            for (int q = 0; q < 8; ++q) {
                const int cq = __popc(bw[4 * q]) + __popc(bw[4 * q + 1]) + __popc(bw[4 * q + 2]) + __popc(bw[4 * q + 3]);
                int pre = cur;
#pragma unroll
                for (int jj = 0; jj < 4; ++jj) {
                    const uint32_t w = bw[4 * q + jj];
                    const int f = (w >> lane) & 1u;
                    const int r = __popc(w & lt);
                    const int32_t row = (int32_t)(row0 + (4 * q + jj) * 32 + lane);
                    if (MODE == 0) {
                        if (f) sw[pre + r] = row;
                    } else {
                        // cursor arithmetic: unconditional store; rows that do
                        // not qualify land past the block's count, overwritten next
                        const int sel_before = pre - cur + r;
                        const int k = f ? pre + r : cur + cq + (jj * 32 + lane - sel_before);
                        sw[k] = row;
                    }
                    pre += __popc(w);
                }
                cur += cq;
            }
            __syncwarp();
            const int tot = cur - a;
            const int ngr = (a + tot + 3) >> 2;
            int32_t* ob = out + gc - a;  // 16-byte aligned
            for (int v = lane; v < ngr; v += 32) {
                const int4 x = *reinterpret_cast<const int4*>(sw + 4 * v);
                if (4 * v >= a && 4 * v + 4 <= a + tot) {
                    __stcs(reinterpret_cast<int4*>(ob) + v, x);
                } else {
                    const int32_t xs[4] = {x.x, x.y, x.z, x.w};
#pragma unroll
                    for (int e = 0; e < 4; ++e) {
                        const int kk = 4 * v + e;
                        if (kk >= a && kk < a + tot) __stcs(ob + kk, xs[e]);
                    }
                }
            }
            __syncwarp();
            gc += cj;
        }
    }
}

static size_t sel_coop_smem(size_t tsize) {
    const size_t ring = (size_t)SC_STAGES * SC_CHUNKS * 1024 * tsize;
    const size_t p2 = (size_t)SC_P2W * SC_STG * 4 + (size_t)SC_MAXCH * 4 + (size_t)SC_P2W * 128 * 4;  // stages, offsets, words
    return std::max(ring, p2) + 2 * SC_STAGES * 8 + (size_t)SC_MAXCH * 2;
}

// VD_SELECT_COOP=0 keeps the 4-launch bitmap path (comparison runs)
static bool use_sel_coop() {
    static const bool off = [] {
        const char* e = getenv("VD_SELECT_COOP");
        return e && strcmp(e, "0") == 0;
    }();
    return !off;
}

template <int MODE, typename T>
static cudaError_t run_select_coop(const T* col, T lo, T hi, int64_t n, int32_t* out_pos, int64_t* out_count,
                                   void* ws, cudaStream_t s, int* nl) {
    if (n == 0) return cudaMemsetAsync(out_count, 0, sizeof(int64_t), s);
    const int64_t nchunks = (n + 1023) / 1024;
    char* w = (char*)ws;
    unsigned int* bar = (unsigned int*)w;
    int64_t* counts = (int64_t*)(w + 256);
    uint32_t* bits = (uint32_t*)(w + 256 + al256((size_t)4096 * 8));
    const size_t sm = sel_coop_smem(sizeof(T));
    auto kern = k_sel_coop<MODE, T>;
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm);
    int per_sm = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, SC_THREADS, sm) != cudaSuccess || per_sm < 1)
        return cudaErrorCooperativeLaunchTooLarge;
    int grid = (int)std::min<int64_t>((int64_t)num_sms() * per_sm, std::min<int64_t>(nchunks, 4096));
    if ((nchunks + grid - 1) / grid > SC_MAXCH) return cudaErrorNotSupported;  // caller falls back
    cudaError_t e = cudaMemsetAsync(bar, 0, 4, s);
    if (e != cudaSuccess) return e;
    // VD_SELECT_PHASE1=1 (diagnostics only: positions are NOT written) times
    // the stream + barrier half of the kernel
    static const int p1 = [] {
        const char* e = getenv("VD_SELECT_PHASE1");
        return e && strcmp(e, "1") == 0 ? 1 : 0;
    }();
    int phase1_only = p1;
    // branching groups with <= round_max positions take the staged lane-owned
    // path, denser ones the ballot-block stage (VD_SELECT_ROUND_MAX: comparison
    // runs; <= SC_ROUND).  Storing dense groups straight from the ballot
    // blocks (no stage) was measured slower: 1.51 vs 1.26 ms at s = 0.5.
    static const int rmax = [] {
        const char* e = getenv("VD_SELECT_ROUND_MAX");
        const int v = e ? atoi(e) : SC_ROUND;
        return v < 0 ? 0 : (v > SC_ROUND ? SC_ROUND : v);
    }();
    int round_max = rmax;
    void* args[] = {(void*)&col, (void*)&lo, (void*)&hi, (void*)&n, (void*)&out_pos, (void*)&out_count,
                    (void*)&bits, (void*)&counts, (void*)&bar, (void*)&phase1_only, (void*)&round_max};
    e = cudaLaunchCooperativeKernel((const void*)kern, dim3(grid), dim3(SC_THREADS), args, sm, s);
    ++*nl;
    return e;
}
static size_t sel_coop_ws_bytes(int64_t n) {
    const int64_t nchunks = (n + 1023) / 1024;
    return 256 + al256((size_t)4096 * 8) + al256((size_t)nchunks * 32 * 4);
}


// Per-row predicates (several columns, run heads): ballot j is word j.
template <class F>
__global__ void __launch_bounds__(BM_THREADS) k_sel_bits_bal(F fl, int64_t n, uint32_t* __restrict__ bits,
                                                             int32_t* __restrict__ counts, int64_t nchunks) {
    const int lane = threadIdx.x & 31;
    const int64_t gw = ((int64_t)blockIdx.x * BM_THREADS + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * BM_THREADS) >> 5;
    for (int64_t c = gw; c < nchunks; c += nw) {
        uint32_t mine = 0;
#pragma unroll 4
        for (int j = 0; j < 32; ++j) {
            const uint32_t b = __ballot_sync(VD_FULL, fl.eval1(c * BM_CHUNK + j * 32 + lane, n));
            if (lane == j) mine = b;
        }
        bits[c * 32 + lane] = mine;
        int cnt = __popc(mine);
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) cnt += __shfl_xor_sync(VD_FULL, cnt, o);
        if (lane == 0) counts[c] = cnt;
    }
}

__global__ void k_sel_total(const int64_t* __restrict__ offs, const int32_t* __restrict__ counts, int64_t nchunks,
                            int64_t* __restrict__ out_count) {
    *out_count = nchunks > 0 ? offs[nchunks - 1] + counts[nchunks - 1] : 0;
}

// Position pass: lane w owns word w (rows 32w..32w+31 of the chunk); the
// chunk's positions are assembled in a shared-memory stage and stream out
// with coalesced stores.
//   branching : only the qualifying rows are written to the stage;
//   predicated: cursor arithmetic -- every row is written, qualifying rows
//               at the lane's cursor and the others past the chunk's count.
template <int MODE>
__global__ void __launch_bounds__(BM_THREADS) k_sel_write(const uint32_t* __restrict__ bits,
                                                          const int64_t* __restrict__ offs, int64_t nchunks,
                                                          int32_t* __restrict__ out) {
    // stage index k is stored at k + k/32 (one pad word per 32): lanes whose
    // cursors are 32 apart hit different banks
    __shared__ int32_t s_stage[(BM_THREADS / 32) * (BM_CHUNK + BM_CHUNK / 32 + 4)];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int64_t gw = ((int64_t)blockIdx.x * BM_THREADS + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * BM_THREADS) >> 5;
    int32_t* st = s_stage + warp * (BM_CHUNK + BM_CHUNK / 32 + 4);
    // the bitmap words and offsets of the warp's next SW_PF chunks are in
    // flight while this one is decoded (a register queue shifted each step):
    // at low selectivity the pass is otherwise one L2/HBM round trip per chunk
    constexpr int SW_PF = 4;
    uint32_t wq[SW_PF];
    int64_t bq[SW_PF];
#pragma unroll
    for (int u = 0; u < SW_PF; ++u) {
        const int64_t cu = gw + u * nw;
        wq[u] = cu < nchunks ? __ldcs(&bits[cu * 32 + lane]) : 0u;
        bq[u] = cu < nchunks ? __ldcs(&offs[cu]) : 0;
    }
    for (int64_t c = gw; c < nchunks; c += nw) {
        const uint32_t w = wq[0];
        const int64_t base = bq[0];
#pragma unroll
        for (int u = 0; u + 1 < SW_PF; ++u) {
            wq[u] = wq[u + 1];
            bq[u] = bq[u + 1];
        }
        const int64_t cn = c + SW_PF * nw;
        wq[SW_PF - 1] = cn < nchunks ? __ldcs(&bits[cn * 32 + lane]) : 0u;
        bq[SW_PF - 1] = cn < nchunks ? __ldcs(&offs[cn]) : 0;
        const int pc = __popc(w);
        int incl = pc;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const int u = __shfl_up_sync(VD_FULL, incl, o);
            if (lane >= o) incl += u;
        }
        const int excl = incl - pc;
        const int total = __shfl_sync(VD_FULL, incl, 31);
        const int32_t row0 = (int32_t)(c * BM_CHUNK + lane * 32);
        // output index k sits at stage index j = k + a (a = the output's
        // misalignment in words), physically j + j/32: the 16-byte groups of
        // the output are 4-word groups of the stage that never straddle a pad
        const int a = (int)(((uintptr_t)(out + base) >> 2) & 3);
        if (MODE == 0) {
            uint32_t m = w;
            int k = excl + a;
            while (m) {
                st[k + (k >> 5)] = row0 + (__ffs(m) - 1);
                ++k;
                m &= m - 1;
            }
        } else {
            int sel = excl + a, unsel = total + (lane * 32 - excl) + a;
#pragma unroll
            for (int i = 0; i < 32; ++i) {
                const int f = (w >> i) & 1u;
                const int k = f ? sel : unsel;
                st[k + (k >> 5)] = row0 + i;
                sel += f;
                unsel += 1 - f;
            }
        }
        __syncwarp();
        // flush: scalar stores up to the first 16-byte boundary of the output
        // (any 4-byte aligned out_pos), then
        // one 128-bit streaming store per lane per 128 positions, scalar tail
        const int h = min(total, (4 - a) & 3);
        if (lane < h) __stcs(&out[base + lane], st[lane + a]);  // j < 32: no pad yet
        const int nv = (total - h) >> 2;
        int4* o4 = reinterpret_cast<int4*>(out + base + h);
        for (int v = lane; v < nv; v += 32) {
            const int j = h + a + 4 * v;  // a multiple of 4
            const int32_t* g = st + j + (j >> 5);
            __stcs(o4 + v, make_int4(g[0], g[1], g[2], g[3]));
        }
        for (int k = h + 4 * nv + lane; k < total; k += 32) {
            const int j = k + a;
            __stcs(&out[base + k], st[j + (j >> 5)]);
        }
        __syncwarp();
    }
}

struct BmLayout {
    int64_t nchunks;
    uint32_t* bits;
    int32_t* counts;
    int64_t* offs;
    void* scan_ws;
};
static BmLayout bm_layout(int64_t n, void* ws) {
    BmLayout L;
    L.nchunks = (n + BM_CHUNK - 1) / BM_CHUNK;
    char* w = (char*)ws;
    L.bits = (uint32_t*)w;
    w += al256((size_t)L.nchunks * 32 * 4);
    L.counts = (int32_t*)w;
    w += al256((size_t)L.nchunks * 4);
    L.offs = (int64_t*)w;
    w += al256((size_t)L.nchunks * 8);
    L.scan_ws = w;
    return L;
}
static size_t bm_ws_bytes(int64_t n) {
    int64_t nc = (n + BM_CHUNK - 1) / BM_CHUNK;
    return al256((size_t)nc * 32 * 4) + al256((size_t)nc * 4) + al256((size_t)nc * 8) + scan_ws_bytes(nc) + 256;
}
// One resident wave: blocks per SM from the kernel's occupancy (registers,
// shared memory), times the SM count -- a grid-stride loop over a grid
// larger than one wave leaves its last partial wave running alone.
template <class K>
static int bm_grid(K kern, int64_t nchunks) {
    int per_sm = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, BM_THREADS, 0) != cudaSuccess || per_sm < 1)
        per_sm = 1;
    int64_t g = (int64_t)num_sms() * per_sm;
    int64_t need = (nchunks * 32 + BM_THREADS - 1) / BM_THREADS;
    if (g > need) g = need;
    return (int)(g < 1 ? 1 : g);
}

template <int MODE, class LaunchBits>
static cudaError_t run_select_bitmap(LaunchBits launch_bits, int64_t n, int32_t* out_pos, int64_t* out_count,
                                     void* ws, cudaStream_t s, int* nl) {
    BmLayout L = bm_layout(n, ws);
    if (L.nchunks == 0) return cudaMemsetAsync(out_count, 0, sizeof(int64_t), s);
    launch_bits(L);
    ++*nl;
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return e;
    if ((e = launch_scan_i32(L.counts, L.nchunks, L.offs, L.scan_ws, s, nl)) != cudaSuccess) return e;
    k_sel_total<<<1, 1, 0, s>>>(L.offs, L.counts, L.nchunks, out_count);
    k_sel_write<MODE><<<bm_grid(k_sel_write<MODE>, L.nchunks), BM_THREADS, 0, s>>>(L.bits, L.offs, L.nchunks, out_pos);
    *nl += 2;
    return cudaGetLastError();
}

// ---- lagged single-pass selection (default for single interval terms on aligned 4-byte columns) ----
// One cooperative persistent kernel, one CTA per SM; tile t = k*G + blockIdx
// (SL_CW 1024-row chunks each, round robin over the grid):
//   producer warp   in iteration k: loads tile k through a TMA ring (lane 0);
//                   publishes tile k - SL_PUB (its chunk offsets to shared
//                   memory, its count to a global table cnt[k][blockIdx]);
//                   computes the output base of tile k - SL_BASE = the sum of
//                   every earlier table row (a running total) + the earlier
//                   CTAs' entries of its row, all published SL_BASE - SL_PUB
//                   iterations before -- a row is read whole, no look-back chain;
//   consumer warp w counts chunk w of tile k (lane L builds the bitmap word
//                   of rows 32L..32L+31 out of the TMA stage: the predicate
//                   materialised, Fig 8's break, kept in a per-lane REGISTER
//                   queue of LAG words, never written to memory), then decodes
//                   chunk w of tile k - LAG + 1 (positions staged in shared
//                   memory, 16-byte stores).
// Handoffs are mbarriers (counted[slot]: the SL_CW chunk counts; ready[slot]:
// offsets + base), so no warp waits on the CTA's other warps per iteration,
// and reads of tile k overlap position writes of tile k - LAG + 1 in every
// SM.  k_sel_coop (below) decodes only after a grid barrier; a striped
// counting/decoding warp split (k_sel_stream, round 2) and a per-iteration
// CTA barrier instead of mbarriers were measured slower.
// Deadlock-free under a cooperative launch: producer iteration k depends only
// on producer iterations < k of every CTA (row k - SL_BASE is published at
// iteration k - SL_BASE + SL_PUB), and consumers only on their producer.
constexpr int SL_CW = 15;                     // consumer warps = chunks per tile
constexpr int SL_THREADS = (SL_CW + 1) * 32;  // + the producer warp
constexpr int SL_STAGES = 3;                  // 3 x 60 KB in flight per SM
constexpr int SL_NS = 32;                     // per-tile shared slots (>= LAG + SL_STAGES + 1)
constexpr int SL_LAG = 12;                    // default LAG: iterations between counting and decoding a tile
                                              // (VD_SEL_LAG=16: a longer-lag instance)
constexpr int SL_PUB = 2;                     // producer: publishes tile k - SL_PUB in iteration k
constexpr int SL_BASE = 8;                    // ... and computes the base of tile k - SL_BASE
constexpr int SL_STG = 512 + 128 + 60;        // per-warp position stage (ints): half a chunk + garbage, or
                                              // VD_SEL_MID lane-owned positions + pad; the last 32: the words
static_assert(3 + 512 + 128 + 4 <= SL_STG - 32, "dense stage");
constexpr int SL_SPARSE = 48;                 // defaults: branching chunks this sparse store directly,
constexpr int SL_UNROLL = 160;                // ... this sparse: lane-owned rows, a per-bit loop (staged),
constexpr int SL_MID = 640;                   // ... this sparse: lane-owned rows, a fixed 32-row loop with
                                              //     predicated stores (staged); denser: ballot blocks
constexpr int SL_MID_PRED = 640;              // predicated chunks this sparse: lane-owned cursor arithmetic
                                              // (VD_SEL_SPARSE / VD_SEL_UNROLL / VD_SEL_MID override;
                                              // measured at s = 0.5: predicated 0.89 ms lane-owned vs 1.05 ms
                                              // ballot blocks; branching 0.87 ms with the fixed loop vs 0.97
                                              // per-bit loop or ballot blocks, profiles/round2s3_fig1_selpos_lag.md)
static_assert(640 + 4 + (640 + 4) / 32 + 4 <= SL_STG - 32, "lane-owned stage (VD_SEL_MID <= 640)");

struct SlShared {
    uint64_t full[SL_STAGES], empty[SL_STAGES];
    uint64_t counted[SL_NS];  // per slot: the SL_CW chunk counts are in cc
    uint64_t ready[SL_NS];    // per slot: off (producer, publish) and base (producer, table row) are set
    uint16_t cc[SL_NS][16];   // chunk counts of the tile in slot k % SL_NS
    uint16_t off[SL_NS][16];  // their exclusive prefix within the tile
    int64_t base[SL_NS]; // the tile's output base
};

__device__ __forceinline__ uint32_t ld_relaxed_u32(const unsigned int* p) {
    uint32_t v;
    asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_relaxed_u32(unsigned int* p, uint32_t v) {
    asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// `bit` if lo <= x <= hi (NaN / INT_MIN never: A9), else 0 -- two compares
// into one predicate and one select
__device__ __forceinline__ uint32_t ivl_bit(float x, float lo, float hi, uint32_t bit) {
    uint32_t r;
    asm("{\n\t.reg .pred p;\n\tsetp.ge.f32 p, %1, %2;\n\tsetp.le.and.f32 p, %1, %3, p;\n\tselp.b32 %0, %4, 0, p;\n\t}"
        : "=r"(r) : "f"(x), "f"(lo), "f"(hi), "r"(bit));
    return r;
}
__device__ __forceinline__ uint32_t ivl_bit(int32_t x, int32_t lo, int32_t hi, uint32_t bit) {
    uint32_t r;
    asm("{\n\t.reg .pred p;\n\tsetp.ge.s32 p, %1, %2;\n\tsetp.le.and.s32 p, %1, %3, p;\n\tselp.b32 %0, %4, 0, p;\n\t}"
        : "=r"(r) : "r"(x), "r"(lo), "r"(hi), "r"(bit));
    return r;
}

// Flush stage[a, a + tot) to o[0, tot) (o - a is 16-byte aligned): 16-byte
// streaming stores, the ragged head / tail element-wise.
__device__ __forceinline__ void sl_flush(const int32_t* sw, int a, int tot, int32_t* o, int lane) {
    const int ngr = (a + tot + 3) >> 2;
    int32_t* ob = o - a;
    for (int v = lane; v < ngr; v += 32) {
        const int4 x = *reinterpret_cast<const int4*>(sw + 4 * v);
        if (4 * v >= a && 4 * v + 4 <= a + tot) {
            __stcs(reinterpret_cast<int4*>(ob) + v, x);
        } else {
            const int32_t xs[4] = {x.x, x.y, x.z, x.w};
#pragma unroll
            for (int e = 0; e < 4; ++e) {
                const int kk = 4 * v + e;
                if (kk >= a && kk < a + tot) __stcs(ob + kk, xs[e]);
            }
        }
    }
}

// Positions of one 1024-row chunk: lane L holds word L (bit i <-> row
// row0 + 32 L + i), `cnt` its population, o = the chunk's first output.
template <int MODE>
__device__ __forceinline__ void sl_decode(uint32_t word, int cnt, int32_t* __restrict__ o, int32_t row0,
                                          int32_t* __restrict__ sw, int lane, int sparse_max, int mid_max,
                                          int unroll_min) {
    const unsigned lt = lanemask_lt();
    if (MODE == 1 && cnt <= mid_max) {
        // predicated, lane-owned rows: cursor arithmetic over the lane's 32
        // rows -- every row stored at the lane's cursor, the cursor advancing
        // by the predicate (no branch).  A lane's writes past its last
        // qualifying row land on the next lane's first slot; that lane
        // re-stores its first position once all stores are done.
        const int pc = __popc(word);
        int incl = pc;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            const int u = __shfl_up_sync(VD_FULL, incl, d);
            if (lane >= d) incl += u;
        }
        const int a = (int)(((uintptr_t)o >> 2) & 3);
        const int k0 = incl - pc + a;
        int cur = k0;
        const int32_t r = row0 + 32 * lane;
#pragma unroll
        for (int i = 0; i < 32; ++i) {
            sw[cur] = r + i;
            cur += (word >> i) & 1u;
        }
        __syncwarp();
        if (pc) sw[k0] = r + __ffs(word) - 1;
        __syncwarp();
        sl_flush(sw, a, cnt, o, lane);
        __syncwarp();
        return;
    }
    if (MODE == 0 && cnt <= mid_max) {
        const int pc = __popc(word);
        int incl = pc;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            const int u = __shfl_up_sync(VD_FULL, incl, d);
            if (lane >= d) incl += u;
        }
        int k = incl - pc;
        const int32_t r = row0 + 32 * lane - 1;
        uint32_t m = word;
        if (cnt <= sparse_max) {  // few positions: straight to global memory
            while (m) {
                __stcs(o + k, r + __ffs(m));
                ++k;
                m &= m - 1;
            }
            return;
        }
        if (cnt > unroll_min) {
            // denser lane-owned chunks: the lane walks all 32 rows with the
            // store under the row's predicate (only qualifying rows are
            // written: branching) -- a fixed loop, no divergence on the
            // per-lane bit counts; then 16-byte stores
            const int a = (int)(((uintptr_t)o >> 2) & 3);
            int cur = k + a;
#pragma unroll
            for (int i = 0; i < 32; ++i) {
                const uint32_t f = (word >> i) & 1u;
                if (f) sw[cur] = r + 1 + i;
                cur += f;
            }
            __syncwarp();
            sl_flush(sw, a, cnt, o, lane);
            __syncwarp();
            return;
        }
        // lane-owned rows staged (index x at x + x/32: lanes 32 apart hit
        // different banks), then 16-byte stores
        const int a = (int)(((uintptr_t)o >> 2) & 3);
        while (m) {
            const int x = k + a;
            sw[x + (x >> 5)] = r + __ffs(m);
            ++k;
            m &= m - 1;
        }
        __syncwarp();
        const int ngr = (a + cnt + 3) >> 2;
        int32_t* ob = o - a;
        for (int v = lane; v < ngr; v += 32) {
            const int x = 4 * v;  // a multiple of 4: the group never straddles a pad word
            const int32_t* q = sw + x + (x >> 5);
            if (x >= a && x + 4 <= a + cnt) {
                __stcs(reinterpret_cast<int4*>(ob) + v, make_int4(q[0], q[1], q[2], q[3]));
            } else {
#pragma unroll
                for (int e = 0; e < 4; ++e)
                    if (x + e >= a && x + e < a + cnt) __stcs(ob + x + e, q[e]);
            }
        }
        __syncwarp();
        return;
    }
    // dense chunks (and every predicated chunk): word j broadcast to the warp,
    // lane L places row 32j + L at the running rank (branching: qualifying
    // lanes only; predicated: cursor arithmetic -- every lane stores, rows that
    // do not qualify past the 128-row block's count, overwritten later)
    const int32_t rl = row0 + lane;
    uint32_t* ww = reinterpret_cast<uint32_t*>(sw + SL_STG - 32);  // the chunk's words, read back as broadcasts
    ww[lane] = word;
    __syncwarp();
#pragma unroll
    for (int h = 0; h < 2; ++h) {  // two 512-row halves, each staged and flushed
    const int a = (int)(((uintptr_t)o >> 2) & 3);
    int cur = a;
#pragma unroll
    for (int q = 4 * h; q < 4 * h + 4; ++q) {
        const uint4 b4 = *reinterpret_cast<const uint4*>(ww + 4 * q);
        const uint32_t bw[4] = {b4.x, b4.y, b4.z, b4.w};
        const int cq = __popc(bw[0]) + __popc(bw[1]) + __popc(bw[2]) + __popc(bw[3]);
        int pre = cur;
#pragma unroll
        for (int jj = 0; jj < 4; ++jj) {
            const uint32_t w = bw[jj];
            const bool f = (w >> lane) & 1u;
            const int r = __popc(w & lt);
            const int32_t row = rl + 32 * (4 * q + jj);
            if (MODE == 0) {
                if (f) sw[pre + r] = row;
            } else {
                const int sel_before = pre - cur + r;
                sw[f ? pre + r : cur + cq + (jj * 32 + lane - sel_before)] = row;
            }
            pre += __popc(w);
        }
        cur += cq;
    }
    __syncwarp();
    sl_flush(sw, a, cur - a, o, lane);
    __syncwarp();
    o += cur - a;
    }
}

template <int MODE, typename T, int LAG>
__global__ void __launch_bounds__(SL_THREADS, 1) k_sel_lag(const T* __restrict__ col, T lo, T hi, int64_t n,
                                                           int32_t* __restrict__ out, int64_t* __restrict__ out_count,
                                                           unsigned int* __restrict__ cnt /* [nk][G], zeroed */,
                                                           int sparse_max, int mid_max, int unroll_min) {
    static_assert(sizeof(T) == 4, "k_sel_lag: 4-byte columns (f32 / i32)");
    static_assert(SL_PUB < SL_BASE && SL_BASE < LAG && LAG + SL_STAGES + 1 <= SL_NS, "k_sel_lag: lags / shared slots");
    constexpr uint32_t TB = SL_CW * 1024 * sizeof(T);
    extern __shared__ __align__(128) uint8_t smem[];
    int32_t* stages = reinterpret_cast<int32_t*>(smem + (size_t)SL_STAGES * TB);
    SlShared& H = *reinterpret_cast<SlShared*>(stages + SL_CW * SL_STG);
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int G = gridDim.x, c = blockIdx.x;
    const int64_t nchunks = (n + 1023) / 1024;
    const int64_t ntiles = (nchunks + SL_CW - 1) / SL_CW;
    const int64_t myk = ntiles > c ? (ntiles - c + G - 1) / G : 0;  // this CTA's tiles: k < myk
    if (threadIdx.x == 0) {
        for (int i = 0; i < SL_STAGES; ++i) {
            mbar_init(&H.full[i], 1);
            mbar_init(&H.empty[i], SL_CW);
        }
        for (int i = 0; i < SL_NS; ++i) {
            mbar_init(&H.counted[i], SL_CW);
            mbar_init(&H.ready[i], 2);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (warp == SL_CW) {
        // ---- producer / bookkeeping warp: in iteration k it
        //   loads tile k (lane 0, TMA),
        //   publishes tile k - SL_PUB: chunk offsets to shared memory, the
        //     tile's count to the table,
        //   computes the base of tile k - SL_BASE from table row k - SL_BASE
        //     (published by every CTA SL_BASE - SL_PUB iterations earlier),
        // and the two halves of ready[tile] let its decoders go.
        const uint64_t pol = policy_evict_first();
        int st = 0;
        uint32_t ph = 0;
        int64_t run = 0;  // the totals of the rows read so far
        for (int64_t k = 0; k < myk + SL_BASE; ++k) {
            if (k < myk) {
                if (lane == 0) {
                    if (k >= SL_STAGES) mbar_wait(&H.empty[st], ph ^ 1u);
                    const int64_t r0 = (k * G + c) * (int64_t)SL_CW * 1024;
                    if (r0 + (int64_t)SL_CW * 1024 <= n) {
                        mbar_expect_tx(&H.full[st], TB);
                        tma_load_1d(smem + (size_t)st * TB, col + r0, TB, &H.full[st], pol);
                    } else {
                        mbar_arrive(&H.full[st]);  // the column's last, partial tile: consumers load it directly
                    }
                }
                if (++st == SL_STAGES) { st = 0; ph ^= 1u; }
                __syncwarp();
            }
            const int64_t kp = k - SL_PUB;
            if (kp >= 0 && kp < myk) {
                const int sp = (int)(kp & (SL_NS - 1));
                mbar_wait(&H.counted[sp], (uint32_t)(kp / SL_NS) & 1u);
                const int x = lane < SL_CW ? H.cc[sp][lane] : 0;
                int incl = x;
#pragma unroll
                for (int d = 1; d < 32; d <<= 1) {
                    const int u = __shfl_up_sync(VD_FULL, incl, d);
                    if (lane >= d) incl += u;
                }
                if (lane < SL_CW) H.off[sp][lane] = (uint16_t)(incl - x);
                if (lane == 31) st_relaxed_u32(cnt + kp * G + c, (uint32_t)incl + 1u);
                __syncwarp();
                if (lane == 0) mbar_arrive(&H.ready[sp]);
            }
            const int64_t kb = k - SL_BASE;
            if (kb >= 0 && kb < myk) {
                uint32_t rv[5];
#pragma unroll
                for (int i = 0; i < 5; ++i) {
                    const int j = lane + 32 * i;
                    rv[i] = (j < G && kb * G + j < ntiles) ? ld_relaxed_u32(cnt + kb * G + j) : 1u;  // absent: 0
                }
                int pre = 0, tot = 0;
#pragma unroll
                for (int i = 0; i < 5; ++i) {
                    const int j = lane + 32 * i;
                    while (rv[i] == 0u) {
                        __nanosleep(20);
                        rv[i] = ld_relaxed_u32(cnt + kb * G + j);
                    }
                    const int x = (int)rv[i] - 1;
                    tot += x;
                    pre += j < c ? x : 0;
                }
#pragma unroll
                for (int d = 16; d; d >>= 1) {
                    pre += __shfl_xor_sync(VD_FULL, pre, d);
                    tot += __shfl_xor_sync(VD_FULL, tot, d);
                }
                const int sb = (int)(kb & (SL_NS - 1));
                if (lane == 0) {
                    H.base[sb] = run + pre;
                    mbar_arrive(&H.ready[sb]);
                }
                run += tot;
            }
        }
        // CTA 0 owns a tile in every row: its run is the grand total
        if (c == 0 && lane == 0) *out_count = run;
        return;
    }
    // ---- consumer warps: count chunk `warp` of tile k, decode it LAG iterations later ----
    int32_t* sw = stages + warp * SL_STG;
    uint32_t q[LAG];
#pragma unroll
    for (int i = 0; i < LAG; ++i) q[i] = 0;
    int st = 0;
    uint32_t ph = 0;
    for (int64_t k = 0; k < myk + LAG; ++k) {
        if (k < myk) {
            const int slot = (int)(k & (SL_NS - 1));
            uint32_t word = 0;
            mbar_wait(&H.full[st], ph);
            const int64_t t = k * G + c;
            const int64_t ch = t * SL_CW + warp;
            if (ch < nchunks) {
                if ((t + 1) * (int64_t)SL_CW * 1024 <= n) {
                    // lane L: rows 32L .. 32L+31 of the chunk in 8 16-byte loads,
                    // rotated by L so the 8 lanes of a load phase hit 8
                    // different 16-byte bank groups (conflict-free)
                    const T* src = reinterpret_cast<const T*>(smem + (size_t)st * TB) + warp * 1024 + 32 * lane;
#pragma unroll
                    for (int m = 0; m < 8; ++m) {
                        const int mm = (m + lane) & 7;
                        T x[4];
                        Vec4Lds<T>::ld(src + 4 * mm, x);
                        const uint32_t nib = ivl_bit(x[0], lo, hi, 1u) | ivl_bit(x[1], lo, hi, 2u) |
                                             ivl_bit(x[2], lo, hi, 4u) | ivl_bit(x[3], lo, hi, 8u);
                        word |= nib << (4 * mm);
                    }
                } else {
                    for (int i = 0; i < 32; ++i) {
                        const int64_t r = ch * 1024 + 32 * lane + i;
                        if (r < n) {
                            const T v = __ldg(col + r);
                            word |= (uint32_t)(v >= lo && v <= hi) << i;
                        }
                    }
                }
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&H.empty[st]);
            if (++st == SL_STAGES) { st = 0; ph ^= 1u; }
            int cw = __popc(word);
#pragma unroll
            for (int d = 16; d; d >>= 1) cw += __shfl_xor_sync(VD_FULL, cw, d);
            if (lane == 0) {
                H.cc[slot][warp] = (uint16_t)cw;
                mbar_arrive(&H.counted[slot]);  // release: the count is visible to the producer's wait
            }
#pragma unroll
            for (int i = 0; i + 1 < LAG; ++i) q[i] = q[i + 1];
            q[LAG - 1] = word;
        } else {
#pragma unroll
            for (int i = 0; i + 1 < LAG; ++i) q[i] = q[i + 1];
            q[LAG - 1] = 0;
        }
        // decode chunk `warp` of tile k - LAG + 1 (q[0])
        const int64_t kd = k - LAG + 1;
        if (kd >= 0 && kd < myk) {
            const int ds = (int)(kd & (SL_NS - 1));
            mbar_wait(&H.ready[ds], (uint32_t)(kd / SL_NS) & 1u);
            const int cd = H.cc[ds][warp];
            if (cd > 0) {
                const int64_t ob = H.base[ds] + H.off[ds][warp];
                const int32_t row0 = (int32_t)(((kd * G + c) * SL_CW + warp) * 1024);
                sl_decode<MODE>(q[0], cd, out + ob, row0, sw, lane, sparse_max, mid_max, unroll_min);
            }
        }
    }
}

static size_t sel_lag_smem() {
    return (size_t)SL_STAGES * SL_CW * 1024 * 4 + (size_t)SL_CW * SL_STG * 4 + sizeof(SlShared);
}
static size_t sel_lag_ws_bytes(int64_t n) {
    const int64_t ntiles = ((n + 1023) / 1024 + SL_CW - 1) / SL_CW;
    return al256((size_t)(ntiles + 4096) * 4);
}

// VD_SELECT_KERNEL=coop: the single-barrier kernel instead (comparison runs;
// read per call: tests switch kernels inside one process)
static int sel_kernel_choice() {
    const char* e = getenv("VD_SELECT_KERNEL");
    return (e && strcmp(e, "coop") == 0) ? 1 : 0;
}

template <int MODE, typename T>
static cudaError_t run_select_lag(const T* col, T lo, T hi, int64_t n, int32_t* out_pos, int64_t* out_count,
                                  void* ws, cudaStream_t s, int* nl) {
    if (n == 0) return cudaMemsetAsync(out_count, 0, sizeof(int64_t), s);
    const int64_t ntiles = ((n + 1023) / 1024 + SL_CW - 1) / SL_CW;
    const size_t sm = sel_lag_smem();
    const char* lv = getenv("VD_SEL_LAG");
    auto kern = (lv && atoi(lv) == 16) ? k_sel_lag<MODE, T, 16> : k_sel_lag<MODE, T, SL_LAG>;
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm);
    int per_sm = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, SL_THREADS, sm) != cudaSuccess || per_sm < 1)
        return cudaErrorNotSupported;
    // one CTA per SM, at most one per tile (small inputs: one tile each, the
    // table a single row); a table row = 5 loads per lane
    const int G = (int)std::min<int64_t>(std::min<int64_t>((int64_t)num_sms() * per_sm, 160), ntiles);
    if (n > (int64_t)INT32_MAX) return cudaErrorNotSupported;
    const int64_t nk = (ntiles + G - 1) / G;
    unsigned int* cnt = (unsigned int*)ws;
    cudaError_t e = cudaMemsetAsync(cnt, 0, (size_t)nk * G * 4, s);
    if (e != cudaSuccess) return e;
    auto knob = [](const char* name, int dflt, int hi) {
        const char* v = getenv(name);
        const int x = v ? atoi(v) : dflt;
        return x < 0 ? 0 : (x > hi ? hi : x);
    };
    // lane-owned chunks must fit the stage: x + x/32 + 4 < SL_STG
    int sparse_max = knob("VD_SEL_SPARSE", SL_SPARSE, 1024), mid_max = knob("VD_SEL_MID", MODE ? SL_MID_PRED : SL_MID, 640);
    int unroll_min = knob("VD_SEL_UNROLL", SL_UNROLL, 1024);  // branching lane-owned chunks above this: the fixed loop
    void* args[] = {(void*)&col,       (void*)&lo,  (void*)&hi,         (void*)&n,       (void*)&out_pos,
                    (void*)&out_count, (void*)&cnt, (void*)&sparse_max, (void*)&mid_max, (void*)&unroll_min};
    e = cudaLaunchCooperativeKernel((const void*)kern, dim3(G), dim3(SL_THREADS), args, sm, s);
    ++*nl;
    return e;
}

size_t select_ws_bytes(int64_t n) {
    int64_t ntiles = (n + SEL_TILE - 1) / SEL_TILE;
    size_t b = 256 + (size_t)ntiles * 8;
    size_t lb = (b + 255) & ~(size_t)255;
    size_t bm = std::max(std::max(bm_ws_bytes(n), sel_lag_ws_bytes(n)), sel_coop_ws_bytes(n));
    return lb > bm ? lb : bm;
}

static bool use_lookback() {
    const char* v = getenv("VD_SELECT_VARIANT");
    return v && strcmp(v, "lookback") == 0;
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

// Interval form [lo, hi] of one comparison on a column of T (epsilon
// excluded); false for NE / IN.
template <typename T>
static bool term_interval_t(const DevTerm& t, T* lo, T* hi) {
    if (IsFloat<T>::value) {
        // exact for f32 / f64 values against a double constant
        const double c = t.fv;
        double l = -HUGE_VAL, h = HUGE_VAL;
        auto down = [](double x) { T f = (T)x; if ((double)f > x) f = nextafter(f, (T)-HUGE_VAL); return f; };
        auto up = [](double x) { T f = (T)x; if ((double)f < x) f = nextafter(f, (T)HUGE_VAL); return f; };
        switch (t.cmp) {
        case VD_CMP_GT: l = (double)nextafter(down(c), (T)HUGE_VAL); break;
        case VD_CMP_GE: l = (double)up(c); break;
        case VD_CMP_LT: h = (double)nextafter(up(c), (T)-HUGE_VAL); break;
        case VD_CMP_LE: h = (double)down(c); break;
        case VD_CMP_EQ: if ((double)(T)c != c) { l = 1; h = 0; } else { l = h = c; } break;
        default: return false;
        }
        *lo = (T)l;
        *hi = (T)h;
        return true;
    }
    const int64_t tmin = std::is_same<T, uint8_t>::value ? 0 : (std::is_same<T, int32_t>::value ? INT32_MIN + 1 : INT64_MIN + 1);
    const int64_t tmax = std::is_same<T, uint8_t>::value ? 0xFE : (std::is_same<T, int32_t>::value ? INT32_MAX : INT64_MAX);
    int64_t l = tmin, h = tmax;
    const int64_t c = t.iv;
    switch (t.cmp) {
    case VD_CMP_GT: if (c >= tmax) { l = 1; h = 0; } else l = std::max(l, c + 1); break;
    case VD_CMP_GE: l = std::max(l, c); break;
    case VD_CMP_LT: if (c <= tmin) { l = 1; h = 0; } else h = std::min(h, c - 1); break;
    case VD_CMP_LE: h = std::min(h, c); break;
    case VD_CMP_EQ: l = std::max(l, c); h = std::min(h, c); break;
    default: return false;
    }
    if (l > h) { l = 1; h = 0; }
    if (std::is_same<T, uint8_t>::value && l > h) { *lo = (T)1; *hi = (T)0; return true; }
    *lo = (T)l;
    *hi = (T)h;
    return true;
}

// TMA flag pass: 1- and 4-byte columns (16-byte aligned, checked by the
// caller); VD_SELECT_BITS=ldg forces the LDG pass (kept for comparison)
template <typename T>
static bool use_bits_tma() {
    if (sizeof(T) != 4 && sizeof(T) != 1) return false;
    static const bool ldg = [] {
        const char* e = getenv("VD_SELECT_BITS");
        return e && strcmp(e, "ldg") == 0;
    }();
    return !ldg;
}

template <int MODE, typename T>
static cudaError_t dispatch_term(const void* p, const DevTerm& t, int64_t n, int32_t* out_pos, int64_t* out_count,
                                 void* ws, cudaStream_t s, int* nl) {
    size_t vecbytes = sizeof(T) * 4 > 16 ? 16 : sizeof(T) * 4;
    bool aligned = ((uintptr_t)p % vecbytes) == 0;
    T ilo = T(0), ihi = T(0);
    const int ivl = term_interval_t<T>(t, &ilo, &ihi) ? 1 : 0;
    if (aligned) {
        TermFlags<T, true> f{(const T*)p, t.cmp, t.iv, t.fv, ivl, ilo, ihi};
        if (use_lookback()) {
            set_fragment("sel_lookback");
            return run_select<MODE>(f, n, out_pos, out_count, ws, s, nl);
        }
        if constexpr (sizeof(T) == 4) {
            if (ivl && use_sel_coop() && ((uintptr_t)p & 15) == 0) {
                const int kc = sel_kernel_choice();
                if (kc == 0) {
                    set_fragment("sel_lag");
                    cudaError_t e = run_select_lag<MODE, T>((const T*)p, ilo, ihi, n, out_pos, out_count, ws, s, nl);
                    if (e != cudaErrorNotSupported) return e;  // else: small, the single-barrier kernel
                }
                set_fragment("sel_coop");
                cudaError_t e = run_select_coop<MODE, T>((const T*)p, ilo, ihi, n, out_pos, out_count, ws, s, nl);
                if (e != cudaErrorNotSupported) return e;  // else: more chunks per CTA than fit, bitmap path
            }
        }
        set_fragment("sel_bitmap");
        return run_select_bitmap<MODE>(
            [&](const BmLayout& L) {
                bool tma_done = false;
                if constexpr (sizeof(T) == 4 || sizeof(T) == 1) {
                if (ivl && use_bits_tma<T>() && ((uintptr_t)p & 15) == 0) {
                    // full tiles through the TMA ring, the rest (< BT_CW chunks + ragged tail) by LDG
                    const int64_t ntiles = n / ((int64_t)BT_CW * BM_CHUNK);
                    if (ntiles > 0) {
                        const size_t sm = (size_t)BT_STAGES * BT_CW * BM_CHUNK * sizeof(T) + 2 * BT_STAGES * 8;
                        cudaFuncSetAttribute(k_sel_bits_tma<T>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm);
                        const int g = (int)std::min<int64_t>(ntiles, num_sms());
                        k_sel_bits_tma<T><<<g, BT_THREADS, sm, s>>>((const T*)p, ilo, ihi, ntiles, L.bits, L.counts);
                        ++*nl;
                    }
                    const int64_t c0 = ntiles * BT_CW;
                    if (c0 < L.nchunks)
                        k_sel_bits_vec<T, true, true><<<bm_grid(k_sel_bits_vec<T, true, true>, L.nchunks - c0), BM_THREADS, 0, s>>>(f, n, L.bits, L.counts, L.nchunks, c0);
                    else
                        --*nl;  // run_select_bitmap counts one flag launch
                    tma_done = true;
                }
                }
                if (tma_done) {
                } else if (ivl) k_sel_bits_vec<T, true, true><<<bm_grid(k_sel_bits_vec<T, true, true>, L.nchunks), BM_THREADS, 0, s>>>(f, n, L.bits, L.counts, L.nchunks);
                else k_sel_bits_vec<T, true, false><<<bm_grid(k_sel_bits_vec<T, true, false>, L.nchunks), BM_THREADS, 0, s>>>(f, n, L.bits, L.counts, L.nchunks);
            },
            n, out_pos, out_count, ws, s, nl);
    }
    TermFlags<T, false> f{(const T*)p, t.cmp, t.iv, t.fv, ivl, ilo, ihi};
    if (use_lookback()) return run_select<MODE>(f, n, out_pos, out_count, ws, s, nl);
    return run_select_bitmap<MODE>(
        [&](const BmLayout& L) {
            k_sel_bits_vec<T, false, false><<<bm_grid(k_sel_bits_vec<T, false, false>, L.nchunks), BM_THREADS, 0, s>>>(f, n, L.bits, L.counts, L.nchunks);
        },
        n, out_pos, out_count, ws, s, nl);
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
    if (use_lookback()) return run_select<MODE>(g, n, out_pos, out_count, ws, s, nl);
    return run_select_bitmap<MODE>(
        [&](const BmLayout& L) {
            k_sel_bits_bal<GenericFlags><<<bm_grid(k_sel_bits_bal<GenericFlags>, L.nchunks), BM_THREADS, 0, s>>>(g, n, L.bits, L.counts, L.nchunks);
        },
        n, out_pos, out_count, ws, s, nl);
}

cudaError_t launch_select(int mode, const DevCols& cols, const DevPred& pred, int64_t n, int32_t* out_pos,
                          int64_t* out_count, void* ws, size_t, cudaStream_t s, int* nl) {
    if (mode == VD_SEL_PREDICATED) return select_mode<1>(cols, pred, n, out_pos, out_count, ws, s, nl);
    return select_mode<0>(cols, pred, n, out_pos, out_count, ws, s, nl);
}

cudaError_t launch_select_heads(const CtrlInfo& ci, int64_t n, int32_t* out_pos, int64_t* out_count, void* ws,
                                size_t, cudaStream_t s, int* nl) {
    HeadFlags h{ci.mat, ci.mat_dtype, ci.from, ci.num, ci.den, ci.cap};
    if (use_lookback()) return run_select<0>(h, n, out_pos, out_count, ws, s, nl);
    return run_select_bitmap<0>(
        [&](const BmLayout& L) {
            k_sel_bits_bal<HeadFlags><<<bm_grid(k_sel_bits_bal<HeadFlags>, L.nchunks), BM_THREADS, 0, s>>>(h, n, L.bits, L.counts, L.nchunks);
        },
        n, out_pos, out_count, ws, s, nl);
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
