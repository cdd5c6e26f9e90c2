// k_scatter.cu -- Scatter and Partition (§8(a) a5).
//
// Scatter(V1, V2, .kp2, V3, .pos) (Table 2): an output of the
// requested size whose slots are filled by placing each value of V1 at its
// position; "values are overwritten on conflict ... in order within a run".
// Canonical reading A12: the later input index wins.  Unique positions (a
// Partition output) need no arbitration; otherwise a claim pass keeps, per
// output slot, the largest writing index (REDG.MAX on a 32-bit claim word)
// and only that index stores its value.
//
// Partition(.out, V1, .v, V2, .pv) (Fig 11): stable range
// partition -> scatter positions.  Three passes over warp tiles:
//   k_part_hist    per-tile bucket counts, bucket-major matrix
//   k_scan_i32     exclusive scan of that matrix (decoupled look-back)
//   k_part_place   per-tile stable ranks via __match_any_sync + per-warp
//                  running bucket counters, position = offset + rank.
#include "vd_common.cuh"
#include "vd_internal.h"
#include "vd_lookback.cuh"

namespace vd {

// ---- Scatter ----------------------------------------------------------------
template <typename T>
__global__ void k_fill_eps(T* __restrict__ out, int64_t n) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) out[i] = Eps<T>::value();
}

__global__ void k_scatter_claim(const int32_t* __restrict__ pos, int64_t n, int64_t out_len, int* __restrict__ claim) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        int32_t p = __ldg(pos + i);
        if (p >= 0 && (int64_t)p < out_len) atomicMax(claim + p, (int)i);
    }
}

template <typename T, bool UNIQUE>
__global__ void k_scatter_write(const T* __restrict__ src, const int32_t* __restrict__ pos, int64_t n, int64_t out_len,
                                const int* __restrict__ claim, T* __restrict__ out) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        int32_t p = __ldg(pos + i);
        if (p < 0 || (int64_t)p >= out_len) continue;
        if (UNIQUE || __ldg(claim + p) == (int)i) out[p] = __ldg(src + i);
    }
}

size_t scatter_ws_bytes(int64_t out_len) { return (((size_t)out_len * 4 + 255) & ~(size_t)255) + 256; }

static int grid_for(int64_t n, int per = 256) {
    int64_t b = (n + per - 1) / per;
    int64_t cap = (int64_t)num_sms() * 8;
    if (b > cap) b = cap;
    return (int)(b < 1 ? 1 : b);
}

template <typename T>
static cudaError_t scatter_typed(const vd_column& src, const int32_t* pos, int64_t n, void* out, int64_t out_len,
                                 bool unique, void* ws, cudaStream_t s, int* nl) {
    if (out_len > 0) {
        k_fill_eps<T><<<grid_for(out_len), 256, 0, s>>>((T*)out, out_len);
        ++*nl;
    }
    if (n == 0 || out_len == 0) return cudaGetLastError();
    int* claim = (int*)ws;
    if (!unique) {
        cudaError_t e = cudaMemsetAsync(claim, 0xFF, (size_t)out_len * 4, s);  // -1
        if (e != cudaSuccess) return e;
        k_scatter_claim<<<grid_for(n), 256, 0, s>>>(pos, n, out_len, claim);
        ++*nl;
        k_scatter_write<T, false><<<grid_for(n), 256, 0, s>>>((const T*)src.data, pos, n, out_len, claim, (T*)out);
    } else {
        k_scatter_write<T, true><<<grid_for(n), 256, 0, s>>>((const T*)src.data, pos, n, out_len, claim, (T*)out);
    }
    ++*nl;
    return cudaGetLastError();
}

cudaError_t launch_scatter(const vd_column& src, const int32_t* pos, int64_t n, void* out, int64_t out_len,
                           bool unique, void* ws, cudaStream_t s, int* nl) {
    switch (src.dtype) {
    case VD_U8: return scatter_typed<uint8_t>(src, pos, n, out, out_len, unique, ws, s, nl);
    case VD_I32: return scatter_typed<int32_t>(src, pos, n, out, out_len, unique, ws, s, nl);
    case VD_I64: return scatter_typed<int64_t>(src, pos, n, out, out_len, unique, ws, s, nl);
    case VD_F32: return scatter_typed<float>(src, pos, n, out, out_len, unique, ws, s, nl);
    default: return scatter_typed<double>(src, pos, n, out, out_len, unique, ws, s, nl);
    }
}

// ---- Partition ---------------------------------------------------------------
constexpr int PART_THREADS = 256;
constexpr int PART_WARPS = PART_THREADS / 32;
constexpr int PART_MAXP = 1024;

template <typename T>
__device__ __forceinline__ int bucket_of(T x, int64_t from, int64_t npiv) {
    if (Eps<T>::is(x)) return -1;
    int64_t b = (int64_t)x - from;
    if (b < 0) b = 0;
    if (b >= npiv) b = npiv - 1;
    return (int)b;
}

// One warp per tile of `tw` rows, counts[b * ntiles + tile].
template <typename T>
__global__ void __launch_bounds__(PART_THREADS) k_part_hist(const T* __restrict__ v, int64_t n, int64_t from, int npiv,
                                                            int64_t tw, int64_t ntiles, int32_t* __restrict__ counts) {
    extern __shared__ int s_cnt[];  // [PART_WARPS][npiv]
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    int* c = s_cnt + warp * npiv;
    const int64_t gw = (int64_t)blockIdx.x * PART_WARPS + warp;
    const int64_t nw = (int64_t)gridDim.x * PART_WARPS;
    for (int64_t tile = gw; tile < ntiles; tile += nw) {
        for (int b = lane; b < npiv; b += 32) c[b] = 0;
        __syncwarp();
        int64_t a = tile * tw, e = a + tw < n ? a + tw : n;
        for (int64_t i = a + lane; i < e; i += 32) {
            int b = bucket_of(__ldg(v + i), from, npiv);
            if (b >= 0) atomicAdd(c + b, 1);
        }
        __syncwarp();
        for (int b = lane; b < npiv; b += 32) counts[(int64_t)b * ntiles + tile] = c[b];
        __syncwarp();
    }
}

// Exclusive scan of int32 counts into int64 offsets, one pass (look-back).
constexpr int SCAN_THREADS = 256;
constexpr int SCAN_ITEMS = 8;
constexpr int SCAN_TILE = SCAN_THREADS * SCAN_ITEMS;

__global__ void __launch_bounds__(SCAN_THREADS) k_scan_i32(const int32_t* __restrict__ in, int64_t m,
                                                           int64_t* __restrict__ out, uint64_t* __restrict__ status,
                                                           unsigned long long* __restrict__ ctr, int64_t ntiles) {
    __shared__ int64_t s_tile, s_base;
    __shared__ int64_t s_warp[SCAN_THREADS / 32];
    const int t = threadIdx.x, warp = t >> 5, lane = t & 31;
    for (;;) {
        if (t == 0) s_tile = (int64_t)atomicAdd(ctr, 1ull);
        __syncthreads();
        int64_t tile = s_tile;
        if (tile >= ntiles) break;
        int64_t r0 = tile * SCAN_TILE + (int64_t)t * SCAN_ITEMS;
        int64_t x[SCAN_ITEMS], sum = 0;
#pragma unroll
        for (int j = 0; j < SCAN_ITEMS; ++j) {
            x[j] = (r0 + j < m) ? (int64_t)in[r0 + j] : 0;
            sum += x[j];
        }
        int64_t incl = sum;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            int64_t u = __shfl_up_sync(VD_FULL, incl, o);
            if (lane >= o) incl += u;
        }
        if (lane == 31) s_warp[warp] = incl;
        __syncthreads();
        if (warp == 0) {
            int64_t w = lane < SCAN_THREADS / 32 ? s_warp[lane] : 0;
            int64_t wi = w;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                int64_t u = __shfl_up_sync(VD_FULL, wi, o);
                if (lane >= o) wi += u;
            }
            if (lane < SCAN_THREADS / 32) s_warp[lane] = wi - w;
            int64_t agg = __shfl_sync(VD_FULL, wi, SCAN_THREADS / 32 - 1);
            int64_t base = lookback_exclusive(status, tile, agg, lane);
            if (lane == 0) s_base = base;
        }
        __syncthreads();
        int64_t run = s_base + s_warp[warp] + incl - sum;
#pragma unroll
        for (int j = 0; j < SCAN_ITEMS; ++j) {
            if (r0 + j < m) out[r0 + j] = run;
            run += x[j];
        }
        __syncthreads();
    }
}

size_t scan_ws_bytes(int64_t m) { return 256 + ((((size_t)(m + SCAN_TILE - 1) / SCAN_TILE) * 8 + 255) & ~(size_t)255); }

cudaError_t launch_scan_i32(const int32_t* in, int64_t m, int64_t* out, void* ws, cudaStream_t s, int* nl) {
    if (m <= 0) return cudaSuccess;
    int64_t st = (m + SCAN_TILE - 1) / SCAN_TILE;
    cudaError_t e = cudaMemsetAsync(ws, 0, 256 + (size_t)st * 8, s);
    if (e != cudaSuccess) return e;
    int sg = (int)(st < (int64_t)num_sms() * 4 ? st : (int64_t)num_sms() * 4);
    k_scan_i32<<<sg, SCAN_THREADS, 0, s>>>(in, m, out, (uint64_t*)((char*)ws + 256), (unsigned long long*)ws, st);
    ++*nl;
    return cudaGetLastError();
}

template <typename T>
__global__ void __launch_bounds__(PART_THREADS) k_part_place(const T* __restrict__ v, int64_t n, int64_t from, int npiv,
                                                             int64_t tw, int64_t ntiles,
                                                             const int64_t* __restrict__ offs,
                                                             int32_t* __restrict__ out) {
    extern __shared__ int s_cnt[];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    int* c = s_cnt + warp * npiv;
    const unsigned lt = lanemask_lt();
    const int64_t gw = (int64_t)blockIdx.x * PART_WARPS + warp;
    const int64_t nw = (int64_t)gridDim.x * PART_WARPS;
    for (int64_t tile = gw; tile < ntiles; tile += nw) {
        for (int b = lane; b < npiv; b += 32) c[b] = 0;
        __syncwarp();
        int64_t a = tile * tw, e = a + tw < n ? a + tw : n;
        for (int64_t i0 = a; i0 < e; i0 += 32) {
            int64_t i = i0 + lane;
            int b = (i < e) ? bucket_of(__ldg(v + i), from, npiv) : -2;
            unsigned m = __match_any_sync(VD_FULL, b);
            int rank = __popc(m & lt);
            int before = (b >= 0) ? c[b] : 0;
            __syncwarp();
            if (b >= 0) {
                out[i] = (int32_t)(offs[(int64_t)b * ntiles + tile] + before + rank);
                if (rank == __popc(m) - 1) c[b] = before + __popc(m);  // last lane of the group advances
            } else if (b == -1) {
                out[i] = -1;  // epsilon key: no position
            }
            __syncwarp();
        }
    }
}

struct PartGeom {
    int64_t tw, ntiles, m;
};
static PartGeom part_geom(int64_t n, int64_t npiv) {
    PartGeom g;
    g.tw = 1024;
    // keep the count matrix <= 2^24 entries
    while (npiv * ((n + g.tw - 1) / g.tw) > (1ll << 24)) g.tw *= 2;
    g.ntiles = (n + g.tw - 1) / g.tw;
    g.m = npiv * g.ntiles;
    return g;
}

size_t partition_ws_bytes(int64_t n, int64_t npiv) {
    PartGeom g = part_geom(n, npiv);
    size_t cnt = ((size_t)g.m * 4 + 255) & ~(size_t)255;
    size_t off = ((size_t)g.m * 8 + 255) & ~(size_t)255;
    int64_t st = (g.m + SCAN_TILE - 1) / SCAN_TILE;
    size_t stb = 256 + (((size_t)st * 8 + 255) & ~(size_t)255);
    return cnt + off + stb + 256;
}

template <typename T>
static cudaError_t partition_typed(const vd_column& v, int64_t from, int64_t npiv, int32_t* out_pos,
                                   int64_t* out_counts, void* ws, cudaStream_t s, int* nl) {
    const int64_t n = v.len;
    PartGeom g = part_geom(n, npiv);
    char* w = (char*)ws;
    int32_t* counts = (int32_t*)w;
    w += ((size_t)g.m * 4 + 255) & ~(size_t)255;
    int64_t* offs = (int64_t*)w;
    w += ((size_t)g.m * 8 + 255) & ~(size_t)255;
    unsigned long long* ctr = (unsigned long long*)w;
    uint64_t* status = (uint64_t*)(w + 256);
    int64_t st = (g.m + SCAN_TILE - 1) / SCAN_TILE;
    size_t smem = (size_t)PART_WARPS * npiv * sizeof(int);
    int grid = grid_for(g.ntiles * 32, PART_THREADS);
    if (n > 0) {
        k_part_hist<T><<<grid, PART_THREADS, smem, s>>>((const T*)v.data, n, from, (int)npiv, g.tw, g.ntiles, counts);
        ++*nl;
        cudaError_t e = cudaMemsetAsync(w, 0, 256 + (size_t)st * 8, s);
        if (e != cudaSuccess) return e;
        int sg = (int)(st < (int64_t)num_sms() * 4 ? st : (int64_t)num_sms() * 4);
        k_scan_i32<<<sg, SCAN_THREADS, 0, s>>>(counts, g.m, offs, status, ctr, st);
        ++*nl;
        k_part_place<T><<<grid, PART_THREADS, smem, s>>>((const T*)v.data, n, from, (int)npiv, g.tw, g.ntiles, offs,
                                                          out_pos);
        ++*nl;
    }
    if (out_counts && n == 0) return cudaMemsetAsync(out_counts, 0, (size_t)npiv * 8, s);
    return cudaGetLastError();
}

__global__ void k_bucket_totals2(const int64_t* __restrict__ offs, const int32_t* __restrict__ counts, int64_t ntiles,
                                 int npiv, int64_t* __restrict__ out) {
    int b = blockIdx.x * blockDim.x + threadIdx.x;
    if (b >= npiv) return;
    int64_t m = (int64_t)npiv * ntiles;
    int64_t s = offs[(int64_t)b * ntiles];
    int64_t e = (b + 1 < npiv) ? offs[(int64_t)(b + 1) * ntiles] : offs[m - 1] + counts[m - 1];
    out[b] = e - s;
}

cudaError_t launch_partition(const vd_column& v, int64_t from, int64_t npiv, int32_t* out_pos, int64_t* out_counts,
                             void* ws, cudaStream_t s, int* nl) {
    cudaError_t e;
    switch (v.dtype) {
    case VD_U8: e = partition_typed<uint8_t>(v, from, npiv, out_pos, out_counts, ws, s, nl); break;
    case VD_I32: e = partition_typed<int32_t>(v, from, npiv, out_pos, out_counts, ws, s, nl); break;
    default: e = partition_typed<int64_t>(v, from, npiv, out_pos, out_counts, ws, s, nl); break;
    }
    if (e != cudaSuccess || !out_counts || v.len == 0) return e;
    PartGeom g = part_geom(v.len, npiv);
    int32_t* counts = (int32_t*)ws;
    int64_t* offs = (int64_t*)((char*)ws + (((size_t)g.m * 4 + 255) & ~(size_t)255));
    k_bucket_totals2<<<(int)((npiv + 255) / 256), 256, 0, s>>>(offs, counts, g.ntiles, (int)npiv, out_counts);
    ++*nl;
    return cudaGetLastError();
}

}  // namespace vd
