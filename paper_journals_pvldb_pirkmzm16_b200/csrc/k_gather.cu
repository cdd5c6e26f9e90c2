// k_gather.cu -- positional Gather (§8(a) a4).
//
// Gather(V1, V2, .pos) (Table 2): output of |pos| slots,
// out[i] = V1[pos[i]]; out-of-bounds positions give the empty value.  A
// foreign key is a position into the target vector; with dense
// keys and min/max metadata the lookup is identity hashing pos = fk - bias
// (P:L1054-1056).  One pass resolves the positions into up to
// VD_MAX_GATHERS target columns (the "Single Loop" of Fig 14,
// P:L1164-1166).  Each thread keeps GATHER_ILP independent random loads in
// flight per column (latency-bound access, Guideline 7).
#include <algorithm>

#include "vd_common.cuh"
#include "vd_internal.h"

namespace vd {

constexpr int GATHER_THREADS = 256;
constexpr int GATHER_ILP = 4;

struct GatherArgs {
    const void* src[VD_MAX_GATHERS];
    int64_t len[VD_MAX_GATHERS];
    int32_t dt[VD_MAX_GATHERS];
    void* out[VD_MAX_GATHERS];
    int32_t nsrc;
};

template <typename T>
__device__ __forceinline__ void gather_one(const T* __restrict__ src, int64_t len, T* __restrict__ out,
                                           const int64_t (&p)[GATHER_ILP], const int64_t (&i)[GATHER_ILP], int64_t n) {
    T v[GATHER_ILP];
#pragma unroll
    for (int u = 0; u < GATHER_ILP; ++u) {
        bool ok = i[u] < n && p[u] >= 0 && p[u] < len;
        v[u] = ok ? ldg64b(src + p[u]) : Eps<T>::value();
    }
#pragma unroll
    for (int u = 0; u < GATHER_ILP; ++u)
        if (i[u] < n) out[i[u]] = v[u];
}

__global__ void __launch_bounds__(GATHER_THREADS) k_gather(GatherArgs g, const int32_t* __restrict__ pos, int64_t n,
                                                           int64_t bias) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x * GATHER_ILP;
    for (int64_t base = (int64_t)blockIdx.x * blockDim.x * GATHER_ILP + threadIdx.x; base < n; base += stride) {
        int64_t i[GATHER_ILP], p[GATHER_ILP];
#pragma unroll
        for (int u = 0; u < GATHER_ILP; ++u) {
            i[u] = base + (int64_t)u * blockDim.x;
            int32_t q = i[u] < n ? __ldg(pos + i[u]) : -1;
            p[u] = q < 0 ? -1 : (int64_t)q - bias;  // negative position = epsilon
        }
        for (int k = 0; k < g.nsrc; ++k) {
            switch (g.dt[k]) {
            case VD_U8: gather_one((const uint8_t*)g.src[k], g.len[k], (uint8_t*)g.out[k], p, i, n); break;
            case VD_I32: gather_one((const int32_t*)g.src[k], g.len[k], (int32_t*)g.out[k], p, i, n); break;
            case VD_I64: gather_one((const int64_t*)g.src[k], g.len[k], (int64_t*)g.out[k], p, i, n); break;
            case VD_F32: gather_one((const float*)g.src[k], g.len[k], (float*)g.out[k], p, i, n); break;
            default: gather_one((const double*)g.src[k], g.len[k], (double*)g.out[k], p, i, n); break;
            }
        }
    }
}

// Same-dtype sources (the common case): NSRC x GU_ILP independent loads in
// flight per thread, issued before the first use.
constexpr int GU_ILP = 8;

template <typename T, int NSRC>
__global__ void __launch_bounds__(GATHER_THREADS) k_gather_u(GatherArgs g, const int32_t* __restrict__ pos, int64_t n,
                                                             int64_t bias) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x * GU_ILP;
    for (int64_t base = (int64_t)blockIdx.x * blockDim.x * GU_ILP + threadIdx.x; base - (threadIdx.x & 31) < n;
         base += stride) {
        int64_t i[GU_ILP], p[GU_ILP];
#pragma unroll
        for (int u = 0; u < GU_ILP; ++u) {
            i[u] = base + (int64_t)u * blockDim.x;
            const int32_t q = i[u] < n ? __ldcs(pos + i[u]) : -1;
            p[u] = q < 0 ? -1 : (int64_t)q - bias;  // negative position = epsilon
        }
        T v[NSRC][GU_ILP];
#pragma unroll
        for (int k = 0; k < NSRC; ++k)
#pragma unroll
            for (int u = 0; u < GU_ILP; ++u) {
                const bool ok = p[u] >= 0 && p[u] < g.len[k];
                v[k][u] = ok ? ldg64b((const T*)g.src[k] + p[u]) : Eps<T>::value();
            }
        __syncwarp();  // all loads issued before the first store
#pragma unroll
        for (int k = 0; k < NSRC; ++k)
#pragma unroll
            for (int u = 0; u < GU_ILP; ++u)
                if (i[u] < n) __stcs((T*)g.out[k] + i[u], v[k][u]);
    }
}

template <typename T>
static void launch_gather_u(const GatherArgs& g, int nsrc, int blocks, const int32_t* pos, int64_t n, int64_t bias,
                            cudaStream_t s) {
    switch (nsrc) {
    case 1: k_gather_u<T, 1><<<blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias); break;
    case 2: k_gather_u<T, 2><<<blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias); break;
    case 3: k_gather_u<T, 3><<<blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias); break;
    default: k_gather_u<T, 4><<<blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias); break;
    }
}

cudaError_t launch_gather(const vd_column* srcs, int nsrc, const int32_t* pos, int64_t n, int64_t bias,
                          void* const* outs, cudaStream_t s, int* nl) {
    if (n == 0) return cudaSuccess;
    GatherArgs g;
    g.nsrc = nsrc;
    for (int k = 0; k < nsrc; ++k) {
        g.src[k] = srcs[k].data;
        g.len[k] = srcs[k].len;
        g.dt[k] = srcs[k].dtype;
        g.out[k] = outs[k];
    }
    bool same = true;
    for (int k = 1; k < nsrc; ++k) same = same && srcs[k].dtype == srcs[0].dtype;
    if (same) {
        const int64_t blocks = std::min<int64_t>((n + GATHER_THREADS * GU_ILP - 1) / (GATHER_THREADS * GU_ILP),
                                                 (int64_t)num_sms() * 8);
        switch (srcs[0].dtype) {
        case VD_U8: launch_gather_u<uint8_t>(g, nsrc, (int)blocks, pos, n, bias, s); break;
        case VD_I32: launch_gather_u<int32_t>(g, nsrc, (int)blocks, pos, n, bias, s); break;
        case VD_F32: launch_gather_u<float>(g, nsrc, (int)blocks, pos, n, bias, s); break;
        case VD_I64: launch_gather_u<int64_t>(g, nsrc, (int)blocks, pos, n, bias, s); break;
        default: launch_gather_u<double>(g, nsrc, (int)blocks, pos, n, bias, s); break;
        }
        ++*nl;
        return cudaGetLastError();
    }
    int64_t blocks = (n + GATHER_THREADS * GATHER_ILP - 1) / (GATHER_THREADS * GATHER_ILP);
    int64_t cap = (int64_t)num_sms() * 8;
    if (blocks > cap) blocks = cap;
    k_gather<<<(int)blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias);
    ++*nl;
    return cudaGetLastError();
}

// ---------------------------------------------------------------------------
// Layout Transform (Fig 14): Zip + materialise into rows, then
// one lookup per row.  A row is <= 32 bytes and its stride a power of two,
// so a random lookup touches one sector instead of one per column.
// ---------------------------------------------------------------------------
static int dsize(int dt) { return dt == VD_U8 ? 1 : (dt == VD_I32 || dt == VD_F32) ? 4 : 8; }

bool row_layout(const int32_t* dtypes, int nfields, int32_t* offsets, int32_t* stride) {
    int off = 0;
    for (int k = 0; k < nfields; ++k) {
        const int sz = dsize(dtypes[k]);
        off = (off + sz - 1) / sz * sz;
        offsets[k] = off;
        off += sz;
    }
    int st = 8;
    while (st < off) st *= 2;
    *stride = st;
    return off <= 32;
}

struct RowArgs {
    const void* col[VD_MAX_GATHERS];
    void* out[VD_MAX_GATHERS];
    int32_t dt[VD_MAX_GATHERS];
    int32_t off[VD_MAX_GATHERS];
    int32_t nf;
};

// one row = NW 8-byte words (NW = stride / 8)
template <int NW>
__global__ void __launch_bounds__(256) k_zip(const __grid_constant__ RowArgs a, int64_t n, uint64_t* __restrict__ rows) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x) {
        uint64_t w[NW];
#pragma unroll
        for (int k = 0; k < NW; ++k) w[k] = 0;
        for (int f = 0; f < a.nf; ++f) {
            uint64_t v;
            switch (a.dt[f]) {
            case VD_U8: v = __ldcs((const uint8_t*)a.col[f] + i); break;
            case VD_I32: case VD_F32: v = (uint32_t)__ldcs((const int32_t*)a.col[f] + i); break;
            default: v = (uint64_t)__ldcs((const long long*)a.col[f] + i); break;
            }
            const int o = a.off[f];
#pragma unroll
            for (int k = 0; k < NW; ++k)
                if ((o >> 3) == k) w[k] |= v << ((o & 7) * 8);
        }
        if (NW == 1) {
            rows[i] = w[0];
        } else if (NW == 2) {
            reinterpret_cast<ulonglong2*>(rows)[i] = make_ulonglong2(w[0], w[1]);
        } else {
#pragma unroll
            for (int k = 0; k < NW; k += 2)
                reinterpret_cast<ulonglong2*>(rows)[i * (NW / 2) + k / 2] = make_ulonglong2(w[k], w[k + 1]);
        }
    }
}

template <int NW>
__device__ __forceinline__ void load_row(const uint64_t* rows, int64_t p, bool ok, uint64_t (&w)[NW]) {
    if (NW == 1) {
        w[0] = ok ? ldg64b(rows + p) : 0;
    } else {
#pragma unroll
        for (int k = 0; k < NW; k += 2) {
            ulonglong2 x = make_ulonglong2(0, 0);
            if (ok) x = __ldg(reinterpret_cast<const ulonglong2*>(rows) + p * (NW / 2) + k / 2);
            w[k] = x.x;
            w[k + 1] = x.y;
        }
    }
}

constexpr int ROW_ILP = 8;

template <int NW>
__global__ void __launch_bounds__(256) k_gather_rows(const __grid_constant__ RowArgs a, const uint64_t* __restrict__ rows,
                                                     int64_t nrows, const int32_t* __restrict__ pos, int64_t n,
                                                     int64_t bias) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x * ROW_ILP;
    for (int64_t base = (int64_t)blockIdx.x * blockDim.x * ROW_ILP + threadIdx.x; base - (threadIdx.x & 31) < n;
         base += stride) {
        int64_t i[ROW_ILP], p[ROW_ILP];
        bool ok[ROW_ILP];
#pragma unroll
        for (int u = 0; u < ROW_ILP; ++u) {
            i[u] = base + (int64_t)u * blockDim.x;
            const int32_t q = i[u] < n ? __ldcs(pos + i[u]) : -1;
            p[u] = (int64_t)q - bias;
            ok[u] = q >= 0 && p[u] >= 0 && p[u] < nrows;  // negative position = epsilon
        }
        uint64_t w[ROW_ILP][NW];
#pragma unroll
        for (int u = 0; u < ROW_ILP; ++u) load_row<NW>(rows, ok[u] ? p[u] : 0, ok[u], w[u]);
        __syncwarp();  // all ROW_ILP row loads are issued before the first use
#pragma unroll
        for (int u = 0; u < ROW_ILP; ++u) {
            if (i[u] >= n) continue;
            for (int f = 0; f < a.nf; ++f) {
                const int o = a.off[f];
                uint64_t x = 0;
#pragma unroll
                for (int k = 0; k < NW; ++k)
                    if ((o >> 3) == k) x = w[u][k] >> ((o & 7) * 8);
                switch (a.dt[f]) {
                case VD_U8: ((uint8_t*)a.out[f])[i[u]] = ok[u] ? (uint8_t)x : Eps<uint8_t>::value(); break;
                case VD_I32: ((int32_t*)a.out[f])[i[u]] = ok[u] ? (int32_t)(uint32_t)x : Eps<int32_t>::value(); break;
                case VD_F32: ((uint32_t*)a.out[f])[i[u]] = ok[u] ? (uint32_t)x : 0x7fc00000u; break;
                case VD_I64: ((int64_t*)a.out[f])[i[u]] = ok[u] ? (int64_t)x : Eps<int64_t>::value(); break;
                default: ((uint64_t*)a.out[f])[i[u]] = ok[u] ? x : 0x7ff8000000000000ull; break;
                }
            }
        }
    }
}

cudaError_t launch_zip(const vd_column* cols, int ncols, void* out_rows, cudaStream_t s, int* nl) {
    RowArgs a;
    int32_t dts[VD_MAX_GATHERS], st;
    for (int k = 0; k < ncols; ++k) dts[k] = cols[k].dtype;
    row_layout(dts, ncols, a.off, &st);
    a.nf = ncols;
    for (int k = 0; k < ncols; ++k) {
        a.col[k] = cols[k].data;
        a.dt[k] = cols[k].dtype;
        a.out[k] = nullptr;
    }
    const int64_t n = cols[0].len;
    if (n == 0) return cudaSuccess;
    int64_t blocks = std::min<int64_t>((n + 255) / 256, (int64_t)num_sms() * 8);
    switch (st) {
    case 8: k_zip<1><<<(int)blocks, 256, 0, s>>>(a, n, (uint64_t*)out_rows); break;
    case 16: k_zip<2><<<(int)blocks, 256, 0, s>>>(a, n, (uint64_t*)out_rows); break;
    default: k_zip<4><<<(int)blocks, 256, 0, s>>>(a, n, (uint64_t*)out_rows); break;
    }
    ++*nl;
    return cudaGetLastError();
}

cudaError_t launch_gather_rows(const void* rows, int64_t nrows, const int32_t* dtypes, int nfields,
                               const int32_t* pos, int64_t n, int64_t bias, void* const* outs, cudaStream_t s, int* nl) {
    if (n == 0) return cudaSuccess;
    RowArgs a;
    int32_t st;
    row_layout(dtypes, nfields, a.off, &st);
    a.nf = nfields;
    for (int k = 0; k < nfields; ++k) {
        a.col[k] = nullptr;
        a.dt[k] = dtypes[k];
        a.out[k] = outs[k];
    }
    int64_t blocks = std::min<int64_t>((n + 256 * ROW_ILP - 1) / (256 * ROW_ILP), (int64_t)num_sms() * 8);
    switch (st) {
    case 8: k_gather_rows<1><<<(int)blocks, 256, 0, s>>>(a, (const uint64_t*)rows, nrows, pos, n, bias); break;
    case 16: k_gather_rows<2><<<(int)blocks, 256, 0, s>>>(a, (const uint64_t*)rows, nrows, pos, n, bias); break;
    default: k_gather_rows<4><<<(int)blocks, 256, 0, s>>>(a, (const uint64_t*)rows, nrows, pos, n, bias); break;
    }
    ++*nl;
    return cudaGetLastError();
}

}  // namespace vd
