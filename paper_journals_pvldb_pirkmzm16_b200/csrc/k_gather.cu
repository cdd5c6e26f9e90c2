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
        v[u] = ok ? __ldg(src + p[u]) : Eps<T>::value();
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
    int64_t blocks = (n + GATHER_THREADS * GATHER_ILP - 1) / (GATHER_THREADS * GATHER_ILP);
    int64_t cap = (int64_t)num_sms() * 8;
    if (blocks > cap) blocks = cap;
    k_gather<<<(int)blocks, GATHER_THREADS, 0, s>>>(g, pos, n, bias);
    ++*nl;
    return cudaGetLastError();
}

}  // namespace vd
