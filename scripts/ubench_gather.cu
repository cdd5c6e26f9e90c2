// Micro-benchmark (not part of the product): random 1-byte lookups into a
// 1 MiB dimension table (Q9's s_nationkey at SF100) by four routes --
//   0: global memory (L2-resident table, LDG.U8)
//   1: distributed shared memory, table split over an 8-CTA cluster (128 KiB
//      per CTA), ld.shared::cluster.u8 through mapa
//   2: local shared memory only (128 KiB per CTA, the upper bound)
//   3: half of the lookups through DSMEM, half through L2
// and the L2 slice throughput on B200 (k_l2): random 4-byte loads (one
// sector each) and sequential 16-byte loads over a 64 MiB L2-resident buffer.
// Prints lookups (sectors) per ns for the whole GPU.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_gather scripts/ubench_gather.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

constexpr int TBL = 1 << 20;
constexpr int SLICE = TBL / 8;  // 128 KiB per CTA
constexpr int THREADS = 512;
constexpr int ITERS = 2048;
constexpr int UNR = 8;

__device__ __forceinline__ uint32_t hsh(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}
__device__ __forceinline__ uint32_t mapa(uint32_t saddr, uint32_t cta) {
    uint32_t r;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(saddr), "r"(cta));
    return r;
}
__device__ __forceinline__ uint32_t ld_dsmem_u8(uint32_t addr) {
    uint16_t v;
    asm volatile("ld.shared::cluster.u8 %0, [%1];" : "=h"(v) : "r"(addr));
    return v;
}
__device__ __forceinline__ void cluster_sync() {
    asm volatile("barrier.cluster.arrive.release.aligned;\nbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}

template <int MODE>
__global__ void __cluster_dims__(8, 1, 1) __launch_bounds__(THREADS, 1)
    k_gather(const uint8_t* __restrict__ tbl, uint32_t* __restrict__ sink) {
    extern __shared__ __align__(16) uint8_t s[];
    uint32_t rank;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(rank));
    for (int i = threadIdx.x; i < SLICE / 4; i += THREADS)
        reinterpret_cast<uint32_t*>(s)[i] = reinterpret_cast<const uint32_t*>(tbl + rank * SLICE)[i];
    cluster_sync();
    const uint32_t sbase = (uint32_t)__cvta_generic_to_shared(s);
    uint32_t acc = 0;
    uint32_t seed = (blockIdx.x * THREADS + threadIdx.x) * 0x9E3779B9u;
    for (int it = 0; it < ITERS; it += UNR) {
        uint32_t v[UNR];
#pragma unroll
        for (int u = 0; u < UNR; ++u) {
            const uint32_t idx = hsh(seed + it + u) & (TBL - 1);
            if (MODE == 0 || (MODE == 3 && (u & 1))) {
                v[u] = __ldg(tbl + idx);
            } else if (MODE == 2) {
                v[u] = s[idx & (SLICE - 1)];
            } else {
                v[u] = ld_dsmem_u8(mapa(sbase + (idx & (SLICE - 1)), idx >> 17));
            }
        }
#pragma unroll
        for (int u = 0; u < UNR; ++u) acc += v[u];
    }
    cluster_sync();  // no CTA may exit while its slice is being read
    if (acc == 0xFFFFFFFFu) sink[0] = acc;
}

template <int SEQ>
__global__ void __launch_bounds__(512) k_l2(const uint32_t* __restrict__ buf, uint32_t nwords, uint32_t* sink) {
    uint32_t acc = 0;
    const uint32_t tid = blockIdx.x * 512 + threadIdx.x;
    if (SEQ) {
        const uint4* b4 = reinterpret_cast<const uint4*>(buf);
        const uint32_t nv = nwords / 4, stride = gridDim.x * 512;
        for (int rep = 0; rep < 4; ++rep)
            for (uint32_t i = tid; i < nv; i += stride * UNR) {
                uint4 v[UNR];
#pragma unroll
                for (int u = 0; u < UNR; ++u) v[u] = i + u * stride < nv ? __ldcg(b4 + i + u * stride) : make_uint4(0, 0, 0, 0);
#pragma unroll
                for (int u = 0; u < UNR; ++u) acc += v[u].x ^ v[u].w;
            }
    } else {
        uint32_t seed = tid * 0x9E3779B9u;
        for (int it = 0; it < ITERS; it += UNR) {
            uint32_t v[UNR];
#pragma unroll
            for (int u = 0; u < UNR; ++u) v[u] = __ldcg(buf + (hsh(seed + it + u) & (nwords - 1)));
#pragma unroll
            for (int u = 0; u < UNR; ++u) acc += v[u];
        }
    }
    if (acc == 0xFFFFFFFFu) sink[0] = acc;
}

int main() {
    uint8_t* tbl;
    uint32_t* sink;
    cudaMalloc(&tbl, TBL);
    cudaMalloc(&sink, 4);
    cudaMemset(tbl, 7, TBL);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const int grid = (sms / 8) * 8;
    const size_t smem = SLICE;
    auto run = [&](auto kern, const char* name) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        for (int w = 0; w < 3; ++w) kern<<<grid, THREADS, smem>>>(tbl, sink);
        cudaEvent_t a, b;
        cudaEventCreate(&a);
        cudaEventCreate(&b);
        const int reps = 10;
        cudaEventRecord(a);
        for (int r = 0; r < reps; ++r) kern<<<grid, THREADS, smem>>>(tbl, sink);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms = 0;
        cudaEventElapsedTime(&ms, a, b);
        cudaError_t e = cudaGetLastError();
        const double lookups = (double)grid * THREADS * ITERS * reps;
        printf("{\"route\": \"%s\", \"grid\": %d, \"lookups_per_ns\": %.2f, \"err\": \"%s\"}\n", name, grid,
               lookups / (ms * 1e6), cudaGetErrorString(e));
    };
    run(k_gather<0>, "l2_ldg");
    run(k_gather<1>, "dsmem_cluster8");
    run(k_gather<2>, "local_smem");
    run(k_gather<3>, "half_dsmem_half_l2");
    {
        const uint32_t nwords = 16u << 20;  // 64 MiB
        uint32_t* buf;
        cudaMalloc(&buf, (size_t)nwords * 4);
        cudaMemset(buf, 3, (size_t)nwords * 4);
        const int g = sms * 4;
        for (int mode = 0; mode < 2; ++mode) {
            auto kern = mode ? k_l2<1> : k_l2<0>;
            for (int w = 0; w < 3; ++w) kern<<<g, 512>>>(buf, nwords, sink);
            cudaEvent_t a, b;
            cudaEventCreate(&a);
            cudaEventCreate(&b);
            cudaEventRecord(a);
            for (int r = 0; r < 10; ++r) kern<<<g, 512>>>(buf, nwords, sink);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms = 0;
            cudaEventElapsedTime(&ms, a, b);
            const double sectors = mode ? 4.0 * nwords * 4 / 32 * 10 : (double)g * 512 * ITERS * 10;
            printf("{\"route\": \"%s\", \"sectors_per_ns\": %.1f, \"GBps\": %.1f, \"err\": \"%s\"}\n",
                   mode ? "l2_seq_ldg128" : "l2_random_sector", sectors / (ms * 1e6), sectors * 32 / (ms * 1e6),
                   cudaGetErrorString(cudaGetLastError()));
        }
    }
    return 0;
}
