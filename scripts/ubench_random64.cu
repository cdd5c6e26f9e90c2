// Micro-benchmark (not part of the product): the throughput ceiling of
// independent random 64-byte block reads on B200 -- the access pattern the
// algorithmic models of the FK-lookup fragments count (readings A31 / A33 /
// A34: one 64-byte block per random lookup).  Each thread issues U
// independent loads per iteration (memory-level parallelism), each from a
// random 64-byte-aligned block of an 8 GiB buffer (far beyond L2), with
// `ld.global.nc.L2::64B` (the DRAM fetch is the 64-byte block, not the
// 128-byte line: profiles/round2_traffic.md).  Block indices come from a
// counter-based mix with a power-of-two mask (no 64-bit modulo on the
// critical path).  Reported: probes per ns and the equivalent GB/s at 64 B
// per probe, by loads in flight per thread and by grid size; plus the
// sequential 16-byte-per-lane read of the same buffer for reference.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_random64 scripts/ubench_random64.cu
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cuda_runtime.h>

__device__ __forceinline__ uint64_t mix(uint64_t x) {
    x ^= x >> 30; x *= 0xBF58476D1CE4E5B9ull; x ^= x >> 27; x *= 0x94D049BB133111EBull; x ^= x >> 31;
    return x;
}

__device__ __forceinline__ int4 ld64b(const void* p) {
    int4 v;
    asm volatile("ld.global.nc.L2::64B.v4.s32 {%0,%1,%2,%3}, [%4];"
                 : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "l"(p));
    return v;
}

template <int U>
__global__ void k_rand(const int4* __restrict__ buf, uint64_t mask, uint64_t m, int* out) {
    int acc = 0;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x * U;
    for (uint64_t i = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) * U; i < m; i += stride) {
        int4 v[U];
#pragma unroll
        for (int u = 0; u < U; ++u) v[u] = ld64b(buf + (mix(i + u) & mask) * 4);  // block b = 4 int4s
#pragma unroll
        for (int u = 0; u < U; ++u) acc += v[u].x ^ v[u].w;
    }
    if (acc == 0x7fffffff) out[0] = acc;
}

__global__ void k_seq(const int4* __restrict__ buf, uint64_t n16, int* out) {
    int acc = 0;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n16; i += (uint64_t)gridDim.x * blockDim.x) {
        const int4 v = __ldcs(buf + i);
        acc += v.x ^ v.w;
    }
    if (acc == 0x7fffffff) out[0] = acc;
}

int main(int argc, char** argv) {
    // buffer size in GiB (a power of two): 8 by default; 1 = the Fig 16 target
    const size_t bytes = (size_t)(argc > 1 ? atoi(argv[1]) : 8) << 30;
    int4* buf;
    int* out;
    if (cudaMalloc(&buf, bytes) != cudaSuccess || cudaMalloc(&out, 4) != cudaSuccess) return 1;
    cudaMemset(buf, 1, bytes);
    const uint64_t nblocks = bytes / 64, mask = nblocks - 1, m = (uint64_t)256 << 20;  // 256 Mi probes = 16 GB of blocks
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    int nsm = 148;
    cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
    auto timeit = [&](auto launch) {
        launch();
        cudaEventRecord(e0);
        launch();
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        return ms;
    };
#define RUN(U, BPS)                                                                                          \
    {                                                                                                        \
        const float ms = timeit([&] { k_rand<U><<<nsm * BPS, 256>>>(buf, mask, m, out); });                  \
        printf("{\"kind\": \"random64\", \"buffer_GiB\": %zu, \"loads_per_thread\": %d, \"ctas_per_sm\": %d, " \
               "\"probes\": %llu, \"ms\": %.4f, \"probes_per_ns\": %.2f, \"GBps_at_64B\": %.1f}\n",            \
               bytes >> 30, U, BPS, (unsigned long long)m, ms, m / (ms * 1e6), m * 64.0 / (ms * 1e6));      \
    }
    RUN(1, 8) RUN(2, 8) RUN(4, 8) RUN(8, 8) RUN(16, 8) RUN(4, 4) RUN(8, 4) RUN(16, 4) RUN(32, 4) RUN(8, 2)
    {
        const float ms = timeit([&] { k_seq<<<nsm * 8, 256>>>(buf, bytes / 16, out); });
        printf("{\"kind\": \"sequential\", \"bytes\": %zu, \"ms\": %.4f, \"GBps\": %.1f}\n", bytes, ms, bytes / (ms * 1e6));
    }
    printf("{\"err\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
