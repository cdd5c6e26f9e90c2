// Micro-benchmark (not part of the product): the DRAM bytes one isolated
// 4-byte load costs on B200, by load flavour -- the granularity question
// behind the late-materialisation fragments (Q19 late, Q15 group fold, Fig 16
// branching), whose algorithmic model counts 64-byte blocks (readings
// A31/A33/A34).  Each kernel reads ONE int32 from each of M distinct random
// 256-byte-aligned blocks of an 8 GiB buffer (far beyond L2, no reuse).
// Run under `ncu --metrics dram__bytes_read.sum,lts__t_sectors_srcunit_tex_op_read.sum`:
// dram bytes / M = the effective DRAM granularity of that flavour.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_dram_gran scripts/ubench_dram_gran.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ uint64_t mix(uint64_t x) {
    x ^= x >> 30; x *= 0xBF58476D1CE4E5B9ull; x ^= x >> 27; x *= 0x94D049BB133111EBull; x ^= x >> 31;
    return x;
}

template <int FLAVOUR>
__device__ __forceinline__ int ld(const int* p) {
    int v;
    if (FLAVOUR == 0) asm volatile("ld.global.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 1) asm volatile("ld.global.nc.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 2) asm volatile("ld.global.nc.L2::64B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 3) asm volatile("ld.global.nc.L2::128B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 4) asm volatile("ld.global.cs.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 5) asm volatile("ld.global.nc.L1::no_allocate.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else if (FLAVOUR == 6) asm volatile("ld.global.nc.L2::256B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    else {
        uint64_t pol;
        asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
        asm volatile("ld.global.nc.L2::cache_hint.u32 %0, [%1], %2;" : "=r"(v) : "l"(p), "l"(pol));
    }
    return v;
}

template <int FLAVOUR>
__global__ void k_probe(const int* __restrict__ buf, uint64_t nblocks, uint64_t m, int* out) {
    int acc = 0;
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < m; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t b = mix(i * 0x9E3779B97F4A7C15ull + 12345) % nblocks;  // a random 256-byte block
        acc += ld<FLAVOUR>(buf + b * 64 + (i & 7) * 4);  // one int32 at an offset inside the first 128 B
    }
    if (acc == 0x7fffffff) out[0] = acc;
}

int main() {
    const size_t bytes = (size_t)8 << 30;
    int* buf;
    int* out;
    if (cudaMalloc(&buf, bytes) != cudaSuccess || cudaMalloc(&out, 4) != cudaSuccess) return 1;
    cudaMemset(buf, 1, bytes);
    const uint64_t nblocks = bytes / 256, m = 8 << 20;  // 8 Mi probes: 0.25% of the blocks touched twice at most
    const char* names[8] = {"ld.global", "ld.global.nc", "nc.L2::64B", "nc.L2::128B", "ld.global.cs",
                            "nc.L1::no_allocate", "nc.L2::256B", "nc.L2::cache_hint(evict_first)"};
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
#define RUN(F)                                                                                 \
    {                                                                                          \
        k_probe<F><<<148 * 8, 256>>>(buf, nblocks, m, out);                                    \
        cudaEventRecord(e0);                                                                   \
        k_probe<F><<<148 * 8, 256>>>(buf, nblocks, m, out);                                    \
        cudaEventRecord(e1);                                                                   \
        cudaEventSynchronize(e1);                                                              \
        float ms;                                                                              \
        cudaEventElapsedTime(&ms, e0, e1);                                                     \
        printf("{\"flavour\": \"%s\", \"probes\": %llu, \"ms\": %.4f, \"probes_per_ns\": %.2f}\n", names[F], \
               (unsigned long long)m, ms, m / (ms * 1e6));                                    \
    }
    RUN(0) RUN(1) RUN(2) RUN(3) RUN(4) RUN(5) RUN(6) RUN(7)
    printf("{\"err\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
