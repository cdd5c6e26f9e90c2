// Micro-benchmark (not part of the product): HBM read bandwidth of 1D TMA
// bulk-copy streams into a shared-memory ring (the staging every fused
// fragment uses), by access pattern.  A 4 GiB buffer, one CTA per SM, one
// producer lane issuing cp.async.bulk into an S-stage mbarrier ring and 8
// consumer warps that only release the stages (no compute).  Patterns:
//   rr K : the buffer seen as K equal "columns"; stage t holds one slice of
//          every column (K bulk copies), tiles round-robin over the CTAs --
//          the Q1 fragment reads 7 columns this way;
//   cta K: each CTA owns a contiguous range of every column.
// The question: why the 7-column Q1 fragment streams at 7.39 TB/s while a
// single-column stream (selective sum, selection phase 1) stays at 6.4-6.5.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_tma_read scripts/ubench_tma_read.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
    asm volatile(
        "{\n\t.reg .pred P1;\nW_%=:\n\tmbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n\t@P1 bra D_%=;\n\tbra W_%=;\nD_%=:\n\t}" ::"r"(
            smem_u32(bar)),
        "r"(parity)
        : "memory");
}
__device__ __forceinline__ void tma_load_1d(void* dst, const void* src, uint32_t bytes, uint64_t* bar, uint64_t pol) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::"r"(
            smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(pol)
        : "memory");
}

constexpr int CW = 16;

// stage = K slices of `slice` bytes; `ntiles` tiles per column
// work: 0 = release at once; 1 = selective-sum consumer (float4 loads to
// registers, release, then 2 compares + an f64 add per row); 2 = the same
// work done BEFORE releasing the stage (the stage is held during compute)
__global__ void __launch_bounds__(CW * 32 + 32, 1) k_tma_read(const uint8_t* buf, int64_t colbytes, int K, int slice,
                                                              int stages, int64_t ntiles, int contiguous, int work,
                                                              double* sink) {
    extern __shared__ __align__(128) uint8_t smem[];
    const int SB = K * slice;
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + (size_t)stages * SB);
    uint64_t* empty = full + stages;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < stages; ++s) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], CW);
        }
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    const int64_t per = (ntiles + gridDim.x - 1) / gridDim.x;
    auto tile_of = [&](int64_t it) -> int64_t {
        if (contiguous) {
            const int64_t t = blockIdx.x * per + it;
            return (it < per && t < ntiles) ? t : -1;
        }
        const int64_t t = blockIdx.x + it * gridDim.x;
        return t < ntiles ? t : -1;
    };
    if (warp == CW) {
        if (lane == 0) {
            uint64_t pol;
            asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
            int s = 0;
            uint32_t ph = 0;
            for (int64_t it = 0;; ++it) {
                const int64_t t = tile_of(it);
                if (t < 0) break;
                if (it >= stages) mbar_wait(&empty[s], ph ^ 1u);
                mbar_expect_tx(&full[s], SB);
                for (int k = 0; k < K; ++k)
                    tma_load_1d(smem + (size_t)s * SB + k * slice, buf + k * colbytes + t * slice, slice, &full[s], pol);
                if (++s == stages) { s = 0; ph ^= 1u; }
            }
        }
        return;
    }
    int s = 0;
    uint32_t ph = 0;
    double sum = 0;
    const int nv = SB / 16 / (CW * 32);  // float4 per thread per stage
    for (int64_t it = 0;; ++it) {
        if (tile_of(it) < 0) break;
        mbar_wait(&full[s], ph);
        if (work == 0) {
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
        } else {
            const float4* st = reinterpret_cast<const float4*>(smem + (size_t)s * SB);
            float4 x[8];
            for (int k = 0; k < nv && k < 8; ++k) x[k] = st[threadIdx.x + k * CW * 32];
            if (work == 1) { __syncwarp(); if (lane == 0) mbar_arrive(&empty[s]); }
            for (int k = 0; k < nv && k < 8; ++k) {
                const float v[4] = {x[k].x, x[k].y, x[k].z, x[k].w};
                for (int j = 0; j < 4; ++j) sum += (v[j] >= 0.25f && v[j] <= 0.75f) ? (double)v[j] : 0.0;
            }
            if (work == 2) { __syncwarp(); if (lane == 0) mbar_arrive(&empty[s]); }
        }
        if (++s == stages) { s = 0; ph ^= 1u; }
    }
    if (sum == 12345.0) sink[0] = sum;
}

int main() {
    const size_t bytes = 4ull << 30;
    uint8_t* buf;
    if (cudaMalloc(&buf, bytes) != cudaSuccess) return 1;
    cudaMemset(buf, 1, bytes);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    struct Cfg { int K, slice, stages, contiguous, work; };
    double* sink;
    cudaMalloc(&sink, 8);
    const Cfg cfgs[] = {
        {1, 32768, 6, 0, 0}, {1, 32768, 6, 0, 1}, {1, 32768, 6, 0, 2}, {1, 65536, 3, 0, 0}, {1, 65536, 3, 0, 1},
        {1, 65536, 3, 0, 2}, {1, 16384, 12, 0, 1}, {1, 16384, 8, 0, 1}, {1, 65536, 3, 1, 1}, {1, 32768, 6, 1, 1},
    };
    for (const Cfg& c : cfgs) {
        const int64_t colbytes = bytes / c.K;
        const int64_t ntiles = colbytes / c.slice;
        const size_t smem = (size_t)c.stages * c.K * c.slice + 2 * c.stages * 8;
        cudaFuncSetAttribute(k_tma_read, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        for (int w = 0; w < 2; ++w)
            k_tma_read<<<sms, CW * 32 + 32, smem>>>(buf, colbytes, c.K, c.slice, c.stages, ntiles, c.contiguous, c.work, sink);
        cudaEventRecord(a);
        for (int r = 0; r < 10; ++r)
            k_tma_read<<<sms, CW * 32 + 32, smem>>>(buf, colbytes, c.K, c.slice, c.stages, ntiles, c.contiguous, c.work, sink);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms = 0;
        cudaEventElapsedTime(&ms, a, b);
        printf("{\"K\": %d, \"slice\": %d, \"stages\": %d, \"inflight_KB\": %zu, \"pattern\": \"%s\", \"work\": %d, \"GBps\": %.1f, \"err\": \"%s\"}\n",
               c.K, c.slice, c.stages, smem / 1024, c.contiguous ? "cta" : "rr", c.work, (double)bytes * 10.0 / (ms * 1e6),
               cudaGetErrorString(cudaGetLastError()));
    }
    return 0;
}
