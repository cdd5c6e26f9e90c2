// Micro-benchmark (not part of the product): HBM read bandwidth of a 4 GiB
// buffer read as K interleaved streams (K = 1, 2, 4, 8): the buffer is cut
// into K equal segments and every thread reads one 16-byte vector from each
// segment per step, so K DRAM regions are open at once.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_read scripts/ubench_read.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

template <int K>
__global__ void __launch_bounds__(256) k_read(const int4* __restrict__ p, int64_t nvec, int* sink) {
    const int64_t seg = nvec / K;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    int acc = 0;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < seg; i += stride * 2) {
        int4 v[2 * K];
#pragma unroll
        for (int k = 0; k < K; ++k) {
            v[2 * k] = __ldcs(p + k * seg + i);
            v[2 * k + 1] = (i + stride < seg) ? __ldcs(p + k * seg + i + stride) : make_int4(0, 0, 0, 0);
        }
#pragma unroll
        for (int k = 0; k < 2 * K; ++k) acc ^= v[k].x ^ v[k].y ^ v[k].z ^ v[k].w;
    }
    if (acc == 0x12345678) sink[0] = acc;
}

int main() {
    const size_t bytes = 4ull << 30;
    int4* p;
    int* sink;
    cudaMalloc(&p, bytes);
    cudaMalloc(&sink, 4);
    cudaMemset(p, 1, bytes);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const int64_t nvec = bytes / 16;
    auto run = [&](auto kern, int K) {
        int per = 0;
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, kern, 256, 0);
        const int grid = sms * per;
        for (int w = 0; w < 3; ++w) kern<<<grid, 256>>>(p, nvec, sink);
        cudaEvent_t a, b;
        cudaEventCreate(&a);
        cudaEventCreate(&b);
        cudaEventRecord(a);
        for (int r = 0; r < 10; ++r) kern<<<grid, 256>>>(p, nvec, sink);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms = 0;
        cudaEventElapsedTime(&ms, a, b);
        printf("{\"streams\": %d, \"grid\": %d, \"GBps\": %.1f, \"err\": \"%s\"}\n", K, grid, bytes * 10.0 / (ms * 1e6),
               cudaGetErrorString(cudaGetLastError()));
    };
    run(k_read<1>, 1);
    run(k_read<2>, 2);
    run(k_read<4>, 4);
    run(k_read<8>, 8);
    return 0;
}
