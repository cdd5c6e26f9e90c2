// gen/vdgen.cu -- host and device fill entry points of the shared input
// generator (gen/vd_gen.h).  Built into gen/libvdgen.so.  No method
// arithmetic lives here: only the per-row draws of vd_gen.h.
#include <cuda_runtime.h>
#include <stdint.h>
#include <string.h>

#include "vd_gen.h"

template <typename T>
static void fill_host_int(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, int64_t row0, int64_t n, T* out) {
    for (int64_t i = 0; i < n; ++i) out[i] = (T)vdg_value_i(col, seed, sf, p0, p1, row0 + i);
}

extern "C" int vdg_fill_host(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, double fscale, int64_t row0,
                             int64_t n, void* out) {
    switch (vdg_col_dtype(col)) {
    case 0: fill_host_int(col, seed, sf, p0, p1, row0, n, (uint8_t*)out); return 0;
    case 1: fill_host_int(col, seed, sf, p0, p1, row0, n, (int32_t*)out); return 0;
    case 2: fill_host_int(col, seed, sf, p0, p1, row0, n, (int64_t*)out); return 0;
    case 3: {
        float* o = (float*)out;
        for (int64_t i = 0; i < n; ++i) o[i] = (float)vdg_value_f(col, seed, fscale, row0 + i);
        return 0;
    }
    case 4: {
        double* o = (double*)out;
        for (int64_t i = 0; i < n; ++i) o[i] = vdg_value_f(col, seed, fscale, row0 + i);
        return 0;
    }
    default: return -1;
    }
}

template <typename T>
__global__ void k_fill_int(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, int64_t row0, int64_t n, T* out) {
    int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        out[i] = (T)vdg_value_i(col, seed, sf, p0, p1, row0 + i);
}

template <typename T>
__global__ void k_fill_flt(int col, uint64_t seed, double fscale, int64_t row0, int64_t n, T* out) {
    int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        out[i] = (T)vdg_value_f(col, seed, fscale, row0 + i);
}

extern "C" int vdg_fill_device(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, double fscale,
                               int64_t row0, int64_t n, void* out, void* stream) {
    if (n <= 0) return 0;
    cudaStream_t s = (cudaStream_t)stream;
    int dev = 0, sms = 148;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    int64_t blocks = (n + 255) / 256;
    int64_t cap = (int64_t)sms * 16;
    int grid = (int)(blocks < cap ? blocks : cap);
    switch (vdg_col_dtype(col)) {
    case 0: k_fill_int<<<grid, 256, 0, s>>>(col, seed, sf, p0, p1, row0, n, (uint8_t*)out); break;
    case 1: k_fill_int<<<grid, 256, 0, s>>>(col, seed, sf, p0, p1, row0, n, (int32_t*)out); break;
    case 2: k_fill_int<<<grid, 256, 0, s>>>(col, seed, sf, p0, p1, row0, n, (int64_t*)out); break;
    case 3: k_fill_flt<<<grid, 256, 0, s>>>(col, seed, fscale, row0, n, (float*)out); break;
    case 4: k_fill_flt<<<grid, 256, 0, s>>>(col, seed, fscale, row0, n, (double*)out); break;
    default: return -1;
    }
    return cudaGetLastError() == cudaSuccess ? 0 : -2;
}
