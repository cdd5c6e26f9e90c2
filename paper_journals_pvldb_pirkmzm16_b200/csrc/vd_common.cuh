// vd_common.cuh -- device helpers shared by the libvd kernels (sm_100a).
// Product code: nothing here is shared with oracle/.
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>

#include "vd.h"

typedef __int128 i128;
typedef unsigned __int128 u128;

#define VD_FULL 0xFFFFFFFFu

namespace vd {

// ---- empty-slot sentinels (include/vd.h "Empty slots") -------------------
template <typename T> struct Eps;
template <> struct Eps<uint8_t> {
    static __host__ __device__ __forceinline__ bool is(uint8_t v) { return v == 0xFF; }
    static __host__ __device__ __forceinline__ uint8_t value() { return 0xFF; }
};
template <> struct Eps<int32_t> {
    static __host__ __device__ __forceinline__ bool is(int32_t v) { return v == INT32_MIN; }
    static __host__ __device__ __forceinline__ int32_t value() { return INT32_MIN; }
};
template <> struct Eps<int64_t> {
    static __host__ __device__ __forceinline__ bool is(int64_t v) { return v == INT64_MIN; }
    static __host__ __device__ __forceinline__ int64_t value() { return INT64_MIN; }
};
template <> struct Eps<float> {
    static __host__ __device__ __forceinline__ bool is(float v) { return v != v; }
    static __device__ __forceinline__ float value() { return __int_as_float(0x7fc00000); }
};
template <> struct Eps<double> {
    static __host__ __device__ __forceinline__ bool is(double v) { return v != v; }
    static __device__ __forceinline__ double value() { return __longlong_as_double(0x7ff8000000000000ll); }
};

template <typename T> struct IsFloat { static constexpr bool value = false; };
template <> struct IsFloat<float> { static constexpr bool value = true; };
template <> struct IsFloat<double> { static constexpr bool value = true; };

// ---- loads ---------------------------------------------------------------
// Read-only path, allocating in L1 (neighbouring lanes' sectors are reused
// by the sibling vector loads of a thread).
template <typename T> __device__ __forceinline__ T ldg(const T* p) { return __ldg(p); }
template <> __device__ __forceinline__ uint8_t ldg<uint8_t>(const uint8_t* p) { return __ldg(p); }

// Streaming 16-byte load that does not allocate in L1 (single-use data).
__device__ __forceinline__ int4 ld_stream16(const void* p) {
    int4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.s32 {%0,%1,%2,%3}, [%4];"
                 : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w)
                 : "l"(p));
    return r;
}
// Isolated (late / random) loads: by default an L1 miss fetches the whole
// 128-byte line from DRAM (scripts/ubench_dram_gran.cu: 125 B of DRAM per
// random 4-byte load); the .L2::64B prefetch size makes it one 64-byte block
// (63 B per load) -- the granule of the algorithmic byte models A31 / A33.
__device__ __forceinline__ uint32_t ld64b_u8(const void* p) {
    uint16_t v;
    asm volatile("ld.global.nc.L2::64B.u8 %0, [%1];" : "=h"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld64b_u32(const void* p) {
    uint32_t v;
    asm volatile("ld.global.nc.L2::64B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint64_t ld64b_u64(const void* p) {
    uint64_t v;
    asm volatile("ld.global.nc.L2::64B.u64 %0, [%1];" : "=l"(v) : "l"(p));
    return v;
}
template <typename T>
__device__ __forceinline__ T ldg64b(const T* p) {
    static_assert(sizeof(T) == 1 || sizeof(T) == 4 || sizeof(T) == 8, "1-, 4- or 8-byte element");
    T v;
    if (sizeof(T) == 1) { const uint8_t x = (uint8_t)ld64b_u8(p); memcpy(&v, &x, 1); }
    else if (sizeof(T) == 4) { const uint32_t x = ld64b_u32(p); memcpy(&v, &x, 4); }
    else { const uint64_t x = ld64b_u64(p); memcpy(&v, &x, 8); }
    return v;
}
// 128-bit streaming load with an L2 eviction-policy hint (evict_first for a
// single-use scan, so it does not push out a table other rows update)
__device__ __forceinline__ int4 ld_stream16_hint(const void* p, uint64_t pol) {
    int4 r;
    asm volatile("ld.global.nc.L1::no_allocate.L2::cache_hint.v4.s32 {%0,%1,%2,%3}, [%4], %5;"
                 : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w)
                 : "l"(p), "l"(pol));
    return r;
}
// global reductions with an L2 eviction-policy hint (evict_last: a grouping
// table that must stay L2-resident under a streaming scan)
__device__ __forceinline__ void red_add_u64_hint(unsigned long long* p, unsigned long long v, uint64_t pol) {
    asm volatile("red.relaxed.gpu.global.add.L2::cache_hint.u64 [%0], %1, %2;" ::"l"(p), "l"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void red_add_f64_hint(double* p, double v, uint64_t pol) {
    asm volatile("red.relaxed.gpu.global.add.L2::cache_hint.f64 [%0], %1, %2;" ::"l"(p), "d"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void red_min_s64_hint(long long* p, long long v, uint64_t pol) {
    asm volatile("red.relaxed.gpu.global.min.L2::cache_hint.s64 [%0], %1, %2;" ::"l"(p), "l"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void red_max_s64_hint(long long* p, long long v, uint64_t pol) {
    asm volatile("red.relaxed.gpu.global.max.L2::cache_hint.s64 [%0], %1, %2;" ::"l"(p), "l"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ int2 ld_stream8(const void* p) {
    int2 r;
    asm volatile("ld.global.nc.L1::no_allocate.v2.s32 {%0,%1}, [%2];" : "=r"(r.x), "=r"(r.y) : "l"(p));
    return r;
}
__device__ __forceinline__ int ld_stream4(const void* p) {
    int r;
    asm volatile("ld.global.nc.L1::no_allocate.s32 %0, [%1];" : "=r"(r) : "l"(p));
    return r;
}

// ---- gpu-scope acquire/release on 64-bit status words ---------------------
// Eight predicated read-only gathers (default value where !pred) in one
// inline-PTX block: every address is ready before the first load issues, so
// all eight are in flight together (left to itself the compiler consumes each
// gather before computing the next address).
// Eight predicated random loads issued back to back (memory-level
// parallelism); each moves one 64-byte block (.L2::64B, see ld64b_*).
__device__ __forceinline__ void gather8(const int64_t* const* p, const bool* pr, int64_t dflt, int64_t* v) {
    asm volatile("{\n\t.reg .pred q<8>;\n\tsetp.ne.b32 q0, %16, 0;\n\tsetp.ne.b32 q1, %17, 0;\n\tsetp.ne.b32 q2, %18, 0;\n\tsetp.ne.b32 q3, %19, 0;\n\tsetp.ne.b32 q4, %20, 0;\n\tsetp.ne.b32 q5, %21, 0;\n\tsetp.ne.b32 q6, %22, 0;\n\tsetp.ne.b32 q7, %23, 0;\n\tmov.b64 %0, %24;\n\tmov.b64 %1, %24;\n\tmov.b64 %2, %24;\n\tmov.b64 %3, %24;\n\tmov.b64 %4, %24;\n\tmov.b64 %5, %24;\n\tmov.b64 %6, %24;\n\tmov.b64 %7, %24;\n\t@q0 ld.global.nc.L2::64B.b64 %0, [%8];\n\t@q1 ld.global.nc.L2::64B.b64 %1, [%9];\n\t@q2 ld.global.nc.L2::64B.b64 %2, [%10];\n\t@q3 ld.global.nc.L2::64B.b64 %3, [%11];\n\t@q4 ld.global.nc.L2::64B.b64 %4, [%12];\n\t@q5 ld.global.nc.L2::64B.b64 %5, [%13];\n\t@q6 ld.global.nc.L2::64B.b64 %6, [%14];\n\t@q7 ld.global.nc.L2::64B.b64 %7, [%15];\n\t}"
                 : "=l"(v[0]), "=l"(v[1]), "=l"(v[2]), "=l"(v[3]), "=l"(v[4]), "=l"(v[5]), "=l"(v[6]), "=l"(v[7])
                 : "l"(p[0]), "l"(p[1]), "l"(p[2]), "l"(p[3]), "l"(p[4]), "l"(p[5]), "l"(p[6]), "l"(p[7]), "r"((int)pr[0]), "r"((int)pr[1]), "r"((int)pr[2]), "r"((int)pr[3]), "r"((int)pr[4]), "r"((int)pr[5]), "r"((int)pr[6]), "r"((int)pr[7]), "l"(dflt));
}
__device__ __forceinline__ void gather8(const int32_t* const* p, const bool* pr, int32_t dflt, int32_t* v) {
    asm volatile("{\n\t.reg .pred q<8>;\n\tsetp.ne.b32 q0, %16, 0;\n\tsetp.ne.b32 q1, %17, 0;\n\tsetp.ne.b32 q2, %18, 0;\n\tsetp.ne.b32 q3, %19, 0;\n\tsetp.ne.b32 q4, %20, 0;\n\tsetp.ne.b32 q5, %21, 0;\n\tsetp.ne.b32 q6, %22, 0;\n\tsetp.ne.b32 q7, %23, 0;\n\tmov.b32 %0, %24;\n\tmov.b32 %1, %24;\n\tmov.b32 %2, %24;\n\tmov.b32 %3, %24;\n\tmov.b32 %4, %24;\n\tmov.b32 %5, %24;\n\tmov.b32 %6, %24;\n\tmov.b32 %7, %24;\n\t@q0 ld.global.nc.L2::64B.b32 %0, [%8];\n\t@q1 ld.global.nc.L2::64B.b32 %1, [%9];\n\t@q2 ld.global.nc.L2::64B.b32 %2, [%10];\n\t@q3 ld.global.nc.L2::64B.b32 %3, [%11];\n\t@q4 ld.global.nc.L2::64B.b32 %4, [%12];\n\t@q5 ld.global.nc.L2::64B.b32 %5, [%13];\n\t@q6 ld.global.nc.L2::64B.b32 %6, [%14];\n\t@q7 ld.global.nc.L2::64B.b32 %7, [%15];\n\t}"
                 : "=r"(v[0]), "=r"(v[1]), "=r"(v[2]), "=r"(v[3]), "=r"(v[4]), "=r"(v[5]), "=r"(v[6]), "=r"(v[7])
                 : "l"(p[0]), "l"(p[1]), "l"(p[2]), "l"(p[3]), "l"(p[4]), "l"(p[5]), "l"(p[6]), "l"(p[7]), "r"((int)pr[0]), "r"((int)pr[1]), "r"((int)pr[2]), "r"((int)pr[3]), "r"((int)pr[4]), "r"((int)pr[5]), "r"((int)pr[6]), "r"((int)pr[7]), "r"(dflt));
}

__device__ __forceinline__ uint64_t ld_acquire_u64(const uint64_t* p) {
    uint64_t v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ uint32_t ld_acquire_u32(const unsigned int* p) {
    uint32_t v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
// named barrier `id` over `nthreads` threads (a multiple of 32)
__device__ __forceinline__ void bar_sync_n(int id, int nthreads) {
    asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}
__device__ __forceinline__ void st_release_u64(uint64_t* p, uint64_t v) {
    asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ uint64_t ld_relaxed_u64(const uint64_t* p) {
    uint64_t v;
    asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

// ---- warp reductions -------------------------------------------------------
__device__ __forceinline__ int64_t warp_sum_i64(int64_t v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(VD_FULL, v, o);
    return v;
}
__device__ __forceinline__ double warp_sum_f64(double v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(VD_FULL, v, o);
    return v;
}
__device__ __forceinline__ i128 shfl_xor_i128(i128 v, int o) {
    uint64_t lo = (uint64_t)(u128)v, hi = (uint64_t)((u128)v >> 64);
    lo = __shfl_xor_sync(VD_FULL, lo, o);
    hi = __shfl_xor_sync(VD_FULL, hi, o);
    return (i128)(((u128)hi << 64) | lo);
}
__device__ __forceinline__ i128 warp_sum_i128(i128 v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += shfl_xor_i128(v, o);
    return v;
}

__device__ __forceinline__ unsigned lanemask_lt() {
    unsigned m;
    asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m));
    return m;
}

// ---- 128-bit global accumulation via 64-bit atomics ----------------------
// Adds a signed 64-bit value into a little-endian two's-complement 128-bit
// integer {lo, hi}: the carry out of the low word is derived from the value
// the atomic returned, so the high word receives every carry exactly and
// the final sum is independent of the order of the adds.
__device__ __forceinline__ void atomic_add_i128_i64(unsigned long long* p, int64_t v) {
    unsigned long long add = (unsigned long long)v;
    unsigned long long old = atomicAdd(p, add);
    unsigned long long carry = (old + add) < old ? 1ull : 0ull;
    unsigned long long hi = (v < 0 ? ~0ull : 0ull) + carry;
    if (hi) atomicAdd(p + 1, hi);
}
__device__ __forceinline__ void atomic_add_i128(unsigned long long* p, i128 v) {
    unsigned long long lo = (unsigned long long)(u128)v;
    unsigned long long hi = (unsigned long long)((u128)v >> 64);
    unsigned long long old = atomicAdd(p, lo);
    unsigned long long carry = (old + lo) < old ? 1ull : 0ull;
    hi += carry;
    if (hi) atomicAdd(p + 1, hi);
}

__device__ __forceinline__ void st_i128(void* p, i128 v) {
    uint64_t* q = (uint64_t*)p;
    q[0] = (uint64_t)(u128)v;
    q[1] = (uint64_t)((u128)v >> 64);
}
__device__ __forceinline__ i128 ld_i128(const void* p) {
    const uint64_t* q = (const uint64_t*)p;
    return (i128)(((u128)q[1] << 64) | q[0]);
}

// ---- calendar year of a day number (days since 1970-01-01) ---------------
// Civil-from-days in integer arithmetic (proleptic Gregorian), valid for
// all int32 day numbers >= -719468.
__host__ __device__ __forceinline__ int32_t year_of_day(int32_t z) {
    z += 719468;
    int32_t era = (z >= 0 ? z : z - 146096) / 146097;
    int32_t doe = z - era * 146097;
    int32_t yoe = (doe - doe / 1460 + doe / 36524 - doe / 146096) / 365;
    int32_t y = yoe + era * 400;
    int32_t doy = doe - (365 * yoe + yoe / 4 - yoe / 100);
    int32_t mp = (5 * doy + 2) / 153;
    int32_t m = mp < 10 ? mp + 3 : mp - 9;
    return y + (m <= 2 ? 1 : 0);
}

// ---- mbarrier + 1D TMA bulk copies (sm_90+; SASS UBLKCP / SYNCS) ------------
__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void fence_mbar_init() { asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }
__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
    asm volatile(
        "{\n\t.reg .pred P1;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n\t"
        "@P1 bra DONE_%=;\n\t"
        "bra WAIT_%=;\n"
        "DONE_%=:\n\t}" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
}
// L2 eviction policy for single-use streaming data.
// L2 eviction policy for data re-read by other rows (lookups, group tables).
__device__ __forceinline__ uint64_t policy_evict_last() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ uint64_t policy_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
// 1D bulk copy global -> shared, completion counted on `bar` (bytes % 16 == 0,
// both addresses 16-byte aligned).
__device__ __forceinline__ void tma_load_1d(void* smem_dst, const void* gsrc, uint32_t bytes, uint64_t* bar,
                                            uint64_t policy) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::"r"(
            smem_u32(smem_dst)),
        "l"(gsrc), "r"(bytes), "r"(smem_u32(bar)), "l"(policy)
        : "memory");
}

// Bulk prefetch global -> L2 (no shared-memory destination, no completion):
// keeps HBM requests in flight beyond what the shared-memory ring can hold.
__device__ __forceinline__ void prefetch_l2_bulk(const void* gsrc, uint32_t bytes) {
    asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(gsrc), "r"(bytes) : "memory");
}

}  // namespace vd
