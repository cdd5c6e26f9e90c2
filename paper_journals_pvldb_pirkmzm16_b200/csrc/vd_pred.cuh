// vd_pred.cuh -- device evaluation of vd_pred (Greater/Equals compositions,
// P:L495-498; reading A8) over typed columns.  Product code.
#pragma once

#include "vd_common.cuh"
#include "vd_internal.h"

namespace vd {

__device__ __forceinline__ bool cmp_int(int cmp, int64_t x, int64_t c) {
    switch (cmp) {
    case VD_CMP_GT: return x > c;
    case VD_CMP_LT: return x < c;
    case VD_CMP_EQ: return x == c;
    case VD_CMP_GE: return x >= c;
    case VD_CMP_LE: return x <= c;
    case VD_CMP_NE: return x != c;
    case VD_CMP_IN: return (uint64_t)x < 64ull && (((uint64_t)c >> (uint64_t)x) & 1ull);
    default: return false;
    }
}

__device__ __forceinline__ bool cmp_flt(int cmp, double x, double c) {
    switch (cmp) {
    case VD_CMP_GT: return x > c;
    case VD_CMP_LT: return x < c;
    case VD_CMP_EQ: return x == c;
    case VD_CMP_GE: return x >= c;
    case VD_CMP_LE: return x <= c;
    case VD_CMP_NE: return x != c;
    default: return false;
    }
}

// A typed value fetched from a column: epsilon flag + int or float payload.
struct Val {
    bool eps;
    bool isf;
    int64_t i;
    double f;
};

__device__ __forceinline__ Val fetch_typed(const void* p, int32_t dt, int64_t row) {
    Val v;
    v.isf = false;
    v.i = 0;
    v.f = 0;
    switch (dt) {
    case VD_U8: { uint8_t x = __ldg((const uint8_t*)p + row); v.eps = Eps<uint8_t>::is(x); v.i = x; break; }
    case VD_I32: { int32_t x = __ldg((const int32_t*)p + row); v.eps = Eps<int32_t>::is(x); v.i = x; break; }
    case VD_I64: { int64_t x = __ldg((const long long*)p + row); v.eps = Eps<int64_t>::is(x); v.i = x; break; }
    case VD_F32: { float x = __ldg((const float*)p + row); v.eps = Eps<float>::is(x); v.isf = true; v.f = x; break; }
    default: { double x = __ldg((const double*)p + row); v.eps = Eps<double>::is(x); v.isf = true; v.f = x; break; }
    }
    return v;
}

// The same, for an isolated (late / random) row: the load moves one 64-byte
// block, not the default 128-byte line (ld64b_*, vd_common.cuh).
__device__ __forceinline__ Val fetch_typed_64b(const void* p, int32_t dt, int64_t row) {
    Val v;
    v.isf = false;
    v.i = 0;
    v.f = 0;
    switch (dt) {
    case VD_U8: { uint8_t x = (uint8_t)ld64b_u8((const uint8_t*)p + row); v.eps = Eps<uint8_t>::is(x); v.i = x; break; }
    case VD_I32: { int32_t x = (int32_t)ld64b_u32((const int32_t*)p + row); v.eps = Eps<int32_t>::is(x); v.i = x; break; }
    case VD_I64: { int64_t x = (int64_t)ld64b_u64((const int64_t*)p + row); v.eps = Eps<int64_t>::is(x); v.i = x; break; }
    case VD_F32: { float x = __uint_as_float(ld64b_u32((const float*)p + row)); v.eps = Eps<float>::is(x); v.isf = true; v.f = x; break; }
    default: { double x = __longlong_as_double((long long)ld64b_u64((const double*)p + row)); v.eps = Eps<double>::is(x); v.isf = true; v.f = x; break; }
    }
    return v;
}

__device__ __forceinline__ bool term_true(const DevTerm& t, const Val& v) {
    if (v.eps) return false;  // a predicate on epsilon is "not selected" (reading A9)
    return v.isf ? cmp_flt(t.cmp, v.f, t.fv) : cmp_int(t.cmp, v.i, t.iv);
}

// Row predicate over plain columns.
__device__ __forceinline__ bool eval_pred_row(const DevPred& P, const DevCols& C, int64_t row) {
    if (P.nconj == 0) return true;
    for (int c = 0; c < P.nconj; ++c) {
        bool ok = true;
        for (int k = 0; k < P.nterms[c] && ok; ++k) {
            const DevTerm& t = P.t[c][k];
            ok = term_true(t, fetch_typed(C.p[t.col], C.dt[t.col], row));
        }
        if (ok) return true;
    }
    return false;
}

}  // namespace vd
