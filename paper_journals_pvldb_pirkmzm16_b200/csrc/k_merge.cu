// k_merge.cu -- the cross-GPU step of the hierarchical fold and the Fig 11
// compaction, on the device.  Product code.
//
// Fig 3 folds partial aggregates level by level; one level above
// the CTAs of a pipeline launch sit the GPUs of the row-range partition
// (SURVEY §8(e)): each rank's vd_partials ([ngroups][naggs+1] 16-byte slots)
// is all-gathered, and every rank combines them in rank order -- exact in
// 128 bits for integer SUM/COUNT, f64 for float SUM, MIN/MAX over the ranks
// where the group is non-empty.  The result is then compacted as in Fig 11
// (P:L866-928): FoldSelect over the row counts keeps the non-empty groups,
// in ascending key order (reading A16), and Gather moves their aggregates
// to the front.  One CTA: ngroups <= VD_MAX_GROUPS (4096) and nparts <= a
// few dozen, so the kernel is a few microseconds of latency, launched on the
// pipeline's stream right behind it (no host round trip).
#include <cuda_runtime.h>

#include "vd_common.cuh"
#include "vd_internal.h"

namespace vd {

constexpr int MG_THREADS = 256;

struct MergeArgs {
    const unsigned long long* parts;  // nparts x [G][NA+1] x 2 words
    int32_t nparts, naggs;
    int64_t ngroups;
    int32_t kind[VD_MAX_AGGS];
    int32_t isf[VD_MAX_AGGS];
    int64_t* keys;
    unsigned long long* aggs;  // [cap][NA] x 2 words
    int64_t* rows;
    int64_t* ngroups_out;
};

__device__ __forceinline__ i128 slot_i128(const unsigned long long* p) {
    return (i128)(((u128)p[1] << 64) | p[0]);
}

__global__ void __launch_bounds__(MG_THREADS) k_merge_partials(const __grid_constant__ MergeArgs a) {
    __shared__ int s_warp[MG_THREADS / 32];
    __shared__ int64_t s_base;
    const int NA = a.naggs;
    const int64_t stride = (int64_t)a.ngroups * (NA + 1) * 2;  // words per partial
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    if (threadIdx.x == 0) s_base = 0;
    __syncthreads();
    for (int64_t g0 = 0; g0 < a.ngroups; g0 += MG_THREADS) {
        const int64_t g = g0 + threadIdx.x;
        const int64_t base = g * (NA + 1) * 2;
        i128 rows = 0;
        if (g < a.ngroups)
            for (int r = 0; r < a.nparts; ++r) rows += slot_i128(a.parts + r * stride + base + 2 * NA);
        const bool keep = rows != 0;
        // FoldSelect over the row counts: block-wide exclusive prefix of `keep`
        const unsigned m = __ballot_sync(0xFFFFFFFFu, keep);
        if (lane == 0) s_warp[warp] = __popc(m);
        __syncthreads();
        int64_t off = s_base;
        for (int w = 0; w < warp; ++w) off += s_warp[w];
        off += __popc(m & ((1u << lane) - 1u));
        if (keep) {
            for (int ag = 0; ag < NA; ++ag) {
                const int kind = a.kind[ag];
                const bool fl = a.isf[ag] && kind != VD_AGG_COUNT;
                i128 vi = 0;
                double vf = 0;
                bool have = false;
                for (int r = 0; r < a.nparts; ++r) {  // rank order (deterministic)
                    const unsigned long long* q = a.parts + r * stride + base;
                    if (slot_i128(q + 2 * NA) == 0) continue;  // group empty on rank r
                    const unsigned long long* x = q + 2 * ag;
                    if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                        if (fl) vf += __longlong_as_double((long long)x[0]);
                        else vi += slot_i128(x);
                    } else if (fl) {
                        const double d = __longlong_as_double((long long)x[0]);
                        if (!have || (kind == VD_AGG_MIN ? d < vf : d > vf)) vf = d;
                    } else {
                        const i128 y = slot_i128(x);
                        if (!have || (kind == VD_AGG_MIN ? y < vi : y > vi)) vi = y;
                    }
                    have = true;
                }
                unsigned long long* o = a.aggs + 2 * (off * NA + ag);
                if (a.nparts == 1) {  // a single partial: the slot verbatim
                    o[0] = a.parts[base + 2 * ag];
                    o[1] = a.parts[base + 2 * ag + 1];
                } else if (fl) {
                    o[0] = (unsigned long long)__double_as_longlong(vf);
                    o[1] = 0;
                } else {
                    o[0] = (unsigned long long)(u128)vi;
                    o[1] = (unsigned long long)((u128)vi >> 64);
                }
            }
            a.keys[off] = g;
            a.rows[off] = (int64_t)rows;
        }
        __syncthreads();
        if (threadIdx.x == 0) {
            int t = 0;
            for (int w = 0; w < MG_THREADS / 32; ++w) t += s_warp[w];
            s_base += t;
        }
        __syncthreads();
    }
    if (threadIdx.x == 0) *a.ngroups_out = s_base;
}

cudaError_t launch_merge_partials(const vd_pipeline* plan, const int32_t* isf, const void* parts, int nparts,
                                  const vd_result& out, cudaStream_t s, int* nl) {
    MergeArgs a;
    a.parts = (const unsigned long long*)parts;
    a.nparts = nparts;
    a.naggs = plan->naggs;
    a.ngroups = plan->ngroups;
    for (int k = 0; k < VD_MAX_AGGS; ++k) {
        a.kind[k] = k < plan->naggs ? plan->aggs[k].kind : 0;
        a.isf[k] = k < plan->naggs ? isf[k] : 0;
    }
    a.keys = out.keys;
    a.aggs = (unsigned long long*)out.aggs;
    a.rows = out.rows;
    a.ngroups_out = out.ngroups;
    k_merge_partials<<<1, MG_THREADS, 0, s>>>(a);
    *nl += 1;
    return cudaGetLastError();
}

}  // namespace vd
