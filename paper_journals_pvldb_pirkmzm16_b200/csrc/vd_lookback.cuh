// vd_lookback.cuh -- single-pass decoupled look-back over per-tile status
// words (used by selection, partition and scans).  Product code.
#pragma once

#include "vd_common.cuh"

namespace vd {

constexpr uint64_t ST_AGG = 1ull << 62;
constexpr uint64_t ST_PFX = 2ull << 62;
constexpr uint64_t ST_MASK = (1ull << 62) - 1;

// Decoupled look-back, executed by one full warp.  Publishes this tile's
// aggregate, accumulates predecessors until one with an inclusive prefix,
// publishes the inclusive prefix, returns the exclusive prefix.
static __device__ __noinline__ int64_t lookback_exclusive(uint64_t* status, int64_t tile, int64_t agg, int lane) {
    if (tile == 0) {
        if (lane == 0) st_release_u64(&status[0], ST_PFX | (uint64_t)agg);
        return 0;
    }
    if (lane == 0) st_release_u64(&status[tile], ST_AGG | (uint64_t)agg);
    int64_t excl = 0;
    int64_t end = tile - 1;
    for (;;) {
        int64_t idx = end - lane;
        uint64_t w = ST_PFX;  // before tile 0: prefix 0
        if (idx >= 0) {
            do { w = ld_acquire_u64(&status[idx]); } while ((w >> 62) == 0);
        }
        unsigned pm = __ballot_sync(VD_FULL, (w >> 62) == 2);
        int stop = pm ? (__ffs(pm) - 1) : 31;
        int64_t v = (lane <= stop) ? (int64_t)(w & ST_MASK) : 0;
        excl += warp_sum_i64(v);
        if (pm) break;
        end -= 32;
    }
    if (lane == 0) st_release_u64(&status[tile], ST_PFX | (uint64_t)(excl + agg));
    return excl;
}

}  // namespace vd
