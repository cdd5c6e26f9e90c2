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

// Wide decoupled look-back: each lane inspects 4 consecutive predecessors,
// so one L2 round trip covers a 128-tile window (the throughput of a
// look-back chain is bounded by window x tile bytes per round trip).
static __device__ __noinline__ int64_t lookback_exclusive_w128(uint64_t* status, int64_t tile, int64_t agg,
                                                               int lane) {
    // The status word carries its own payload, so relaxed (volatile) loads
    // suffice; all four polls of a lane are issued back to back so one
    // window costs one L2 round trip.
    if (tile == 0) {
        if (lane == 0) st_release_u64(&status[0], ST_PFX | (uint64_t)agg);
        return 0;
    }
    if (lane == 0) st_release_u64(&status[tile], ST_AGG | (uint64_t)agg);
    int64_t excl = 0;
    int64_t end = tile - 1;
    for (;;) {
        uint64_t w[4];
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const int64_t idx = end - (lane * 4 + j);
            w[j] = idx >= 0 ? ld_relaxed_u64(&status[idx]) : ST_PFX;
        }
        for (;;) {  // re-poll only the predecessors that have not published yet
            bool ready = true;
#pragma unroll
            for (int j = 0; j < 4; ++j) ready = ready && (w[j] >> 62) != 0;
            if (ready) break;
#pragma unroll
            for (int j = 0; j < 4; ++j)
                if ((w[j] >> 62) == 0) w[j] = ld_relaxed_u64(&status[end - (lane * 4 + j)]);
        }
        int first = 4;  // first predecessor (by distance) of this lane holding a prefix
#pragma unroll
        for (int j = 3; j >= 0; --j)
            if ((w[j] >> 62) == 2) first = j;
        const unsigned pm = __ballot_sync(VD_FULL, first < 4);
        const int stop_lane = pm ? (__ffs(pm) - 1) : 32;
        const int stop_j = __shfl_sync(VD_FULL, first, pm ? stop_lane : 0);
        int64_t v = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const bool take = (lane < stop_lane) || (lane == stop_lane && j <= stop_j);
            if (take) v += (int64_t)(w[j] & ST_MASK);
        }
        excl += warp_sum_i64(v);
        if (pm) break;
        end -= 128;
    }
    if (lane == 0) st_release_u64(&status[tile], ST_PFX | (uint64_t)(excl + agg));
    return excl;
}

}  // namespace vd
