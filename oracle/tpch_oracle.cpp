// oracle/tpch_oracle.cpp -- layer 2 of the CPU oracle: brute-force
// SQL-equivalent loops (SURVEY.md §8(c) "Oracle queries").
//
// TEST INFRASTRUCTURE ONLY (see oracle.h).  Written independently of the
// interpreter (layer 1) so that each pins the other.  Single-threaded, one
// pass, 128-bit integer accumulators, long-double float accumulators.
//
// Fixed point [ext: TPC-H / MonetDB storage, P:L1031-1033]: DECIMAL(15,2)
// is an integer scaled by 10^2; a product of two decimals has scale 10^4,
// of three 10^6; no intermediate rounding (reading A17).
#include <algorithm>
#include <cstring>
#include <string>
#include <vector>

#include "oracle.h"

typedef __int128 i128;

static void put128(i128 v, int64_t* lo, int64_t* hi) {
    unsigned __int128 u = (unsigned __int128)v;
    *lo = (int64_t)(uint64_t)u;
    *hi = (int64_t)(uint64_t)(u >> 64);
}

extern "C" void or_q1(int64_t n, const int32_t* ship, const uint8_t* rf, const uint8_t* ls, const int64_t* qty,
                      const int64_t* ext, const int64_t* disc, const int64_t* tax, int32_t ship_max,
                      int64_t* out_lo, int64_t* out_hi) {
    // TPC-H Q1 [ext]: WHERE l_shipdate <= date '1998-12-01' - interval DELTA day
    // GROUP BY l_returnflag, l_linestatus.
    i128 acc[6][6];
    std::memset(acc, 0, sizeof(acc));
    for (int64_t i = 0; i < n; ++i) {
        if (!(ship[i] <= ship_max)) continue;
        int k = (int)rf[i] * 2 + (int)ls[i];
        i128 dp = (i128)ext[i] * (100 - disc[i]);          // extendedprice*(1-discount), scale 1e4
        acc[k][0] += qty[i];
        acc[k][1] += ext[i];
        acc[k][2] += dp;
        acc[k][3] += dp * (100 + tax[i]);                  // *(1+tax), scale 1e6
        acc[k][4] += disc[i];
        acc[k][5] += 1;
    }
    for (int k = 0; k < 6; ++k)
        for (int a = 0; a < 6; ++a) put128(acc[k][a], &out_lo[k * 6 + a], &out_hi[k * 6 + a]);
}

extern "C" void or_q6(int64_t n, const int32_t* ship, const int64_t* disc, const int64_t* qty, const int64_t* ext,
                      int32_t d0, int32_t d1, int64_t dlo, int64_t dhi, int64_t qmax, int64_t* rev_lo,
                      int64_t* rev_hi, int64_t* count) {
    // TPC-H Q6 [ext]: shipdate in [DATE, DATE + 1 year), discount between
    // DISCOUNT -/+ 0.01, quantity < QUANTITY; sum(extendedprice*discount).
    i128 rev = 0;
    int64_t c = 0;
    for (int64_t i = 0; i < n; ++i) {
        if (ship[i] >= d0 && ship[i] < d1 && disc[i] >= dlo && disc[i] <= dhi && qty[i] < qmax) {
            rev += (i128)ext[i] * disc[i];
            ++c;
        }
    }
    put128(rev, rev_lo, rev_hi);
    *count = c;
}

extern "C" int64_t or_q15(int64_t n, const int32_t* ship, const int32_t* suppkey, const int64_t* ext,
                          const int64_t* disc, int32_t d0, int32_t d1, int64_t* out_key, int64_t* out_lo,
                          int64_t* out_hi, int64_t* out_cnt) {
    // TPC-H Q15's revenue view [ext]: shipdate in [DATE, DATE + 3 months),
    // GROUP BY l_suppkey, SUM(l_extendedprice * (1 - l_discount)) -- here
    // ext * (100 - disc) at scale 1e4 (reading A17).  A std::map keyed by the
    // supplier key: ascending key order, only suppliers that occur (the
    // SQL GROUP BY result, reading A16).  Returns the number of groups.
    // collect the qualifying (key, value) pairs, stable-sort by key, sum runs
    std::vector<std::pair<int64_t, i128>> rows;
    for (int64_t i = 0; i < n; ++i)
        if (ship[i] >= d0 && ship[i] < d1) rows.push_back({(int64_t)suppkey[i], (i128)ext[i] * (100 - disc[i])});
    std::stable_sort(rows.begin(), rows.end(),
                     [](const std::pair<int64_t, i128>& a, const std::pair<int64_t, i128>& b) { return a.first < b.first; });
    int64_t g = -1;
    i128 rev = 0;
    int64_t cnt = 0;
    for (size_t k = 0; k <= rows.size(); ++k) {
        if (k == rows.size() || (k > 0 && rows[k].first != rows[k - 1].first)) {
            if (k > 0) {
                ++g;
                out_key[g] = rows[k - 1].first;
                put128(rev, &out_lo[g], &out_hi[g]);
                out_cnt[g] = cnt;
            }
            rev = 0;
            cnt = 0;
        }
        if (k == rows.size()) break;
        rev += rows[k].second;
        ++cnt;
    }
    return g + 1;
}

extern "C" int64_t or_select_f32(int64_t n, const float* v, float t, int op, int32_t* pos, double* sum_hi,
                                 double* sum_lo) {
    // Fig 1: filter a list of values with a predicate; the output
    // is the ascending list of qualifying positions (std::copy_if on indices).
    long double s = 0;
    int64_t c = 0;
    for (int64_t i = 0; i < n; ++i) {
        bool p = (op == 0) ? (v[i] < t) : (v[i] > t);
        if (p) {
            if (pos) pos[c] = (int32_t)i;
            ++c;
            s += (long double)v[i];
        }
    }
    *sum_hi = (double)s;
    *sum_lo = (double)(s - (long double)*sum_hi);
    return c;
}

extern "C" int32_t or_year_of_day(int32_t day) {
    // Count whole years from 1970 (proleptic Gregorian); plain loop.
    int32_t y = 1970, d = day;
    for (;;) {
        bool leap = (y % 4 == 0 && y % 100 != 0) || (y % 400 == 0);
        int32_t len = leap ? 366 : 365;
        if (d < len) return y;
        d -= len;
        ++y;
    }
}

// Dictionary of p_container [ext: TPC-H 4.2.2.13]: syllable1 x syllable2,
// codes are ranks in sorted order (order-preserving dictionary).
static int container_code(const std::string& s) {
    const char* s1[] = {"SM", "LG", "MED", "JUMBO", "WRAP"};
    const char* s2[] = {"CASE", "BOX", "BAG", "JAR", "PKG", "PACK", "CAN", "DRUM"};
    std::vector<std::string> all;
    for (auto a : s1)
        for (auto b : s2) all.push_back(std::string(a) + " " + b);
    std::sort(all.begin(), all.end());
    for (size_t k = 0; k < all.size(); ++k)
        if (all[k] == s) return (int)k;
    return -1;
}

static int brand_code(int m, int nn) { return (m - 1) * 5 + (nn - 1); }  // Brand#MN, sorted

extern "C" void or_fkj(int variant, int64_t n, const int32_t* partkey, const int32_t* suppkey, const int64_t* qty,
                       const int64_t* ext, const int64_t* disc, const uint8_t* shipmode,
                       const uint8_t* shipinstruct, const int32_t* ship, int64_t nparts, const uint8_t* p_brand,
                       const uint8_t* p_container, const int32_t* p_size, int64_t nsupp, const uint8_t* s_nation,
                       int64_t* out_lo, int64_t* out_hi) {
    // C5: lineitem x part (x supplier) through dense FK
    // positions pos = key - 1 (identity hashing P:L1054-1056).
    i128 rev[175], cnt[175];
    std::memset(rev, 0, sizeof(rev));
    std::memset(cnt, 0, sizeof(cnt));
    // Q19 [ext] constants: Brand#12/#23/#34, quantity 1/10/20 (+10),
    // sizes 1..5/10/15, shipmode in ('AIR','AIR REG'), 'DELIVER IN PERSON'.
    const char* cont[3][4] = {{"SM CASE", "SM BOX", "SM PACK", "SM PKG"},
                              {"MED BAG", "MED BOX", "MED PKG", "MED PACK"},
                              {"LG CASE", "LG BOX", "LG PACK", "LG PKG"}};
    int brand[3] = {brand_code(1, 2), brand_code(2, 3), brand_code(3, 4)};
    int qlo[3] = {1, 10, 20};
    int smax[3] = {5, 10, 15};
    int ccode[3][4];
    for (int g = 0; g < 3; ++g)
        for (int j = 0; j < 4; ++j) ccode[g][j] = container_code(cont[g][j]);
    // shipmode dictionary (sorted): AIR FOB MAIL RAIL "REG AIR" SHIP TRUCK;
    // 'AIR REG' is not a dbgen value, so it matches nothing (reading A26).
    const int MODE_AIR = 0;
    const int INSTR_DELIVER_IN_PERSON = 1;  // COLLECT COD, DELIVER IN PERSON, NONE, TAKE BACK RETURN
    for (int64_t i = 0; i < n; ++i) {
        int64_t p = (int64_t)partkey[i] - 1;
        int64_t s = (int64_t)suppkey[i] - 1;
        if (p < 0 || p >= nparts || s < 0 || s >= nsupp) continue;  // FK miss (never with dbgen data)
        int g = 0;
        if (variant == 0) {
            bool ok = false;
            for (int b = 0; b < 3 && !ok; ++b) {
                bool cm = false;
                for (int j = 0; j < 4; ++j) cm = cm || ((int)p_container[p] == ccode[b][j]);
                ok = (int)p_brand[p] == brand[b] && cm && qty[i] >= (int64_t)qlo[b] * 100 &&
                     qty[i] <= (int64_t)(qlo[b] + 10) * 100 && p_size[p] >= 1 && p_size[p] <= smax[b] &&
                     (int)shipmode[i] == MODE_AIR && (int)shipinstruct[i] == INSTR_DELIVER_IN_PERSON;
            }
            if (!ok) continue;
        } else {
            int y = or_year_of_day(ship[i]);
            g = (int)s_nation[s] * 7 + (y - 1992);
            if (g < 0 || g >= 175) continue;
        }
        rev[g] += (i128)ext[i] * (100 - disc[i]);
        cnt[g] += 1;
    }
    for (int g = 0; g < 175; ++g) {
        put128(rev[g], &out_lo[g * 2], &out_hi[g * 2]);
        put128(cnt[g], &out_lo[g * 2 + 1], &out_hi[g * 2 + 1]);
    }
}
