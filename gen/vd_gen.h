/*
 * gen/vd_gen.h -- seeded, counter-based, partition-invariant input generator.
 *
 * This is the ONLY module shared by the oracle side (host) and the CUDA side
 * (device).  It holds random draws and the TPC-H dbgen-shaped value recipes
 * (DESIGN.md "Input recipe"), and NONE of the Voodoo method's arithmetic:
 * no predicate, fold, gather, scatter or partition lives here.
 *
 * Every value is a pure function of (seed, column id, row index), so a row
 * range [row0, row0+n) generated on any device / host / rank is bit-identical
 * to the same rows of a whole-table generation (SURVEY.md §8(d) "RNG").
 *
 * Shapes follow the TPC-H spec §4.2.3 distributions [ext] as restated in
 * SURVEY.md §8(d):
 *   orders     : lines per order ~ U[1,7], o_orderdate ~ 8035 + U[0,2405]
 *                (1992-01-01 .. 1998-08-02, days since 1970-01-01)
 *   lineitem   : l_shipdate = orderdate + U[1,121]; receipt = ship + U[1,30]
 *                l_returnflag = receipt <= 9298 ? {A,R} : N  (codes A=0,N=1,R=2)
 *                l_linestatus = ship > 9298 ? O : F          (codes F=0,O=1)
 *                l_quantity U[1,50] (x100), l_partkey U[1,200000*SF],
 *                l_extendedprice = qty * retail(partkey) (cents),
 *                l_discount U[0,10], l_tax U[0,8] (x100),
 *                l_suppkey U[1,10000*SF], l_shipmode U{7}, l_shipinstruct U{4}
 *   part       : p_brand U{25}, p_container U{40}, p_size U[1,50]
 *   supplier   : s_nationkey U[0,24]
 *   f32 column : v = (u >> 40) * 2^-24 in [0,1)
 *
 * Order structure without a global prefix sum: lineitem rows are grouped in
 * blocks of VDG_OBLOCK consecutive rows; inside a block, orders of U[1,7]
 * lines are laid end to end (the last one truncated at the block edge).
 * Consecutive rows therefore share an order (and its o_orderdate) exactly as
 * dbgen's lineitem does, yet row i depends only on (seed, i).
 */
#ifndef VD_GEN_H
#define VD_GEN_H

#include <stdint.h>

#if defined(__CUDACC__)
#define VDG_HD __host__ __device__ __forceinline__
#else
#define VDG_HD static inline
#endif

#ifdef __cplusplus
extern "C" {
#endif

/* Column ids (also the RNG stream ids). */
enum {
    VDG_L_SHIPDATE = 1,      /* i32 days since 1970-01-01            */
    VDG_L_RETURNFLAG = 2,    /* u8  A=0 N=1 R=2                      */
    VDG_L_LINESTATUS = 3,    /* u8  F=0 O=1                          */
    VDG_L_QUANTITY = 4,      /* i64 DECIMAL(15,2) scaled 10^2        */
    VDG_L_EXTENDEDPRICE = 5, /* i64 scaled 10^2                      */
    VDG_L_DISCOUNT = 6,      /* i64 scaled 10^2                      */
    VDG_L_TAX = 7,           /* i64 scaled 10^2                      */
    VDG_L_PARTKEY = 8,       /* i32 1-based                          */
    VDG_L_SUPPKEY = 9,       /* i32 1-based                          */
    VDG_L_SHIPMODE = 10,     /* u8 dictionary code 0..6              */
    VDG_L_SHIPINSTRUCT = 11, /* u8 dictionary code 0..3              */
    VDG_P_BRAND = 12,        /* u8 0..24                             */
    VDG_P_CONTAINER = 13,    /* u8 0..39                             */
    VDG_P_SIZE = 14,         /* i32 1..50                            */
    VDG_S_NATIONKEY = 15,    /* u8 0..24                             */
    VDG_F32_UNIFORM = 16,    /* f32 U[0,1)                           */
    VDG_I32_UNIFORM = 17,    /* i32 U[lo,hi] (params)                */
    VDG_I32_PERM = 18,       /* i32 permutation of [0,n) (param n)   */
    VDG_I64_UNIFORM = 19,    /* i64 U[lo,hi] (params)                */
    VDG_F64_UNIFORM = 20,    /* f64 U[0,1) * scale (param)           */
    /* internal streams */
    VDG_S_ORDLINES = 100,
    VDG_S_ORDDATE = 101,
    VDG_S_SHIPOFF = 102,
    VDG_S_RECEIPTOFF = 103,
    VDG_S_RFLAG_AR = 104,
    VDG_S_PERM = 105
};

#define VDG_OBLOCK 32
#define VDG_DEFAULT_SEED 0x5EEDC0DEull

/* Dates (days since 1970-01-01). */
#define VDG_STARTDATE 8035   /* 1992-01-01 */
#define VDG_ODATE_SPAN 2405  /* .. 1998-08-02 */
#define VDG_CURRENTDATE 9298 /* 1995-06-17 */

VDG_HD uint64_t vdg_splitmix(uint64_t z) {
    z += 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

/* One 64-bit draw of stream `stream` at counter `idx`. */
VDG_HD uint64_t vdg_draw(uint64_t seed, uint64_t stream, uint64_t idx) {
    uint64_t key = vdg_splitmix(seed ^ (stream * 0xD1B54A32D192ED03ull));
    return vdg_splitmix(key + idx * 0x9E3779B97F4A7C15ull);
}

/* Uniform integer in [lo, hi] (multiply-shift on the high 32 bits). */
VDG_HD int64_t vdg_uniform(uint64_t seed, uint64_t stream, uint64_t idx, int64_t lo, int64_t hi) {
    uint64_t range = (uint64_t)(hi - lo) + 1ull;
    uint64_t u = vdg_draw(seed, stream, idx);
    if (range <= 0xFFFFFFFFull) return lo + (int64_t)(((u >> 32) * range) >> 32);
    return lo + (int64_t)(u % range);
}

/* Table cardinalities for a scale factor (rounded, >= 1). */
VDG_HD int64_t vdg_lineitem_rows(double sf) { int64_t n = (int64_t)(6000000.0 * sf + 0.5); return n; }
VDG_HD int64_t vdg_part_rows(double sf) { int64_t n = (int64_t)(200000.0 * sf + 0.5); return n < 1 ? 1 : n; }
VDG_HD int64_t vdg_supplier_rows(double sf) { int64_t n = (int64_t)(10000.0 * sf + 0.5); return n < 1 ? 1 : n; }

/* o_orderdate of the order that lineitem row `row` belongs to. */
VDG_HD int32_t vdg_orderdate_of_row(uint64_t seed, int64_t row) {
    int64_t blk = row / VDG_OBLOCK;
    int32_t off = (int32_t)(row - blk * VDG_OBLOCK);
    int32_t cum = 0, k = 0;
    for (;;) {
        int32_t lines = (int32_t)vdg_uniform(seed, VDG_S_ORDLINES, (uint64_t)(blk * VDG_OBLOCK + k), 1, 7);
        if (off < cum + lines) break;
        cum += lines;
        ++k;
    }
    return (int32_t)vdg_uniform(seed, VDG_S_ORDDATE, (uint64_t)(blk * VDG_OBLOCK + k), VDG_STARTDATE,
                                VDG_STARTDATE + VDG_ODATE_SPAN);
}

VDG_HD int32_t vdg_shipdate(uint64_t seed, int64_t row) {
    return vdg_orderdate_of_row(seed, row) + (int32_t)vdg_uniform(seed, VDG_S_SHIPOFF, (uint64_t)row, 1, 121);
}

VDG_HD int32_t vdg_receiptdate_from_ship(uint64_t seed, int64_t row, int32_t ship) {
    return ship + (int32_t)vdg_uniform(seed, VDG_S_RECEIPTOFF, (uint64_t)row, 1, 30);
}

/* retail price of part `pk` in cents (TPC-H 4.2.3: 90000 + ((pk/10) mod 20001) + 100*(pk mod 1000)). */
VDG_HD int64_t vdg_retail_cents(int64_t pk) { return 90000 + ((pk / 10) % 20001) + 100 * (pk % 1000); }

VDG_HD int64_t vdg_quantity_units(uint64_t seed, int64_t row) {
    return vdg_uniform(seed, VDG_L_QUANTITY, (uint64_t)row, 1, 50);
}

VDG_HD int32_t vdg_partkey(uint64_t seed, int64_t row, double sf) {
    return (int32_t)vdg_uniform(seed, VDG_L_PARTKEY, (uint64_t)row, 1, vdg_part_rows(sf));
}

/* Generic per-row value of a lineitem/part/supplier/synthetic column, widened
 * to int64 (floats are returned through vdg_value_f). `p0`,`p1` are the
 * column parameters (lo/hi for *_UNIFORM, n for PERM, unused otherwise). */
VDG_HD uint32_t vdg_perm_round(uint64_t seed, int r, uint32_t x, uint32_t mask) {
    return (uint32_t)(vdg_draw(seed, VDG_S_PERM + 16 * (uint64_t)r, x) & mask);
}

/* Counter-based permutation of [0,n) (balanced Feistel + cycle walking). */
VDG_HD int64_t vdg_perm(uint64_t seed, int64_t n, int64_t i) {
    if (n <= 1) return 0;
    int bits = 0;
    while ((1ll << bits) < n) ++bits;
    if (bits & 1) ++bits;
    int half = bits / 2;
    uint32_t mask = (half >= 32) ? 0xFFFFFFFFu : ((1u << half) - 1u);
    uint64_t x = (uint64_t)i;
    do {
        uint32_t L = (uint32_t)(x >> half) & mask, R = (uint32_t)x & mask;
        for (int r = 0; r < 4; ++r) {
            uint32_t t = L ^ vdg_perm_round(seed, r, R, mask);
            L = R;
            R = t;
        }
        x = ((uint64_t)L << half) | R;
    } while ((int64_t)x >= n);
    return (int64_t)x;
}

VDG_HD int64_t vdg_value_i(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, int64_t row) {
    switch (col) {
    case VDG_L_SHIPDATE: return vdg_shipdate(seed, row);
    case VDG_L_RETURNFLAG: {
        int32_t ship = vdg_shipdate(seed, row);
        int32_t rec = vdg_receiptdate_from_ship(seed, row, ship);
        if (rec <= VDG_CURRENTDATE) return vdg_uniform(seed, VDG_S_RFLAG_AR, (uint64_t)row, 0, 1) ? 2 : 0;
        return 1;
    }
    case VDG_L_LINESTATUS: return vdg_shipdate(seed, row) > VDG_CURRENTDATE ? 1 : 0;
    case VDG_L_QUANTITY: return 100 * vdg_quantity_units(seed, row);
    case VDG_L_EXTENDEDPRICE: return vdg_quantity_units(seed, row) * vdg_retail_cents(vdg_partkey(seed, row, sf));
    case VDG_L_DISCOUNT: return vdg_uniform(seed, VDG_L_DISCOUNT, (uint64_t)row, 0, 10);
    case VDG_L_TAX: return vdg_uniform(seed, VDG_L_TAX, (uint64_t)row, 0, 8);
    case VDG_L_PARTKEY: return vdg_partkey(seed, row, sf);
    case VDG_L_SUPPKEY: return vdg_uniform(seed, VDG_L_SUPPKEY, (uint64_t)row, 1, vdg_supplier_rows(sf));
    case VDG_L_SHIPMODE: return vdg_uniform(seed, VDG_L_SHIPMODE, (uint64_t)row, 0, 6);
    case VDG_L_SHIPINSTRUCT: return vdg_uniform(seed, VDG_L_SHIPINSTRUCT, (uint64_t)row, 0, 3);
    case VDG_P_BRAND: return vdg_uniform(seed, VDG_P_BRAND, (uint64_t)row, 0, 24);
    case VDG_P_CONTAINER: return vdg_uniform(seed, VDG_P_CONTAINER, (uint64_t)row, 0, 39);
    case VDG_P_SIZE: return vdg_uniform(seed, VDG_P_SIZE, (uint64_t)row, 1, 50);
    case VDG_S_NATIONKEY: return vdg_uniform(seed, VDG_S_NATIONKEY, (uint64_t)row, 0, 24);
    case VDG_I32_UNIFORM:
    case VDG_I64_UNIFORM: return vdg_uniform(seed, (uint64_t)col, (uint64_t)row, p0, p1);
    case VDG_I32_PERM: return vdg_perm(seed, p0, row);
    default: return 0;
    }
}

VDG_HD double vdg_value_f(int col, uint64_t seed, double scale, int64_t row) {
    uint64_t u = vdg_draw(seed, (uint64_t)col, (uint64_t)row);
    if (col == VDG_F32_UNIFORM) return (double)(float)((double)(u >> 40) * (1.0 / 16777216.0));
    return (double)(u >> 11) * (1.0 / 9007199254740992.0) * scale;
}

/* Storage dtype of each column: 0=u8 1=i32 2=i64 3=f32 4=f64 (matches vd_dtype). */
VDG_HD int vdg_col_dtype(int col) {
    switch (col) {
    case VDG_L_RETURNFLAG: case VDG_L_LINESTATUS: case VDG_L_SHIPMODE: case VDG_L_SHIPINSTRUCT:
    case VDG_P_BRAND: case VDG_P_CONTAINER: case VDG_S_NATIONKEY: return 0;
    case VDG_L_SHIPDATE: case VDG_L_PARTKEY: case VDG_L_SUPPKEY: case VDG_P_SIZE:
    case VDG_I32_UNIFORM: case VDG_I32_PERM: return 1;
    case VDG_L_QUANTITY: case VDG_L_EXTENDEDPRICE: case VDG_L_DISCOUNT: case VDG_L_TAX:
    case VDG_I64_UNIFORM: return 2;
    case VDG_F32_UNIFORM: return 3;
    case VDG_F64_UNIFORM: return 4;
    default: return -1;
    }
}

/* Fill one column, host side. Returns 0 on success, -1 on unknown column. */
int vdg_fill_host(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, double fscale, int64_t row0,
                  int64_t n, void* out);
/* Fill one column on the current CUDA device (stream may be 0). */
int vdg_fill_device(int col, uint64_t seed, double sf, int64_t p0, int64_t p1, double fscale, int64_t row0,
                    int64_t n, void* out_dev, void* stream);

#ifdef __cplusplus
}
#endif

#endif /* VD_GEN_H */
