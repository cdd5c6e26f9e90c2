/*
 * oracle/oracle.h -- C API of the CPU oracle.
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and
 * bench.py's cpu_baseline / --impl reference legs may load liboracle.so.
 * The product path (paper_journals_pvldb_pirkmzm16_b200/) never links,
 * imports or calls anything here, and this code shares nothing with it.
 *
 * Two independent layers:
 *   1. or_ctx_* : a literal, single-threaded interpreter of Voodoo programs
 *      (§2.2 Table 2).  Every intermediate vector is
 *      materialised in its epsilon-padded logical form, as the paper's own
 *      interpreter backend does.
 *   2. or_q1 / or_q6 / or_fkj / or_select : brute-force SQL-equivalent loops
 *      over the same columns (TPC-H SQL [ext]), written independently of
 *      layer 1, used to pin it.
 *
 * Integers are carried as signed 128-bit (returned as lo/hi int64 pairs),
 * floats as long double; nothing is rounded before the caller reads it.
 */
#ifndef VD_ORACLE_H
#define VD_ORACLE_H
#include <stdint.h>
#ifdef __cplusplus
extern "C" {
#endif

/* ---- layer 1: interpreter -------------------------------------------- */
void* or_ctx_new(void);
void or_ctx_free(void* ctx);
/* Bind an input attribute "vec.attr" (or "vec" = single attribute "vec").
 * eps may be NULL (no empty slots).  dtype: 0 = integer (int64 values),
 * 1 = float (double values). */
int or_ctx_set_i64(void* ctx, const char* name, const int64_t* v, const uint8_t* eps, int64_t n);
int or_ctx_set_f64(void* ctx, const char* name, const double* v, const uint8_t* eps, int64_t n);
/* Execute a program (one statement per line, "x := Op(args)", // comments).
 * Returns 0 on success, else nonzero with a message in err. */
int or_ctx_run(void* ctx, const char* program, char* err, int errlen);
/* Inspect a result attribute ("vec.attr" or "vec"). */
int64_t or_ctx_len(void* ctx, const char* name);          /* -1: unknown */
int or_ctx_is_float(void* ctx, const char* name);          /* 1 float, 0 int, -1 unknown */
/* Copy out: ints as (lo, hi) pairs of the 128-bit value; floats as double
 * (and, if fl != NULL, the long-double value's residual v - (double)v). */
int or_ctx_get_i128(void* ctx, const char* name, int64_t* lo, int64_t* hi, uint8_t* eps);
int or_ctx_get_f64(void* ctx, const char* name, double* v, double* resid, uint8_t* eps);

/* ---- layer 2: brute-force loops -------------------------------------- */
/* TPC-H Q1 [ext: TPC-H spec]: for every row with ship <= ship_max, group
 * k = rf*2 + ls (rf: A=0,N=1,R=2; ls: F=0,O=1), accumulate
 *   agg 0 sum_qty, 1 sum_base_price, 2 sum_disc_price (scale 1e4),
 *   3 sum_charge (scale 1e6), 4 sum_disc, 5 count
 * into out[k*6 + agg] as 128-bit (lo/hi). 6 slots. */
void or_q1(int64_t n, const int32_t* ship, const uint8_t* rf, const uint8_t* ls, const int64_t* qty,
           const int64_t* ext, const int64_t* disc, const int64_t* tax, int32_t ship_max, int64_t* out_lo,
           int64_t* out_hi);
/* TPC-H Q6: rev = sum(ext*disc) over ship in [d0,d1), disc in [dlo,dhi],
 * qty < qmax. out[0] = revenue (scale 1e4, 128-bit lo/hi), *count. */
void or_q6(int64_t n, const int32_t* ship, const int64_t* disc, const int64_t* qty, const int64_t* ext, int32_t d0,
           int32_t d1, int64_t dlo, int64_t dhi, int64_t qmax, int64_t* rev_lo, int64_t* rev_hi, int64_t* count);
/* TPC-H Q15 revenue view: for rows with ship in [d0, d1), group by suppkey
 * (ascending, only keys that occur): out_key[g], revenue sum(ext*(100-disc))
 * (scale 1e4, 128-bit lo/hi), out_cnt[g] rows.  Capacity n groups; returns
 * the number of groups. */
int64_t or_q15(int64_t n, const int32_t* ship, const int32_t* suppkey, const int64_t* ext, const int64_t* disc,
               int32_t d0, int32_t d1, int64_t* out_key, int64_t* out_lo, int64_t* out_hi, int64_t* out_cnt);
/* Float selection micro-benchmark (Fig 1): positions i (ascending)
 * with v[i] < t (op=0) or v[i] > t (op=1); returns count, writes positions
 * and the long-double sum of selected values (split into hi + lo doubles). */
int64_t or_select_f32(int64_t n, const float* v, float t, int op, int32_t* pos, double* sum_hi, double* sum_lo);
/* FK gather join + grouped fold (C5, SURVEY §8(c) "C5 FKJ").
 * variant 0 = Q19-style scalar (group 0), 1 = Q9-style group nation*7+(year-1992).
 * out[g*2+0] = sum(ext*(100-disc)) (scale 1e4), out[g*2+1] = count; 175 groups. */
void or_fkj(int variant, int64_t n, const int32_t* partkey, const int32_t* suppkey, const int64_t* qty,
            const int64_t* ext, const int64_t* disc, const uint8_t* shipmode, const uint8_t* shipinstruct,
            const int32_t* ship, int64_t nparts, const uint8_t* p_brand, const uint8_t* p_container,
            const int32_t* p_size, int64_t nsupp, const uint8_t* s_nation, int64_t* out_lo, int64_t* out_hi);
/* Calendar year of a day number (days since 1970-01-01), proleptic Gregorian. */
int32_t or_year_of_day(int32_t day);

#ifdef __cplusplus
}
#endif
#endif
