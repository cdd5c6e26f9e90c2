/*
 * include/vd.h -- C ABI of libvd.so, the B200-native hot path of Voodoo's
 * compiled vector algebra (Pirk, Moll, Zaharia, Madden, PVLDB 9(14) 2016).
 *
 * Citations: "P:Lx" = line x of the paper text, with the section,
 * figure or table it belongs to.  Readings "Ann" are listed in DESIGN.md
 * (SURVEY.md §8(c)).
 *
 * Conventions shared by every entry point
 * ---------------------------------------
 *  - Memory.  Every data pointer is a DEVICE pointer on the current CUDA
 *    device unless the parameter name ends in _host.  The caller owns every
 *    buffer (inputs, outputs, workspace); the library never allocates, frees
 *    or retains a pointer beyond the call's stream-ordered lifetime.
 *  - Streams.  `stream` is a cudaStream_t passed as void* (NULL = legacy
 *    default stream).  Calls are asynchronous: they enqueue kernels and
 *    return; results are valid once the stream reaches that point.
 *  - Errors.  Argument / metadata validation happens before any launch and
 *    returns a VD_E_* code synchronously, with detail in vd_last_error()
 *    (thread-local).  A launch failure returns VD_E_CUDA.  Nothing throws
 *    across the ABI.  There is no CPU fallback: without a CUDA device every
 *    compute call returns VD_E_CUDA.
 *  - Workspace.  Calls taking (ws, ws_bytes) need a device scratch buffer of
 *    at least vd_workspace_bytes(op, n, ...) bytes, 256-byte aligned; its
 *    contents need not be initialised and are garbage afterwards.
 *  - Empty slots (epsilon, §2.1).  Device data encodes epsilon by
 *    MonetDB-style reserved values: u8 0xFF, i32 INT32_MIN,
 *    i64 INT64_MIN, f32/f64 any NaN (written as the canonical quiet NaN),
 *    positions: any negative value.
 *  - Results of folds are in the empty-slot-SUPPRESSED form of §3.1.2
 *    (reading A4): one slot per run, in run order, instead of the
 *    logical epsilon-padded vector whose result sits at each run start.
 */
#ifndef VD_H
#define VD_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
    VD_OK = 0,
    VD_E_NULL = 1,        /* a required pointer is NULL                          */
    VD_E_DTYPE = 2,       /* unsupported dtype for this operator                 */
    VD_E_SHAPE = 3,       /* length / size / alignment / count out of range      */
    VD_E_CTRL = 4,        /* invalid control vector (den <= 0, negative step ...) */
    VD_E_DOMAIN = 5,      /* group-key domain overflows (ctrl/data bit conflict) */
    VD_E_OVERFLOW = 6,    /* min/max metadata cannot prove int64 partial sums exact */
    VD_E_WORKSPACE = 7,   /* workspace missing or smaller than vd_workspace_bytes */
    VD_E_CUDA = 8,        /* CUDA launch / runtime error (or no device)           */
    VD_E_UNSUPPORTED = 9, /* valid request outside what this build implements     */
    VD_E_ARG = 10         /* other invalid argument                               */
} vd_status;

typedef enum { VD_U8 = 0, VD_I32 = 1, VD_I64 = 2, VD_F32 = 3, VD_F64 = 4 } vd_dtype;

#define VD_EPS_U8 ((uint8_t)0xFF)
#define VD_EPS_I32 ((int32_t)INT32_MIN)
#define VD_EPS_I64 ((int64_t)INT64_MIN)

/* A typed, non-owning device view of one attribute of a Structured Vector
 * (§2.1).  `min`/`max` are the value metadata the paper's
 * frontend exploits: identity-hashed table
 * sizes and proofs that narrow / int64 arithmetic is exact. */
typedef struct {
    const void* data;   /* device pointer to `len` elements of `dtype`        */
    int64_t len;        /* number of slots                                     */
    int32_t dtype;      /* vd_dtype                                            */
    int32_t scale;      /* decimal scale: value = data / 10^scale (0 = plain)  */
    int64_t min, max;   /* inclusive bounds of the non-epsilon values          */
    int32_t has_minmax; /* 1 if min/max are valid                              */
    int32_t flags;      /* VD_COL_* metadata bits (0 = nothing known)          */
} vd_column;

/* vd_column.flags: VD_COL_NOEPS -- the metadata producer has verified that
 * no slot in [0, len) is epsilon (MonetDB's "nonil" column property).  Like
 * min/max it is a promise by the caller; fused fragments use it (with
 * min/max) to drop per-row epsilon / bounds checks.  A false promise gives
 * unspecified results (never an out-of-bounds access: gathers still need
 * min/max to prove their positions in range). */
#define VD_COL_NOEPS 1

/* Control vector (§2.2 Controlled Folding).  Runs = maximal
 * blocks of ADJACENT equal values (reading A3).
 *   materialized == NULL : virtual, never computed; its values
 *       follow the run metadata of §3.1.1 (reading A2):
 *           v[i] = (from + floor(i * step_num / step_den)) mod cap
 *       (cap == 0: no modulo).  Divide(Range, R) is {0, 1, R, 0}: runs of R.
 *   materialized != NULL : a device vector of `len` int32/int64 values
 *       (mat_dtype VD_I32 / VD_I64) whose adjacent-equal blocks are the runs.
 * A NULL vd_ctrl* means the constant control vector: one run over all slots
 * (Fig 3 line 9). */
typedef struct {
    int64_t from;
    int64_t step_num, step_den; /* step = num/den, num >= 0, den > 0 */
    int64_t cap;                /* 0 = none                           */
    const void* materialized;
    int32_t mat_dtype;
    int32_t reserved;
} vd_ctrl;

/* Predicates.  The algebra has only Greater and Equals combined
 * with LogicalAnd/Or; other comparisons are their compositions
 * (reading A8): LT(c) = Greater(c, x), GE(c) = Greater(x, c-1) on integers,
 * LE(c) = Greater(c+1, x), NE = not Equals, IN = OR of Equals over a small
 * dictionary (bit k of `ival` set <=> code k, codes 0..63).  A term over an
 * epsilon slot is false (reading A9). */
typedef enum { VD_CMP_GT = 0, VD_CMP_LT = 1, VD_CMP_EQ = 2, VD_CMP_GE = 3, VD_CMP_LE = 4, VD_CMP_NE = 5,
               VD_CMP_IN = 6 } vd_cmp;

#define VD_MAX_TERMS 8
#define VD_MAX_CONJ 4

typedef struct {
    int32_t col;  /* index into the call's column list                       */
    int32_t cmp;  /* vd_cmp                                                  */
    int64_t ival; /* constant for integer columns (IN: 64-bit code mask)      */
    double fval;  /* constant for float columns                              */
} vd_term;

typedef struct {
    int32_t nterms; /* 0..VD_MAX_TERMS, AND-ed */
    int32_t reserved;
    vd_term terms[VD_MAX_TERMS];
} vd_conj;

typedef struct {
    int32_t nconj; /* 0 = always true; else OR of nconj conjunctions */
    int32_t reserved;
    vd_conj conj[VD_MAX_CONJ];
} vd_pred;

/* How a selection / fused pipeline realises the predicate (Fig 1,
 * P:L98-108; Fig 15/16):
 *   BRANCH     : data-dependent control -- only qualifying rows are
 *                written / accumulated, and (in fused pipelines) columns only
 *                used by qualifying rows are loaded only for them;
 *   PREDICATED : branch-free cursor arithmetic -- every row is written at the
 *                output cursor and the cursor advances by the predicate
 *                (selection); every row is loaded and its contribution is
 *                multiplied by the 0/1 predicate (aggregation: "Predicated
 *                Aggregation" of Fig 16);
 *   PREDICATED_LOOKUP : (pipelines with gathers) the FK position is
 *                multiplied by the predicate before the lookup, so rows that
 *                do not qualify all read position 0 -- one "very hot" cache
 *                line -- and their contribution is still multiplied by the
 *                predicate ("Predicated Lookups").
 * All modes return identical results. */
typedef enum { VD_SEL_BRANCH = 0, VD_SEL_PREDICATED = 1, VD_SEL_PREDICATED_LOOKUP = 2 } vd_sel_mode;

/* ---------------------------------------------------------------------- */
/* Misc                                                                    */
/* ---------------------------------------------------------------------- */
const char* vd_status_str(vd_status s);
/* Detail of the last error on this thread ("" if none). */
const char* vd_last_error(void);
/* Library version string. */
const char* vd_version(void);

/* Number of runs of a control vector over n slots.  Virtual controls are
 * counted on the host; a materialized control returns VD_E_UNSUPPORTED
 * (its run count is data dependent and returned on the device by the fold
 * calls).  ctrl == NULL -> 1 (0 if n == 0). */
vd_status vd_ctrl_runs(const vd_ctrl* ctrl, int64_t n, int64_t* nruns_host);

/* Operator ids for vd_workspace_bytes. */
typedef enum { VD_OP_SELECT = 0, VD_OP_FOLD = 1, VD_OP_SCATTER = 2, VD_OP_PIPELINE = 3, VD_OP_FOLD_SELECT = 4,
               VD_OP_PARTITION = 5, VD_OP_FOLD_SCAN = 6 } vd_op;
/* Scratch bytes needed by `op` over n input slots (out_len for SCATTER;
 * ngroups*naggs for PIPELINE is taken from `plan`, which may be NULL
 * otherwise; a materialising plan also needs its intermediate vector: n
 * bytes for VD_MAT_BREAK, 4 bytes per row + 4 per chunk for VD_MAT_CHUNKS). */
struct vd_pipeline;
vd_status vd_workspace_bytes(int32_t op, int64_t n, const vd_ctrl* ctrl, const struct vd_pipeline* plan,
                             size_t* bytes_host);

/* ---------------------------------------------------------------------- */
/* a1  Load (Table 2 "Load(.keypath)"; MonetDB binary columns,     */
/*     P:L1031-1033)                                                        */
/* ---------------------------------------------------------------------- */
/* Copy `len` host elements of `dtype` into the caller's device buffer
 * `dev_dst` (async on `stream`; `host_src` should be pinned for overlap) and
 * fill the view *out (data = dev_dst).  If compute_minmax != 0 the value
 * bounds are computed on the host from host_src while the copy runs and
 * stored in out->min/max (epsilon values excluded; floats: has_minmax = 0),
 * and VD_COL_NOEPS is set in out->flags if no slot is epsilon. */
vd_status vd_load_column(const void* host_src, int64_t len, int32_t dtype, int32_t scale, void* dev_dst,
                         int32_t compute_minmax, void* stream, vd_column* out);

/* ---------------------------------------------------------------------- */
/* a2+a3  Selection -> position list (FoldSelect P:L524-525, cursor        */
/*        arithmetic P:L101-108, order preserving P:L580-582)               */
/* ---------------------------------------------------------------------- */
/* Evaluate `pred` over rows [0, n) of cols[0..ncols) (all of length >= n)
 * and write the ascending int32 positions of the qualifying rows to
 * out_pos[0 .. count) (capacity n).  *out_count_dev (device int64) receives
 * the count.  With a control vector the positions are aligned to its runs
 * (Fig 9): the suppressed form is the same ascending list plus, if
 * out_run_off != NULL, out_run_off[r] = number of positions in runs before
 * run r, for r in [0, nruns] (capacity nruns+1; for a materialized control
 * nruns <= n).  *out_nruns_dev (nullable) receives the run count.
 * Branch and predicated variants return identical results.
 * n <= 2^31 - 1. */
vd_status vd_select_branch(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, const vd_ctrl* ctrl,
                           int32_t* out_pos, int64_t* out_count_dev, int64_t* out_run_off, int64_t* out_nruns_dev,
                           void* ws, size_t ws_bytes, void* stream);
vd_status vd_select_predicated(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred,
                               const vd_ctrl* ctrl, int32_t* out_pos, int64_t* out_count_dev, int64_t* out_run_off,
                               int64_t* out_nruns_dev, void* ws, size_t ws_bytes, void* stream);

/* ---------------------------------------------------------------------- */
/* a6  Controlled folds (Table 2; Fig 7; §2.2)       */
/* ---------------------------------------------------------------------- */
/* FoldSelect(.out, V1, .fold, .s): positions of slots with s != 0 and not
 * epsilon, aligned to the runs of `ctrl` -- identical output contract to
 * vd_select_*, with the predicate "s != 0". */
vd_status vd_fold_select(const vd_column* s, const vd_ctrl* ctrl, int32_t sel_mode, int32_t* out_pos,
                         int64_t* out_count_dev, int64_t* out_run_off, int64_t* out_nruns_dev, void* ws,
                         size_t ws_bytes, void* stream);

/* FoldSum / FoldCount / FoldMin / FoldMax(.out, V1, .fold, .agg) over
 * vals->len slots: one result per run of `ctrl`, in run order.
 *   out (capacity nruns):
 *     sum  : integer input -> 16-byte signed 128-bit integers (two's
 *            complement, little endian: lo int64 then hi int64), exact;
 *            float input   -> f64, accumulated in f64.
 *     count: int64 (number of non-epsilon slots, reading A6).
 *     min/max: same dtype as the input; epsilon if the run has no
 *            non-epsilon slot (reading A5).
 *   out_counts (nullable, int64, capacity nruns): non-epsilon slots per run.
 *   out_nruns_dev (nullable, device int64): number of runs.
 * Epsilon inputs are skipped; an all-epsilon run sums / counts to 0. */
vd_status vd_fold_sum(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts,
                      int64_t* out_nruns_dev, void* ws, size_t ws_bytes, void* stream);
vd_status vd_fold_count(const vd_column* vals, const vd_ctrl* ctrl, int64_t* out, int64_t* out_nruns_dev, void* ws,
                        size_t ws_bytes, void* stream);
vd_status vd_fold_min(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts,
                      int64_t* out_nruns_dev, void* ws, size_t ws_bytes, void* stream);
vd_status vd_fold_max(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts,
                      int64_t* out_nruns_dev, void* ws, size_t ws_bytes, void* stream);

/* FoldScan(.out, V1, .fold, .s) (Table 2): out[i] = sum of the
 * non-epsilon vals[j] for j <= i in the same run of `ctrl` as i -- the
 * prefix sum restarts at every run (inclusive, reading A27); an epsilon
 * slot stays epsilon in out.  out has vals->len slots: integer input ->
 * int64 (epsilon INT64_MIN; an i64 column needs min/max metadata proving
 * |value| * len < 2^63, else VD_E_OVERFLOW), float input -> f64 (epsilon
 * NaN; the association order is fixed per launch shape).
 * ws: vd_workspace_bytes(VD_OP_FOLD_SCAN, len, ...). */
vd_status vd_fold_scan(const vd_column* vals, const vd_ctrl* ctrl, void* out, void* ws, size_t ws_bytes,
                       void* stream);

/* ---------------------------------------------------------------------- */
/* a4  Gather (Table 2; FK as position P:L452-456)              */
/* ---------------------------------------------------------------------- */
/* out[i] = src[pos[i] - bias] for i in [0, n); a negative (epsilon) or
 * out-of-bounds position gives epsilon (reading A11).  `out` has src's
 * dtype and n slots.  vd_gather_multi resolves the same positions into
 * nsrc columns in one pass (the "Single Loop" of Fig 14);
 * outs[k] receives srcs[k]. */
vd_status vd_gather(const vd_column* src, const int32_t* pos, int64_t n, int64_t bias, void* out, void* stream);
vd_status vd_gather_multi(const vd_column* srcs, int32_t nsrc, const int32_t* pos, int64_t n, int64_t bias,
                          void* const* outs_host, void* stream);

/* Just-in-time layout transformation (Fig 14 "Layout Transform",
 * P:L1156-1193): Zip + materialise the target columns into row-wise storage
 * (P:L1185-1188), then resolve positions with one lookup per row.
 *
 * vd_row_layout (host only, no device work): the row format shared by
 * vd_zip and vd_gather_rows.  Field k (dtypes[k], 1 <= nfields <= 4) sits at
 * offsets[k] bytes, each field aligned to its own size, in declaration
 * order; *stride = the packed size rounded up to a power of two >= 8, so a
 * row never straddles a 32-byte sector.  VD_E_UNSUPPORTED if the packed
 * size exceeds 32 bytes.
 *
 * vd_zip: rows[i] (stride bytes at out_rows + i*stride) = the fields
 * cols[0..ncols)[i]; every column has cols[0].len rows; out_bytes >=
 * len*stride; padding bytes are zero; epsilon values are copied as is.
 *
 * vd_gather_rows: for i in [0, n), p = pos[i] - bias: outs_host[k][i] =
 * field k of row p (dtype dtypes[k]); a negative (epsilon) or out-of-bounds
 * position gives epsilon in every field (reading A11).  outs_host is a host
 * array of nfields device pointers. */
vd_status vd_row_layout(const int32_t* dtypes, int32_t nfields, int32_t* offsets, int32_t* stride);
vd_status vd_zip(const vd_column* cols, int32_t ncols, void* out_rows, int64_t out_bytes, void* stream);
vd_status vd_gather_rows(const void* rows, int64_t nrows, const int32_t* dtypes, int32_t nfields, const int32_t* pos,
                         int64_t n, int64_t bias, void* const* outs_host, void* stream);

/* ---------------------------------------------------------------------- */
/* a5  Scatter / Partition (Table 2; §3.1.3)        */
/* ---------------------------------------------------------------------- */
/* out (out_len slots of src's dtype) is first set to epsilon; then for i in
 * [0, n) src[i] is placed at pos[i]; out-of-bounds / negative positions are
 * dropped; on conflict the later input index wins (reading A12), an epsilon
 * value is placed like any value.  flags & VD_SCATTER_UNIQUE asserts the
 * in-bounds positions are distinct (e.g. a Partition output), which skips
 * the conflict-claim pass. */
#define VD_SCATTER_UNIQUE 1
vd_status vd_scatter(const vd_column* src, const int32_t* pos, int64_t n, void* out, int64_t out_len,
                     int32_t flags, void* ws, size_t ws_bytes, void* stream);

/* Partition(.out, V1, .v, V2, .pv) for the pivot vector Range(pivot_from,
 * npivots, 1): out_pos[i] = (number of rows in earlier buckets) + (rank of
 * row i among its bucket's rows in input order), bucket = clamp(v - from,
 * 0, npivots-1) (stable range partition, reading A13, pinned by Fig 11).
 * Integer columns only; epsilon rows get position -1 and occupy no bucket.
 * npivots <= 4096.  out_bucket_counts (nullable, int64, npivots). */
vd_status vd_partition(const vd_column* v, int64_t pivot_from, int64_t npivots, int32_t* out_pos,
                       int64_t* out_bucket_counts, void* ws, size_t ws_bytes, void* stream);

/* ---------------------------------------------------------------------- */
/* a7+a8+a9  Fused pipeline (fragments, §3.1; Fig 8 Fragment 1, */
/*           P:L831-865; grouped fold Fig 10/11)              */
/* ---------------------------------------------------------------------- */
/* One Voodoo fragment compiled ahead of time: scan the n rows of cols[],
 * optionally resolve FK gathers into dimension columns, evaluate `pred`,
 * compute the group key, and fold the aggregates per group -- with no
 * intermediate vector materialised (the Partition/Scatter of the grouped
 * fold stay virtual, §3.1.3).  The hierarchical fold (Fig 3) happens inside:
 * per-thread -> per-CTA -> grid (the global-barrier Fragment 2, P:L929-931,
 * is the last CTA to finish).
 *
 * Column references in terms / factors / key parts: index c < ncols is
 * cols[c]; c = ncols + g is the g-th gathered column
 * dims[gathers[g].dim_col][cols[gathers[g].fk_col][i] - gathers[g].bias].
 *
 * group key = sum_k (fn_k(col_k) - sub_k) * mult_k, fn: 0 identity,
 * 1 calendar year of a day number; must lie in [0, ngroups) for every
 * qualifying row (else VD_E_DOMAIN is possible when metadata shows it).
 *
 * aggregate value of a row = prod_j (a_j + b_j * col_j) over its factors
 * (factor col = -1: the constant a_j).  SUM/MIN/MAX of that value, COUNT of
 * rows.  Integer columns: exact (int64 per thread, proven by min/max
 * metadata, else VD_E_OVERFLOW; 128-bit above); float columns: f64.
 */
typedef enum { VD_AGG_SUM = 0, VD_AGG_COUNT = 1, VD_AGG_MIN = 2, VD_AGG_MAX = 3 } vd_agg_kind;

#define VD_MAX_AGGS 8
#define VD_MAX_FACTORS 3
#define VD_MAX_GATHERS 4
#define VD_MAX_KEYPARTS 3
#define VD_MAX_GROUPS 4096

typedef struct {
    int32_t col; /* -1 = constant */
    int32_t reserved;
    int64_t a, b; /* factor = a + b * col */
} vd_factor;

typedef struct {
    int32_t kind;     /* vd_agg_kind */
    int32_t nfactors; /* 1..VD_MAX_FACTORS (ignored by COUNT) */
    vd_factor f[VD_MAX_FACTORS];
} vd_agg;

typedef struct {
    int32_t col;
    int32_t fn; /* 0 identity, 1 year(day number since 1970-01-01) */
    int64_t sub, mult;
} vd_keypart;

typedef struct {
    int32_t fk_col;  /* index into cols (int32 column)            */
    int32_t dim_col; /* index into dims                           */
    int64_t bias;    /* position = fk - bias (1 for 1-based keys) */
} vd_gatherspec;

/* Pipeline breakers (Table 2; Fig 8; Fig 15
 * "Vectorized" P:L1202-1230).  The default fuses the whole chain into one
 * kernel with no intermediate vector.  The two materialising plans split it
 * at the operator the paper inserts:
 *   VD_MAT_BREAK  : Break(pred) -- the predicate is evaluated fully
 *       data-parallel and materialised in memory (one byte per row, the
 *       workspace); a second kernel folds the rows whose flag is set.
 *   VD_MAT_CHUNKS : Materialize(positions, Divide(Range, mat_chunk)) -- the
 *       X100-style vectorized plan: per chunk of mat_chunk rows (one run of
 *       the control vector) the ascending positions of the qualifying rows
 *       are written, in order, to the chunk's slice of a position buffer in
 *       memory (the workspace); a second loop resolves them (Gather) and
 *       folds.  mat_chunk: a multiple of 32 in [32, 2^24] (0 = 1024).
 * All plans return identical results (floating-point sums up to the
 * association order). */
typedef enum { VD_MAT_NONE = 0, VD_MAT_BREAK = 1, VD_MAT_CHUNKS = 2 } vd_materialize;

typedef struct vd_pipeline {
    vd_pred pred;
    int32_t sel_mode; /* vd_sel_mode */
    int32_t ngathers;
    vd_gatherspec gathers[VD_MAX_GATHERS];
    int32_t nkeyparts; /* 0 = scalar (one group) */
    int32_t reserved;
    vd_keypart key[VD_MAX_KEYPARTS];
    int64_t ngroups; /* key domain size, 1..VD_MAX_GROUPS */
    int32_t naggs;
    int32_t force_generic; /* 1: bypass the specialised fragments (testing) */
    vd_agg aggs[VD_MAX_AGGS];
    int32_t materialize; /* vd_materialize (0 = fused)                        */
    int32_t reserved2;
    int64_t mat_chunk;   /* VD_MAT_CHUNKS: rows per chunk (run of the control) */
} vd_pipeline;

/* Per-device partial result of a pipeline ("vd_partials"): a device buffer
 * of ngroups * (naggs + 1) slots of 16 bytes; slot [g][a] holds aggregate a
 * of group g (SUM/COUNT of integers: signed 128-bit; SUM of floats: f64 in
 * the low 8 bytes; MIN/MAX: int64 or f64 in the low 8 bytes), slot
 * [g][naggs] the group's row count (128-bit).  A group with row count 0 is
 * empty (dropped by the compaction, Fig 11).  Size: vd_partials_bytes(). */
size_t vd_partials_bytes(const vd_pipeline* plan);

vd_status vd_run_pipeline(const vd_pipeline* plan, const vd_column* cols, int32_t ncols, int64_t n,
                          const vd_column* dims, int32_t ndims, void* out_partials, void* ws, size_t ws_bytes,
                          void* stream);

/* Grouped fold over a LARGE key domain.  The
 * paper's frontend sizes grouping tables from min/max metadata and
 * addresses them by identity hashing: row i belongs to group
 * key[i] - key.min in [0, D), D = key.max - key.min + 1 (<= VD_MAX_DOMAIN).
 * Fig 10/11's chain Partition -> Scatter -> FoldSum/FoldCount/... ->
 * FoldSelect compaction with the Partition/Scatter virtual
 * (§3.1.3): every qualifying row folds into a D-slot table in the
 * workspace (global reductions: the shared-memory tables of
 * vd_run_pipeline spilled), then the non-empty slots are compacted.
 *   cols[0..ncols), n, pred : as vd_run_pipeline (no gathers); epsilon
 *       never qualifies (A9).
 *   key_col : an i32/i64 column WITH min/max metadata (VD_E_DOMAIN
 *       without); an epsilon key has no group.
 *   aggs[0..naggs) : SUM (integer: exact, int64 table slots proven from
 *       the factors' min/max x n, else VD_E_OVERFLOW; float: f64, summed
 *       in an unspecified order), COUNT(*), MIN / MAX (integer only).  An
 *       epsilon factor makes the row's value epsilon: skipped (A5).
 *   outputs (device, capacity D groups; only *out_ngroups are written), in
 *       ascending key order with empty groups dropped (A16):
 *       out_keys[g] int64, out_aggs[g*naggs + a] 16-byte slots as in
 *       vd_partials (integer SUM/COUNT: int128; MIN/MAX: int64 sign-
 *       extended, epsilon INT64_MIN if the group had no non-epsilon value;
 *       float SUM: f64 in the low 8 bytes), out_rows[g] int64 row count,
 *       *out_ngroups_dev int64.
 *   ws : vd_group_fold_ws_bytes(D, naggs) bytes. */
#define VD_MAX_DOMAIN ((int64_t)1 << 31)
vd_status vd_group_fold_ws_bytes(int64_t domain, int32_t naggs, size_t* bytes_host);
vd_status vd_group_fold(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, int32_t key_col,
                        const vd_agg* aggs, int32_t naggs, int64_t* out_keys, void* out_aggs, int64_t* out_rows,
                        int64_t* out_ngroups_dev, void* ws, size_t ws_bytes, void* stream);

/* Grouped fold over SPARSE keys: when the key domain
 * max - min + 1 is far larger than the number of distinct keys (64-bit
 * surrogate or hashed keys), identity hashing over min..max (vd_group_fold,
 * P:L1054-1056) cannot size its table.  Here the open-addressing table is
 * sized from `max_groups`, an upper bound on the distinct qualifying keys
 * (capacity: the power of two >= 2 x max_groups), and keys are placed by a
 * 64-bit mixing hash with linear probing: each CTA folds into a private
 * shared-memory table first and SPILLS to the global table (workspace,
 * global reductions) when a key finds no free slot there; the CTA's table
 * is flushed into the global one at its end.  Then the FoldSelect
 * compaction of the occupied slots (Fig 11).
 *   cols, n, pred, key_col (i32/i64, no metadata needed), aggs : as
 *       vd_group_fold (integer SUMs proven int64-exact from min/max x n, else
 *       VD_E_OVERFLOW; float SUM f64 in an unspecified order; integer MIN /
 *       MAX; epsilon keys have no group; epsilon factors are skipped).
 *   outputs: as vd_group_fold, but the groups come in TABLE order (a hash
 *       table has no key order; vd_group_fold is the ascending-key variant).
 *       *out_ngroups_dev = -1 if more than the capacity's distinct keys
 *       arrived (the table filled up; results are then incomplete).
 *   ws : vd_hash_group_fold_ws_bytes(max_groups, naggs) bytes. */
#define VD_MAX_HASH_GROUPS ((int64_t)1 << 28)
vd_status vd_hash_group_fold_ws_bytes(int64_t max_groups, int32_t naggs, size_t* bytes_host);
vd_status vd_hash_group_fold(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, int32_t key_col,
                             const vd_agg* aggs, int32_t naggs, int64_t max_groups, int64_t* out_keys, void* out_aggs,
                             int64_t* out_rows, int64_t* out_ngroups_dev, void* ws, size_t ws_bytes, void* stream);

/* Cross-GPU merge of COMPACTED groups (the Fig 3 hierarchical fold one
 * level above GPUs, for high-cardinality grouping): nparts
 * blocks of `stride` groups each -- e.g. every rank's vd_group_fold /
 * vd_hash_group_fold output after an all-gather of fixed-size buffers,
 * block r holding counts_dev[r] valid groups and padding after them -- are
 * re-inserted into one hash table: equal keys combine (integer SUM / COUNT
 * exactly in 128 bits, float SUM in f64 in an unspecified order, MIN / MAX
 * over the non-epsilon values, row counts added) and the result is
 * compacted in table order.
 *   keys / aggs / rows : device, [nparts * stride] groups in the
 *       vd_group_fold output layout (16-byte aggregate slots, naggs each).
 *   counts_dev : device int64 [nparts], valid groups per block (<= stride).
 *   kinds_host[a] / isf_host[a] : aggregate kind and whether it is f64.
 *   max_groups : bound on the distinct keys; *out_ngroups_dev = -1 if exceeded.
 *   ws : vd_merge_groups_ws_bytes(max_groups, naggs). */
vd_status vd_merge_groups_ws_bytes(int64_t max_groups, int32_t naggs, size_t* bytes_host);
vd_status vd_merge_groups(const int64_t* keys, const void* aggs, const int64_t* rows, const int64_t* counts_dev,
                          int32_t nparts, int64_t stride, const int32_t* kinds_host, const int32_t* isf_host,
                          int32_t naggs, int64_t max_groups, int64_t* out_keys, void* out_aggs, int64_t* out_rows,
                          int64_t* out_ngroups_dev, void* ws, size_t ws_bytes, void* stream);

/* Compacted result of a pipeline: the FoldSelect compaction of Fig 11
 * applied to the merged partials -- the non-empty groups
 * (row count > 0), in ascending key order (reading A16), empty groups
 * dropped.  Every pointer is caller-owned; HOST memory for
 * vd_merge_partials, DEVICE memory for vd_merge_partials_device.
 *   keys    : int64 [capacity], the group key (index in [0, plan->ngroups))
 *   aggs    : [capacity][plan->naggs] 16-byte slots, encoded as in
 *             vd_partials (integer SUM/COUNT int128; float SUM f64 in the
 *             low 8 bytes; MIN/MAX int64 / f64 in the low 8 bytes)
 *   rows    : int64 [capacity], the group's row count (> 0)
 *   ngroups : int64 scalar, the number of groups written
 * capacity >= plan->ngroups (else VD_E_SHAPE). */
typedef struct {
    int64_t capacity;
    int64_t* keys;
    void* aggs;
    int64_t* rows;
    int64_t* ngroups;
} vd_result;

/* Merge of per-device partials, the cross-GPU step of the hierarchical fold
 * (Fig 3 one level up), followed by the Fig 11 compaction:
 * parts_host[r] points to rank r's vd_partials copied to the host; they are
 * combined in rank order (SUM/COUNT exact in 128 bits or f64; MIN/MAX over
 * the ranks where the group is non-empty) and the non-empty groups are
 * written to *out (host buffers).  cols / dims are the column views the plan
 * ran with: only their dtypes are read (they decide which aggregates are
 * f64); they may be NULL when nparts == 1 (a single partial is compacted,
 * nothing is added). */
vd_status vd_merge_partials(const vd_pipeline* plan, const vd_column* cols, int32_t ncols, const vd_column* dims,
                            int32_t ndims, const void* const* parts_host, int32_t nparts, const vd_result* out);

/* The same merge + compaction on the device, in one kernel (one CTA) on
 * `stream`: parts_dev holds nparts vd_partials buffers back to back (e.g.
 * the output of an all-gather of every rank's partials, rank order), and
 * *out's buffers are device memory.  For nparts == 1 it is the device-side
 * finalisation of a single GPU's pipeline.  Stream-ordered: nothing is
 * synchronised; *out->ngroups is valid once the stream reaches the kernel's
 * end.  cols/dims as vd_merge_partials. */
vd_status vd_merge_partials_device(const vd_pipeline* plan, const vd_column* cols, int32_t ncols,
                                   const vd_column* dims, int32_t ndims, const void* parts_dev, int32_t nparts,
                                   const vd_result* out, void* stream);

/* Rows whose group key fell outside [0, ngroups) in the last generic-path
 * vd_run_pipeline on `ws` (device int64 at ws + 128; read after the stream
 * synchronises).  They are dropped, not folded. */
#define VD_WS_DOMAIN_ERRORS_OFFSET 128

/* sizeof() of the ABI structs, for binding self-checks: out[0..8] =
 * vd_column, vd_ctrl, vd_term, vd_conj, vd_pred, vd_agg, vd_keypart,
 * vd_pipeline, vd_result.  Returns the number written (<= n). */
int32_t vd_abi_struct_sizes(size_t* out, int32_t n);

/* Name of the fragment the last vd_run_pipeline on this thread ran:
 * "q1_tma", "q1_ldg", "scalar_tma", "scalar_ldg", "selsum_tma", "gather_fold",
 * "generic", "break" or "mat_chunks" (the last two: materialising plans);
 * after a single-term selection (vd_select_*): "sel_stream" (striped
 * warp-specialised kernel), "sel_coop" (single grid barrier), "sel_bitmap"
 * (bitmap + scan launches) or "sel_lookback". */
const char* vd_last_fragment(void);

/* Number of kernel launches the last successful call on this thread
 * enqueued (for launch accounting in benchmarks). */
int32_t vd_last_launch_count(void);

#ifdef __cplusplus
}
#endif

#endif /* VD_H */
