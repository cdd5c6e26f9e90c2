// vd_internal.h -- host-side declarations shared by the ABI layer
// (vd_api.cpp) and the kernel launchers (*.cu).  Product code.
#pragma once

#include <cuda_runtime.h>
#include <stddef.h>
#include <stdint.h>

#include <string>

#include "vd.h"

namespace vd {

// Thread-local error detail + launch accounting (vd_api.cpp).
void set_error(const std::string& msg);
void count_launches(int k);
void reset_launches();
void set_fragment(const char* name);

size_t dtype_size(int32_t dt);

// ---- control-vector run classes (include/vd.h vd_ctrl) -------------------
enum RunClass { RUNS_ONE = 0, RUNS_FIXED = 1, RUNS_GENERAL = 2 };

struct CtrlInfo {
    RunClass cls;
    int64_t R;       // RUNS_FIXED: run length
    int64_t nruns;   // host-known count (-1 for materialized)
    // virtual parameters (RUNS_GENERAL virtual)
    int64_t from, num, den, cap;
    const void* mat;  // materialized values or NULL
    int32_t mat_dtype;
};
vd_status classify_ctrl(const vd_ctrl* c, int64_t n, CtrlInfo* out);

// ---- device-side predicate descriptor ------------------------------------
struct DevTerm {
    int32_t col, cmp;
    int64_t iv;
    double fv;
};
struct DevPred {
    int32_t nconj;
    int32_t nterms[VD_MAX_CONJ];
    DevTerm t[VD_MAX_CONJ][VD_MAX_TERMS];
};
#define VD_MAX_DEVCOLS 24
struct DevCols {
    const void* p[VD_MAX_DEVCOLS];
    int32_t dt[VD_MAX_DEVCOLS];
    int32_t ncols;
};
void make_devpred(const vd_pred* p, DevPred* d);

// ---- launchers (implemented in the .cu files); return cudaError_t ---------
// k_scatter.cu: exclusive scan of int32 counts into int64 offsets (look-back)
size_t scan_ws_bytes(int64_t m);
cudaError_t launch_scan_i32(const int32_t* in, int64_t m, int64_t* out, void* ws, cudaStream_t s, int* nl);

// k_select.cu
size_t select_ws_bytes(int64_t n);
cudaError_t launch_select(int mode, const DevCols& cols, const DevPred& pred, int64_t n, int32_t* out_pos,
                          int64_t* out_count, void* ws, size_t ws_bytes, cudaStream_t s, int* nlaunch);
// select of run heads of a GENERAL control (positions i where v[i] != v[i-1], plus 0)
cudaError_t launch_select_heads(const CtrlInfo& ci, int64_t n, int32_t* out_pos, int64_t* out_count, void* ws,
                                size_t ws_bytes, cudaStream_t s, int* nlaunch);
// run offsets by binary search of run starts in the selected positions
cudaError_t launch_run_offsets(const CtrlInfo& ci, int64_t n, const int32_t* pos, const int64_t* count,
                               const int32_t* run_starts, const int64_t* nruns_dev, int64_t* out_run_off,
                               int64_t* out_nruns, cudaStream_t s, int* nlaunch);

// k_fold.cu
enum FoldOp { FOLD_SUM = 0, FOLD_COUNT = 1, FOLD_MIN = 2, FOLD_MAX = 3 };
size_t fold_ws_bytes(int64_t n);
cudaError_t launch_fold(FoldOp op, const vd_column& vals, const CtrlInfo& ci, void* out, int64_t* out_counts,
                        int64_t* out_nruns, void* ws, size_t ws_bytes, cudaStream_t s, int* nlaunch);

size_t fold_scan_ws_bytes(int64_t n);
cudaError_t launch_fold_scan(const vd_column& vals, const CtrlInfo& ci, void* out, void* ws, cudaStream_t s, int* nl);

// k_gather.cu
cudaError_t launch_gather(const vd_column* srcs, int nsrc, const int32_t* pos, int64_t n, int64_t bias,
                          void* const* outs, cudaStream_t s, int* nlaunch);
bool row_layout(const int32_t* dtypes, int nfields, int32_t* offsets, int32_t* stride);
cudaError_t launch_zip(const vd_column* cols, int ncols, void* out_rows, cudaStream_t s, int* nl);
cudaError_t launch_gather_rows(const void* rows, int64_t nrows, const int32_t* dtypes, int nfields,
                               const int32_t* pos, int64_t n, int64_t bias, void* const* outs, cudaStream_t s, int* nl);
// k_scatter.cu
size_t scatter_ws_bytes(int64_t out_len);
cudaError_t launch_scatter(const vd_column& src, const int32_t* pos, int64_t n, void* out, int64_t out_len,
                           bool unique, void* ws, cudaStream_t s, int* nlaunch);
size_t partition_ws_bytes(int64_t n, int64_t npiv);
cudaError_t launch_partition(const vd_column& v, int64_t from, int64_t npiv, int32_t* out_pos,
                             int64_t* out_counts, void* ws, cudaStream_t s, int* nlaunch);

// k_pipeline.cu
size_t pipeline_ws_bytes(const vd_pipeline* plan, int64_t n);
vd_status run_pipeline(const vd_pipeline* plan, const vd_column* cols, int32_t ncols, int64_t n,
                       const vd_column* dims, int32_t ndims, void* out, void* ws, size_t ws_bytes, cudaStream_t s,
                       int* nlaunch);

// k_group.cu (NEXT-4)
size_t group_ws_bytes(int64_t D, int naggs);
cudaError_t launch_group_fold(const DevCols& cols, const DevPred& pred, int64_t n, int key_col, int64_t kmin,
                              int64_t D, const vd_agg* aggs, const int32_t* isf, int naggs, int64_t* out_keys,
                              void* out_aggs, int64_t* out_rows, int64_t* out_ng, void* ws, cudaStream_t s,
                              int* nl);

// k_merge.cu: rank-order merge of nparts device partials + Fig 11 compaction
cudaError_t launch_merge_partials(const vd_pipeline* plan, const int32_t* isf, const void* parts, int nparts,
                                  const vd_result& out, cudaStream_t s, int* nl);

// k_hash.cu (NEXT-4, sparse keys)
size_t hash_group_ws_bytes(int64_t max_groups, int naggs, bool wide);
cudaError_t launch_hash_group_fold(const DevCols& cols, const DevPred& pred, int64_t n, int key_col,
                                   const vd_agg* aggs, const int32_t* isf, int naggs, int64_t max_groups,
                                   int64_t* out_keys, void* out_aggs, int64_t* out_rows, int64_t* out_ng, void* ws,
                                   cudaStream_t s, int* nl);
cudaError_t launch_merge_groups(const int64_t* keys, const void* aggs, const int64_t* rows, const int64_t* counts,
                                int nparts, int64_t stride, const int32_t* kinds, const int32_t* isf, int naggs,
                                int64_t max_groups, int64_t* out_keys, void* out_aggs, int64_t* out_rows,
                                int64_t* out_ng, void* ws, cudaStream_t s, int* nl);

int num_sms();

}  // namespace vd
