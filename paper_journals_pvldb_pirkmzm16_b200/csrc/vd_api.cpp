// vd_api.cpp -- the C ABI of libvd.so (include/vd.h): argument / metadata
// validation, workspace sizing, control-vector classification and dispatch
// to the kernel launchers.  No computation on the host except vd_load_column's
// optional min/max scan and vd_merge_partials (the cross-device merge).
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <cstring>
#include <string>

#include "vd.h"
#include "vd_internal.h"

namespace vd {

static thread_local std::string t_err;
static thread_local int t_launches = 0;
static thread_local const char* t_fragment = "";

void set_error(const std::string& msg) { t_err = msg; }
void count_launches(int k) { t_launches += k; }
void reset_launches() { t_launches = 0; }
void set_fragment(const char* name) { t_fragment = name; }

size_t dtype_size(int32_t dt) {
    switch (dt) {
    case VD_U8: return 1;
    case VD_I32: return 4;
    case VD_I64: return 8;
    case VD_F32: return 4;
    case VD_F64: return 8;
    default: return 0;
    }
}

int num_sms() {
    static thread_local int dev_cached = -1, sms_cached = 148;
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess) return sms_cached;
    if (dev != dev_cached) {
        int s = 0;
        if (cudaDeviceGetAttribute(&s, cudaDevAttrMultiProcessorCount, dev) == cudaSuccess && s > 0) sms_cached = s;
        dev_cached = dev;
    }
    return sms_cached;
}

void make_devpred(const vd_pred* p, DevPred* d) {
    std::memset(d, 0, sizeof(*d));
    if (!p) return;
    d->nconj = p->nconj;
    for (int c = 0; c < p->nconj; ++c) {
        d->nterms[c] = p->conj[c].nterms;
        for (int k = 0; k < p->conj[c].nterms; ++k) {
            d->t[c][k].col = p->conj[c].terms[k].col;
            d->t[c][k].cmp = p->conj[c].terms[k].cmp;
            d->t[c][k].iv = p->conj[c].terms[k].ival;
            d->t[c][k].fv = p->conj[c].terms[k].fval;
        }
    }
}

vd_status classify_ctrl(const vd_ctrl* c, int64_t n, CtrlInfo* o) {
    std::memset(o, 0, sizeof(*o));
    o->den = 1;
    if (!c) {
        o->cls = RUNS_ONE;
        o->nruns = n > 0 ? 1 : 0;
        return VD_OK;
    }
    if (c->materialized) {
        if (c->mat_dtype != VD_I32 && c->mat_dtype != VD_I64) {
            set_error("materialized control vector must be int32 or int64");
            return VD_E_DTYPE;
        }
        o->cls = RUNS_GENERAL;
        o->nruns = -1;
        o->mat = c->materialized;
        o->mat_dtype = c->mat_dtype;
        return VD_OK;
    }
    if (c->step_den <= 0 || c->step_num < 0 || c->cap < 0) {
        set_error("control vector needs step_num >= 0, step_den > 0, cap >= 0");
        return VD_E_CTRL;
    }
    o->from = c->from;
    o->num = c->step_num;
    o->den = c->step_den;
    o->cap = c->cap;
    if (c->step_num == 0 || c->cap == 1) {  // constant values: one run
        o->cls = RUNS_ONE;
        o->nruns = n > 0 ? 1 : 0;
        return VD_OK;
    }
    if (c->step_num == 1) {  // Divide(Range, R): runs of R
        int64_t R = c->step_den;
        if (R >= n) { o->cls = RUNS_ONE; o->nruns = n > 0 ? 1 : 0; return VD_OK; }
        o->cls = RUNS_FIXED;
        o->R = R;
        o->nruns = (n + R - 1) / R;
        return VD_OK;
    }
    if (c->step_num % c->step_den == 0) {  // integer step k: runs of 1 unless k = 0 mod cap
        int64_t k = c->step_num / c->step_den;
        if (c->cap != 0 && k % c->cap == 0) { o->cls = RUNS_ONE; o->nruns = n > 0 ? 1 : 0; return VD_OK; }
        if (n <= 1) { o->cls = RUNS_ONE; o->nruns = n; return VD_OK; }
        o->cls = RUNS_FIXED;
        o->R = 1;
        o->nruns = n;
        return VD_OK;
    }
    o->cls = RUNS_GENERAL;  // irregular virtual runs: run starts computed on the device
    o->nruns = -1;
    return VD_OK;
}

static bool valid_dtype(int32_t dt) { return dt >= VD_U8 && dt <= VD_F64; }
static bool is_int(int32_t dt) { return dt == VD_U8 || dt == VD_I32 || dt == VD_I64; }

static vd_status check_col(const vd_column* c, int64_t need, const char* what) {
    if (!c) { set_error(std::string(what) + ": NULL column"); return VD_E_NULL; }
    if (!valid_dtype(c->dtype)) { set_error(std::string(what) + ": bad dtype"); return VD_E_DTYPE; }
    if (c->len < need) { set_error(std::string(what) + ": column shorter than n"); return VD_E_SHAPE; }
    if (need > 0 && !c->data) { set_error(std::string(what) + ": NULL data"); return VD_E_NULL; }
    return VD_OK;
}

static vd_status check_ws(void* ws, size_t have, size_t need) {
    if (need == 0) return VD_OK;
    if (!ws || have < need) {
        set_error("workspace smaller than vd_workspace_bytes (" + std::to_string(need) + " bytes)");
        return VD_E_WORKSPACE;
    }
    return VD_OK;
}

static vd_status cuda_status(cudaError_t e) {
    if (e == cudaSuccess) return VD_OK;
    set_error(std::string("CUDA: ") + cudaGetErrorString(e));
    return VD_E_CUDA;
}

static vd_status check_device() {
    int n = 0;
    cudaError_t e = cudaGetDeviceCount(&n);
    if (e != cudaSuccess || n == 0) {
        set_error("no CUDA device: libvd has no CPU fallback");
        return VD_E_CUDA;
    }
    return VD_OK;
}

static vd_status check_pred(const vd_pred* p, const int32_t* dts, int ncols) {
    if (!p) return VD_OK;
    if (p->nconj < 0 || p->nconj > VD_MAX_CONJ) { set_error("pred.nconj out of range"); return VD_E_ARG; }
    for (int c = 0; c < p->nconj; ++c) {
        if (p->conj[c].nterms < 0 || p->conj[c].nterms > VD_MAX_TERMS) { set_error("nterms out of range"); return VD_E_ARG; }
        for (int k = 0; k < p->conj[c].nterms; ++k) {
            const vd_term& t = p->conj[c].terms[k];
            if (t.col < 0 || t.col >= ncols) { set_error("predicate term column out of range"); return VD_E_ARG; }
            if (t.cmp < VD_CMP_GT || t.cmp > VD_CMP_IN) { set_error("bad comparison"); return VD_E_ARG; }
            if (t.cmp == VD_CMP_IN && !is_int(dts[t.col])) { set_error("IN needs an integer column"); return VD_E_DTYPE; }
        }
    }
    return VD_OK;
}

static size_t align256(size_t b) { return (b + 255) & ~(size_t)255; }

static size_t select_total_ws(int64_t n, const CtrlInfo& ci) {
    size_t b = select_ws_bytes(n);
    if (ci.cls == RUNS_GENERAL) b += align256((size_t)n * 4) + 256;
    return b;
}

static size_t fold_total_ws(int64_t n, const CtrlInfo& ci) {
    size_t b = fold_ws_bytes(n);
    if (ci.cls == RUNS_GENERAL) b += select_ws_bytes(n) + align256((size_t)n * 4) + 256;
    return b;
}

// Selection with an optional control vector (shared by vd_select_* and
// vd_fold_select).
static vd_status do_select(int mode, const DevCols& dc, const DevPred& dp, int64_t n, const vd_ctrl* ctrl,
                           int32_t* out_pos, int64_t* out_count, int64_t* out_run_off, int64_t* out_nruns, void* ws,
                           size_t ws_bytes, cudaStream_t s) {
    CtrlInfo ci;
    vd_status st = classify_ctrl(ctrl, n, &ci);
    if (st != VD_OK) return st;
    st = check_ws(ws, ws_bytes, select_total_ws(n, ci));
    if (st != VD_OK) return st;
    int nl = 0;
    const int32_t* starts = nullptr;
    const int64_t* nstarts = nullptr;
    size_t sel = select_ws_bytes(n);
    if (ci.cls == RUNS_GENERAL && (out_run_off || out_nruns)) {
        int32_t* st_pos = (int32_t*)((char*)ws + sel);
        int64_t* ns = (int64_t*)((char*)ws + sel + align256((size_t)n * 4));
        st = cuda_status(launch_select_heads(ci, n, st_pos, ns, ws, sel, s, &nl));
        if (st != VD_OK) return st;
        starts = st_pos;
        nstarts = ns;
    }
    st = cuda_status(launch_select(mode, dc, dp, n, out_pos, out_count, ws, sel, s, &nl));
    if (st != VD_OK) return st;
    if (out_run_off || out_nruns) {
        st = cuda_status(launch_run_offsets(ci, n, out_pos, out_count, starts, nstarts, out_run_off, out_nruns, s, &nl));
        if (st != VD_OK) return st;
    }
    count_launches(nl);
    return VD_OK;
}

static vd_status select_entry(int mode, const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred,
                              const vd_ctrl* ctrl, int32_t* out_pos, int64_t* out_count, int64_t* out_run_off,
                              int64_t* out_nruns, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    if (n < 0 || n > INT32_MAX) { set_error("n must be in [0, 2^31-1]"); return VD_E_SHAPE; }
    if (ncols < 0 || ncols > VD_MAX_DEVCOLS || (ncols > 0 && !cols)) { set_error("bad column list"); return VD_E_ARG; }
    if (!out_count || (n > 0 && !out_pos)) { set_error("out_pos / out_count required"); return VD_E_NULL; }
    DevCols dc;
    std::memset(&dc, 0, sizeof(dc));
    dc.ncols = ncols;
    for (int c = 0; c < ncols; ++c) {
        vd_status st = check_col(&cols[c], n, "select");
        if (st != VD_OK) return st;
        dc.p[c] = cols[c].data;
        dc.dt[c] = cols[c].dtype;
    }
    vd_status st = check_pred(pred, dc.dt, ncols);
    if (st != VD_OK) return st;
    if (ctrl && ctrl->materialized == nullptr && ctrl->step_den <= 0) { set_error("bad ctrl"); return VD_E_CTRL; }
    if ((st = check_device()) != VD_OK) return st;
    DevPred dp;
    make_devpred(pred, &dp);
    return do_select(mode, dc, dp, n, ctrl, out_pos, out_count, out_run_off, out_nruns, ws, ws_bytes,
                     (cudaStream_t)stream);
}

static vd_status fold_entry(FoldOp op, const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts,
                            int64_t* out_nruns, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    vd_status st = check_col(vals, 0, "fold");
    if (st != VD_OK) return st;
    if (vals->len > 0 && !out) { set_error("fold: NULL out"); return VD_E_NULL; }
    if (vals->len > INT32_MAX) { set_error("fold: n must be < 2^31"); return VD_E_SHAPE; }
    CtrlInfo ci;
    if ((st = classify_ctrl(ctrl, vals->len, &ci)) != VD_OK) return st;
    st = check_ws(ws, ws_bytes, fold_total_ws(vals->len, ci));
    if (st != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_fold(op, *vals, ci, out, out_counts, out_nruns, ws, ws_bytes, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

}  // namespace vd

using namespace vd;

extern "C" {

const char* vd_status_str(vd_status s) {
    switch (s) {
    case VD_OK: return "VD_OK";
    case VD_E_NULL: return "VD_E_NULL";
    case VD_E_DTYPE: return "VD_E_DTYPE";
    case VD_E_SHAPE: return "VD_E_SHAPE";
    case VD_E_CTRL: return "VD_E_CTRL";
    case VD_E_DOMAIN: return "VD_E_DOMAIN";
    case VD_E_OVERFLOW: return "VD_E_OVERFLOW";
    case VD_E_WORKSPACE: return "VD_E_WORKSPACE";
    case VD_E_CUDA: return "VD_E_CUDA";
    case VD_E_UNSUPPORTED: return "VD_E_UNSUPPORTED";
    case VD_E_ARG: return "VD_E_ARG";
    default: return "VD_E_?";
    }
}

const char* vd_last_error(void) { return t_err.c_str(); }
const char* vd_version(void) { return "voodoo-b200 0.1 (sm_100a)"; }
int32_t vd_last_launch_count(void) { return t_launches; }
const char* vd_last_fragment(void) { return t_fragment; }

int32_t vd_abi_struct_sizes(size_t* out, int32_t n) {
    const size_t v[9] = {sizeof(vd_column), sizeof(vd_ctrl),     sizeof(vd_term),
                         sizeof(vd_conj),   sizeof(vd_pred),     sizeof(vd_agg),
                         sizeof(vd_keypart), sizeof(vd_pipeline), sizeof(vd_result)};
    int32_t k = 0;
    for (; k < n && k < 9; ++k) out[k] = v[k];
    return k;
}

vd_status vd_ctrl_runs(const vd_ctrl* ctrl, int64_t n, int64_t* nruns_host) {
    if (!nruns_host) return VD_E_NULL;
    CtrlInfo ci;
    vd_status st = classify_ctrl(ctrl, n, &ci);
    if (st != VD_OK) return st;
    if (ci.cls == RUNS_GENERAL) {
        set_error("run count of this control vector is data dependent");
        return VD_E_UNSUPPORTED;
    }
    *nruns_host = ci.nruns;
    return VD_OK;
}

vd_status vd_workspace_bytes(int32_t op, int64_t n, const vd_ctrl* ctrl, const struct vd_pipeline* plan,
                             size_t* bytes) {
    if (!bytes) return VD_E_NULL;
    if (n < 0) return VD_E_SHAPE;
    CtrlInfo ci;
    vd_status st = classify_ctrl(ctrl, n, &ci);
    if (st != VD_OK) return st;
    switch (op) {
    case VD_OP_SELECT:
    case VD_OP_FOLD_SELECT: *bytes = select_total_ws(n, ci); return VD_OK;
    case VD_OP_FOLD: *bytes = fold_total_ws(n, ci); return VD_OK;
    case VD_OP_SCATTER: *bytes = scatter_ws_bytes(n); return VD_OK;
    case VD_OP_PARTITION: *bytes = partition_ws_bytes(n, 1024); return VD_OK;
    case VD_OP_FOLD_SCAN: *bytes = fold_scan_ws_bytes(n); return VD_OK;
    case VD_OP_PIPELINE:
        if (!plan) return VD_E_NULL;
        if (plan->ngroups < 1 || plan->ngroups > VD_MAX_GROUPS || plan->naggs < 0 || plan->naggs > VD_MAX_AGGS)
            return VD_E_ARG;
        if (plan->materialize < VD_MAT_NONE || plan->materialize > VD_MAT_CHUNKS) return VD_E_ARG;
        *bytes = pipeline_ws_bytes(plan, n);
        return VD_OK;
    default: set_error("unknown op"); return VD_E_ARG;
    }
}

vd_status vd_load_column(const void* host_src, int64_t len, int32_t dtype, int32_t scale, void* dev_dst,
                         int32_t compute_minmax, void* stream, vd_column* out) {
    reset_launches();
    if (!out) return VD_E_NULL;
    if (!valid_dtype(dtype)) { set_error("bad dtype"); return VD_E_DTYPE; }
    if (len < 0) return VD_E_SHAPE;
    if (len > 0 && (!host_src || !dev_dst)) { set_error("NULL buffer"); return VD_E_NULL; }
    vd_status st = check_device();
    if (st != VD_OK) return st;
    size_t bytes = (size_t)len * dtype_size(dtype);
    if (bytes) {
        st = cuda_status(cudaMemcpyAsync(dev_dst, host_src, bytes, cudaMemcpyHostToDevice, (cudaStream_t)stream));
        if (st != VD_OK) return st;
    }
    std::memset(out, 0, sizeof(*out));
    out->data = dev_dst;
    out->len = len;
    out->dtype = dtype;
    out->scale = scale;
    if (compute_minmax && is_int(dtype) && len > 0) {
        // host scan of the source while the copy is in flight (MonetDB keeps
        // such min/max metadata per column)
        int64_t mn = INT64_MAX, mx = INT64_MIN;
        bool any = false;
        int64_t neps = 0;
        for (int64_t i = 0; i < len; ++i) {
            int64_t v;
            if (dtype == VD_U8) { uint8_t x = ((const uint8_t*)host_src)[i]; if (x == VD_EPS_U8) { ++neps; continue; } v = x; }
            else if (dtype == VD_I32) { int32_t x = ((const int32_t*)host_src)[i]; if (x == VD_EPS_I32) { ++neps; continue; } v = x; }
            else { int64_t x = ((const int64_t*)host_src)[i]; if (x == VD_EPS_I64) { ++neps; continue; } v = x; }
            mn = std::min(mn, v);
            mx = std::max(mx, v);
            any = true;
        }
        if (any) { out->min = mn; out->max = mx; out->has_minmax = 1; }
        if (neps == 0) out->flags |= VD_COL_NOEPS;
    }
    return VD_OK;
}

vd_status vd_select_branch(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, const vd_ctrl* ctrl,
                           int32_t* out_pos, int64_t* out_count, int64_t* out_run_off, int64_t* out_nruns, void* ws,
                           size_t ws_bytes, void* stream) {
    return select_entry(VD_SEL_BRANCH, cols, ncols, n, pred, ctrl, out_pos, out_count, out_run_off, out_nruns, ws,
                        ws_bytes, stream);
}

vd_status vd_select_predicated(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred,
                               const vd_ctrl* ctrl, int32_t* out_pos, int64_t* out_count, int64_t* out_run_off,
                               int64_t* out_nruns, void* ws, size_t ws_bytes, void* stream) {
    return select_entry(VD_SEL_PREDICATED, cols, ncols, n, pred, ctrl, out_pos, out_count, out_run_off, out_nruns,
                        ws, ws_bytes, stream);
}

vd_status vd_fold_select(const vd_column* s, const vd_ctrl* ctrl, int32_t sel_mode, int32_t* out_pos,
                         int64_t* out_count, int64_t* out_run_off, int64_t* out_nruns, void* ws, size_t ws_bytes,
                         void* stream) {
    if (!s) return VD_E_NULL;
    // FoldSelect(.fold, .s): positions with s != 0 (epsilon never selected)
    vd_pred p;
    std::memset(&p, 0, sizeof(p));
    p.nconj = 1;
    p.conj[0].nterms = 1;
    p.conj[0].terms[0].col = 0;
    p.conj[0].terms[0].cmp = VD_CMP_NE;
    p.conj[0].terms[0].ival = 0;
    p.conj[0].terms[0].fval = 0.0;
    return select_entry(sel_mode == VD_SEL_PREDICATED ? VD_SEL_PREDICATED : VD_SEL_BRANCH, s, 1, s->len, &p, ctrl,
                        out_pos, out_count, out_run_off, out_nruns, ws, ws_bytes, stream);
}

vd_status vd_fold_sum(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts, int64_t* out_nruns,
                      void* ws, size_t ws_bytes, void* stream) {
    return fold_entry(FOLD_SUM, vals, ctrl, out, out_counts, out_nruns, ws, ws_bytes, stream);
}
vd_status vd_fold_count(const vd_column* vals, const vd_ctrl* ctrl, int64_t* out, int64_t* out_nruns, void* ws,
                        size_t ws_bytes, void* stream) {
    return fold_entry(FOLD_COUNT, vals, ctrl, out, nullptr, out_nruns, ws, ws_bytes, stream);
}
vd_status vd_fold_min(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts, int64_t* out_nruns,
                      void* ws, size_t ws_bytes, void* stream) {
    return fold_entry(FOLD_MIN, vals, ctrl, out, out_counts, out_nruns, ws, ws_bytes, stream);
}
vd_status vd_fold_max(const vd_column* vals, const vd_ctrl* ctrl, void* out, int64_t* out_counts, int64_t* out_nruns,
                      void* ws, size_t ws_bytes, void* stream) {
    return fold_entry(FOLD_MAX, vals, ctrl, out, out_counts, out_nruns, ws, ws_bytes, stream);
}

vd_status vd_fold_scan(const vd_column* vals, const vd_ctrl* ctrl, void* out, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    vd_status st = check_col(vals, 0, "fold_scan");
    if (st != VD_OK) return st;
    if (vals->len > 0 && (!out || !vals->data)) { set_error("fold_scan: NULL out / data"); return VD_E_NULL; }
    if (vals->len > INT32_MAX) { set_error("fold_scan: n must be < 2^31"); return VD_E_SHAPE; }
    if (vals->dtype == VD_I64) {
        // int64 running sums: |value| * n must stay below 2^63 (metadata)
        const double b = std::max(std::fabs((double)vals->min), std::fabs((double)vals->max)) * (double)vals->len;
        if (!vals->has_minmax || b >= 9.2e18) {
            set_error("fold_scan: min/max metadata cannot prove int64 running sums exact");
            return VD_E_OVERFLOW;
        }
    }
    CtrlInfo ci;
    if ((st = classify_ctrl(ctrl, vals->len, &ci)) != VD_OK) return st;
    if ((st = check_ws(ws, ws_bytes, fold_scan_ws_bytes(vals->len))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_fold_scan(*vals, ci, out, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_gather_multi(const vd_column* srcs, int32_t nsrc, const int32_t* pos, int64_t n, int64_t bias,
                          void* const* outs, void* stream) {
    reset_launches();
    if (nsrc < 1 || nsrc > VD_MAX_GATHERS || !srcs || !outs) { set_error("gather: 1..4 sources"); return VD_E_ARG; }
    if (n < 0) return VD_E_SHAPE;
    if (n > 0 && !pos) { set_error("gather: NULL pos"); return VD_E_NULL; }
    for (int k = 0; k < nsrc; ++k) {
        vd_status st = check_col(&srcs[k], 0, "gather");
        if (st != VD_OK) return st;
        if (srcs[k].len > 0 && !srcs[k].data) { set_error("gather: NULL source"); return VD_E_NULL; }
        if (n > 0 && !outs[k]) { set_error("gather: NULL out"); return VD_E_NULL; }
    }
    vd_status st = check_device();
    if (st != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_gather(srcs, nsrc, pos, n, bias, outs, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_gather(const vd_column* src, const int32_t* pos, int64_t n, int64_t bias, void* out, void* stream) {
    void* outs[1] = {out};
    return vd_gather_multi(src, 1, pos, n, bias, outs, stream);
}

vd_status vd_row_layout(const int32_t* dtypes, int32_t nfields, int32_t* offsets, int32_t* stride) {
    if (!dtypes || !offsets || !stride) return VD_E_NULL;
    if (nfields < 1 || nfields > VD_MAX_GATHERS) { set_error("row layout: 1..4 fields"); return VD_E_ARG; }
    for (int k = 0; k < nfields; ++k)
        if (!valid_dtype(dtypes[k])) { set_error("row layout: bad dtype"); return VD_E_DTYPE; }
    if (!row_layout(dtypes, nfields, offsets, stride)) {
        set_error("row layout: a row must fit 32 bytes");
        return VD_E_UNSUPPORTED;
    }
    return VD_OK;
}

vd_status vd_zip(const vd_column* cols, int32_t ncols, void* out_rows, int64_t out_bytes, void* stream) {
    reset_launches();
    if (!cols) return VD_E_NULL;
    if (ncols < 1 || ncols > VD_MAX_GATHERS) { set_error("zip: 1..4 columns"); return VD_E_ARG; }
    int32_t dts[VD_MAX_GATHERS], offs[VD_MAX_GATHERS], stride;
    for (int k = 0; k < ncols; ++k) {
        vd_status st = check_col(&cols[k], cols[0].len, "zip");
        if (st != VD_OK) return st;
        dts[k] = cols[k].dtype;
    }
    vd_status st = vd_row_layout(dts, ncols, offs, &stride);
    if (st != VD_OK) return st;
    if (out_bytes < cols[0].len * (int64_t)stride) { set_error("zip: output smaller than len * stride"); return VD_E_SHAPE; }
    if (cols[0].len > 0 && !out_rows) return VD_E_NULL;
    if (((uintptr_t)out_rows % 16) != 0) { set_error("zip: rows must be 16-byte aligned"); return VD_E_ARG; }
    st = check_device();
    if (st != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_zip(cols, ncols, out_rows, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_gather_rows(const void* rows, int64_t nrows, const int32_t* dtypes, int32_t nfields, const int32_t* pos,
                         int64_t n, int64_t bias, void* const* outs, void* stream) {
    reset_launches();
    int32_t offs[VD_MAX_GATHERS], stride;
    vd_status st = vd_row_layout(dtypes, nfields, offs, &stride);
    if (st != VD_OK) return st;
    if (n < 0 || nrows < 0) return VD_E_SHAPE;
    if (n > 0 && (!pos || !outs)) { set_error("gather_rows: NULL pos/outs"); return VD_E_NULL; }
    if (nrows > 0 && !rows) return VD_E_NULL;
    if (((uintptr_t)rows % 16) != 0) { set_error("gather_rows: rows must be 16-byte aligned"); return VD_E_ARG; }
    for (int k = 0; k < nfields && n > 0; ++k)
        if (!outs[k]) { set_error("gather_rows: NULL out"); return VD_E_NULL; }
    st = check_device();
    if (st != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_gather_rows(rows, nrows, dtypes, nfields, pos, n, bias, outs, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_scatter(const vd_column* src, const int32_t* pos, int64_t n, void* out, int64_t out_len, int32_t flags,
                     void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    vd_status st = check_col(src, n, "scatter");
    if (st != VD_OK) return st;
    if (n < 0 || out_len < 0 || n > INT32_MAX || out_len > (int64_t)INT32_MAX + 1) { set_error("scatter: sizes"); return VD_E_SHAPE; }
    if ((n > 0 && !pos) || (out_len > 0 && !out)) { set_error("scatter: NULL buffer"); return VD_E_NULL; }
    bool unique = (flags & VD_SCATTER_UNIQUE) != 0;
    if (!unique && (st = check_ws(ws, ws_bytes, scatter_ws_bytes(out_len))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_scatter(*src, pos, n, out, out_len, unique, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_partition(const vd_column* v, int64_t pivot_from, int64_t npivots, int32_t* out_pos,
                       int64_t* out_bucket_counts, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    vd_status st = check_col(v, 0, "partition");
    if (st != VD_OK) return st;
    if (!is_int(v->dtype)) { set_error("partition: integer column required"); return VD_E_DTYPE; }
    if (npivots < 1 || npivots > 1024) { set_error("partition: npivots in [1, 1024]"); return VD_E_UNSUPPORTED; }
    if (v->len > INT32_MAX) return VD_E_SHAPE;
    if (v->len > 0 && !out_pos) return VD_E_NULL;
    if ((st = check_ws(ws, ws_bytes, partition_ws_bytes(v->len, npivots))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_partition(*v, pivot_from, npivots, out_pos, out_bucket_counts, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

size_t vd_partials_bytes(const vd_pipeline* plan) {
    if (!plan || plan->ngroups < 1 || plan->naggs < 0) return 0;
    return (size_t)plan->ngroups * (size_t)(plan->naggs + 1) * 16;
}

static int plan_col_dtype(const vd_pipeline* p, const vd_column* cols, int ncols, const vd_column* dims, int ndims,
                          int c) {
    if (c < 0) return -1;
    if (c < ncols) return cols[c].dtype;
    int g = c - ncols;
    if (g >= p->ngathers) return -1;
    int d = p->gathers[g].dim_col;
    if (d < 0 || d >= ndims) return -1;
    return dims[d].dtype;
}

static bool plan_col_bounds(const vd_pipeline* p, const vd_column* cols, int ncols, const vd_column* dims, int c,
                            int64_t* lo, int64_t* hi) {
    const vd_column* col = c < ncols ? &cols[c] : &dims[p->gathers[c - ncols].dim_col];
    if (!col->has_minmax || !is_int(col->dtype)) return false;
    *lo = col->min;
    *hi = col->max;
    return true;
}

vd_status vd_run_pipeline(const vd_pipeline* plan, const vd_column* cols, int32_t ncols, int64_t n,
                          const vd_column* dims, int32_t ndims, void* out, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    if (!plan || !out) { set_error("pipeline: NULL plan / out"); return VD_E_NULL; }
    if (n < 0) return VD_E_SHAPE;
    if (ncols < 0 || ncols + plan->ngathers > VD_MAX_DEVCOLS || (ncols > 0 && !cols)) { set_error("pipeline: columns"); return VD_E_ARG; }
    if (plan->ngroups < 1 || plan->ngroups > VD_MAX_GROUPS) { set_error("pipeline: ngroups in [1, 4096]"); return VD_E_ARG; }
    if (plan->naggs < 0 || plan->naggs > VD_MAX_AGGS) { set_error("pipeline: naggs in [0, 8]"); return VD_E_ARG; }
    if (plan->ngathers < 0 || plan->ngathers > VD_MAX_GATHERS) { set_error("pipeline: ngathers in [0, 4]"); return VD_E_ARG; }
    if (plan->nkeyparts < 0 || plan->nkeyparts > VD_MAX_KEYPARTS) { set_error("pipeline: nkeyparts in [0, 3]"); return VD_E_ARG; }
    if (plan->nkeyparts == 0 && plan->ngroups != 1) { set_error("pipeline: scalar plans have ngroups = 1"); return VD_E_ARG; }
    if (plan->sel_mode < VD_SEL_BRANCH || plan->sel_mode > VD_SEL_PREDICATED_LOOKUP) { set_error("pipeline: sel_mode"); return VD_E_ARG; }
    if (plan->ngathers > 0 && (!dims || ndims < 1)) { set_error("pipeline: gathers need dims"); return VD_E_NULL; }
    vd_status st;
    for (int c = 0; c < ncols; ++c)
        if ((st = check_col(&cols[c], n, "pipeline")) != VD_OK) return st;
    for (int g = 0; g < plan->ngathers; ++g) {
        const vd_gatherspec& gs = plan->gathers[g];
        if (gs.fk_col < 0 || gs.fk_col >= ncols || !is_int(cols[gs.fk_col].dtype)) { set_error("gather fk column"); return VD_E_ARG; }
        if (gs.dim_col < 0 || gs.dim_col >= ndims) { set_error("gather dim column"); return VD_E_ARG; }
        if ((st = check_col(&dims[gs.dim_col], 0, "dim")) != VD_OK) return st;
        if (dims[gs.dim_col].len > 0 && !dims[gs.dim_col].data) return VD_E_NULL;
    }
    const int nref = ncols + plan->ngathers;
    int32_t dts[VD_MAX_DEVCOLS];
    for (int c = 0; c < nref; ++c) dts[c] = plan_col_dtype(plan, cols, ncols, dims, ndims, c);
    if ((st = check_pred(&plan->pred, dts, nref)) != VD_OK) return st;
    // key parts: integer columns; domain proof from metadata
    bool known = true;
    double klo = 0, khi = 0;
    for (int k = 0; k < plan->nkeyparts; ++k) {
        const vd_keypart& kp = plan->key[k];
        if (kp.col < 0 || kp.col >= nref) { set_error("key column out of range"); return VD_E_ARG; }
        if (!is_int(dts[kp.col])) { set_error("key column must be integer"); return VD_E_DTYPE; }
        if (kp.fn != 0 && kp.fn != 1) { set_error("key fn must be 0 or 1"); return VD_E_ARG; }
        int64_t lo, hi;
        if (!plan_col_bounds(plan, cols, ncols, dims, kp.col, &lo, &hi)) { known = false; continue; }
        double a = (double)lo, b = (double)hi;
        if (kp.fn == 1) {
            auto yr = [](int64_t d) {  // civil year (host copy of the device helper)
                int64_t z = d + 719468;
                int64_t era = (z >= 0 ? z : z - 146096) / 146097;
                int64_t doe = z - era * 146097;
                int64_t yoe = (doe - doe / 1460 + doe / 36524 - doe / 146096) / 365;
                int64_t doy = doe - (365 * yoe + yoe / 4 - yoe / 100);
                int64_t mp = (5 * doy + 2) / 153;
                int64_t m = mp < 10 ? mp + 3 : mp - 9;
                return (double)(yoe + era * 400 + (m <= 2 ? 1 : 0));
            };
            a = yr(lo);
            b = yr(hi);
        }
        double x1 = (a - (double)kp.sub) * (double)kp.mult, x2 = (b - (double)kp.sub) * (double)kp.mult;
        klo += std::min(x1, x2);
        khi += std::max(x1, x2);
    }
    if (known && plan->nkeyparts > 0 && (klo < 0 || khi >= (double)plan->ngroups)) {
        set_error("group key domain [" + std::to_string((long long)klo) + ", " + std::to_string((long long)khi) +
                  "] exceeds [0, ngroups) (ctrl/data bit conflict, P:L951-956)");
        return VD_E_DOMAIN;
    }
    for (int a = 0; a < plan->naggs; ++a) {
        const vd_agg& g = plan->aggs[a];
        if (g.kind < VD_AGG_SUM || g.kind > VD_AGG_MAX) { set_error("bad aggregate kind"); return VD_E_ARG; }
        if (g.kind == VD_AGG_COUNT) continue;
        if (g.nfactors < 1 || g.nfactors > VD_MAX_FACTORS) { set_error("nfactors in [1, 3]"); return VD_E_ARG; }
        for (int f = 0; f < g.nfactors; ++f)
            if (g.f[f].col < -1 || g.f[f].col >= nref) { set_error("factor column out of range"); return VD_E_ARG; }
    }
    if (plan->materialize < VD_MAT_NONE || plan->materialize > VD_MAT_CHUNKS) {
        set_error("materialize: VD_MAT_NONE / VD_MAT_BREAK / VD_MAT_CHUNKS");
        return VD_E_ARG;
    }
    if (plan->materialize == VD_MAT_CHUNKS && plan->mat_chunk != 0 &&
        (plan->mat_chunk < 32 || plan->mat_chunk > (1 << 24) || plan->mat_chunk % 32 != 0)) {
        set_error("mat_chunk: a multiple of 32 in [32, 2^24] (0 = 1024)");
        return VD_E_ARG;
    }
    if ((st = check_ws(ws, ws_bytes, pipeline_ws_bytes(plan, n))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = run_pipeline(plan, cols, ncols, n, dims, ndims, out, ws, ws_bytes, (cudaStream_t)stream, &nl);
    count_launches(nl);
    return st;
}

// ---- NEXT-4: grouped fold over a large key domain (k_group.cu) --------------
vd_status vd_group_fold_ws_bytes(int64_t domain, int32_t naggs, size_t* bytes) {
    if (!bytes) return VD_E_NULL;
    if (domain < 1 || domain > VD_MAX_DOMAIN || naggs < 0 || naggs > VD_MAX_AGGS) return VD_E_ARG;
    *bytes = group_ws_bytes(domain, naggs);
    return VD_OK;
}

// Aggregates of a grouped fold over int64 table words (vd_group_fold,
// vd_hash_group_fold): factor columns in range, float aggregates SUM only,
// integer SUMs provably exact in int64 over all n rows (min/max metadata).
static vd_status check_group_aggs(const vd_column* cols, int32_t ncols, int64_t n, const vd_agg* aggs, int32_t naggs,
                                  int32_t* isf, const char* tag) {
    for (int a = 0; a < naggs; ++a) {
        const vd_agg& g = aggs[a];
        if (g.kind < VD_AGG_SUM || g.kind > VD_AGG_MAX) { set_error("bad aggregate kind"); return VD_E_ARG; }
        if (g.kind == VD_AGG_COUNT) continue;
        if (g.nfactors < 1 || g.nfactors > VD_MAX_FACTORS) { set_error("nfactors in [1, 3]"); return VD_E_ARG; }
        double mx = 1.0;  // bound of |product|
        bool known = true;
        for (int f = 0; f < g.nfactors; ++f) {
            const vd_factor& fc = g.f[f];
            if (fc.col < -1 || fc.col >= ncols) { set_error("factor column out of range"); return VD_E_ARG; }
            if (fc.col < 0) { mx *= std::fabs((double)fc.a); continue; }
            const vd_column& c = cols[fc.col];
            if (c.dtype == VD_F32 || c.dtype == VD_F64) { isf[a] = 1; continue; }
            if (!c.has_minmax) { known = false; continue; }
            const double x1 = (double)fc.a + (double)fc.b * (double)c.min, x2 = (double)fc.a + (double)fc.b * (double)c.max;
            mx *= std::max(std::fabs(x1), std::fabs(x2));
        }
        if (isf[a] && g.kind != VD_AGG_SUM) {
            set_error(std::string(tag) + ": float MIN/MAX not supported");
            return VD_E_UNSUPPORTED;
        }
        if (isf[a]) continue;
        // int64 table slots: a SUM must be exact over all n rows, MIN/MAX must
        // stay below the table's identity values
        const double lim = g.kind == VD_AGG_SUM ? mx * (double)(n > 0 ? n : 1) : mx;
        if (!known || lim >= 9.2e18) {
            set_error(std::string(tag) + ": min/max metadata cannot prove int64 aggregates exact");
            return VD_E_OVERFLOW;
        }
    }
    return VD_OK;
}

vd_status vd_group_fold(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, int32_t key_col,
                        const vd_agg* aggs, int32_t naggs, int64_t* out_keys, void* out_aggs, int64_t* out_rows,
                        int64_t* out_ngroups, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    if (n < 0) return VD_E_SHAPE;
    if (ncols < 1 || ncols > VD_MAX_DEVCOLS || !cols) { set_error("group_fold: columns"); return VD_E_ARG; }
    if (naggs < 0 || naggs > VD_MAX_AGGS || (naggs > 0 && !aggs)) { set_error("group_fold: naggs in [0, 8]"); return VD_E_ARG; }
    if (!out_keys || !out_rows || !out_ngroups || (naggs > 0 && !out_aggs)) { set_error("group_fold: outputs"); return VD_E_NULL; }
    vd_status st;
    DevCols dc;
    std::memset(&dc, 0, sizeof(dc));
    dc.ncols = ncols;
    for (int c = 0; c < ncols; ++c) {
        if ((st = check_col(&cols[c], n, "group_fold")) != VD_OK) return st;
        dc.p[c] = cols[c].data;
        dc.dt[c] = cols[c].dtype;
    }
    if ((st = check_pred(pred, dc.dt, ncols)) != VD_OK) return st;
    if (key_col < 0 || key_col >= ncols) { set_error("group_fold: key column out of range"); return VD_E_ARG; }
    const vd_column& kc = cols[key_col];
    if (kc.dtype != VD_I32 && kc.dtype != VD_I64) { set_error("group_fold: key must be i32/i64"); return VD_E_DTYPE; }
    // identity hashing: the table is sized from the key's min/max
    if (!kc.has_minmax) { set_error("group_fold: the key column needs min/max metadata"); return VD_E_DOMAIN; }
    const double dspan = (double)kc.max - (double)kc.min + 1.0;
    if (kc.max < kc.min || dspan > (double)VD_MAX_DOMAIN) { set_error("group_fold: key domain exceeds VD_MAX_DOMAIN"); return VD_E_DOMAIN; }
    const int64_t D = kc.max - kc.min + 1;
    int32_t isf[VD_MAX_AGGS] = {0};
    if ((st = check_group_aggs(cols, ncols, n, aggs, naggs, isf, "group_fold")) != VD_OK) return st;
    if ((st = check_ws(ws, ws_bytes, group_ws_bytes(D, naggs))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    DevPred dp;
    make_devpred(pred, &dp);
    int nl = 0;
    st = cuda_status(launch_group_fold(dc, dp, n, key_col, kc.min, D, aggs, isf, naggs, out_keys, out_aggs, out_rows,
                                       out_ngroups, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

// ---- NEXT-4: grouped fold over sparse keys (k_hash.cu) ------------------------
vd_status vd_hash_group_fold_ws_bytes(int64_t max_groups, int32_t naggs, size_t* bytes) {
    if (!bytes) return VD_E_NULL;
    if (max_groups < 1 || max_groups > VD_MAX_HASH_GROUPS || naggs < 0 || naggs > VD_MAX_AGGS) return VD_E_ARG;
    *bytes = hash_group_ws_bytes(max_groups, naggs, false);
    return VD_OK;
}

vd_status vd_hash_group_fold(const vd_column* cols, int32_t ncols, int64_t n, const vd_pred* pred, int32_t key_col,
                             const vd_agg* aggs, int32_t naggs, int64_t max_groups, int64_t* out_keys, void* out_aggs,
                             int64_t* out_rows, int64_t* out_ngroups, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    if (n < 0) return VD_E_SHAPE;
    if (ncols < 1 || ncols > VD_MAX_DEVCOLS || !cols) { set_error("hash_group_fold: columns"); return VD_E_ARG; }
    if (naggs < 0 || naggs > VD_MAX_AGGS || (naggs > 0 && !aggs)) { set_error("hash_group_fold: naggs in [0, 8]"); return VD_E_ARG; }
    if (max_groups < 1 || max_groups > VD_MAX_HASH_GROUPS) { set_error("hash_group_fold: max_groups"); return VD_E_ARG; }
    if (!out_keys || !out_rows || !out_ngroups || (naggs > 0 && !out_aggs)) { set_error("hash_group_fold: outputs"); return VD_E_NULL; }
    vd_status st;
    DevCols dc;
    std::memset(&dc, 0, sizeof(dc));
    dc.ncols = ncols;
    for (int c = 0; c < ncols; ++c) {
        if ((st = check_col(&cols[c], n, "hash_group_fold")) != VD_OK) return st;
        dc.p[c] = cols[c].data;
        dc.dt[c] = cols[c].dtype;
    }
    if ((st = check_pred(pred, dc.dt, ncols)) != VD_OK) return st;
    if (key_col < 0 || key_col >= ncols) { set_error("hash_group_fold: key column out of range"); return VD_E_ARG; }
    if (cols[key_col].dtype != VD_I32 && cols[key_col].dtype != VD_I64) {
        set_error("hash_group_fold: key must be i32/i64");
        return VD_E_DTYPE;
    }
    int32_t isf[VD_MAX_AGGS] = {0};
    if ((st = check_group_aggs(cols, ncols, n, aggs, naggs, isf, "hash_group_fold")) != VD_OK) return st;
    if ((st = check_ws(ws, ws_bytes, hash_group_ws_bytes(max_groups, naggs, false))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    DevPred dp;
    make_devpred(pred, &dp);
    int nl = 0;
    st = cuda_status(launch_hash_group_fold(dc, dp, n, key_col, aggs, isf, naggs, max_groups, out_keys, out_aggs,
                                            out_rows, out_ngroups, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

vd_status vd_merge_groups_ws_bytes(int64_t max_groups, int32_t naggs, size_t* bytes) {
    if (!bytes) return VD_E_NULL;
    if (max_groups < 1 || max_groups > VD_MAX_HASH_GROUPS || naggs < 0 || naggs > VD_MAX_AGGS) return VD_E_ARG;
    *bytes = hash_group_ws_bytes(max_groups, naggs, true);
    return VD_OK;
}

vd_status vd_merge_groups(const int64_t* keys, const void* aggs_in, const int64_t* rows, const int64_t* counts_dev,
                          int32_t nparts, int64_t stride, const int32_t* kinds_host, const int32_t* isf_host,
                          int32_t naggs, int64_t max_groups, int64_t* out_keys, void* out_aggs, int64_t* out_rows,
                          int64_t* out_ngroups, void* ws, size_t ws_bytes, void* stream) {
    reset_launches();
    if (nparts < 0 || stride < 0) return VD_E_SHAPE;
    if (naggs < 0 || naggs > VD_MAX_AGGS || (naggs > 0 && (!kinds_host || !isf_host))) return VD_E_ARG;
    if (max_groups < 1 || max_groups > VD_MAX_HASH_GROUPS) { set_error("merge_groups: max_groups"); return VD_E_ARG; }
    const bool any = nparts > 0 && stride > 0;
    if ((any && (!keys || !rows || !counts_dev || (naggs > 0 && !aggs_in))) || !out_keys || !out_rows ||
        !out_ngroups || (naggs > 0 && !out_aggs))
        return VD_E_NULL;
    for (int a = 0; a < naggs; ++a) {
        if (kinds_host[a] < VD_AGG_SUM || kinds_host[a] > VD_AGG_MAX) { set_error("bad aggregate kind"); return VD_E_ARG; }
        if (isf_host[a] && kinds_host[a] != VD_AGG_SUM && kinds_host[a] != VD_AGG_COUNT) {
            set_error("merge_groups: float MIN/MAX not supported");
            return VD_E_UNSUPPORTED;
        }
    }
    vd_status st;
    if ((st = check_ws(ws, ws_bytes, hash_group_ws_bytes(max_groups, naggs, true))) != VD_OK) return st;
    if ((st = check_device()) != VD_OK) return st;
    int nl = 0;
    st = cuda_status(launch_merge_groups(keys, aggs_in, rows, counts_dev, any ? nparts : 0, any ? stride : 0,
                                         kinds_host, isf_host, naggs, max_groups, out_keys, out_aggs, out_rows,
                                         out_ngroups, ws, (cudaStream_t)stream, &nl));
    count_launches(nl);
    return st;
}

// Which aggregates of `plan` are f64 (a float factor column); cols/dims may
// be NULL (then every aggregate reads as integer: only valid for nparts == 1,
// where nothing is added).
static vd_status merge_prologue(const vd_pipeline* plan, const vd_column* cols, int32_t ncols,
                                const vd_column* dims, int32_t ndims, int32_t nparts, const vd_result* out,
                                int32_t* isf) {
    if (!plan || !out || !out->keys || !out->rows || !out->ngroups || (plan->naggs > 0 && !out->aggs))
        return VD_E_NULL;
    if (plan->ngroups < 1 || plan->ngroups > VD_MAX_GROUPS || plan->naggs < 0 || plan->naggs > VD_MAX_AGGS)
        return VD_E_ARG;
    if (nparts < 1) { set_error("merge: nparts < 1"); return VD_E_SHAPE; }
    if (out->capacity < plan->ngroups) { set_error("vd_result capacity < plan->ngroups"); return VD_E_SHAPE; }
    if (nparts > 1 && !cols && !dims) {  // the dtypes decide int128 vs f64 addition
        for (int a = 0; a < plan->naggs; ++a)
            if (plan->aggs[a].kind != VD_AGG_COUNT && plan->aggs[a].nfactors > 0) {
                set_error("merge of several partials needs the column views (their dtypes)");
                return VD_E_NULL;
            }
    }
    for (int a = 0; a < VD_MAX_AGGS; ++a) isf[a] = 0;
    for (int a = 0; a < plan->naggs; ++a) {
        const vd_agg& g = plan->aggs[a];
        if (g.kind == VD_AGG_COUNT || (!cols && !dims)) continue;
        for (int f = 0; f < g.nfactors; ++f) {
            int dt = plan_col_dtype(plan, cols, ncols, dims, ndims, g.f[f].col);
            if (dt == VD_F32 || dt == VD_F64) isf[a] = 1;
        }
    }
    return VD_OK;
}

vd_status vd_merge_partials(const vd_pipeline* plan, const vd_column* cols, int32_t ncols, const vd_column* dims,
                            int32_t ndims, const void* const* parts, int32_t nparts, const vd_result* out) {
    int32_t isf[VD_MAX_AGGS];
    vd_status st = merge_prologue(plan, cols, ncols, dims, ndims, nparts, out, isf);
    if (st != VD_OK) return st;
    if (!parts) return VD_E_NULL;
    for (int r = 0; r < nparts; ++r)
        if (!parts[r]) return VD_E_NULL;
    const int NA = plan->naggs;
    const int64_t G = plan->ngroups;
    typedef __int128 I;
    auto rd = [](const void* p, int64_t k) {
        const uint64_t* q = (const uint64_t*)p + 2 * k;
        return (I)(((unsigned __int128)q[1] << 64) | q[0]);
    };
    auto rdf = [](const void* p, int64_t k) {
        double d;
        std::memcpy(&d, (const uint64_t*)p + 2 * k, 8);
        return d;
    };
    uint64_t* oa = (uint64_t*)out->aggs;
    int64_t ng = 0;
    for (int64_t g = 0; g < G; ++g) {  // ascending key: the pivot order of Fig 11
        const int64_t base = g * (NA + 1);
        I rows = 0;
        for (int r = 0; r < nparts; ++r) rows += rd(parts[r], base + NA);
        if (rows == 0) continue;  // empty group: dropped by the compaction (A16)
        for (int a = 0; a < NA; ++a) {
            const int kind = plan->aggs[a].kind;
            I vi = 0;
            double vf = 0;
            bool have = false;
            for (int r = 0; r < nparts; ++r) {  // rank order
                if (rd(parts[r], base + NA) == 0) continue;  // empty on that rank
                if (kind == VD_AGG_SUM || kind == VD_AGG_COUNT) {
                    if (isf[a] && kind == VD_AGG_SUM) vf += rdf(parts[r], base + a);
                    else vi += rd(parts[r], base + a);
                } else if (isf[a]) {
                    double x = rdf(parts[r], base + a);
                    if (!have || (kind == VD_AGG_MIN ? x < vf : x > vf)) vf = x;
                } else {
                    I x = rd(parts[r], base + a);
                    if (!have || (kind == VD_AGG_MIN ? x < vi : x > vi)) vi = x;
                }
                have = true;
            }
            uint64_t* q = oa + 2 * (ng * NA + a);
            if (nparts == 1) {  // a single partial: the slot verbatim
                std::memcpy(q, (const uint64_t*)parts[0] + 2 * (base + a), 16);
            } else if (isf[a] && kind != VD_AGG_COUNT) {
                std::memcpy(q, &vf, 8);
                q[1] = 0;
            } else {
                q[0] = (uint64_t)(unsigned __int128)vi;
                q[1] = (uint64_t)((unsigned __int128)vi >> 64);
            }
        }
        out->keys[ng] = g;
        out->rows[ng] = (int64_t)rows;
        ++ng;
    }
    *out->ngroups = ng;
    return VD_OK;
}

vd_status vd_merge_partials_device(const vd_pipeline* plan, const vd_column* cols, int32_t ncols,
                                   const vd_column* dims, int32_t ndims, const void* parts_dev, int32_t nparts,
                                   const vd_result* out, void* stream) {
    reset_launches();
    int32_t isf[VD_MAX_AGGS];
    vd_status st = merge_prologue(plan, cols, ncols, dims, ndims, nparts, out, isf);
    if (st != VD_OK) return st;
    if (!parts_dev) return VD_E_NULL;
    int nl = 0;
    cudaError_t e = launch_merge_partials(plan, isf, parts_dev, nparts, *out, (cudaStream_t)stream, &nl);
    count_launches(nl);
    if (e != cudaSuccess) { set_error(cudaGetErrorString(e)); return VD_E_CUDA; }
    return VD_OK;
}

}  // extern "C"
