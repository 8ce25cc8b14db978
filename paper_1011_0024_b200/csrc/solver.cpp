// solver.cpp — mixed-precision BiCGstab with reliable updates (
// BiCGstab: van der Vorst, ref [8]; reliable updates: Sleijpen & van der Vorst, ref [21]).
//
// "Algorithm R" (reading Q10): the Krylov iteration runs in the sloppy precision
// on the even-odd operator Mhat; the solution accumulates in a sloppy xs that is folded into
// the high-precision x at every reliable update, where the true residual r = bhat - Mhat x is
// recomputed in the high precision.  One Krylov space is kept throughout (p, v continue across
// updates).  The solve stops only on a TRUE residual <= tol ||bhat||.
//
//   setup: x = 0; r = bhat; rs = lo(r); rhat0 = rs; xs = 0; r0Norm = maxrr = maxrx = ||r||
//   iterate:
//     rho' = <rhat0, rs>;  p = rs (first) | rs + beta (p - omega v), beta = (rho'/rho)(alpha/omega)
//     v = Mhat p;  alpha = rho' / <rhat0, v>;  rs -= alpha v
//     t = Mhat rs; omega = <t, rs> / |t|^2
//     xs += alpha p + omega rs;  rs -= omega t;  rNorm = |rs|
//     maxrx = max(maxrx, rNorm); maxrr = max(maxrr, rNorm)
//     updX = rNorm < delta r0Norm && r0Norm <= maxrx
//     updR = (rNorm < delta maxrr && r0Norm <= maxrr) || updX || rNorm <= tol ||bhat||
//     on updR: x += xs; xs = 0; r = bhat - Mhat x (high); rs = lo(r); rNorm = |r|; maxrr = rNorm;
//              rho' = <rhat0, rs> recomputed for the replaced residual;
//              if updX: r0Norm = maxrx = rNorm;  stop if rNorm <= tol ||bhat||
#include <cmath>
#include <complex>
#include <cstdio>
#include <cstring>
#include <string>
#include <vector>

#include "ctx.h"

namespace qx {

using cd = std::complex<double>;

static void *field(qudax_ctx *c, void *&slot, int prec) {
    if (!slot) slot = dalloc(c, spinor_bytes(prec, c->g.stride));
    return slot;
}

// Point a solver workspace at (Pd, Ps): the fields of a precision that changes are released
// (the outer-precision fields survive a change of the sloppy precision alone), so switching
// modes never strands device memory until finalize.
static void ws_select(qudax_ctx *c, qudax_ctx::SolverWs &w, int Pd, int Ps) {
    if (w.prec != Pd) {
        for (void **f : {&w.b_e, &w.b_o, &w.bh, &w.x_e, &w.x_o, &w.r, &w.t_e, &w.t_o}) {
            dfree(c, *f);
            *f = nullptr;
        }
        w.prec = Pd;
    }
    if (w.prec_s != Ps) {
        for (void **f : {&w.rs, &w.xs, &w.p, &w.v, &w.t, &w.r0}) {
            dfree(c, *f);
            *f = nullptr;
        }
        w.prec_s = Ps;
    }
}

static void zero(qudax_ctx *c, void *f, int prec) {
    QX_CUDA(cudaMemsetAsync(f, 0, spinor_bytes(prec, c->g.stride), c->stream));
}
static void copy(qudax_ctx *c, void *dst, const void *src, int prec) {
    QX_CUDA(cudaMemcpyAsync(dst, src, spinor_bytes(prec, c->g.stride), cudaMemcpyDeviceToDevice, c->stream));
}

static double norm2_of(qudax_ctx *c, int prec, void *f) {
    double r;
    void *fs[1] = {f};
    blas_op(c, OP_NORM2, prec, fs, nullptr, &r);
    return r;
}
static cd cdot_of(qudax_ctx *c, int prec, void *a, void *b) {
    double r[2];
    void *fs[2] = {a, b};
    blas_op(c, OP_CDOT, prec, fs, nullptr, r);
    return cd(r[0], r[1]);
}

static SolverScalars *scalars(qudax_ctx *c) {
    if (!c->d_scal) {
        c->d_scal = static_cast<SolverScalars *>(dalloc(c, sizeof(SolverScalars)));
        c->h_scal = static_cast<SolverScalars *>(halloc(c, sizeof(SolverScalars)));
    }
    return c->d_scal;
}

// Capture `body` (stream-ordered work on c->stream, possibly forking to the comm stream for
// the NCCL halo) into an instantiated CUDA graph.  *nlaunch = library kernels per replay;
// *trecs receives the event-bracketed Dslash launches (kernel timing on).
template <typename F>
static cudaGraphExec_t capture_graph(qudax_ctx *c, F &&body, long long *nlaunch,
                                     std::vector<qudax_ctx::TimingRec> *trecs) {
    const long long l0 = c->launches;
    c->capturing = true;
    c->graph_trecs.clear();
    QX_CUDA(cudaStreamBeginCapture(c->stream, cudaStreamCaptureModeThreadLocal));
    try {
        body();
    } catch (...) {
        cudaGraph_t g;
        cudaStreamEndCapture(c->stream, &g);
        if (g) cudaGraphDestroy(g);
        c->capturing = false;
        c->cap_iter = 0;
        c->launches = l0;
        release_graph_timing(c, c->graph_trecs);
        throw;
    }
    cudaGraph_t graph = nullptr;
    const cudaError_t ee = cudaStreamEndCapture(c->stream, &graph);
    c->capturing = false;
    c->cap_iter = 0;
    cudaGraphExec_t exec = nullptr;
    const cudaError_t ie = (ee == cudaSuccess) ? cudaGraphInstantiate(&exec, graph, 0) : ee;
    if (graph) cudaGraphDestroy(graph);
    if (ie != cudaSuccess) {
        c->launches = l0;
        release_graph_timing(c, c->graph_trecs);
        throw Error(QUDAX_ERR_CUDA, std::string("solver graph capture: ") + cudaGetErrorString(ie));
    }
    *nlaunch = c->launches - l0;
    c->launches = l0;
    trecs->swap(c->graph_trecs);
    c->graph_trecs.clear();
    return exec;
}

// Cached solver graphs (ctx.h Graph): at most kMaxGraphs, least recently captured dropped first;
// all of them on gauge_load (their key holds the gauge epoch).
constexpr size_t kMaxGraphs = 24;
void drop_graphs(qudax_ctx *c) {
    for (auto &gr : c->graphs) {
        if (gr.exec) cudaGraphExecDestroy(gr.exec);
        release_graph_timing(c, gr.trecs);
    }
    c->graphs.clear();
}
template <typename F>
static qudax_ctx::Graph *cached_graph(qudax_ctx *c, std::vector<uintptr_t> key, F &&body) {
    key.push_back((uintptr_t)c->gauge_epoch);
    key.push_back((uintptr_t)c->timing);
    for (auto &gr : c->graphs)
        if (gr.key == key) return &gr;
    if (c->graphs.size() >= kMaxGraphs) {
        auto &old = c->graphs.front();
        if (old.exec) cudaGraphExecDestroy(old.exec);
        release_graph_timing(c, old.trecs);
        c->graphs.erase(c->graphs.begin());
    }
    qudax_ctx::Graph gr;
    gr.key = std::move(key);
    try {
        gr.exec = capture_graph(c, body, &gr.launches, &gr.trecs);
    } catch (const Error &e) {
        // a capture the runtime or a transport refuses (e.g. a NCCL build without graph support):
        // the context continues with eager enqueues, which compute the same iterates
        if (e.status != QUDAX_ERR_CUDA && e.status != QUDAX_ERR_NCCL) throw;
        cudaGetLastError();
        std::fprintf(stderr, "qudax: CUDA-graph capture of the solver batch failed (%s); continuing eagerly\n", e.what());
        c->flags |= QUDAX_FLAG_NO_GRAPHS;
        return nullptr;
    }
    c->graphs.push_back(std::move(gr));
    return &c->graphs.back();
}

// Kernel directions of a BiCGstab iteration (QX_SOLVER_ORDER 1): every kernel starts at the end
// of the lattice where the previous one finished, so the first part of the field it reads from
// the previous kernel (p, tmp, v, s, tmp, t) is still in the 126 MB L2 — p update (up), first
// Mhat's clover-inverse kernel (down) and xpay (up), s = r - alpha v (down), second Mhat's
// kernels (up, down), final update (up): six of the seven transitions hot instead of four.
#ifndef QX_SOLVER_ORDER
#define QX_SOLVER_ORDER 1
#endif
constexpr int kCaxpyOp = QX_SOLVER_ORDER ? OP_CAXPY_REV : OP_CAXPY;

// Batch graph (solve_dev): [k_batch_begin] -> WHILE(cond) { one iteration; k_batch_cond } ->
// [k_batch_end].  The WHILE node repeats the captured iteration on the device until k_batch_cond
// clears the condition from what the reduction tail evaluating Algorithm R decided (reliable
// update, convergence, maxiter) or after the batch's `n` iterations: no host round trip and no launch inside a batch, and no kernel
// of a halted iteration is launched at all.  Returns nullptr if the iteration's nodes cannot sit
// in a conditional body (e.g. host nodes a transport adds); the caller then replays one
// iteration per plain graph.
template <typename F>
static cudaGraphExec_t capture_while_graph(qudax_ctx *c, SolverScalars *S, int n, F &&body, long long *outer,
                                           long long *per_iter) {
    cudaGraph_t g = nullptr;
    QX_CUDA(cudaGraphCreate(&g, 0));
    struct Guard {
        cudaGraph_t g;
        ~Guard() { if (g) cudaGraphDestroy(g); }
    } guard{g};
    cudaGraphConditionalHandle h;
    QX_CUDA(cudaGraphConditionalHandleCreate(&h, g, 1u, cudaGraphCondAssignDefault));
    cudaGraph_t cg = g;
    QX_CUDA(cudaStreamBeginCaptureToGraph(c->stream, g, nullptr, nullptr, 0, cudaStreamCaptureModeThreadLocal));
    launch_batch_begin(S, (unsigned long long)h, n, c->stream);
    QX_CUDA(cudaStreamEndCapture(c->stream, &cg));
    cudaGraphNode_t first = nullptr;
    size_t nn = 1;
    QX_CUDA(cudaGraphGetNodes(g, &first, &nn));
    cudaGraphNodeParams cp = {};
    cp.type = cudaGraphNodeTypeConditional;
    cp.conditional.handle = h;
    cp.conditional.type = cudaGraphCondTypeWhile;
    cp.conditional.size = 1;
    cudaGraphNode_t cnode = nullptr;
    QX_CUDA(cudaGraphAddNode(&cnode, g, &first, 1, &cp));
    cudaGraph_t bg = cp.conditional.phGraph_out[0];
    const long long l0 = c->launches;
    c->capturing = true;
    QX_CUDA(cudaStreamBeginCaptureToGraph(c->stream, bg, nullptr, nullptr, 0, cudaStreamCaptureModeThreadLocal));
    try {
        body();
        launch_batch_cond(S, c->stream);
    } catch (...) {
        cudaGraph_t tmp;
        cudaStreamEndCapture(c->stream, &tmp);
        c->capturing = false;
        c->launches = l0;
        throw;
    }
    cudaGraph_t bg2 = bg;
    const cudaError_t ee = cudaStreamEndCapture(c->stream, &bg2);
    c->capturing = false;
    *per_iter = c->launches - l0 + 1;  // + k_batch_cond
    c->launches = l0;
    if (ee != cudaSuccess) {
        std::fprintf(stderr, "qudax: capture of the batch iteration into a WHILE body failed (%s); one iteration per host poll\n",
                     cudaGetErrorString(ee));
        cudaGetLastError();
        return nullptr;
    }
    {  // what a conditional body may hold: kernels, memcpy / memset, empty nodes
        size_t nb = 0;
        QX_CUDA(cudaGraphGetNodes(bg, nullptr, &nb));
        std::vector<cudaGraphNode_t> nodes(nb);
        if (nb) QX_CUDA(cudaGraphGetNodes(bg, nodes.data(), &nb));
        for (auto nd : nodes) {
            cudaGraphNodeType ty;
            QX_CUDA(cudaGraphNodeGetType(nd, &ty));
            if (ty != cudaGraphNodeTypeKernel && ty != cudaGraphNodeTypeMemcpy && ty != cudaGraphNodeTypeMemset &&
                ty != cudaGraphNodeTypeEmpty) {
                std::fprintf(stderr, "qudax: the batch iteration holds a graph node of type %d (of %zu nodes) a WHILE "
                             "body cannot; one iteration per host poll\n", (int)ty, nb);
                return nullptr;
            }
        }
    }
    QX_CUDA(cudaStreamBeginCaptureToGraph(c->stream, g, &cnode, nullptr, 1, cudaStreamCaptureModeThreadLocal));
    launch_batch_end(S, c->stream);
    QX_CUDA(cudaStreamEndCapture(c->stream, &cg));
    cudaGraphExec_t exec = nullptr;
    const cudaError_t ie = cudaGraphInstantiate(&exec, g, 0);
    if (ie != cudaSuccess) {
        std::fprintf(stderr, "qudax: instantiating the WHILE batch graph failed (%s); one iteration per host poll\n",
                     cudaGetErrorString(ie));
        cudaGetLastError();
        return nullptr;
    }
    *outer = 2;
    return exec;
}

template <typename F>
static qudax_ctx::Graph *cached_while_graph(qudax_ctx *c, std::vector<uintptr_t> key, SolverScalars *S, int n,
                                            F &&body) {
    key.push_back((uintptr_t)c->gauge_epoch);
    key.push_back((uintptr_t)c->timing);
    for (auto &gr : c->graphs)
        if (gr.key == key) return gr.no_while ? nullptr : &gr;
    if (c->graphs.size() >= kMaxGraphs) {
        auto &old = c->graphs.front();
        if (old.exec) cudaGraphExecDestroy(old.exec);
        release_graph_timing(c, old.trecs);
        c->graphs.erase(c->graphs.begin());
    }
    qudax_ctx::Graph gr;
    gr.key = std::move(key);
    try {
        gr.exec = capture_while_graph(c, S, n, body, &gr.launches, &gr.per_iter);
    } catch (const Error &e) {
        // a runtime without conditional nodes, or a capture it refuses: one iteration per poll
        if (e.status != QUDAX_ERR_CUDA && e.status != QUDAX_ERR_NCCL) throw;
        cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
        if (cudaStreamIsCapturing(c->stream, &cs) == cudaSuccess && cs != cudaStreamCaptureStatusNone) {
            cudaGraph_t tmp = nullptr;
            cudaStreamEndCapture(c->stream, &tmp);
            if (tmp) cudaGraphDestroy(tmp);
        }
        c->capturing = false;
        cudaGetLastError();
        std::fprintf(stderr, "qudax: WHILE batch graph unavailable (%s); one iteration per host poll\n", e.what());
        gr.exec = nullptr;
    }
    gr.no_while = (gr.exec == nullptr);
    c->graphs.push_back(std::move(gr));
    return c->graphs.back().no_while ? nullptr : &c->graphs.back();
}

// the Schur form matpc_op applies during one solve (restored on every exit path)
struct SchurForm {
    qudax_ctx *c;
    int saved;
    SchurForm(qudax_ctx *c_, bool sym) : c(c_), saved(c_->matpc_sym) { c->matpc_sym = sym ? 1 : 0; }
    ~SchurForm() { c->matpc_sym = saved; }
};

// b (device fp64 DR slab) -> b_e, b_o and the Schur source
//   bhat = b_e + kappa D_eo T_oo^{-1} b_o   (use_schur = 1), T_ee^{-1} of that (use_schur = 2,
//   symmetric form), else bhat = b_e
static void prepare_source(qudax_ctx *c, int Pd, const double *b_dev, void *b_e, void *b_o, void *bh, void *t_e,
                           void *t_o, int use_schur) {
    const Geom &g = c->g;
    launch_spinor_import(Pd, g, 0, b_dev, b_e, c->stream);
    launch_spinor_import(Pd, g, 1, b_dev, b_o, c->stream);
    c->launches += 2;
    if (use_schur) {
        clover_apply_op(c, t_o, b_o, Pd, 1, true);                // T_oo^{-1} b_o
        dslash_op(c, t_e, t_o, nullptr, Pd, 0, 0, QUDAX_HOP, 0);  // D_eo T_oo^{-1} b_o
        void *f[3] = {b_e, t_e, bh};
        double a = c->kappa;
        blas_op(c, OP_XPAY, Pd, f, &a, nullptr);                   // bhat = b_e + kappa (...)
        if (use_schur == 2) {                                          // symmetric: T_ee^{-1} bhat
            clover_apply_op(c, t_e, bh, Pd, 0, true);
            copy(c, bh, t_e, Pd);
        }
    } else {
        copy(c, bh, b_e, Pd);
    }
}

// x_e -> x_o = T_oo^{-1}(b_o + kappa D_oe x_e), the full-system fp64 (if Pd = 8) true residual
// ||b - M x|| / ||b|| and the export of x to the device DR slab x_dev
static void finish_solution(qudax_ctx *c, int Pd, double *x_dev, void *b_e, void *b_o, void *x_e, void *x_o,
                            void *t_e, void *t_o, int use_schur, qudax_solve_stats *st) {
    const Geom &g = c->g;
    const double kappa = c->kappa;
    if (use_schur) {
        dslash_op(c, t_o, x_e, nullptr, Pd, 1, 0, QUDAX_HOP, 0);  // D_oe x_e
        {
            void *f[3] = {b_o, t_o, t_o};
            double a = kappa;
            blas_op(c, OP_XPAY, Pd, f, &a, nullptr);               // b_o + kappa D_oe x_e
        }
        clover_apply_op(c, x_o, t_o, Pd, 1, true);                 // x_o = T_oo^{-1}(...)
        // (M x)_e = T_ee x_e - kappa D_eo x_o.  The odd residual b_o - (T_oo x_o - kappa D_oe x_e)
        // is t_o - T_oo x_o with t_o = b_o + kappa D_oe x_e still at hand: one clover
        // application instead of a second Dslash
        dslash_op(c, t_e, x_o, x_e, Pd, 0, 0, QUDAX_CLOVER_XPAY, -kappa);
        void *tx_o = tmp_odd_field(c, Pd);
        clover_apply_op(c, tx_o, x_o, Pd, 1, false);               // T_oo x_o
        double re2, ro2;
        {
            void *f[2] = {b_e, t_e};
            blas_op(c, OP_BMR_NORM, Pd, f, nullptr, &re2);
        }
        {
            void *f[2] = {t_o, tx_o};
            blas_op(c, OP_BMR_NORM, Pd, f, nullptr, &ro2);          // r_o = t_o - T_oo x_o
        }
        const double bb = norm2_of(c, Pd, b_e) + norm2_of(c, Pd, b_o);
        st->true_res = bb > 0 ? std::sqrt((re2 + ro2) / bb) : 0.0;
        launch_spinor_export(Pd, g, 0, x_e, x_dev, c->stream);
        launch_spinor_export(Pd, g, 1, x_o, x_dev, c->stream);
        c->launches += 2;
    } else {
        st->true_res = st->true_res_schur;
        QX_CUDA(cudaMemsetAsync(x_dev, 0, sizeof(double) * 24 * g.V, c->stream));
        launch_spinor_export(Pd, g, 0, x_e, x_dev, c->stream);
        c->launches += 1;
    }
    QX_CUDA(cudaStreamSynchronize(c->stream));
}

void solve_dev(qudax_ctx *c, double *x_dev, const double *b_dev, const qudax_solve_param *sp, qudax_solve_stats *st) {
    QX_CHECK(sp->use_schur >= 0 && sp->use_schur <= 2, QUDAX_ERR_ARG, "use_schur must be 0, 1 or 2");
    SchurForm form_guard(c, sp->use_schur == 2);
    QX_CHECK(c->gauge_loaded, QUDAX_ERR_STATE, "gauge not loaded");
    const int Pd = sp->prec, Ps = sp->prec_sloppy;
    check_prec(Pd);
    check_prec(Ps);
    QX_CHECK(sp->maxiter >= 0 && sp->tol >= 0 && sp->delta >= 0, QUDAX_ERR_ARG, "solve: bad parameters");
    std::memset(st, 0, sizeof(*st));
    auto &w = c->sws;
    QX_CUDA(cudaStreamSynchronize(c->stream));  // (released buffers may be in flight)
    ws_select(c, w, Pd, Ps);
    const Geom &g = c->g;
    void *b_e = field(c, w.b_e, Pd), *b_o = field(c, w.b_o, Pd), *bh = field(c, w.bh, Pd);
    void *x_e = field(c, w.x_e, Pd), *x_o = field(c, w.x_o, Pd), *r = field(c, w.r, Pd);
    void *t_e = field(c, w.t_e, Pd), *t_o = field(c, w.t_o, Pd);
    void *rs = field(c, w.rs, Ps), *xs = field(c, w.xs, Ps), *p = field(c, w.p, Ps);
    void *v = field(c, w.v, Ps), *t = field(c, w.t, Ps), *r0 = field(c, w.r0, Ps);

    prepare_source(c, Pd, b_dev, b_e, b_o, bh, t_e, t_o, sp->use_schur);

    // ---- Algorithm R
    const double b2 = norm2_of(c, Pd, bh);
    const double bnorm = std::sqrt(b2);
    const double stop = sp->tol * bnorm;
    zero(c, x_e, Pd);
    zero(c, xs, Ps);
    zero(c, v, Ps);
    zero(c, p, Ps);
    copy(c, r, bh, Pd);
    convert_op(c, rs, Ps, r, Pd);
    copy(c, r0, rs, Ps);
    // device-resident scalars: the iteration needs no host round trip (the coefficient
    // recurrences and Algorithm R's update rule run in the reduction tails)
    SolverScalars *S = scalars(c);
    SolverScalars *hS = c->h_scal;  // pinned staging (written only after a synchronisation)
    const int poll = sp->poll_every > 0 ? sp->poll_every : 16;
    QX_CHECK(poll <= kHistRing, QUDAX_ERR_ARG, "poll_every must be <= " + std::to_string(kHistRing));
    {
        const cd rn = cdot_of(c, Ps, r0, rs);
        std::memset(hS, 0, sizeof(*hS));
        hS->rho = make_double2(1, 0);
        hS->rho_new = make_double2(rn.real(), rn.imag());
        hS->alpha = make_double2(1, 0);
        hS->omega = make_double2(1, 0);
        hS->beta = make_double2(0, 0);  // first iteration: p = rs + 0 * (p - omega v) = rs
        hS->rNorm = hS->r0Norm = hS->maxrr = hS->maxrx = bnorm;
        hS->delta = sp->delta;
        hS->stop = stop;
        hS->maxiter = sp->maxiter;
        hS->decide = 1;
        QX_CUDA(cudaMemcpyAsync(S, hS, sizeof(*hS), cudaMemcpyHostToDevice, c->stream));
    }
    int k = 0, updates = 0, restarts = 0, polls = 0, dev_batches = 0;
    bool converged = (bnorm == 0.0);
    const double V_h_all = (double)g.Vh * g.nranks;
    double flops = 0;
    qudax_site_model mm;
    qudax_model(4, 12, -1, &mm);  // 3696 flops / site for Mhat (precision independent)
    const double matpc_flops = mm.flops * V_h_all;
    const double blas_flops_iter = 960.0 * V_h_all;  // reading Q16 (fused BLAS per iteration)

    // one BiCGstab iteration, fully stream-ordered; its scalars stay on the device
    auto enqueue_iteration = [&] {
        {
            void *f[3] = {rs, p, v};
            CoefArg co[2] = {{{0, 0}, &S->beta}, {{0, 0}, &S->omega}};
            blas_op_dev(c, OP_P_UPDATE, Ps, f, co, S, COEF_NONE);      // p = r + beta (p - omega v)
        }
        RedReq red_rv{RED_RHAT_DOT, r0, nullptr, S, COEF_ALPHA};
        matpc_op(c, v, p, Ps, 0, &red_rv, QX_SOLVER_ORDER);           // v = Mhat p; alpha = rho'/<rhat0,v>
        {
            void *f[2] = {v, rs};
            CoefArg co[1] = {{{0, 0}, &S->malpha}};
            blas_op_dev(c, kCaxpyOp, Ps, f, co, S, COEF_NONE);         // s = r - alpha v
        }
        RedReq red_ts{RED_XDOT_NORM, nullptr, nullptr, S, COEF_OMEGA};
        matpc_op(c, t, rs, Ps, 0, &red_ts);                            // t = Mhat s; omega = <t,s>/|t|^2
        {
            void *f[5] = {xs, p, rs, t, r0};
            CoefArg co[2] = {{{0, 0}, &S->alpha}, {{0, 0}, &S->omega}};
            blas_op_dev(c, OP_FINAL, Ps, f, co, S, COEF_RHO);          // x += a p + w s; r = s - w t; rho', beta; decide
        }
    };
    // Batches of up to `poll` iterations run as one cached batch graph (capture_while_graph): the
    // device loops over iterations and the host reads the scalars once per batch.  One iteration
    // per host poll instead: the host transport (its hooks synchronise), eager mode, kernel
    // timing (its event nodes cannot sit in a conditional body), and iterations a WHILE node
    // cannot hold — those replay one iteration as a plain cached graph (or run eagerly).
    const bool host_comm = (c->comm == QUDAX_COMM_HOST);
    const bool use_graph = !host_comm && !(c->flags & QUDAX_FLAG_NO_GRAPHS);
    bool first = true;

    while (!converged && k < sp->maxiter) {
        const std::vector<qudax_ctx::TimingRec> *grecs = nullptr;
        qudax_ctx::Graph *while_graph = nullptr;
        if (!use_graph || first) {
            // eager (the first iteration runs eagerly: it allocates the lazily-created buffers)
            enqueue_iteration();
            first = false;
        } else {
            const std::vector<uintptr_t> key = {1, (uintptr_t)Pd, (uintptr_t)Ps, (uintptr_t)poll, (uintptr_t)rs,
                                                (uintptr_t)xs, (uintptr_t)p, (uintptr_t)v, (uintptr_t)t,
                                                (uintptr_t)r0, (uintptr_t)S, (uintptr_t)c->matpc_sym};
            qudax_ctx::Graph *wg = c->timing ? nullptr : cached_while_graph(c, key, S, poll, enqueue_iteration);
            if (wg) {
                QX_CUDA(cudaGraphLaunch(wg->exec, c->stream));
                c->launches += wg->launches;  // (+ per_iter x the iterations that ran, below)
            } else {
                std::vector<uintptr_t> key1 = key;
                key1[0] = 3;  // one iteration, plain graph
                auto *gr = cached_graph(c, key1, enqueue_iteration);
                if (gr) {
                    QX_CUDA(cudaGraphLaunch(gr->exec, c->stream));
                    c->launches += gr->launches;
                    grecs = &gr->trecs;
                } else {
                    enqueue_iteration();
                }
            }
            while_graph = wg;
        }
        QX_CUDA(cudaMemcpyAsync(hS, S, sizeof(*hS), cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        check_device_error(c);
        ++polls;
        if (while_graph) ++dev_batches;
        const SolverScalars &hs = *hS;
        const int ran = hs.k - k;  // iterations of this batch that ran
        if (grecs) harvest_graph_timing(c, *grecs, ran);
        if (while_graph) c->launches += while_graph->per_iter * ran;
        for (int j = 0; j < ran; ++j) {
            const int kk = k + j + 1;  // 1-based iteration number
            const double rn = hs.hist[(kk - 1) % kHistRing];
            if (c->flags & QUDAX_FLAG_DEBUG_SOLVER)
                std::fprintf(stderr, "qudax it %d: |r| %.6e rho (%.4e,%.4e) alpha (%.4e,%.4e) omega (%.4e,%.4e)\n",
                             kk - 1, rn, hs.rho_new.x, hs.rho_new.y, hs.alpha.x, hs.alpha.y, hs.omega.x, hs.omega.y);
            if (sp->res_history && kk - 1 < sp->history_cap) sp->res_history[kk - 1] = bnorm > 0 ? rn / bnorm : 0.0;
            flops += 2 * matpc_flops + blas_flops_iter;
        }
        k = hs.k;
        if (!hs.halt) continue;
        // ---- reliable update requested by iteration k (Algorithm R; reading R3 for `blown`)
        const double rNorm_it = hs.rNorm;
        const bool blown = hs.blown != 0, updX = hs.updX != 0;
        if (std::isfinite(rNorm_it)) xpy_mixed_op(c, Pd, Ps, xs, x_e);   // x += xs
        zero(c, xs, Ps);
        matpc_op(c, r, x_e, Pd, 0);          // r = Mhat x (high)
        double r2;
        {
            void *f[2] = {bh, r};
            blas_op(c, OP_BMR_NORM, Pd, f, nullptr, &r2);  // r = bhat - r
        }
        flops += matpc_flops;
        convert_op(c, rs, Ps, r, Pd);
        const double rNorm = std::sqrt(r2);
        SolverScalars upd = hs;
        upd.halt = 0;
        upd.updX = upd.blown = 0;
        upd.rNorm = rNorm;
        upd.maxrr = rNorm;
        if (updX || blown) upd.r0Norm = upd.maxrx = rNorm;
        if (blown) {  // restart: rhat0 = r, p = r (beta = 0, v = 0)
            copy(c, r0, rs, Ps);
            zero(c, p, Ps);
            zero(c, v, Ps);
            const cd rn = cdot_of(c, Ps, r0, rs);
            upd.rho = make_double2(1, 0);
            upd.rho_new = make_double2(rn.real(), rn.imag());
            upd.alpha = make_double2(1, 0);
            upd.omega = make_double2(1, 0);
            upd.beta = make_double2(0, 0);
            ++restarts;
        } else {
            // continue the recurrences from the replaced residual: rho' = <rhat0, r>,
            // beta = (rho'/rho)(alpha/omega) with the iteration's rho, alpha, omega
            const cd rn = cdot_of(c, Ps, r0, rs);
            const cd rho(hs.rho.x, hs.rho.y), al(hs.alpha.x, hs.alpha.y), om(hs.omega.x, hs.omega.y);
            const cd beta = (rn / rho) * (al / om);
            upd.rho_new = make_double2(rn.real(), rn.imag());
            upd.beta = make_double2(beta.real(), beta.imag());
        }
        *hS = upd;  // (the stream is idle: blas_op / cdot_of synchronised)
        QX_CUDA(cudaMemcpyAsync(S, hS, sizeof(*hS), cudaMemcpyHostToDevice, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        ++updates;
        if (sp->res_history && k - 1 < sp->history_cap) sp->res_history[k - 1] = bnorm > 0 ? rNorm / bnorm : 0.0;
        if (rNorm <= stop) converged = true;
        st->true_res_schur = bnorm > 0 ? rNorm / bnorm : 0.0;
    }
    st->iters = k;
    st->reliable_updates = updates;
    st->restarts = restarts;
    st->host_polls = polls;
    st->device_batches = dev_batches;
    if (k == 0) st->true_res_schur = bnorm > 0 ? 1.0 : 0.0;

    finish_solution(c, Pd, x_dev, b_e, b_o, x_e, x_o, t_e, t_o, sp->use_schur, st);
    st->flops = flops;
}


// Batched Algorithm R for n <= kMaxRhs right-hand sides ("multi-RHS Dslash /
// block solver"; the paper's tests solve 6 sources per configuration, and production
// calls the solver tens of thousands of times per configuration).  Each system
// keeps its own Krylov space, scalars and reliable-update schedule — the iterates are exactly
// those of n independent solve_dev calls — but the two Mhat applications of an iteration are
// one multi-RHS launch pair for all still-active systems (links and clover streamed once for
// all of them), with the <rhat0, v> and (<t, s>, |t|^2) reductions and scalar recurrences fused
// per right-hand side into the second kernel.  A system leaves the batch when it converges.
void solve_multi_dev(qudax_ctx *c, double *const *x_dev, const double *const *b_dev, int n, const qudax_solve_param *sp,
                     qudax_solve_stats *st) {
    QX_CHECK(n >= 1 && n <= kMaxRhs, QUDAX_ERR_ARG, "nrhs must be 1.." + std::to_string(kMaxRhs));
    QX_CHECK(sp->use_schur >= 0 && sp->use_schur <= 1, QUDAX_ERR_ARG, "multi-RHS solve: use_schur 0 or 1");
    SchurForm form_guard(c, false);
    QX_CHECK(c->gauge_loaded, QUDAX_ERR_STATE, "gauge not loaded");
    const int Pd = sp->prec, Ps = sp->prec_sloppy;
    check_prec(Pd);
    check_prec(Ps);
    QX_CHECK(sp->maxiter >= 0 && sp->tol >= 0 && sp->delta >= 0, QUDAX_ERR_ARG, "solve: bad parameters");
    const Geom &g = c->g;
    if (!c->d_scal_m) {
        c->d_scal_m = static_cast<SolverScalars *>(dalloc(c, sizeof(SolverScalars) * kMaxRhs));
        c->h_scal_m = static_cast<SolverScalars *>(halloc(c, sizeof(SolverScalars) * kMaxRhs));
    }
    struct Sys {
        void *b_e, *b_o, *bh, *x_e, *x_o, *r, *t_e, *t_o, *rs, *xs, *p, *v, *t, *r0;
        SolverScalars *S;
        double bnorm, stop, rNorm, r0Norm, maxrr, maxrx, flops;
        int k, updates, restarts;
        bool converged, active;
    } sys[kMaxRhs];
    qudax_site_model mm;
    qudax_model(4, 12, -1, &mm);
    const double V_h_all = (double)g.Vh * g.nranks;
    const double matpc_flops = mm.flops * V_h_all, blas_flops_iter = 960.0 * V_h_all;
    for (int j = 0; j < n; ++j) {
        auto &w = c->mws[j];
        if (j == 0) QX_CUDA(cudaStreamSynchronize(c->stream));
        ws_select(c, w, Pd, Ps);
        Sys &y = sys[j];
        y.b_e = field(c, w.b_e, Pd); y.b_o = field(c, w.b_o, Pd); y.bh = field(c, w.bh, Pd);
        y.x_e = field(c, w.x_e, Pd); y.x_o = field(c, w.x_o, Pd); y.r = field(c, w.r, Pd);
        y.t_e = field(c, w.t_e, Pd); y.t_o = field(c, w.t_o, Pd);
        y.rs = field(c, w.rs, Ps); y.xs = field(c, w.xs, Ps); y.p = field(c, w.p, Ps);
        y.v = field(c, w.v, Ps); y.t = field(c, w.t, Ps); y.r0 = field(c, w.r0, Ps);
        y.S = c->d_scal_m + j;
        std::memset(&st[j], 0, sizeof(st[j]));
        prepare_source(c, Pd, b_dev[j], y.b_e, y.b_o, y.bh, y.t_e, y.t_o, sp->use_schur);
        y.bnorm = std::sqrt(norm2_of(c, Pd, y.bh));
        y.stop = sp->tol * y.bnorm;
        zero(c, y.x_e, Pd);
        zero(c, y.xs, Ps);
        zero(c, y.v, Ps);
        zero(c, y.p, Ps);
        copy(c, y.r, y.bh, Pd);
        convert_op(c, y.rs, Ps, y.r, Pd);
        copy(c, y.r0, y.rs, Ps);
        y.rNorm = y.r0Norm = y.maxrr = y.maxrx = y.bnorm;
        y.flops = 0;
        y.k = y.updates = y.restarts = 0;
        y.converged = (y.bnorm == 0.0);
        y.active = !y.converged && sp->maxiter > 0;
        SolverScalars h0{};
        const cd rn = cdot_of(c, Ps, y.r0, y.rs);
        h0.rho = make_double2(1, 0);
        h0.rho_new = make_double2(rn.real(), rn.imag());
        h0.alpha = make_double2(1, 0);
        h0.omega = make_double2(1, 0);
        QX_CUDA(cudaMemcpyAsync(y.S, &h0, sizeof(h0), cudaMemcpyHostToDevice, c->stream));
    }
    // one iteration of every active system; all scalars stay on the device
    auto enqueue_iteration = [&](unsigned mask) {
        void *vv[kMaxRhs], *pp[kMaxRhs], *tt[kMaxRhs], *ss[kMaxRhs];
        RedReq red_rv[kMaxRhs], red_ts[kMaxRhs];
        int na = 0;
        for (int j = 0; j < n; ++j) {
            if (!(mask >> j & 1)) continue;
            Sys &y = sys[j];
            void *f[3] = {y.rs, y.p, y.v};
            CoefArg co[2] = {{{0, 0}, &y.S->beta}, {{0, 0}, &y.S->omega}};
            blas_op_dev(c, OP_P_UPDATE, Ps, f, co, y.S, COEF_NONE);  // p = r + beta (p - omega v)
            vv[na] = y.v; pp[na] = y.p; tt[na] = y.t; ss[na] = y.rs;
            red_rv[na] = RedReq{RED_RHAT_DOT, y.r0, nullptr, y.S, COEF_ALPHA};
            red_ts[na] = RedReq{RED_XDOT_NORM, nullptr, nullptr, y.S, COEF_OMEGA};
            ++na;
        }
        matpc_multi_op(c, vv, pp, na, Ps, 0, red_rv, QX_SOLVER_ORDER);  // v = Mhat p; alpha = rho'/<rhat0, v>
        for (int j = 0; j < n; ++j) {
            if (!(mask >> j & 1)) continue;
            void *f[2] = {sys[j].v, sys[j].rs};
            CoefArg co[1] = {{{0, 0}, &sys[j].S->malpha}};
            blas_op_dev(c, kCaxpyOp, Ps, f, co, sys[j].S, COEF_NONE);  // s = r - alpha v
        }
        matpc_multi_op(c, tt, ss, na, Ps, 0, red_ts);  // t = Mhat s; omega = <t,s>/|t|^2
        for (int j = 0; j < n; ++j) {
            if (!(mask >> j & 1)) continue;
            Sys &y = sys[j];
            void *f[5] = {y.xs, y.p, y.rs, y.t, y.r0};
            CoefArg co[2] = {{{0, 0}, &y.S->alpha}, {{0, 0}, &y.S->omega}};
            blas_op_dev(c, OP_FINAL, Ps, f, co, y.S, COEF_RHO);  // x += a p + w s; r = s - w t; rho', beta
        }
        QX_CUDA(cudaMemcpyAsync(c->h_scal_m, c->d_scal_m, sizeof(SolverScalars) * n, cudaMemcpyDeviceToHost, c->stream));
    };
    const bool use_graph = (c->comm != QUDAX_COMM_HOST) && !(c->flags & QUDAX_FLAG_NO_GRAPHS);
    bool first = true;
    for (;;) {
        unsigned mask = 0;
        for (int j = 0; j < n; ++j)
            if (sys[j].active) mask |= 1u << j;
        if (!mask) break;
        const std::vector<qudax_ctx::TimingRec> *grecs = nullptr;
        if (!use_graph || first) {
            enqueue_iteration(mask);  // the first iteration runs eagerly (lazily-created buffers)
            first = false;
        } else {
            // one cached graph per active set (and workspace): every system's fields and scalars
            std::vector<uintptr_t> key = {2, (uintptr_t)Pd, (uintptr_t)Ps, (uintptr_t)mask, (uintptr_t)n,
                                          (uintptr_t)c->d_scal_m};
            for (int j = 0; j < n; ++j)
                for (void *f : {sys[j].rs, sys[j].xs, sys[j].p, sys[j].v, sys[j].t, sys[j].r0}) key.push_back((uintptr_t)f);
            auto *gr = cached_graph(c, key, [&] { enqueue_iteration(mask); });
            if (gr) {
                QX_CUDA(cudaGraphLaunch(gr->exec, c->stream));
                c->launches += gr->launches;
                grecs = &gr->trecs;
            } else {
                enqueue_iteration(mask);
            }
        }
        QX_CUDA(cudaStreamSynchronize(c->stream));
        if (grecs) harvest_graph_timing(c, *grecs, 1);
        for (int j = 0; j < n; ++j) {
            Sys &y = sys[j];
            if (!y.active) continue;
            const SolverScalars &hs = c->h_scal_m[j];
            const double rNorm_it = std::sqrt(hs.r2);
            const bool blown = !std::isfinite(rNorm_it) || rNorm_it > 1e2 * y.maxrr;  // reading R3
            y.rNorm = rNorm_it;
            ++y.k;
            y.flops += 2 * matpc_flops + blas_flops_iter;
            if (!blown) {
                if (y.rNorm > y.maxrx) y.maxrx = y.rNorm;
                if (y.rNorm > y.maxrr) y.maxrr = y.rNorm;
            }
            const bool updX = !blown && (y.rNorm < sp->delta * y.r0Norm) && (y.r0Norm <= y.maxrx);
            const bool updR = blown || ((y.rNorm < sp->delta * y.maxrr) && (y.r0Norm <= y.maxrr)) || updX ||
                              (y.rNorm <= y.stop) || (y.k == sp->maxiter);
            if (updR) {  // reliable update of system j alone (single-RHS high-precision operator)
                if (std::isfinite(rNorm_it)) xpy_mixed_op(c, Pd, Ps, y.xs, y.x_e);
                zero(c, y.xs, Ps);
                matpc_op(c, y.r, y.x_e, Pd, 0);
                double r2;
                {
                    void *f[2] = {y.bh, y.r};
                    blas_op(c, OP_BMR_NORM, Pd, f, nullptr, &r2);
                }
                y.flops += matpc_flops;
                convert_op(c, y.rs, Ps, y.r, Pd);
                y.rNorm = std::sqrt(r2);
                y.maxrr = y.rNorm;
                const bool restart = blown;
                if (updX || restart) y.r0Norm = y.maxrx = y.rNorm;
                SolverScalars upd = hs;
                if (restart) {
                    copy(c, y.r0, y.rs, Ps);
                    zero(c, y.p, Ps);
                    zero(c, y.v, Ps);
                    const cd rn = cdot_of(c, Ps, y.r0, y.rs);
                    upd.rho = make_double2(1, 0);
                    upd.rho_new = make_double2(rn.real(), rn.imag());
                    upd.alpha = make_double2(1, 0);
                    upd.omega = make_double2(1, 0);
                    upd.beta = make_double2(0, 0);
                    ++y.restarts;
                } else {
                    const cd rn = cdot_of(c, Ps, y.r0, y.rs);
                    const cd rho(hs.rho.x, hs.rho.y), al(hs.alpha.x, hs.alpha.y), om(hs.omega.x, hs.omega.y);
                    const cd beta = (rn / rho) * (al / om);
                    upd.rho_new = make_double2(rn.real(), rn.imag());
                    upd.beta = make_double2(beta.real(), beta.imag());
                }
                QX_CUDA(cudaMemcpyAsync(y.S, &upd, sizeof(upd), cudaMemcpyHostToDevice, c->stream));
                QX_CUDA(cudaStreamSynchronize(c->stream));
                ++y.updates;
                if (y.rNorm <= y.stop) y.converged = true;
            }
            if (y.converged || y.k >= sp->maxiter) y.active = false;
            if (j == 0 && sp->res_history && y.k - 1 < sp->history_cap)
                sp->res_history[y.k - 1] = y.bnorm > 0 ? y.rNorm / y.bnorm : 0.0;
        }
    }
    for (int j = 0; j < n; ++j) {
        Sys &y = sys[j];
        st[j].iters = y.k;
        st[j].reliable_updates = y.updates;
        st[j].restarts = y.restarts;
        st[j].true_res_schur = y.bnorm > 0 ? y.rNorm / y.bnorm : 0.0;
        finish_solution(c, Pd, x_dev[j], y.b_e, y.b_o, y.x_e, y.x_o, y.t_e, y.t_o, sp->use_schur, &st[j]);
        st[j].flops = y.flops;
    }
}

// CGNR ("Conjugate Gradients on the normal equations"): CG on the Hermitian
// positive-definite Mhat^dag Mhat x = Mhat^dag bhat, in precision sp->prec (no reliable
// updates).  The stopping test is on the TRUE residual of the original Schur system,
// ||bhat - Mhat x|| <= tol ||bhat||, evaluated whenever the iterated normal-equation residual
// has dropped far enough to make it plausible, and every 50 iterations.
void cgnr_dev(qudax_ctx *c, double *x_dev, const double *b_dev, const qudax_solve_param *sp, qudax_solve_stats *st) {
    QX_CHECK(sp->use_schur >= 0 && sp->use_schur <= 2, QUDAX_ERR_ARG, "use_schur must be 0, 1 or 2");
    SchurForm form_guard(c, sp->use_schur == 2);
    QX_CHECK(c->gauge_loaded, QUDAX_ERR_STATE, "gauge not loaded");
    const int P = sp->prec;
    check_prec(P);
    QX_CHECK(sp->maxiter >= 0 && sp->tol >= 0, QUDAX_ERR_ARG, "cgnr: bad parameters");
    std::memset(st, 0, sizeof(*st));
    auto &w = c->cgws;
    QX_CUDA(cudaStreamSynchronize(c->stream));
    ws_select(c, w, P, P);
    const Geom &g = c->g;
    void *b_e = field(c, w.b_e, P), *b_o = field(c, w.b_o, P), *bh = field(c, w.bh, P);
    void *x_e = field(c, w.x_e, P), *x_o = field(c, w.x_o, P), *r = field(c, w.r, P);
    void *t_e = field(c, w.t_e, P), *t_o = field(c, w.t_o, P);
    void *p = field(c, w.p, P), *ap = field(c, w.v, P), *tmp = field(c, w.t, P);
    prepare_source(c, P, b_dev, b_e, b_o, bh, t_e, t_o, sp->use_schur);
    const double bnorm = std::sqrt(norm2_of(c, P, bh));
    const double stop = sp->tol * bnorm;
    zero(c, x_e, P);
    matpc_op(c, r, bh, P, 1);  // r = Mhat^dag bhat (x = 0)
    copy(c, p, r, P);
    double rr = norm2_of(c, P, r);
    const double rr0 = rr;
    const double V_h_all = (double)g.Vh * g.nranks;
    qudax_site_model mm;
    qudax_model(4, 12, -1, &mm);
    double flops = 0;
    int k = 0;
    double true_res = bnorm;
    bool converged = (bnorm == 0.0);
    auto true_residual = [&]() {  // ||bhat - Mhat x||
        matpc_op(c, tmp, x_e, P, 0);
        double r2;
        void *f[2] = {bh, tmp};
        blas_op(c, OP_BMR_NORM, P, f, nullptr, &r2);
        flops += mm.flops * V_h_all;
        return std::sqrt(r2);
    };
    while (!converged && k < sp->maxiter) {
        matpc_op(c, tmp, p, P, 0);  // Ap = Mhat^dag Mhat p
        matpc_op(c, ap, tmp, P, 1);
        const cd pap = cdot_of(c, P, p, ap);
        const double alpha = rr / pap.real();
        {
            void *f[2] = {p, x_e};
            double co[2] = {alpha, 0.0};
            blas_op(c, OP_CAXPY, P, f, co, nullptr);  // x += alpha p
        }
        {
            void *f[2] = {ap, r};
            double co[2] = {-alpha, 0.0};
            blas_op(c, OP_CAXPY, P, f, co, nullptr);  // r -= alpha Ap
        }
        const double rr_new = norm2_of(c, P, r);
        const double beta = rr_new / rr;
        rr = rr_new;
        {
            void *f[3] = {r, p, p};
            double a = beta;
            blas_op(c, OP_XPAY, P, f, &a, nullptr);  // p = r + beta p
        }
        ++k;
        flops += (4 * mm.flops + 8 * 96) * V_h_all;  // 2 Mhat applications per M^dag M, 4 BLAS
        // the normal-equation residual bounds the true one: |r_true| <= |r_n| / sigma_min
        if (std::sqrt(rr / rr0) <= sp->tol || k % 50 == 0 || k == sp->maxiter) {
            true_res = true_residual();
            if (true_res <= stop) converged = true;
        }
        if (sp->res_history && k - 1 < sp->history_cap) sp->res_history[k - 1] = std::sqrt(rr / rr0);
    }
    if (!converged && k == 0) true_res = true_residual();
    st->iters = k;
    st->true_res_schur = bnorm > 0 ? true_res / bnorm : 0.0;
    finish_solution(c, P, x_dev, b_e, b_o, x_e, x_o, t_e, t_o, sp->use_schur, st);
    st->flops = flops;
}

}  // namespace qx
