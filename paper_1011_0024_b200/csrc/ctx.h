// ctx.h — the runtime context behind the opaque qudax_ctx (host C++).
#pragma once
#include <nccl.h>

#include <string>
#include <vector>

#include "internal.h"

struct qudax_ctx {
    qx::Geom g{};
    int device = 0;
    int comm = QUDAX_COMM_NONE;
    int overlap = 1;
    cudaStream_t stream = nullptr, comm_stream = nullptr;
    bool own_stream = false;
    cudaEvent_t ev_in = nullptr, ev_halo = nullptr;
    // diagnostic halo-overlap timeline (qudax_halo_timeline)
    bool tl_on = false, tl_valid = false;
    cudaEvent_t tl[8] = {};
    ncclComm_t nccl = nullptr;      // halo send/recv (comm stream) and setup exchanges
    ncclComm_t nccl_red = nullptr;  // global sums (compute stream): split from nccl
    qudax_alloc_fn dev_alloc = nullptr;
    qudax_free_fn dev_free = nullptr;
    void *alloc_user = nullptr;
    qudax_exchange_fn host_exchange = nullptr;
    qudax_allreduce_fn host_allreduce = nullptr;
    void *comm_user = nullptr;

    std::string err;
    bool sticky = false;
    long long launches = 0;
    // optional per-launch CUDA-event timing of the Dslash kernels (qudax_kernel_timing)
    int timing = 0;  // 0 off, 1 CUDA events per Dslash launch, 2 events + in-kernel span
    struct TimingRec {
        cudaEvent_t a, b;
        int prec, recon, kind;
        long sites;
        int nrhs = 1;  // multi-RHS launch: links and clover are compulsory once, spinors per RHS
        int red = 0;   // fused reduction kind (RED_RHAT_DOT reads rhat: +1 spinor per site)
        int iter = 0;  // graph-captured launches: solver iteration within the batch
        int span = -1; // slot of the launch's in-kernel span (first-CTA start, last-CTA end)
    };
    std::vector<TimingRec> trecs;
    std::vector<cudaEvent_t> ev_pool;
    // Dslash launches inside a captured CUDA graph: their (external) events are re-recorded at
    // every replay, so they are harvested into running sums after each replay
    std::vector<TimingRec> graph_trecs;
    // solver iteration batches captured as CUDA graphs, cached across solves (keyed by every
    // pointer and parameter the captured launches bake in; gauge_epoch changes on gauge_load)
    struct Graph {
        std::vector<uintptr_t> key;
        cudaGraphExec_t exec = nullptr;
        long long launches = 0;          // library kernels per replay (WHILE graphs: outside the loop)
        long long per_iter = 0;          // WHILE graphs: library kernels per loop iteration
        bool no_while = false;           // this key's iteration cannot sit in a WHILE node
        std::vector<TimingRec> trecs;    // event-bracketed Dslash launches (kernel timing on)
    };
    std::vector<Graph> graphs;
    long long gauge_epoch = 0;
    struct TimingAcc {
        long long launches = 0, sites = 0;
        double ms = 0, flops = 0, bytes_c = 0, bytes_p = 0, span_ms = 0;
    } tacc[3];
    // in-kernel spans of the timed launches (device slots of 4 u64, host copy for harvesting)
    unsigned long long *d_span = nullptr, *h_span = nullptr;
    int span_next = 0;
    bool capturing = false;
    int cap_iter = 0;           // solver iteration (within the captured batch) being captured
    int flags = 0;              // qudax_init_flag bits
    // device error word in mapped pinned host memory (kernel-initiated halo wait timeout)
    int *h_err = nullptr, *d_err = nullptr;
    // the Schur form matpc_op applies: 0 asymmetric (default), 1 symmetric (set by a solve with
    // use_schur = 2 for its duration, and by qudax_matpc_sym)
    int matpc_sym = 0;
    qx::SolverScalars *d_scal = nullptr, *h_scal = nullptr;
    std::vector<void *> allocs;       // device allocations owned by the ctx
    std::vector<void *> host_allocs;  // pinned host allocations

    // gauge + clover
    bool gauge_loaded = false;
    double kappa = 0, csw = 0;
    int t_bc = -1;
    struct GaugeCopy {
        int prec = 0, recon = 0;
        void *d[4][2] = {};
        void *ghost[4][2] = {};  // backward ghost links U_mu(x - mu) at x_mu = -1 per split mu, per parity
    };
    GaugeCopy gcopy[2];
    int ncopies = 0;
    struct Clover {
        bool valid = false;
        void *T[2] = {}, *Tinv[2] = {};
    } clov[3];  // index by prec_idx

    struct Halo {
        bool valid = false;
        size_t bytes = 0;
        void *sb = nullptr, *sf = nullptr, *gb = nullptr, *gf = nullptr;
        void *h_sb = nullptr, *h_sf = nullptr, *h_gb = nullptr, *h_gf = nullptr;
        // partitioned X / Y / Z: projected faces per dimension (send/ghost, back/fwd)
        size_t sbytes[3] = {};
        void *ssb[3] = {}, *ssf[3] = {}, *sgb[3] = {}, *sgf[3] = {};
        void *h_ssb[3] = {}, *h_ssf[3] = {}, *h_sgb[3] = {}, *h_sgf[3] = {};
        // multi-RHS T halo: kMaxRhs faces per buffer, RHS k at k * m_stride (one message per
        // direction carries every right-hand side)
        size_t m_stride = 0;
        void *m_sb = nullptr, *m_sf = nullptr, *m_gb = nullptr, *m_gf = nullptr;
        void *mh_sb = nullptr, *mh_sf = nullptr, *mh_gb = nullptr, *mh_gf = nullptr;
    } halo[3];
    int *blist = nullptr;  // boundary sites (complement of the interior box) when X/Y/Z is split
    // NCCL halo in tail mode: flags[4][2], producer seq, consumer seq, consumer CTA counter (device)
    unsigned *tflags = nullptr;

    // kernel-initiated halo over peer memory (QUDAX_HALO_P2P).  One cudaMalloc region per rank,
    // identical layout on every rank: per precision and split dimension mu ghost_back[2],
    // ghost_fwd[2] (sequence parity), then flags[4][2] (flags[mu][0] raised by the backward
    // neighbour along mu after it filled ghost_back, flags[mu][1] by the forward one after
    // ghost_fwd), the producer (pack) and consumer (Dslash) halo counters and their CTA
    // counters, and the kernel-side allreduce slots.
    struct P2P {
        bool on = false;
        char *base = nullptr;                       // own region (cudaMalloc, IPC-exported)
        char *peer_b[4] = {}, *peer_f[4] = {};           // neighbours' regions per dimension (IPC-mapped or own)
        char *peer[qx::kMaxPeers] = {};                  // every rank's region (nranks <= kMaxPeers)
        std::vector<char *> opened;                      // IPC mappings to close at finalize
        // per precision and split dimension: ghost_back / ghost_fwd (x2 sequence parities)
        size_t off_g[3][4][2] = {}, pdist[3][4] = {};
        size_t off_flags = 0, off_seq = 0, off_count = 0, off_cseq = 0, off_ccount = 0, off_ar = 0, bytes = 0;
    } p2p;
    // kernel-side allreduce descriptor (device memory) of the P2P mode, nullptr otherwise
    qx::DevAllreduce *dar = nullptr;

    // workspace
    void *tmp_odd[3] = {}, *tmp_even[3] = {}, *tmp_sym[3] = {};
    void *tmp_multi[3][qx::kMaxRhs] = {};
    double *partials = nullptr, *red_out = nullptr, *h_red = nullptr;
    double *dpart = nullptr;  // per-CTA partials of Dslash-fused reductions
    unsigned *d_counter = nullptr;  // last-CTA counter of the stream-ordered reductions
    double *dpart_m = nullptr;      // multi-RHS fused reductions: per-RHS CTA slots and counters
    unsigned *dcount_m = nullptr;
    double *stage = nullptr;  // fp64 full-slab staging (V_loc * 24 doubles)
    // pageable host <-> device copies (api.cpp: h2d / d2h): a ring of pinned chunks that CPU
    // threads fill (drain) while the copy engine moves the previous chunk
    struct XferRing {
        char *buf[4] = {};
        cudaEvent_t done[4] = {};
        size_t chunk = 0;
    } xfer;
    int *d_flag = nullptr;

    // solver workspace (lazily allocated per (prec, prec_sloppy))
    struct SolverWs {
        int prec = 0, prec_s = 0;
        void *b_e = nullptr, *b_o = nullptr, *bh = nullptr, *x_e = nullptr, *x_o = nullptr, *r = nullptr, *t_e = nullptr,
             *t_o = nullptr;
        void *rs = nullptr, *xs = nullptr, *p = nullptr, *v = nullptr, *t = nullptr, *r0 = nullptr;
    } sws, cgws, mws[qx::kMaxRhs];
    qx::SolverScalars *d_scal_m = nullptr, *h_scal_m = nullptr;  // batched solver: one set per RHS
};

namespace qx {
inline int prec_idx(int prec) { return prec == 8 ? 0 : (prec == 4 ? 1 : 2); }
void *dalloc(qudax_ctx *c, size_t bytes);
void *halloc(qudax_ctx *c, size_t bytes);
void dfree(qudax_ctx *c, void *p);  // releases a dalloc'ed buffer (no-op for nullptr)
void *tmp_odd_field(qudax_ctx *c, int prec);  // the ctx's odd scratch field of precision prec
void check_prec(int prec);
// optional reduction fused into a Dslash epilogue (see DslashRed); res: 3 global sums (host)
struct RedReq {
    int kind;
    const void *rhat;
    double *res;              // host results (S == nullptr), or
    SolverScalars *S = nullptr; // device: sums land in S->red, then the recurrence coef_mode
    int coef_mode = COEF_NONE;
};
void dslash_op(qudax_ctx *c, void *out, const void *in, const void *x, int prec, int p, int dagger, int kind,
               double a, const RedReq *red = nullptr, int reverse = 0);
// order 0: first kernel bottom-up, second top-down; order 1: the reverse (solver.cpp: each kernel
// starts where the previous one ended, so the first fields it reads are still in L2)
void matpc_op(qudax_ctx *c, void *out, const void *in, int prec, int dagger, const RedReq *red = nullptr,
              int order = 0);
void matpc_sym_op(qudax_ctx *c, void *out, const void *in, int prec, int dagger, const RedReq *red = nullptr);
void dslash_multi_op(qudax_ctx *c, void *const *out, const void *const *in, const void *const *x, int n, int prec,
                     int p, int dagger, int kind, double a, int reverse, const RedReq *reds = nullptr);
void matpc_multi_op(qudax_ctx *c, void *const *out, const void *const *in, int n, int prec, int dagger,
                    const RedReq *reds = nullptr, int order = 0);
void solve_multi_dev(qudax_ctx *c, double *const *x_dev, const double *const *b_dev, int n, const qudax_solve_param *p,
                     qudax_solve_stats *st);
int dslash_threads();
void clover_apply_op(qudax_ctx *c, void *out, const void *in, int prec, int parity, bool inverse);
// run a BLAS op; if it reduces, globally sum and return the values in res (host)
int blas_op(qudax_ctx *c, int op, int prec, void *const *f, const double *coef, double *res);
void blas_op_dev(qudax_ctx *c, int op, int prec, void *const *f, const CoefArg *co, SolverScalars *S, int mode);
void device_sum_coef(qudax_ctx *c, double *dev_vals, int n, SolverScalars *S, int mode);
void xpy_mixed_op(qudax_ctx *c, int pd, int ps, const void *x, void *y);
void convert_op(qudax_ctx *c, void *dst, int pd, const void *src, int ps);
void solve_dev(qudax_ctx *c, double *x_dev, const double *b_dev, const qudax_solve_param *p, qudax_solve_stats *st);
void cgnr_dev(qudax_ctx *c, double *x_dev, const double *b_dev, const qudax_solve_param *p, qudax_solve_stats *st);
void harvest_graph_timing(qudax_ctx *c, const std::vector<qudax_ctx::TimingRec> &recs, int iters);
void release_graph_timing(qudax_ctx *c, std::vector<qudax_ctx::TimingRec> &recs);
// destroy the cached solver graphs (gauge_load: they baked in the old gauge / clover)
void drop_graphs(qudax_ctx *c);
// raise QUDAX_ERR_COMM if a kernel set the device error word (call after a synchronisation)
void check_device_error(qudax_ctx *c);
}  // namespace qx
