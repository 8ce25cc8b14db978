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
    ncclComm_t nccl = nullptr;
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
    bool timing = false;
    struct TimingRec {
        cudaEvent_t a, b;
        int prec, recon, kind;
        long sites;
    };
    std::vector<TimingRec> trecs;
    std::vector<cudaEvent_t> ev_pool;
    std::vector<void *> allocs;       // device allocations owned by the ctx
    std::vector<void *> host_allocs;  // pinned host allocations

    // gauge + clover
    bool gauge_loaded = false;
    double kappa = 0, csw = 0;
    int t_bc = -1;
    struct GaugeCopy {
        int prec = 0, recon = 0;
        void *d[4][2] = {};
        void *ghost[2] = {};
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
    } halo[3];

    // workspace
    void *tmp_odd[3] = {}, *tmp_even[3] = {};
    double *partials = nullptr, *red_out = nullptr, *h_red = nullptr;
    double *stage = nullptr;  // fp64 full-slab staging (V_loc * 24 doubles)
    int *d_flag = nullptr;

    // solver workspace (lazily allocated per (prec, prec_sloppy))
    struct SolverWs {
        int prec = 0, prec_s = 0;
        void *b_e = nullptr, *b_o = nullptr, *bh = nullptr, *x_e = nullptr, *x_o = nullptr, *r = nullptr, *t_e = nullptr,
             *t_o = nullptr;
        void *rs = nullptr, *xs = nullptr, *p = nullptr, *v = nullptr, *t = nullptr, *r0 = nullptr;
    } sws;
};

namespace qx {
inline int prec_idx(int prec) { return prec == 8 ? 0 : (prec == 4 ? 1 : 2); }
void *dalloc(qudax_ctx *c, size_t bytes);
void *halloc(qudax_ctx *c, size_t bytes);
void check_prec(int prec);
void dslash_op(qudax_ctx *c, void *out, const void *in, const void *x, int prec, int p, int dagger, int kind,
               double a);
void matpc_op(qudax_ctx *c, void *out, const void *in, int prec, int dagger);
void clover_apply_op(qudax_ctx *c, void *out, const void *in, int prec, int parity, bool inverse);
// run a BLAS op; if it reduces, globally sum and return the values in res (host)
int blas_op(qudax_ctx *c, int op, int prec, void *const *f, const double *coef, double *res);
void xpy_mixed_op(qudax_ctx *c, int pd, int ps, const void *x, void *y);
void convert_op(qudax_ctx *c, void *dst, int pd, const void *src, int ps);
void solve_dev(qudax_ctx *c, double *x_dev, const double *b_dev, const qudax_solve_param *p, qudax_solve_stats *st);
}  // namespace qx
