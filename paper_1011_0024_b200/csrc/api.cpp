// api.cpp — the extern "C" boundary (include/qudax.h) and the host runtime behind it:
// context, device memory, gauge/clover setup, the T-direction halo orchestration
// (pack -> NCCL send/recv on a comm stream -> interior kernel -> boundary kernel,
// P:692-720), and global reductions.
#include <cuda_runtime.h>
#include <nccl.h>

#include <algorithm>
#include <chrono>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <map>
#include <condition_variable>
#include <functional>
#include <mutex>
#include <thread>
#include <vector>
#include <tuple>

#include "ctx.h"

using qx::Error;

#define QX_NCCL(call)                                                                              \
    do {                                                                                           \
        ncclResult_t r_ = (call);                                                                  \
        if (r_ != ncclSuccess) throw Error(QUDAX_ERR_NCCL, std::string(#call) + ": " + ncclGetErrorString(r_)); \
    } while (0)

namespace qx {

void *dalloc(qudax_ctx *c, size_t bytes) {
    if (bytes == 0) bytes = 16;
    void *p = nullptr;
    if (c->dev_alloc) {
        p = c->dev_alloc(bytes, c->alloc_user);
        if (!p) throw Error(QUDAX_ERR_OOM, "dev_alloc hook returned NULL for " + std::to_string(bytes) + " bytes");
    } else {
        cudaError_t e = cudaMalloc(&p, bytes);
        if (e != cudaSuccess) {
            cudaGetLastError();
            throw Error(QUDAX_ERR_OOM, "cudaMalloc(" + std::to_string(bytes) + "): " + cudaGetErrorString(e));
        }
    }
    c->allocs.push_back(p);
    return p;
}

void *halloc(qudax_ctx *c, size_t bytes) {
    void *p = nullptr;
    QX_CUDA(cudaMallocHost(&p, std::max<size_t>(bytes, 16)));
    c->host_allocs.push_back(p);
    return p;
}

static void hfree(qudax_ctx *c, void *p) {
    if (!p) return;
    auto it = std::find(c->host_allocs.begin(), c->host_allocs.end(), p);
    if (it != c->host_allocs.end()) c->host_allocs.erase(it);
    cudaFreeHost(p);
}

// ---- host <-> device copies of user (typically pageable) host arrays.  A plain cudaMemcpy
// from pageable memory runs at ~11 GB/s H2D / ~18 GB/s D2H on the B200 box (the driver stages
// through its own bounce buffer on one CPU thread), against ~55 GB/s from pinned memory
// (scripts/diag_transfer.py).  Here several CPU threads copy each chunk into (out of) a ring of
// pinned chunks while the copy engine moves the previous one.  Pinned sources / destinations
// (e.g. torch pin_memory tensors) go straight to cudaMemcpyAsync.  Synchronous in both
// directions (the caller's buffer is free / filled on return).
static bool host_is_pinned(const void *p) {
    cudaPointerAttributes at{};
    if (cudaPointerGetAttributes(&at, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return at.type == cudaMemoryTypeHost;
}
// A small persistent pool for the host copies (creating the threads per chunk cost more than
// the copies' parallel speed-up).  Process-wide, started on first use, never torn down
// (detached workers idle on a condition variable).
class CopyPool {
  public:
    explicit CopyPool(int n) : n_(n) {
        for (int t = 0; t < n_ - 1; ++t) std::thread([this, t] { worker(t + 1); }).detach();
    }
    int size() const { return n_; }
    // run f(part) for part = 0 .. n-1 on the pool (part 0 on the caller), then return
    template <typename F>
    void run(F &&f) {
        std::lock_guard<std::mutex> one_job(run_m_);  // contexts used from several host threads
        std::unique_lock<std::mutex> lk(m_);
        job_ = f;
        pending_ = n_ - 1;
        ++gen_;
        lk.unlock();
        cv_.notify_all();
        f(0);
        lk.lock();
        done_.wait(lk, [&] { return pending_ == 0; });
        job_ = nullptr;
    }

  private:
    void worker(int id) {
        unsigned seen = 0;
        for (;;) {
            std::function<void(int)> f;
            {
                std::unique_lock<std::mutex> lk(m_);
                cv_.wait(lk, [&] { return gen_ != seen; });
                seen = gen_;
                f = job_;
            }
            f(id);
            std::lock_guard<std::mutex> lk(m_);
            if (--pending_ == 0) done_.notify_one();
        }
    }
    int n_;
    std::mutex run_m_, m_;
    std::condition_variable cv_, done_;
    std::function<void(int)> job_;
    int pending_ = 0;
    unsigned gen_ = 0;
};
static int g_copy_threads = 0;  // qudax_init_param.copy_threads of the first context (0 = default)
static CopyPool &copy_pool() {
    static CopyPool *pool = [] {
        const int hw = (int)std::thread::hardware_concurrency();
        return new CopyPool(g_copy_threads > 0 ? g_copy_threads : std::max(1, std::min(8, hw)));
    }();
    return *pool;
}
static void par_memcpy(void *dst, const void *src, size_t n) {
    auto &pool = copy_pool();
    const int nt = pool.size();
    if (nt == 1 || n < ((size_t)2 << 20)) {
        std::memcpy(dst, src, n);
        return;
    }
    const size_t part = (n / nt + 63) & ~(size_t)63;
    pool.run([=](int t) {
        const size_t o = (size_t)t * part;
        if (o >= n) return;
        std::memcpy(static_cast<char *>(dst) + o, static_cast<const char *>(src) + o, std::min(part, n - o));
    });
}
static qudax_ctx::XferRing &xfer_ring(qudax_ctx *c) {
    auto &r = c->xfer;
    if (!r.chunk) {
        r.chunk = (size_t)32 << 20;
        for (int k = 0; k < 4; ++k) {
            r.buf[k] = static_cast<char *>(halloc(c, r.chunk));
            QX_CUDA(cudaEventCreateWithFlags(&r.done[k], cudaEventDisableTiming));
        }
    }
    return r;
}
static void h2d(qudax_ctx *c, void *dst, const void *src, size_t n) {
    if (n < ((size_t)8 << 20) || host_is_pinned(src)) {
        QX_CUDA(cudaMemcpyAsync(dst, src, n, cudaMemcpyHostToDevice, c->stream));
        return;
    }
    auto &r = xfer_ring(c);
    size_t k = 0;
    for (size_t o = 0; o < n; o += r.chunk, ++k) {
        const int s = (int)(k % 4);
        const size_t len = std::min(r.chunk, n - o);
        QX_CUDA(cudaEventSynchronize(r.done[s]));  // the copy that last used this slot is done
        par_memcpy(r.buf[s], static_cast<const char *>(src) + o, len);
        QX_CUDA(cudaMemcpyAsync(static_cast<char *>(dst) + o, r.buf[s], len, cudaMemcpyHostToDevice, c->stream));
        QX_CUDA(cudaEventRecord(r.done[s], c->stream));
    }
}
static void d2h(qudax_ctx *c, void *dst, const void *src, size_t n) {
    if (n < ((size_t)8 << 20) || host_is_pinned(dst)) {
        QX_CUDA(cudaMemcpyAsync(dst, src, n, cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        return;
    }
    auto &r = xfer_ring(c);
    const size_t nch = (n + r.chunk - 1) / r.chunk;
    auto issue = [&](size_t k) {
        const size_t o = k * r.chunk, len = std::min(r.chunk, n - o);
        QX_CUDA(cudaMemcpyAsync(r.buf[k % 4], static_cast<const char *>(src) + o, len, cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaEventRecord(r.done[k % 4], c->stream));
    };
    for (size_t k = 0; k < std::min<size_t>(nch, 3); ++k) issue(k);  // copies run ahead of the drain
    for (size_t k = 0; k < nch; ++k) {
        QX_CUDA(cudaEventSynchronize(r.done[k % 4]));
        const size_t o = k * r.chunk, len = std::min(r.chunk, n - o);
        if (k + 3 < nch) issue(k + 3);
        par_memcpy(static_cast<char *>(dst) + o, r.buf[k % 4], len);
    }
}

void dfree(qudax_ctx *c, void *p) {
    if (!p) return;
    auto it = std::find(c->allocs.begin(), c->allocs.end(), p);
    if (it != c->allocs.end()) c->allocs.erase(it);
    if (c->dev_free) c->dev_free(p, c->alloc_user);
    else cudaFree(p);
}

void check_prec(int prec) {
    QX_CHECK(prec == 2 || prec == 4 || prec == 8, QUDAX_ERR_ARG, "precision must be 2, 4 or 8");
}

static qudax_ctx::GaugeCopy &gauge_for(qudax_ctx *c, int prec) {
    QX_CHECK(c->gauge_loaded, QUDAX_ERR_STATE, "gauge field not loaded");
    for (int k = 0; k < c->ncopies; ++k)
        if (c->gcopy[k].prec == prec) return c->gcopy[k];
    throw Error(QUDAX_ERR_ARG, "no gauge copy in precision " + std::to_string(prec));
}

static qudax_ctx::Halo &halo_for(qudax_ctx *c, int prec) {
    auto &h = c->halo[prec_idx(prec)];
    if (!h.valid) {
        const Geom &g = c->g;
        const bool host = c->comm == QUDAX_COMM_HOST;
        if (g.split & 8) {
            h.bytes = face_bytes(prec, g.fstride);
            h.sb = dalloc(c, h.bytes);
            h.sf = dalloc(c, h.bytes);
            h.gb = dalloc(c, h.bytes);
            h.gf = dalloc(c, h.bytes);
            if (host) {
                h.h_sb = halloc(c, h.bytes);
                h.h_sf = halloc(c, h.bytes);
                h.h_gb = halloc(c, h.bytes);
                h.h_gf = halloc(c, h.bytes);
            }
        }
        for (int m = 0; m < 3; ++m) {
            if (!(g.split >> m & 1)) continue;
            const size_t b = sface_bytes(prec, m, g.fsd[m]);
            h.sbytes[m] = b;
            h.ssb[m] = dalloc(c, b);
            h.ssf[m] = dalloc(c, b);
            h.sgb[m] = dalloc(c, b);
            h.sgf[m] = dalloc(c, b);
            if (host) {
                h.h_ssb[m] = halloc(c, b);
                h.h_ssf[m] = halloc(c, b);
                h.h_sgb[m] = halloc(c, b);
                h.h_sgf[m] = halloc(c, b);
            }
        }
        h.valid = true;
    }
    return h;
}

static inline int rank_fwd(const Geom &g) { return g.nbf[3]; }
static inline int rank_back(const Geom &g) { return g.nbb[3]; }

// One neighbour exchange along dimension mu: send_fwd -> nbf[mu], send_back -> nbb[mu],
// recv_back <- nbb[mu], recv_fwd <- nbf[mu].
struct Xfer {
    int mu;
    const void *send_fwd, *send_back;
    void *recv_back, *recv_fwd;
    size_t bytes;
    void *h_sf, *h_sb, *h_gb, *h_gf;  // pinned staging (HOST)
};
// All transfers of one halo: on NCCL one group enqueued on `s` (the messages of different
// dimensions go to different peers, so their order within the group is free); on HOST staged
// through pinned memory, one hook call per dimension, complete before return.  A dimension whose
// neighbour is this rank (loopback on HOST) is a device copy.
static void exchange_all(qudax_ctx *c, const Xfer *x, int n, cudaStream_t s) {
    const Geom &g = c->g;
    if (c->comm == QUDAX_COMM_NCCL) {
        QX_NCCL(ncclGroupStart());
        for (int k = 0; k < n; ++k) {
            const int f = g.nbf[x[k].mu], b = g.nbb[x[k].mu];
            QX_NCCL(ncclSend(x[k].send_fwd, x[k].bytes, ncclChar, f, c->nccl, s));
            QX_NCCL(ncclRecv(x[k].recv_back, x[k].bytes, ncclChar, b, c->nccl, s));
            QX_NCCL(ncclSend(x[k].send_back, x[k].bytes, ncclChar, b, c->nccl, s));
            QX_NCCL(ncclRecv(x[k].recv_fwd, x[k].bytes, ncclChar, f, c->nccl, s));
        }
        QX_NCCL(ncclGroupEnd());
    } else if (c->comm == QUDAX_COMM_HOST) {
        for (int k = 0; k < n; ++k) {
            const Xfer &t = x[k];
            const int f = g.nbf[t.mu], b = g.nbb[t.mu];
            if (f == g.rank && b == g.rank) {
                QX_CUDA(cudaMemcpyAsync(t.recv_back, t.send_fwd, t.bytes, cudaMemcpyDeviceToDevice, s));
                QX_CUDA(cudaMemcpyAsync(t.recv_fwd, t.send_back, t.bytes, cudaMemcpyDeviceToDevice, s));
                continue;
            }
            QX_CUDA(cudaMemcpyAsync(t.h_sf, t.send_fwd, t.bytes, cudaMemcpyDeviceToHost, s));
            QX_CUDA(cudaMemcpyAsync(t.h_sb, t.send_back, t.bytes, cudaMemcpyDeviceToHost, s));
            QX_CUDA(cudaStreamSynchronize(s));
            int rc = c->host_exchange(f, b, t.h_sf, t.h_sb, t.h_gb, t.h_gf, t.bytes, c->comm_user);
            if (rc) throw Error(QUDAX_ERR_COMM, "host_exchange hook failed");
            QX_CUDA(cudaMemcpyAsync(t.recv_back, t.h_gb, t.bytes, cudaMemcpyHostToDevice, s));
            QX_CUDA(cudaMemcpyAsync(t.recv_fwd, t.h_gf, t.bytes, cudaMemcpyHostToDevice, s));
        }
    } else {
        throw Error(QUDAX_ERR_STATE, "exchange without a transport");
    }
}
// T-direction exchange of two device buffers (gauge-free helper used by setup code)
static void exchange(qudax_ctx *c, const void *send_fwd, const void *send_back, void *recv_back, void *recv_fwd,
                     size_t bytes, cudaStream_t s, void *h_sf, void *h_sb, void *h_gb, void *h_gf) {
    Xfer x{3, send_fwd, send_back, recv_back, recv_fwd, bytes, h_sf, h_sb, h_gb, h_gf};
    exchange_all(c, &x, 1, s);
}

static void global_sum(qudax_ctx *c, double *dev_vals, int n, double *res);
// whether a reduction's local sums must go through the transport before they are used: several
// ranks, or the NCCL loopback at one rank (which runs the N > 1 code path on one GPU)
static bool global_sums(const qudax_ctx *c) { return c->g.nranks > 1 || c->comm == QUDAX_COMM_NCCL; }
// whether that global sum happens after the kernel (transport) rather than inside its reduction
// tail (the P2P mode's kernel-side allreduce, DevAllreduce)
static bool sums_after_kernel(const qudax_ctx *c) { return global_sums(c) && !c->dar; }

static cudaEvent_t pool_event(qudax_ctx *c) {
    if (!c->ev_pool.empty()) {
        cudaEvent_t e = c->ev_pool.back();
        c->ev_pool.pop_back();
        return e;
    }
    cudaEvent_t e;
    QX_CUDA(cudaEventCreate(&e));
    return e;
}

static int dslash_blocks_any(int prec, int recon, int dagger, int kind, int nthreads) {
    if (prec == 8) return dslash_blocks_f64(recon, dagger, kind, nthreads);
    if (prec == 4) return dslash_blocks_f32(recon, dagger, kind, nthreads);
    return dslash_blocks_f16(recon, dagger, kind, nthreads);
}

static void launch_dslash_raw(int prec, int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    if (prec == 8) launch_dslash_f64(recon, dagger, kind, a, s);
    else if (prec == 4) launch_dslash_f32(recon, dagger, kind, a, s);
    else launch_dslash_f16(recon, dagger, kind, a, s);
    QX_CUDA(cudaGetLastError());
}

// every Dslash kernel launch goes through here; with timing enabled it is bracketed by CUDA
// events on the launching (compute) stream
constexpr int kSpanSlots = 1 << 14;
static void launch_dslash_ctx(qudax_ctx *c, int prec, int recon, int dagger, int kind, const DslashArgs &a0) {
    if (!c->timing) {
        launch_dslash_raw(prec, recon, dagger, kind, a0, c->stream);
        return;
    }
    if (!c->d_span) {
        c->d_span = static_cast<unsigned long long *>(dalloc(c, sizeof(unsigned long long) * 4 * kSpanSlots));
        QX_CUDA(cudaMemsetAsync(c->d_span, 0, sizeof(unsigned long long) * 4 * kSpanSlots, c->stream));
        c->h_span = static_cast<unsigned long long *>(halloc(c, sizeof(unsigned long long) * 4 * kSpanSlots));
    }
    DslashArgs a = a0;
    int slot = -1;
    if (c->timing == 2) {  // span mode: the kernels stamp their own start / end (a few us each)
        slot = c->span_next;
        c->span_next = (c->span_next + 1) % kSpanSlots;
        a.span = c->d_span + 4 * slot;
    }
    qudax_ctx::TimingRec r{pool_event(c), pool_event(c), prec, recon, kind, (long)a.nthreads, a.nrhs > 1 ? a.nrhs : 1,
                           a.red_kind, c->cap_iter, slot};
    if (c->capturing) {  // graph: external event-record nodes, re-recorded at each replay
        QX_CUDA(cudaEventRecordWithFlags(r.a, c->stream, cudaEventRecordExternal));
        launch_dslash_raw(prec, recon, dagger, kind, a, c->stream);
        QX_CUDA(cudaEventRecordWithFlags(r.b, c->stream, cudaEventRecordExternal));
        c->graph_trecs.push_back(r);
        return;
    }
    QX_CUDA(cudaEventRecord(r.a, c->stream));
    launch_dslash_raw(prec, recon, dagger, kind, a, c->stream);
    QX_CUDA(cudaEventRecord(r.b, c->stream));
    c->trecs.push_back(r);
}
// host copy of the span slots (after a synchronisation); ms of one record's span
static void fetch_spans(qudax_ctx *c) {
    if (c->d_span) QX_CUDA(cudaMemcpy(c->h_span, c->d_span, sizeof(unsigned long long) * 4 * kSpanSlots,
                                      cudaMemcpyDeviceToHost));
}
static double span_ms(const qudax_ctx *c, const qudax_ctx::TimingRec &r) {
    if (r.span < 0 || !c->h_span) return 0.0;
    const unsigned long long t0 = c->h_span[4 * r.span], t1 = c->h_span[4 * r.span + 1];
    return t1 > t0 ? (double)(t1 - t0) * 1e-6 : 0.0;
}

// totals of one recorded launch: flops and bytes over its sites and right-hand sides (links and
// clover are compulsory once per site, spinor reads/writes once per site and RHS)
static void rec_model(const qudax_ctx::TimingRec &r, qudax_site_model *out) {
    qudax_site_model m, hop;
    qudax_model(r.prec, r.recon, r.kind, &m);
    const double w = r.prec, nrm = (r.prec == 2) ? 4 : 0;
    const double sp = 24 * w + nrm;
    const double per_rhs = (r.kind >= QUDAX_CLOVER_XPAY ? 3 : 2) * sp;  // in, out (, x)
    (void)hop;
    out->flops = m.flops * r.sites * r.nrhs;
    out->bytes_compulsory = ((m.bytes_compulsory - per_rhs) + per_rhs * r.nrhs) * r.sites;
    if (r.red == RED_RHAT_DOT) out->bytes_compulsory += sp * r.sites;  // the fused <rhat0, out> reads rhat0
    out->bytes_paper = m.bytes_paper * r.sites * r.nrhs;
}

// QUDAX_FLAG_TIMING_BREAKDOWN (diagnostics): graph-replayed Dslash launch times per (precision,
// kind, fused reduction), printed to stderr at finalize
static std::map<std::tuple<int, int, int>, std::pair<long, double>> g_tbreak;

// the timing records of one replay of a captured graph (only those of the first `iters` solver
// iterations of the batch: the later ones were halted and ran no work)
void harvest_graph_timing(qudax_ctx *c, const std::vector<qudax_ctx::TimingRec> &recs, int iters) {
    if (!recs.empty()) fetch_spans(c);
    for (auto &r : recs) {
        if (r.iter >= iters) continue;
        float ms = 0;
        QX_CUDA(cudaEventElapsedTime(&ms, r.a, r.b));
        if (c->flags & QUDAX_FLAG_TIMING_BREAKDOWN) {
            auto &e = g_tbreak[std::make_tuple(r.prec, r.kind, r.red)];
            e.first += 1;
            e.second += ms;
        }
        qudax_site_model m;
        rec_model(r, &m);
        auto &t = c->tacc[prec_idx(r.prec)];
        t.launches += 1;
        t.sites += r.sites * r.nrhs;
        t.ms += ms;
        t.span_ms += span_ms(c, r);
        t.flops += m.flops;
        t.bytes_c += m.bytes_compulsory;
        t.bytes_p += m.bytes_paper;
    }
}

void check_device_error(qudax_ctx *c) {
    if (c->h_err && *reinterpret_cast<volatile int *>(c->h_err)) {
        *reinterpret_cast<volatile int *>(c->h_err) = 0;
        throw Error(QUDAX_ERR_COMM, "kernel-initiated halo or allreduce: a peer flag did not arrive (wait timed out); "
                                    "the operator result is invalid");
    }
}

void release_graph_timing(qudax_ctx *c, std::vector<qudax_ctx::TimingRec> &recs) {
    for (auto &r : recs) {
        c->ev_pool.push_back(r.a);
        c->ev_pool.push_back(r.b);
    }
    recs.clear();
}

// kernel arguments common to every Dslash launch of (precision, output parity, kind)
static DslashArgs base_args(qudax_ctx *c, const qudax_ctx::GaugeCopy &gc, int prec, int p, int kind, double a,
                            int reverse) {
    const Geom &g = c->g;
    DslashArgs args{};
    args.X = g.X; args.Y = g.Y; args.Z = g.Z; args.T_loc = g.T_loc; args.Xh = g.Xh;
    args.dXh = make_fastdiv(g.Xh); args.dY = make_fastdiv(g.Y); args.dZ = make_fastdiv(g.Z);
    args.Vh = (int)g.Vh; args.F = (int)g.F;
    args.stride = g.stride; args.fstride = g.fstride;
    args.parity = p;
    // the antiperiodic sign belongs to the hops that cross global t = T-1 <-> 0 (reading Q5)
    args.bc_fwd = (g.c[3] == g.P[3] - 1) ? (double)c->t_bc : 1.0;
    args.bc_back = (g.c[3] == 0) ? (double)c->t_bc : 1.0;
    args.a = a;
    args.reverse = reverse;
    args.err = c->d_err;
    args.variant = ((c->flags & QUDAX_FLAG_FORCE_SS) ? kVariantForceSS : 0) |
                   ((c->flags & QUDAX_FLAG_ONE_RHS_PER_THREAD) ? kVariantOneRhsPerThread : 0);
    args.nrhs = 1;
    for (int m = 0; m < 4; ++m)
        for (int q = 0; q < 2; ++q) args.gauge[m][q] = gc.d[m][q];
    args.gauge_ghost = gc.ghost[3][1 - p];
    args.smask = spatial_split(g);
    for (int m = 0; m < 3; ++m) {
        args.sfs[m] = g.fsd[m];
        args.gauge_sghost[m] = gc.ghost[m][1 - p];
    }
    for (int m = 0; m < 4; ++m) {
        args.blo[m] = g.blo[m];
        args.bn[m] = g.bn[m];
    }
    args.blist = c->blist;
    if (kind != QUDAX_HOP) {
        auto &cl = c->clov[prec_idx(prec)];
        QX_CHECK(cl.valid, QUDAX_ERR_STATE, "no clover in this precision");
        args.clover = (kind == QUDAX_CLOVER_XPAY) ? cl.T[p] : cl.Tinv[p];
    }
    return args;
}

void dslash_op(qudax_ctx *c, void *out, const void *in, const void *x, int prec, int p, int dagger, int kind,
               double a, const RedReq *red, int reverse) {
    check_prec(prec);
    QX_CHECK(p == 0 || p == 1, QUDAX_ERR_ARG, "parity must be 0 or 1");
    QX_CHECK(kind >= 0 && kind <= 3, QUDAX_ERR_ARG, "bad dslash kind");
    QX_CHECK(out && in && (kind < QUDAX_CLOVER_XPAY || x), QUDAX_ERR_ARG, "null field");
    QX_CHECK(out != in, QUDAX_ERR_ARG, "dslash cannot run in place");
    auto &gc = gauge_for(c, prec);
    const Geom &g = c->g;
    DslashArgs args = base_args(c, gc, prec, p, kind, a, reverse);
    args.in = in; args.out = out; args.x = x;
    int red_blocks = 0;  // CTA slots used in c->dpart by this call's launches
    const long n_int = g.n_int, n_bnd = g.Vh - g.n_int;
    // NCCL path with overlap: ONE launch whose boundary CTAs (the grid's tail) wait for a flag the
    // comm stream raises after the exchange (tail mode: no separate boundary launch, which ran at
    // a fraction of a wave — 17 us for 1/16 of the sites at 32^3x64, gpurun r02e timeline), or,
    // where the tail layout does not apply (the multi-RHS path), interior + boundary launches
    const bool nccl_ov = c->comm == QUDAX_COMM_NCCL && !c->p2p.on && c->overlap && n_int > 0;
    const bool tail_mode = nccl_ov && (spatial_split(g) ? true : g.T_loc > 2);
    const bool split = nccl_ov && !tail_mode;
    const bool multi = sums_after_kernel(c);  // sums go through the transport before the recurrence
    if (red) {
        QX_CHECK(red->kind != RED_XDOT_NORM || kind >= QUDAX_CLOVER_XPAY, QUDAX_ERR_ARG, "x-dot needs xpay");
        QX_CHECK(red->kind != RED_RHAT_DOT || red->rhat, QUDAX_ERR_ARG, "rhat-dot needs rhat");
        // CTA slots of up to two launches + their group slots (reduce.cuh)
        if (!c->dpart) c->dpart = static_cast<double *>(dalloc(c, sizeof(double) * 3 * (2 * (g.Vh / 32) + 64)));
        args.red_kind = red->kind;
        args.rhat = red->rhat;
        args.tail.partials = c->dpart;
        args.tail.counter = c->d_counter;
        args.tail.total_blocks = split ? dslash_blocks_any(prec, gc.recon, dagger, kind, (int)n_int) +
                                             dslash_blocks_any(prec, gc.recon, dagger, kind, (int)n_bnd)
                                       : dslash_blocks_any(prec, gc.recon, dagger, kind, (int)g.Vh);
        args.tail.out = red->S ? red->S->red : c->red_out;
        args.tail.S = red->S;
        args.tail.coef_mode = (red->S && !multi) ? red->coef_mode : COEF_NONE;
        args.tail.dar = c->dar;
        args.tail.chan = 0;
    }
    auto launch = [&](int range, int nthreads) {
        args.range = range;
        args.nthreads = nthreads;
        args.tail.block_offset = red_blocks;
        launch_dslash_ctx(c, prec, gc.recon, dagger, kind, args);
        red_blocks += dslash_blocks_any(prec, gc.recon, dagger, kind, nthreads);
        c->launches += 1;
    };
    auto finish_red = [&] {
        if (!red) return;
        if (!red->S) global_sum(c, c->red_out, 3, red->res);
        else if (multi) device_sum_coef(c, red->S->red, 3, red->S, red->coef_mode);
    };
    if (c->p2p.on) {  // kernel-initiated halo over peer memory (QUDAX_HALO_P2P), any process grid
        auto &q = c->p2p;
        const int pi = prec_idx(prec);
        args.ghosted = (g.split >> 3) & 1;
        args.ghost_back = q.base + q.off_g[pi][3][0];
        args.ghost_fwd = q.base + q.off_g[pi][3][1];
        args.p2p_pdist = (long)q.pdist[pi][3];
        for (int m = 0; m < 3; ++m) {
            args.sghost_back[m] = q.base + q.off_g[pi][m][0];
            args.sghost_fwd[m] = q.base + q.off_g[pi][m][1];
            args.sp2p_pdist[m] = (long)q.pdist[pi][m];
        }
        args.p2p_cseq = reinterpret_cast<unsigned *>(q.base + q.off_cseq);
        args.p2p_ccount = reinterpret_cast<unsigned *>(q.base + q.off_ccount);
        args.p2p_mask = g.split;
        unsigned *own_flags = reinterpret_cast<unsigned *>(q.base + q.off_flags);
        // our x_mu = 0 face -> the backward neighbour's FORWARD ghost (its flag 2 mu + 1); our
        // x_mu = L-1 face -> the forward neighbour's BACKWARD ghost (its flag 2 mu)
        P2PPackArgs pk{};
        pk.mask = g.split;
        pk.q = 1 - p;
        pk.stride = g.stride;
        for (int m = 0; m < 4; ++m) {
            pk.L[m] = g.L[m];
            pk.Fd[m] = g.Fd[m];
            pk.fsd[m] = g.fsd[m];
            if (!(g.split >> m & 1)) continue;
            pk.dst_b[m] = q.peer_b[m] + q.off_g[pi][m][1];
            pk.dst_f[m] = q.peer_f[m] + q.off_g[pi][m][0];
            pk.pdist[m] = (long)q.pdist[pi][m];
            pk.flag_b[m] = reinterpret_cast<unsigned *>(q.peer_b[m] + q.off_flags) + 2 * m + 1;
            pk.flag_f[m] = reinterpret_cast<unsigned *>(q.peer_f[m] + q.off_flags) + 2 * m;
        }
        pk.seq = reinterpret_cast<unsigned *>(q.base + q.off_seq);
        pk.count = reinterpret_cast<unsigned *>(q.base + q.off_count);
        pk.half_back = dagger ? 0 : 1;  // non-dagger: lower spins go backward (reading Q15)
        pk.half_fwd = dagger ? 1 : 0;
        auto pack = [&](cudaStream_t st) {
            launch_pack_p2p(prec, dagger, pk, in, st);
            c->launches += 1;
        };
        const bool sp = spatial_split(g) != 0;
        // (a split X has no interior box: every site may read a ghost, so every CTA waits)
        const bool tail = c->overlap && (sp ? g.n_int > 0 : g.T_loc > 2);
        if (tail) {
            // ONE Dslash launch (RANGE_TAIL) beside the pack on the high-priority comm stream:
            // interior sites first (T-only: t in [1, T_loc-2]; a grid: the interior box), the
            // boundary CTAs at the grid's tail acquire the neighbours' flags.  The join after it
            // only keeps `in` alive until our own pack has read it.
            QX_CUDA(cudaEventRecord(c->ev_in, c->stream));
            QX_CUDA(cudaStreamWaitEvent(c->comm_stream, c->ev_in, 0));
            pack(c->comm_stream);
            QX_CUDA(cudaEventRecord(c->ev_halo, c->comm_stream));
            args.p2p_flags = own_flags;
            args.reverse = 0;  // the waiting CTAs must be the last ones
            args.tail_ni = sp ? (int)g.n_int : (int)((g.T_loc - 2) * g.F);
            launch(RANGE_TAIL, (int)g.Vh);
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
        } else {
            pack(c->stream);
            args.p2p_flags = own_flags;
            launch(RANGE_ALL, (int)g.Vh);
        }
        finish_red();
        return;
    }
    if (c->comm == QUDAX_COMM_NONE || g.split == 0) {
        args.ghosted = 0;
        launch(RANGE_ALL, (int)g.Vh);
        finish_red();
        return;
    }
    auto &h = halo_for(c, prec);
    args.ghosted = (g.split >> 3) & 1;
    args.ghost_back = h.gb;
    args.ghost_fwd = h.gf;
    Xfer xf[4];
    int nx = 0;
    for (int m = 0; m < 3; ++m) {
        args.sghost_back[m] = h.sgb[m];
        args.sghost_fwd[m] = h.sgf[m];
        if (g.split >> m & 1)
            xf[nx++] = Xfer{m, h.ssf[m], h.ssb[m], h.sgb[m], h.sgf[m], h.sbytes[m], h.h_ssf[m], h.h_ssb[m], h.h_sgb[m], h.h_sgf[m]};
    }
    if (g.split & 8) xf[nx++] = Xfer{3, h.sf, h.sb, h.gb, h.gf, h.bytes, h.h_sf, h.h_sb, h.h_gb, h.h_gf};
    auto pack_all = [&](cudaStream_t st) {
        if (g.split & 8) {
            launch_pack_faces(prec, dagger, g, in, h.sb, h.sf, st);
            c->launches += 1;
        }
        if (spatial_split(g)) {
            launch_pack_spatial(prec, dagger, g, 1 - p, in, h.ssb, h.ssf, st);
            c->launches += 1;
        }
    };
    if (c->comm == QUDAX_COMM_NCCL) {
        // diagnostic overlap timeline (qudax_halo_timeline), eager launches only
        const bool tl = c->tl_on && !c->capturing;
        auto mark = [&](int k, cudaStream_t st) {
            if (tl) QX_CUDA(cudaEventRecord(c->tl[k], st));
        };
        // comm stream: wait for `in` (and for the previous boundary kernel, which read the ghosts)
        mark(0, c->stream);
        QX_CUDA(cudaEventRecord(c->ev_in, c->stream));
        QX_CUDA(cudaStreamWaitEvent(c->comm_stream, c->ev_in, 0));
        mark(1, c->comm_stream);
        pack_all(c->comm_stream);
        mark(2, c->comm_stream);
        exchange_all(c, xf, nx, c->comm_stream);
        mark(3, c->comm_stream);
        if (tail_mode) {
            if (!c->tflags) {
                c->tflags = static_cast<unsigned *>(dalloc(c, sizeof(unsigned) * 16));
                QX_CUDA(cudaMemsetAsync(c->tflags, 0, sizeof(unsigned) * 16, c->stream));
            }
            launch_raise_flags(c->tflags, c->tflags + 8, g.split, c->comm_stream);
            c->launches += 1;
        }
        QX_CUDA(cudaEventRecord(c->ev_halo, c->comm_stream));
        if (tail_mode) {
            args.p2p_flags = c->tflags;
            args.p2p_cseq = c->tflags + 9;
            args.p2p_ccount = c->tflags + 10;
            args.p2p_mask = g.split;
            args.p2p_pdist = 0;
            for (int m = 0; m < 3; ++m) args.sp2p_pdist[m] = 0;
            args.reverse = 0;  // the waiting CTAs must be the last ones
            args.tail_ni = spatial_split(g) ? (int)n_int : (int)((g.T_loc - 2) * g.F);
            mark(4, c->stream);
            launch(RANGE_TAIL, (int)g.Vh);
            mark(5, c->stream);
            mark(6, c->stream);
            mark(7, c->stream);
            // the join keeps the comm stream's next pack behind this Dslash (it overwrites the
            // send buffers only after the ghosts of this one were consumed: ev_in of the next call)
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
        } else if (split) {
            mark(4, c->stream);
            launch(RANGE_INTERIOR, (int)n_int);
            mark(5, c->stream);
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
            mark(6, c->stream);
            launch(RANGE_BOUNDARY, (int)n_bnd);
            mark(7, c->stream);
        } else {
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
            mark(4, c->stream);
            mark(5, c->stream);
            mark(6, c->stream);
            launch(RANGE_ALL, (int)g.Vh);
            mark(7, c->stream);
        }
        if (tl) c->tl_valid = true;
    } else {  // HOST: paper strategy 1 (no overlap)
        pack_all(c->stream);
        exchange_all(c, xf, nx, c->stream);
        launch(RANGE_ALL, (int)g.Vh);
    }
    finish_red();
}

void *tmp_odd_field(qudax_ctx *c, int prec);
static void *tmp_odd(qudax_ctx *c, int prec) { return tmp_odd_field(c, prec); }
void *tmp_odd_field(qudax_ctx *c, int prec) {
    auto &t = c->tmp_odd[prec_idx(prec)];
    if (!t) t = dalloc(c, spinor_bytes(prec, c->g.stride));
    return t;
}
static void *tmp_even(qudax_ctx *c, int prec) {
    auto &t = c->tmp_even[prec_idx(prec)];
    if (!t) t = dalloc(c, spinor_bytes(prec, c->g.stride));
    return t;
}

// Mhat = T_ee - kappa^2 D_eo T_oo^{-1} D_oe (asymmetric Schur form on even sites)
#ifndef QX_MATPC_REVERSE
#define QX_MATPC_REVERSE 1
#endif
// symmetric Schur form: T_ee^{-1} Mhat.  Non-dagger: CLOVER_INV on odd,
// CLOVER_INV_XPAY on even (fused reductions as for Mhat).  Dagger (explicit adjoint, not
// gamma5-Hermitian): T_ee^{-1} in -> CLOVER_INV^dag on odd -> HOP^dag on even -> in - kappa^2 (.)
void matpc_sym_op(qudax_ctx *c, void *out, const void *in, int prec, int dagger, const RedReq *red) {
    void *t = tmp_odd(c, prec);
    if (!dagger) {
        dslash_op(c, t, in, nullptr, prec, 1, 0, QUDAX_CLOVER_INV, 0.0, nullptr);
        dslash_op(c, out, t, in, prec, 0, 0, QUDAX_CLOVER_INV_XPAY, -c->kappa * c->kappa, red, 1);
        return;
    }
    QX_CHECK(!red, QUDAX_ERR_ARG, "symmetric Mhat^dag: no fused reductions");
    QX_CHECK(out != in, QUDAX_ERR_ARG, "matpc_sym dagger cannot run in place");
    auto &ys = c->tmp_sym[prec_idx(prec)];
    if (!ys) ys = dalloc(c, spinor_bytes(prec, c->g.stride));
    void *y = ys;
    clover_apply_op(c, y, in, prec, 0, true);
    dslash_op(c, t, y, nullptr, prec, 1, 1, QUDAX_CLOVER_INV, 0.0, nullptr);
    dslash_op(c, y, t, nullptr, prec, 0, 1, QUDAX_HOP, 0.0, nullptr);
    void *f[3] = {const_cast<void *>(in), y, out};
    const double a = -c->kappa * c->kappa;
    blas_op(c, OP_XPAY, prec, f, &a, nullptr);
}

void matpc_op(qudax_ctx *c, void *out, const void *in, int prec, int dagger, const RedReq *red, int order) {
    if (c->matpc_sym) {
        matpc_sym_op(c, out, in, prec, dagger, red);
        return;
    }
    void *t = tmp_odd(c, prec);
    // the two kernels walk the lattice in opposite directions: the second starts on the
    // timeslices the first touched last (their links, T^{-1} D in and the dirty tmp lines are
    // still in the 126 MB L2)
    dslash_op(c, t, in, nullptr, prec, 1, dagger, QUDAX_CLOVER_INV, 0.0, nullptr, order ? 1 : 0);
    dslash_op(c, out, t, in, prec, 0, dagger, QUDAX_CLOVER_XPAY, -c->kappa * c->kappa, red,
              order ? 0 : QX_MATPC_REVERSE);
}

// Multi-RHS Dslash (SURVEY NEXT row 2, P:748-753 / P:1092-1094: many right-hand sides per
// configuration): one launch for n fields, consecutive CTAs taking the same sites for
// different RHS so the links and clover are read from HBM about once for all of them.
// Partitioned runs (halo exchange per RHS) apply the single-RHS path per field.
void dslash_multi_op(qudax_ctx *c, void *const *out, const void *const *in, const void *const *x, int n, int prec,
                     int p, int dagger, int kind, double a, int reverse, const RedReq *reds) {
    check_prec(prec);
    QX_CHECK(n >= 1 && n <= kMaxRhs, QUDAX_ERR_ARG, "nrhs must be 1.." + std::to_string(kMaxRhs));
    QX_CHECK(p == 0 || p == 1, QUDAX_ERR_ARG, "parity must be 0 or 1");
    QX_CHECK(kind >= 0 && kind <= 3, QUDAX_ERR_ARG, "bad dslash kind");
    for (int k = 0; k < n; ++k) {
        QX_CHECK(out[k] && in[k] && (kind < QUDAX_CLOVER_XPAY || (x && x[k])), QUDAX_ERR_ARG, "null field");
        QX_CHECK(out[k] != in[k], QUDAX_ERR_ARG, "dslash cannot run in place");
    }
    const Geom &g = c->g;
    // partitioned contexts: the multi-RHS halo (T-only split, comm transport) — one exchange per
    // direction carrying every right-hand side's face — else one single-RHS operator per field
    const bool mhalo = (c->comm != QUDAX_COMM_NONE) && !c->p2p.on && g.split == 8;
    if ((c->comm != QUDAX_COMM_NONE && !mhalo) || c->p2p.on || n == 1) {
        for (int k = 0; k < n; ++k)
            dslash_op(c, out[k], in[k], x ? x[k] : nullptr, prec, p, dagger, kind, a, reds ? reds + k : nullptr, reverse);
        return;
    }
    auto &gc = gauge_for(c, prec);
    DslashArgs args = base_args(c, gc, prec, p, kind, a, reverse);
    args.nrhs = n;
    for (int k = 0; k < n; ++k) {
        args.in_m[k] = in[k];
        args.out_m[k] = out[k];
        args.x_m[k] = x ? x[k] : nullptr;
    }
    const bool multi = sums_after_kernel(c);
    const long n_int = g.n_int, n_bnd = g.Vh - g.n_int;
    const bool split = mhalo && c->comm == QUDAX_COMM_NCCL && c->overlap && n_int > 0;
    if (reds) {  // one deterministic reduction (and scalar recurrence) per right-hand side
        const int nb = dslash_blocks_any(prec, gc.recon, dagger, kind, (int)g.Vh);
        const size_t slots = 3 * ((size_t)nb + nb / kGroupHost + 2);
        const size_t ncount = 2 + (size_t)nb / kGroupHost + 2;
        if (!c->dpart_m) {
            c->dpart_m = static_cast<double *>(dalloc(c, sizeof(double) * slots * kMaxRhs));
            c->dcount_m = static_cast<unsigned *>(dalloc(c, sizeof(unsigned) * ncount * kMaxRhs));
            QX_CUDA(cudaMemsetAsync(c->dcount_m, 0, sizeof(unsigned) * ncount * kMaxRhs, c->stream));
        }
        args.red_kind = reds[0].kind;
        for (int k = 0; k < n; ++k) {
            QX_CHECK(reds[k].kind == reds[0].kind && reds[k].S, QUDAX_ERR_ARG, "multi-RHS reductions: one kind, device scalars");
            QX_CHECK(reds[k].kind != RED_XDOT_NORM || kind >= QUDAX_CLOVER_XPAY, QUDAX_ERR_ARG, "x-dot needs xpay");
            QX_CHECK(reds[k].kind != RED_RHAT_DOT || reds[k].rhat, QUDAX_ERR_ARG, "rhat-dot needs rhat");
            args.rhat_m[k] = reds[k].rhat;
            const int tot = split ? dslash_blocks_any(prec, gc.recon, dagger, kind, (int)n_int) +
                                        dslash_blocks_any(prec, gc.recon, dagger, kind, (int)n_bnd)
                                  : nb;
            args.tail_m[k] = RedTail{c->dpart_m + slots * k, c->dcount_m + ncount * k, tot, 0, reds[k].S->red, reds[k].S,
                                     multi ? COEF_NONE : reds[k].coef_mode, c->dar, 1 + k};
        }
    }
    int blk_off = 0;
    auto launch = [&](int range, int nthreads) {
        args.range = range;
        args.nthreads = nthreads;
        for (int k = 0; k < n; ++k) args.tail_m[k].block_offset = blk_off;
        launch_dslash_ctx(c, prec, gc.recon, dagger, kind, args);
        blk_off += dslash_blocks_any(prec, gc.recon, dagger, kind, nthreads);
        c->launches += 1;
    };
    if (!mhalo) {
        args.ghosted = 0;
        launch(RANGE_ALL, (int)g.Vh);
        return;
    }
    // ---- multi-RHS T halo (P:692-720 with every right-hand side in one message per direction)
    auto &h = halo_for(c, prec);
    const bool host = c->comm == QUDAX_COMM_HOST;
    if (!h.m_sb) {
        h.m_stride = (h.bytes + 255) & ~(size_t)255;
        const size_t mb = h.m_stride * kMaxRhs;
        h.m_sb = dalloc(c, mb);
        h.m_sf = dalloc(c, mb);
        h.m_gb = dalloc(c, mb);
        h.m_gf = dalloc(c, mb);
        if (host) {
            h.mh_sb = halloc(c, mb);
            h.mh_sf = halloc(c, mb);
            h.mh_gb = halloc(c, mb);
            h.mh_gf = halloc(c, mb);
        }
    }
    args.ghosted = 1;
    args.ghost_back = h.m_gb;
    args.ghost_fwd = h.m_gf;
    args.ghost_rhs_bytes = (long)h.m_stride;
    Xfer xf{3, h.m_sf, h.m_sb, h.m_gb, h.m_gf, h.m_stride * n, h.mh_sf, h.mh_sb, h.mh_gb, h.mh_gf};
    auto pack_all = [&](cudaStream_t st) {
        for (int k = 0; k < n; ++k) {
            launch_pack_faces(prec, dagger, g, in[k], static_cast<char *>(h.m_sb) + k * h.m_stride,
                              static_cast<char *>(h.m_sf) + k * h.m_stride, st);
            c->launches += 1;
        }
    };
    if (c->comm == QUDAX_COMM_NCCL) {
        QX_CUDA(cudaEventRecord(c->ev_in, c->stream));
        QX_CUDA(cudaStreamWaitEvent(c->comm_stream, c->ev_in, 0));
        pack_all(c->comm_stream);
        exchange_all(c, &xf, 1, c->comm_stream);
        QX_CUDA(cudaEventRecord(c->ev_halo, c->comm_stream));
        if (split) {
            launch(RANGE_INTERIOR, (int)n_int);
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
            launch(RANGE_BOUNDARY, (int)n_bnd);
        } else {
            QX_CUDA(cudaStreamWaitEvent(c->stream, c->ev_halo, 0));
            launch(RANGE_ALL, (int)g.Vh);
        }
    } else {  // HOST transport: exchange first, one launch
        pack_all(c->stream);
        exchange_all(c, &xf, 1, c->stream);
        launch(RANGE_ALL, (int)g.Vh);
    }
    if (reds && multi)
        for (int k = 0; k < n; ++k) device_sum_coef(c, reds[k].S->red, 3, reds[k].S, reds[k].coef_mode);
}

void matpc_multi_op(qudax_ctx *c, void *const *out, const void *const *in, int n, int prec, int dagger,
                    const RedReq *reds, int order) {
    QX_CHECK(n >= 1 && n <= kMaxRhs, QUDAX_ERR_ARG, "nrhs must be 1.." + std::to_string(kMaxRhs));
    void *t[kMaxRhs];
    for (int k = 0; k < n; ++k) {
        auto &slot = c->tmp_multi[prec_idx(prec)][k];
        if (!slot) slot = dalloc(c, spinor_bytes(prec, c->g.stride));
        t[k] = slot;
    }
    QX_CHECK(!c->matpc_sym, QUDAX_ERR_UNSUPPORTED, "multi-RHS Mhat: asymmetric Schur form only");
    // (the same kernel directions as matpc_op, so a batched solve stays bitwise its single ones)
    dslash_multi_op(c, t, in, nullptr, n, prec, 1, dagger, QUDAX_CLOVER_INV, 0.0, order ? 1 : 0, nullptr);
    dslash_multi_op(c, out, t, in, n, prec, 0, dagger, QUDAX_CLOVER_XPAY, -c->kappa * c->kappa,
                    order ? 0 : QX_MATPC_REVERSE, reds);
}

void clover_apply_op(qudax_ctx *c, void *out, const void *in, int prec, int parity, bool inverse) {
    auto &cl = c->clov[prec_idx(prec)];
    QX_CHECK(cl.valid, QUDAX_ERR_STATE, "no clover in this precision");
    launch_clover_apply(prec, c->g, inverse ? cl.Tinv[parity] : cl.T[parity], in, out, c->stream);
    c->launches += 1;
}

static void global_sum(qudax_ctx *c, double *dev_vals, int n, double *res) {
    if (c->dar) {  // the kernel's reduction tail already summed over ranks (DevAllreduce)
        QX_CUDA(cudaMemcpyAsync(c->h_red, dev_vals, sizeof(double) * n, cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        check_device_error(c);
        for (int k = 0; k < n; ++k) res[k] = c->h_red[k];
        return;
    }
    if (c->comm == QUDAX_COMM_NCCL) {  // (one rank: the loopback test of the N > 1 path)
        QX_NCCL(ncclAllReduce(dev_vals, dev_vals, n, ncclDouble, ncclSum, c->nccl_red, c->stream));
    }
    QX_CUDA(cudaMemcpyAsync(c->h_red, dev_vals, sizeof(double) * n, cudaMemcpyDeviceToHost, c->stream));
    QX_CUDA(cudaStreamSynchronize(c->stream));
    if (c->g.nranks > 1 && c->comm == QUDAX_COMM_HOST) {
        if (c->host_allreduce(c->h_red, n, c->comm_user)) throw Error(QUDAX_ERR_COMM, "host_allreduce hook failed");
    }
    for (int k = 0; k < n; ++k) res[k] = c->h_red[k];
}

int blas_op(qudax_ctx *c, int op, int prec, void *const *f, const double *coef, double *res) {
    CoefArg co[2] = {};
    if (coef) {
        co[0].v = make_double2(coef[0], op == OP_XPAY ? 0.0 : coef[1]);
        if (op == OP_P_UPDATE || op == OP_FINAL) co[1].v = make_double2(coef[2], coef[3]);
    }
    RedTail tail{c->partials, c->d_counter, 0, 0, c->red_out, nullptr, COEF_NONE, c->dar, 0};
    int n = blas_run(op, prec, c->g, f, co, tail, c->stream);
    c->launches += 1;
    if (n) global_sum(c, c->red_out, n, res);
    return n;
}

// Global sum of n device doubles in place (stream-ordered, no host round trip for NCCL / one
// rank), then the device-side scalar recurrence `mode` (launch_coef).
void device_sum_coef(qudax_ctx *c, double *dev_vals, int n, SolverScalars *S, int mode) {
    if (c->comm == QUDAX_COMM_NCCL) {  // (one rank: the loopback test of the N > 1 path)
        QX_NCCL(ncclAllReduce(dev_vals, dev_vals, n, ncclDouble, ncclSum, c->nccl_red, c->stream));
    } else if (c->g.nranks > 1 && c->comm == QUDAX_COMM_HOST) {
        QX_CUDA(cudaMemcpyAsync(c->h_red, dev_vals, sizeof(double) * n, cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        if (c->host_allreduce(c->h_red, n, c->comm_user)) throw Error(QUDAX_ERR_COMM, "host_allreduce hook failed");
        QX_CUDA(cudaMemcpyAsync(dev_vals, c->h_red, sizeof(double) * n, cudaMemcpyHostToDevice, c->stream));
    }
    if (mode != COEF_NONE) {
        launch_coef(S, mode, c->stream);
        c->launches += 1;
    }
}

// BLAS op whose coefficients may live on the device; its reduction (if any) goes to S->red,
// is summed over ranks and fed to the scalar recurrence `mode` — all stream-ordered.
void blas_op_dev(qudax_ctx *c, int op, int prec, void *const *f, const CoefArg *co, SolverScalars *S, int mode) {
    const bool multi = sums_after_kernel(c);
    RedTail tail{c->partials, c->d_counter, 0, 0, S->red, S, multi ? COEF_NONE : mode, c->dar, 0};
    int n = blas_run(op, prec, c->g, f, co, tail, c->stream);
    c->launches += 1;
    if (n && multi) device_sum_coef(c, S->red, n, S, mode);
}

void xpy_mixed_op(qudax_ctx *c, int pd, int ps, const void *x, void *y) {
    blas_xpy_mixed(pd, ps, c->g, x, y, c->stream);
    c->launches += 1;
}

void convert_op(qudax_ctx *c, void *dst, int pd, const void *src, int ps) {
    launch_spinor_convert(pd, ps, c->g, dst, src, c->stream);
    c->launches += 1;
}

static void gauge_load(qudax_ctx *c, const double *host, const qudax_gauge_param *p) {
    QX_CHECK(host && p, QUDAX_ERR_ARG, "null gauge or param");
    const Geom &g = c->g;
    for (int k = 0; k < 2; ++k) {
        int pr = k ? p->prec_sloppy : p->prec, rc = k ? p->recon_sloppy : p->recon;
        check_prec(pr);
        QX_CHECK(rc == 18 || rc == 12 || rc == 8, QUDAX_ERR_ARG, "recon must be 18, 12 or 8");
    }
    QX_CHECK(p->t_boundary == 1 || p->t_boundary == -1, QUDAX_ERR_ARG, "t_boundary must be +1 or -1");
    // drop a previous configuration's copies (fields of the previous load are released)
    for (int k = 0; k < c->ncopies; ++k) {
        for (int m = 0; m < 4; ++m)
            for (int q = 0; q < 2; ++q) {
                dfree(c, c->gcopy[k].d[m][q]);
                dfree(c, c->gcopy[k].ghost[m][q]);
            }
        c->gcopy[k] = qudax_ctx::GaugeCopy{};
    }
    for (auto &cl : c->clov) {
        if (!cl.valid) continue;
        for (int q = 0; q < 2; ++q) { dfree(c, cl.T[q]); dfree(c, cl.Tinv[q]); }
        cl = qudax_ctx::Clover{};
    }
    c->ncopies = 0;
    c->gauge_loaded = false;
    c->gauge_epoch += 1;  // cached solver graphs baked in the old gauge / clover pointers
    drop_graphs(c);
    c->kappa = p->kappa;
    c->csw = p->csw;
    c->t_bc = p->t_boundary;

    // 1. upload the box and scatter it into the extended site-major fp64 buffer
    //    ext[Et][Ez][Ey][Ex][4][18] (one-site halo on every split dimension)
    double *ext = static_cast<double *>(dalloc(c, sizeof(double) * 72 * ext_sites(g)));
    {
        double *box = static_cast<double *>(dalloc(c, sizeof(double) * 72 * g.V));
        h2d(c, box, host, sizeof(double) * 72 * g.V);
        launch_ext_fill(g, box, ext, c->stream);
        QX_CUDA(cudaStreamSynchronize(c->stream));
        dfree(c, box);
    }
    // 2. gauge ghost + clover halo: along each split dimension in turn, the first and
    //    last interior cross-sections (with the halos already received: corners) go to the
    //    neighbours and come back as the two halo cross-sections.  Once per configuration.
    for (int mu = 0; mu < 4; ++mu) {
        if (!(g.split >> mu & 1)) continue;
        const long n = ext_slice_doubles(g, mu);
        const size_t bytes = sizeof(double) * n;
        double *buf = static_cast<double *>(dalloc(c, 4 * bytes));
        double *s_lo = buf, *s_hi = buf + n, *r_lo = buf + 2 * n, *r_hi = buf + 3 * n;
        launch_ext_slice(g, ext, mu, 1, s_lo, true, c->stream);             // local x_mu = 0
        launch_ext_slice(g, ext, mu, g.L[mu], s_hi, true, c->stream);       // local x_mu = L-1
        if (c->comm == QUDAX_COMM_NONE || (g.nbf[mu] == g.rank && g.nbb[mu] == g.rank)) {
            QX_CUDA(cudaMemcpyAsync(r_lo, s_hi, bytes, cudaMemcpyDeviceToDevice, c->stream));
            QX_CUDA(cudaMemcpyAsync(r_hi, s_lo, bytes, cudaMemcpyDeviceToDevice, c->stream));
        } else {
            void *hs[4] = {nullptr, nullptr, nullptr, nullptr};
            if (c->comm == QUDAX_COMM_HOST)
                for (auto &q : hs) q = halloc(c, bytes);
            Xfer x{mu, s_hi, s_lo, r_lo, r_hi, bytes, hs[0], hs[1], hs[2], hs[3]};
            exchange_all(c, &x, 1, c->stream);
            QX_CUDA(cudaStreamSynchronize(c->stream));
            for (auto &q : hs) hfree(c, q);
        }
        launch_ext_slice(g, ext, mu, 0, r_lo, false, c->stream);            // local x_mu = -1
        launch_ext_slice(g, ext, mu, g.L[mu] + 1, r_hi, false, c->stream);  // local x_mu = L
        QX_CUDA(cudaStreamSynchronize(c->stream));
        dfree(c, buf);
    }
    // 3. pack each (precision, reconstruct) copy
    int *bad = c->d_flag;
    QX_CUDA(cudaMemsetAsync(bad, 0, sizeof(int), c->stream));
    for (int k = 0; k < 2; ++k) {
        int pr = k ? p->prec_sloppy : p->prec, rc = k ? p->recon_sloppy : p->recon;
        if (k == 1 && pr == p->prec) break;  // sloppy == outer precision: one copy
        auto &gc = c->gcopy[c->ncopies++];
        gc.prec = pr;
        gc.recon = rc;
        const size_t b = soa_bytes(pr, rc, g.stride);
        for (int m = 0; m < 4; ++m)
            for (int q = 0; q < 2; ++q) gc.d[m][q] = dalloc(c, b);
        for (int m = 0; m < 4; ++m)
            if (g.split >> m & 1)
                for (int q = 0; q < 2; ++q) gc.ghost[m][q] = dalloc(c, soa_bytes(pr, rc, g.fsd[m]));
        launch_gauge_pack2(pr, rc, g, ext, gc.d, gc.ghost, bad, c->stream);
        c->launches += 1;
    }
    // 4. clover T and T^{-1} in fp64, then each working precision
    double *T64[2], *I64[2];
    for (int q = 0; q < 2; ++q) {
        T64[q] = static_cast<double *>(dalloc(c, sizeof(double) * 72 * g.Vh));
        I64[q] = static_cast<double *>(dalloc(c, sizeof(double) * 72 * g.Vh));
    }
    int *bad_clover = c->d_flag + 1;
    QX_CUDA(cudaMemsetAsync(bad_clover, 0, sizeof(int), c->stream));
    launch_clover_build(g, ext, p->kappa, p->csw, T64, I64, bad_clover, c->stream);
    c->launches += 1;
    for (int k = 0; k < c->ncopies; ++k) {
        int pr = c->gcopy[k].prec;
        auto &cl = c->clov[prec_idx(pr)];
        if (cl.valid) continue;
        for (int q = 0; q < 2; ++q) {
            cl.T[q] = dalloc(c, clover_bytes(pr, g.stride));
            cl.Tinv[q] = dalloc(c, clover_bytes(pr, g.stride));
            launch_clover_pack(pr, g, T64[q], cl.T[q], c->stream);
            launch_clover_pack(pr, g, I64[q], cl.Tinv[q], c->stream);
            c->launches += 2;
        }
        cl.valid = true;
    }
    int hbad[2];
    QX_CUDA(cudaMemcpyAsync(hbad, c->d_flag, sizeof(hbad), cudaMemcpyDeviceToHost, c->stream));
    QX_CUDA(cudaStreamSynchronize(c->stream));
    for (int q = 0; q < 2; ++q) { dfree(c, T64[q]); dfree(c, I64[q]); }
    dfree(c, ext);
    QX_CHECK(hbad[1] == 0, QUDAX_ERR_ARG, "clover term singular on " + std::to_string(hbad[1]) + " chiral blocks");
    bool r8 = (p->recon == 8) || (p->recon_sloppy == 8 && p->prec_sloppy != p->prec);
    if (r8 && hbad[0]) {
        throw Error(QUDAX_ERR_UNSUPPORTED, "reconstruct 8 rejected: " + std::to_string(hbad[0]) +
                                               " links with |u01|^2+|u02|^2 < 1e-6 (e.g. unit gauge)");
    }
    c->gauge_loaded = true;
}

}  // namespace qx

// ============================================================================ C ABI
using namespace qx;

namespace {
template <typename F>
qudax_status guard(qudax_ctx *c, F &&fn) {
    if (c && c->sticky) return QUDAX_ERR_STATE;
    try {
        fn();
        return QUDAX_OK;
    } catch (const Error &e) {
        if (c) {
            c->err = e.what();
            if (e.status == QUDAX_ERR_CUDA || e.status == QUDAX_ERR_NCCL) c->sticky = true;
        }
        return e.status;
    } catch (const std::exception &e) {
        if (c) c->err = e.what();
        return QUDAX_ERR_STATE;
    } catch (...) {
        if (c) c->err = "unknown exception";
        return QUDAX_ERR_STATE;
    }
}

// Process-grid bookkeeping (multi-dimensional split: SURVEY 8(f) item 4).
// halo_p2p: the init's halo kind (a P2P halo at one rank defaults to a T loopback).
qudax_status fill_partition(const int gd[4], const int grid_in[4], int nranks, int rank, int split_mask, int comm,
                            int halo_p2p, qudax_partition *o) {
    if (!gd || !o || nranks < 1 || rank < 0 || rank >= nranks) return QUDAX_ERR_ARG;
    int P[4] = {1, 1, 1, nranks};
    if (grid_in && (grid_in[0] | grid_in[1] | grid_in[2] | grid_in[3])) {
        for (int k = 0; k < 4; ++k) P[k] = grid_in[k];
    }
    long prod = 1;
    for (int k = 0; k < 4; ++k) {
        if (gd[k] < 1 || P[k] < 1 || gd[k] % P[k]) return QUDAX_ERR_ARG;
        prod *= P[k];
    }
    if (prod != nranks) return QUDAX_ERR_ARG;
    int L[4], c[4];
    for (int k = 0; k < 4; ++k) L[k] = gd[k] / P[k];
    {
        int r = rank;
        for (int k = 0; k < 4; ++k) {
            c[k] = r % P[k];
            r /= P[k];
        }
    }
    int split = 0;
    for (int k = 0; k < 4; ++k)
        if (P[k] > 1) split |= 1 << k;
    if (split_mask) {
        if ((split_mask & split) != split || (split_mask & ~15)) return QUDAX_ERR_ARG;
        split = split_mask;
    } else if (split == 0 && (comm != QUDAX_COMM_NONE || halo_p2p)) {
        split = 8;  // one rank with a transport: T loopback (the split path at N = 1)
    }
    if (L[0] % 2) return QUDAX_ERR_ARG;
    if (L[3] < 2 || L[3] % 2) return QUDAX_ERR_ARG;
    for (int k = 0; k < 4; ++k)
        if ((split >> k & 1) && (L[k] < 2 || L[k] % 2)) return QUDAX_ERR_ARG;
    if ((split & 1) && L[1] % 2) return QUDAX_ERR_ARG;  // X faces pair their sites along y
    std::memset(o, 0, sizeof(*o));
    o->T_loc = L[3];
    o->t0 = c[3] * L[3];
    o->V_s = (long)L[0] * L[1] * L[2];
    o->V_loc = o->V_s * L[3];
    o->V_h = o->V_loc / 2;
    o->face_sites = o->V_s / 2;
    o->applies_bc_fwd = (c[3] == P[3] - 1);
    o->applies_bc_back = (c[3] == 0);
    o->face_bytes[0] = (size_t)o->face_sites * (12 * 2 + 4);
    o->face_bytes[1] = (size_t)o->face_sites * 12 * 4;
    o->face_bytes[2] = (size_t)o->face_sites * 12 * 8;
    auto rank_of = [&](const int cc[4]) { return ((cc[3] * P[2] + cc[2]) * P[1] + cc[1]) * P[0] + cc[0]; };
    for (int k = 0; k < 4; ++k) {
        o->proc_grid[k] = P[k];
        o->coords[k] = c[k];
        o->local_dims[k] = L[k];
        o->origin[k] = c[k] * L[k];
        int cf[4] = {c[0], c[1], c[2], c[3]}, cb[4] = {c[0], c[1], c[2], c[3]};
        cf[k] = (c[k] + 1) % P[k];
        cb[k] = (c[k] - 1 + P[k]) % P[k];
        o->nb_fwd[k] = rank_of(cf);
        o->nb_back[k] = rank_of(cb);
        o->face_sites_dim[k] = o->V_loc / L[k] / 2;
    }
    o->rank_fwd = o->nb_fwd[3];
    o->rank_back = o->nb_back[3];
    o->split_mask = split;
    return QUDAX_OK;
}
}  // namespace

extern "C" {

int qudax_abi_version(void) { return QUDAX_ABI_VERSION; }

const char *qudax_status_string(int s) {
    switch (s) {
        case QUDAX_OK: return "ok";
        case QUDAX_ERR_ARG: return "invalid argument";
        case QUDAX_ERR_STATE: return "invalid state";
        case QUDAX_ERR_CUDA: return "CUDA error";
        case QUDAX_ERR_NCCL: return "NCCL error";
        case QUDAX_ERR_UNSUPPORTED: return "unsupported";
        case QUDAX_ERR_NOT_CONVERGED: return "not converged";
        case QUDAX_ERR_OOM: return "out of device memory";
        case QUDAX_ERR_COMM: return "host transport failed";
        default: return "unknown status";
    }
}

qudax_status qudax_partition_info(const int global_dims[4], const int proc_grid[4], int nranks, int rank,
                                  int split_mask, qudax_partition *out) {
    return fill_partition(global_dims, proc_grid, nranks, rank, split_mask, QUDAX_COMM_NONE, 0, out);
}

qudax_status qudax_model(int prec, int recon, int kind, qudax_site_model *o) {
    if (!o || (prec != 2 && prec != 4 && prec != 8) || (recon != 18 && recon != 12 && recon != 8) || kind < -2 ||
        kind > 3)
        return QUDAX_ERR_ARG;
    const double w = prec;
    const double norm = (prec == 2) ? 4 : 0;
    const double sp = 24 * w + norm, hsp = 12 * w + norm, link = recon * w, clov = 72 * w + (prec == 2 ? 8 : 0);
    auto one = [&](int k, qudax_site_model *m) {
        const double cl = (k == QUDAX_HOP) ? 0 : clov;
        const double xs = (k >= QUDAX_CLOVER_XPAY) ? sp : 0;
        m->flops = 1320 + (k == QUDAX_HOP ? 0 : 504) + (k >= QUDAX_CLOVER_XPAY ? 48 : 0);
        m->bytes_paper = 6 * sp + 2 * hsp + 8 * link + cl + xs + sp;
        m->bytes_compulsory = 8 * link + sp + cl + xs + sp;
    };
    if (kind >= 0) {
        one(kind, o);
    } else {
        qudax_site_model a, b;
        one(QUDAX_CLOVER_INV, &a);
        one(QUDAX_CLOVER_XPAY, &b);
        o->flops = a.flops + b.flops;
        o->bytes_paper = a.bytes_paper + b.bytes_paper;
        o->bytes_compulsory = a.bytes_compulsory + b.bytes_compulsory;
        if (kind == -2) {
            // single-launch (fused) Mhat: the links are compulsory once, both clover terms,
            // the input (also the xpay x), the output, and the intermediate written once
            o->bytes_compulsory = 8 * link + 2 * clov + 3 * sp;
        }
    }
    return QUDAX_OK;
}

qudax_status qudax_nccl_unique_id(void *out128) {
    if (!out128) return QUDAX_ERR_ARG;
    ncclUniqueId id;
    if (ncclGetUniqueId(&id) != ncclSuccess) return QUDAX_ERR_NCCL;
    static_assert(sizeof(id) == 128, "ncclUniqueId size");
    std::memcpy(out128, &id, 128);
    return QUDAX_OK;
}

// Allgather of one small record per rank over the comm transport: NCCL (device buffers), or the
// host hooks — the allreduce hook sums doubles, so each rank places its bytes, as exact 16-bit
// integers, in its own slice of a zero array (sums of one non-zero term are exact).
static void allgather_small(qudax_ctx *c, const void *mine, size_t n, void *all) {
    const Geom &g = c->g;
    if (c->comm == QUDAX_COMM_NCCL) {
        char *d = static_cast<char *>(dalloc(c, n * (g.nranks + 1)));
        QX_CUDA(cudaMemcpyAsync(d, mine, n, cudaMemcpyHostToDevice, c->stream));
        QX_NCCL(ncclAllGather(d, d + n, n, ncclChar, c->nccl_red, c->stream));
        QX_CUDA(cudaMemcpyAsync(all, d + n, n * g.nranks, cudaMemcpyDeviceToHost, c->stream));
        QX_CUDA(cudaStreamSynchronize(c->stream));
        dfree(c, d);
    } else if (c->comm == QUDAX_COMM_HOST) {
        const size_t w = (n + 1) / 2;  // 16-bit words per record
        std::vector<double> v(w * g.nranks, 0.0);
        const unsigned char *m = static_cast<const unsigned char *>(mine);
        for (size_t k = 0; k < w; ++k)
            v[w * g.rank + k] = (double)(m[2 * k] | ((2 * k + 1 < n ? m[2 * k + 1] : 0) << 8));
        if (c->host_allreduce(v.data(), (int)v.size(), c->comm_user))
            throw Error(QUDAX_ERR_COMM, "host_allreduce hook failed (allgather)");
        unsigned char *o = static_cast<unsigned char *>(all);
        for (int r = 0; r < g.nranks; ++r)
            for (size_t k = 0; k < n; ++k) {
                const unsigned u = (unsigned)v[w * r + k / 2];
                o[n * r + k] = (unsigned char)((k & 1) ? (u >> 8) : (u & 255));
            }
    } else {
        throw Error(QUDAX_ERR_ARG, "P2P mode with nranks > 1 needs a comm transport for the handle exchange");
    }
}

// QUDAX_HALO_P2P setup: one IPC-exportable region per rank with the same layout everywhere
// (ctx.h P2P): the halo ghosts and flags, and the slot area of the kernel-side allreduce
// (internal.h DevAllreduce).  Every rank's {IPC handle, PCI bus id} is allgathered; the
// T-neighbours' regions (and, for nranks <= kMaxPeers, every rank's, for the allreduce) are
// mapped.  A rank on another GPU must be reachable by peer access (NVLink / NVSwitch on a B200
// node), else UNSUPPORTED: the comm path (NCCL) is for GPUs without peer access.
static void setup_p2p(qudax_ctx *c) {
    auto &q = c->p2p;
    const Geom &g = c->g;
    auto up = [](size_t v) { return (v + 255) & ~(size_t)255; };
    size_t cur = 0;
    const int precs[3] = {8, 4, 2};
    for (int k = 0; k < 3; ++k) {
        const int pi = prec_idx(precs[k]);
        for (int m = 0; m < 4; ++m) {  // ghosts of every split dimension, two sequence parities each
            if (!(g.split >> m & 1)) continue;
            q.pdist[pi][m] = up(m == 3 ? face_bytes(precs[k], g.fstride) : sface_bytes(precs[k], m, g.fsd[m]));
            q.off_g[pi][m][0] = cur;
            cur += 2 * q.pdist[pi][m];
            q.off_g[pi][m][1] = cur;
            cur += 2 * q.pdist[pi][m];
        }
    }
    q.off_flags = cur;
    q.off_seq = cur + 64;
    q.off_count = cur + 128;
    q.off_cseq = cur + 192;
    q.off_ccount = cur + 256;
    q.off_ar = cur + 512;
    q.bytes = q.off_ar + sizeof(double) * 4 * kArChannels * 2 * kMaxPeers;
    void *base = nullptr;
    QX_CUDA(cudaMalloc(&base, q.bytes));  // not the caller's allocator: IPC exports whole allocations
    q.base = static_cast<char *>(base);
    QX_CUDA(cudaMemset(q.base, 0, q.bytes));
    QX_CUDA(cudaDeviceSynchronize());
    for (int r = 0; r < kMaxPeers; ++r) q.peer[r] = nullptr;
    if (g.nranks > 1) {
        static_assert(sizeof(cudaIpcMemHandle_t) == 64, "IPC handle size");
        struct Rec {
            cudaIpcMemHandle_t h;
            char bus[64];
        };
        Rec mine{};
        QX_CUDA(cudaIpcGetMemHandle(&mine.h, q.base));
        QX_CUDA(cudaDeviceGetPCIBusId(mine.bus, sizeof(mine.bus), c->device));
        std::vector<Rec> all(g.nranks);
        allgather_small(c, &mine, sizeof(Rec), all.data());
        const bool map_all = g.nranks <= kMaxPeers;
        q.opened.assign(g.nranks, nullptr);
        auto is_nb = [&](int r) {
            for (int m = 0; m < 4; ++m)
                if ((g.split >> m & 1) && (r == g.nbf[m] || r == g.nbb[m])) return true;
            return false;
        };
        for (int r = 0; r < g.nranks; ++r) {
            if (r == g.rank || !(map_all || is_nb(r))) continue;
            const Rec &rec = all[r];
            if (std::strncmp(rec.bus, mine.bus, sizeof(mine.bus)) != 0) {  // another GPU (else test mode)
                int peer = -1, can = 0;
                if (cudaDeviceGetByPCIBusId(&peer, rec.bus) != cudaSuccess) {
                    cudaGetLastError();  // the peer GPU is not visible to this process: no peer access
                    throw Error(QUDAX_ERR_UNSUPPORTED, std::string("P2P: rank ") + std::to_string(r) + "'s GPU " +
                                                           rec.bus + " not visible here");
                }
                QX_CUDA(cudaDeviceCanAccessPeer(&can, c->device, peer));
                if (!can)
                    throw Error(QUDAX_ERR_UNSUPPORTED, std::string("P2P: no peer access to rank ") + std::to_string(r) +
                                                           "'s GPU " + rec.bus);
            }
            void *pr = nullptr;
            QX_CUDA(cudaIpcOpenMemHandle(&pr, rec.h, cudaIpcMemLazyEnablePeerAccess));
            q.opened[r] = static_cast<char *>(pr);
        }
        auto region = [&](int r) { return r == g.rank ? q.base : q.opened[r]; };
        for (int m = 0; m < 4; ++m) {
            q.peer_b[m] = region(g.nbb[m]);
            q.peer_f[m] = region(g.nbf[m]);
        }
        if (map_all)
            for (int r = 0; r < g.nranks; ++r) q.peer[r] = region(r);
    } else {  // loopback: the neighbour is this rank
        for (int m = 0; m < 4; ++m) q.peer_b[m] = q.peer_f[m] = q.base;
        q.peer[0] = q.base;
    }
    // kernel-side allreduce descriptor (device memory), when every rank is mapped
    if (g.nranks <= kMaxPeers) {
        DevAllreduce d{};
        for (int r = 0; r < g.nranks; ++r) d.slots[r] = reinterpret_cast<double *>(q.peer[r] + q.off_ar);
        d.seq = static_cast<unsigned *>(dalloc(c, sizeof(unsigned) * kArChannels));
        QX_CUDA(cudaMemset(d.seq, 0, sizeof(unsigned) * kArChannels));
        d.nranks = g.nranks;
        d.rank = g.rank;
        d.err = c->d_err;
        c->dar = static_cast<DevAllreduce *>(dalloc(c, sizeof(DevAllreduce)));
        QX_CUDA(cudaMemcpy(c->dar, &d, sizeof(d), cudaMemcpyHostToDevice));
    }
}

qudax_status qudax_init(qudax_ctx **out, const qudax_init_param *p) {
    if (!out || !p) return QUDAX_ERR_ARG;
    *out = nullptr;
    if (p->comm < 0 || p->comm > 2) return QUDAX_ERR_ARG;
    if (p->halo != QUDAX_HALO_COMM && p->halo != QUDAX_HALO_P2P) return QUDAX_ERR_ARG;
    qudax_partition part;
    if (fill_partition(p->global_dims, p->proc_grid, p->nranks, p->rank, p->split_mask, p->comm,
                       p->halo == QUDAX_HALO_P2P, &part) != QUDAX_OK)
        return QUDAX_ERR_ARG;
    if (p->comm == QUDAX_COMM_NONE && p->nranks != 1) return QUDAX_ERR_ARG;
    if (p->comm == QUDAX_COMM_NCCL && !p->nccl_id) return QUDAX_ERR_ARG;
    if (p->comm == QUDAX_COMM_HOST && (!p->host_exchange || !p->host_allreduce)) return QUDAX_ERR_ARG;
    // a loopback dimension without a transport has nobody to move its faces
    if (p->comm == QUDAX_COMM_NONE && p->halo != QUDAX_HALO_P2P && part.split_mask) return QUDAX_ERR_ARG;
    auto *c = new qudax_ctx();
    qudax_status st = guard(c, [&] {
        Geom &g = c->g;
        for (int k = 0; k < 4; ++k) {
            g.G[k] = p->global_dims[k];
            g.L[k] = part.local_dims[k];
            g.P[k] = part.proc_grid[k];
            g.c[k] = part.coords[k];
            g.o[k] = part.origin[k];
            g.nbf[k] = part.nb_fwd[k];
            g.nbb[k] = part.nb_back[k];
            g.Fd[k] = part.face_sites_dim[k];
            g.fsd[k] = pad64(g.Fd[k]);
        }
        g.split = part.split_mask;
        g.X = g.L[0]; g.Y = g.L[1]; g.Z = g.L[2]; g.T = p->global_dims[3];
        g.nranks = p->nranks; g.rank = p->rank;
        g.T_loc = part.T_loc; g.t0 = part.t0;
        g.Xh = g.X / 2;
        g.Vs = part.V_s; g.V = part.V_loc; g.Vh = part.V_h; g.F = part.face_sites;
        g.stride = pad64(g.Vh);
        g.fstride = pad64(g.F);
        // interior box in (xh, y, z, t): one site off every split face.  A split X has no
        // overlapped interior: its face sites are one per row, so a boundary launch over them is
        // uncoalesced (measured at 32^3x64 fp32: ~150 us for 1/8 of the sites, as long as the
        // whole-lattice kernel) — the exchange then precedes one coalesced launch (n_int = 0).
        {
            const int ext[4] = {g.Xh, g.Y, g.Z, g.T_loc};
            g.n_int = 1;
            for (int k = 0; k < 4; ++k) {
                const int s = (g.split >> k) & 1;
                g.blo[k] = s;
                g.bn[k] = std::max(0, ext[k] - 2 * s);
                g.n_int *= g.bn[k];
            }
            if (g.split & 1) g.n_int = 0;
        }
        QX_CHECK(g.V < (1L << 30), QUDAX_ERR_ARG, "local volume too large for 32-bit site indexing");
        c->device = p->device;
        c->flags = p->flags;
        if (p->copy_threads > 0 && g_copy_threads == 0) g_copy_threads = p->copy_threads;
        c->comm = p->comm;
        c->overlap = p->overlap;
        c->dev_alloc = p->dev_alloc; c->dev_free = p->dev_free; c->alloc_user = p->alloc_user;
        c->host_exchange = p->host_exchange; c->host_allreduce = p->host_allreduce; c->comm_user = p->comm_user;
        QX_CUDA(cudaSetDevice(p->device));
        if (p->stream) {
            c->stream = reinterpret_cast<cudaStream_t>(p->stream);
        } else {
            QX_CUDA(cudaStreamCreateWithFlags(&c->stream, cudaStreamNonBlocking));
            c->own_stream = true;
        }
        int lo, hi;
        QX_CUDA(cudaDeviceGetStreamPriorityRange(&lo, &hi));
        QX_CUDA(cudaStreamCreateWithPriority(&c->comm_stream, cudaStreamNonBlocking, hi));
        QX_CUDA(cudaEventCreateWithFlags(&c->ev_in, cudaEventDisableTiming));
        QX_CUDA(cudaEventCreateWithFlags(&c->ev_halo, cudaEventDisableTiming));
        if (c->comm == QUDAX_COMM_NCCL) {
            ncclUniqueId id;
            std::memcpy(&id, p->nccl_id, sizeof(id));
            QX_NCCL(ncclCommInitRank(&c->nccl, g.nranks, id, g.rank));
            // a second communicator for the global sums: the halo's send/recv run on the comm
            // stream and the allreduces on the compute stream, so neither has to be ordered
            // against the other inside one communicator (NCCL serialises a communicator's
            // operations in issue order, whatever stream they were issued to)
            QX_NCCL(ncclCommSplit(c->nccl, 0, g.rank, &c->nccl_red, nullptr));
        }
        c->partials = static_cast<double *>(dalloc(c, sizeof(double) * 4 * blas_partial_blocks()));
        c->red_out = static_cast<double *>(dalloc(c, sizeof(double) * 8));
        c->h_red = static_cast<double *>(halloc(c, sizeof(double) * 8));
        c->d_flag = static_cast<int *>(dalloc(c, sizeof(int) * 4));
        {  // device error word, readable by the host after any synchronisation without a copy
            void *h = nullptr;
            QX_CUDA(cudaHostAlloc(&h, 64, cudaHostAllocMapped));
            c->host_allocs.push_back(h);
            c->h_err = static_cast<int *>(h);
            *c->h_err = 0;
            void *d = nullptr;
            QX_CUDA(cudaHostGetDevicePointer(&d, h, 0));
            c->d_err = static_cast<int *>(d);
        }
        // reduction tail counters: [0] groups done, [1 + g] CTAs done in group g (reduce.cuh)
        const size_t ncount = 2 + (size_t)(g.Vh / 32) / 64 + 64;
        c->d_counter = static_cast<unsigned *>(dalloc(c, sizeof(unsigned) * ncount));
        QX_CUDA(cudaMemsetAsync(c->d_counter, 0, sizeof(unsigned) * ncount, c->stream));
        if (p->halo == QUDAX_HALO_P2P) {
            setup_p2p(c);
            c->p2p.on = true;
        }
        if (spatial_split(g) && g.n_int > 0) {  // boundary sites of a multi-dimensional split: the box complement
            std::vector<int> bl;
            bl.reserve((size_t)(g.Vh - g.n_int));
            for (long i = 0; i < g.Vh; ++i) {
                long r = i;
                const int xh = (int)(r % g.Xh);
                r /= g.Xh;
                const int y = (int)(r % g.Y);
                r /= g.Y;
                const int z = (int)(r % g.Z);
                const int t = (int)(r / g.Z);
                const int cc[4] = {xh, y, z, t};
                bool in = true;
                for (int k = 0; k < 4; ++k) in &= cc[k] >= g.blo[k] && cc[k] < g.blo[k] + g.bn[k];
                if (!in) bl.push_back((int)i);
            }
            QX_CHECK((long)bl.size() == g.Vh - g.n_int, QUDAX_ERR_STATE, "boundary list size");
            c->blist = static_cast<int *>(dalloc(c, sizeof(int) * std::max<size_t>(bl.size(), 1)));
            QX_CUDA(cudaMemcpy(c->blist, bl.data(), sizeof(int) * bl.size(), cudaMemcpyHostToDevice));
        }
    });
    if (st != QUDAX_OK) {
        qudax_finalize(c);
        return st;
    }
    *out = c;
    return QUDAX_OK;
}

qudax_status qudax_finalize(qudax_ctx *c) {
    if (!c) return QUDAX_ERR_ARG;
    if (c->flags & QUDAX_FLAG_TIMING_BREAKDOWN)
        for (auto &kv : g_tbreak)
            std::fprintf(stderr, "qudax timing: prec %d kind %d red %d: %ld launches, %.2f us avg\n", std::get<0>(kv.first),
                         std::get<1>(kv.first), std::get<2>(kv.first), kv.second.first, 1e3 * kv.second.second / kv.second.first);
    if (c->stream) cudaStreamSynchronize(c->stream);
    if (c->comm_stream) cudaStreamSynchronize(c->comm_stream);
    // the cached solver graphs first: graphs that captured NCCL operations hold references on
    // the communicators (CUDA user objects), and ncclCommDestroy waits for them — with the graphs
    // still alive it never returned (gpurun r02e: every NCCL-loopback solve test hung in close)
    drop_graphs(c);  // (their timing events go back to the pool, destroyed below)
    cudaDeviceSynchronize();  // lets the user objects' release callbacks run
    for (char *m : c->p2p.opened)
        if (m) cudaIpcCloseMemHandle(m);
    if (c->p2p.base) cudaFree(c->p2p.base);
    if (c->nccl_red) ncclCommDestroy(c->nccl_red);
    if (c->nccl) ncclCommDestroy(c->nccl);
    for (void *p : c->allocs) {
        if (c->dev_free) c->dev_free(p, c->alloc_user);
        else cudaFree(p);
    }
    for (void *p : c->host_allocs) cudaFreeHost(p);
    for (auto &r : c->trecs) { cudaEventDestroy(r.a); cudaEventDestroy(r.b); }
    for (auto &r : c->graph_trecs) { cudaEventDestroy(r.a); cudaEventDestroy(r.b); }
    for (auto e : c->ev_pool) cudaEventDestroy(e);
    for (auto e : c->xfer.done)
        if (e) cudaEventDestroy(e);
    for (auto e : c->tl)
        if (e) cudaEventDestroy(e);
    if (c->ev_in) cudaEventDestroy(c->ev_in);
    if (c->ev_halo) cudaEventDestroy(c->ev_halo);
    if (c->comm_stream) cudaStreamDestroy(c->comm_stream);
    if (c->own_stream && c->stream) cudaStreamDestroy(c->stream);
    delete c;
    return QUDAX_OK;
}

const char *qudax_last_error(const qudax_ctx *c) { return c ? c->err.c_str() : "null context"; }

qudax_status qudax_sync(qudax_ctx *c) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CUDA(cudaStreamSynchronize(c->stream));
        QX_CUDA(cudaStreamSynchronize(c->comm_stream));
        check_device_error(c);
    });
}

long long qudax_launch_count(const qudax_ctx *c) { return c ? c->launches : -1; }

qudax_status qudax_get_partition(const qudax_ctx *c, qudax_partition *out) {
    if (!c || !out) return QUDAX_ERR_ARG;
    return fill_partition(c->g.G, c->g.P, c->g.nranks, c->g.rank, c->g.split, c->comm, c->p2p.on, out);
}

qudax_status qudax_kernel_timing(qudax_ctx *c, int enable) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CUDA(cudaStreamSynchronize(c->stream));
        for (auto &r : c->trecs) {
            c->ev_pool.push_back(r.a);
            c->ev_pool.push_back(r.b);
        }
        c->trecs.clear();
        for (auto &t : c->tacc) t = qudax_ctx::TimingAcc{};
        c->timing = enable == 2 ? 2 : (enable != 0 ? 1 : 0);
    });
}

qudax_status qudax_get_kernel_stats(qudax_ctx *c, int prec_filter, qudax_kernel_stats *o) {
    if (!c || !o) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CUDA(cudaStreamSynchronize(c->stream));
        std::memset(o, 0, sizeof(*o));
        fetch_spans(c);
        for (auto &r : c->trecs) {
            if (prec_filter && r.prec != prec_filter) continue;
            float ms = 0;
            QX_CUDA(cudaEventElapsedTime(&ms, r.a, r.b));
            qudax_site_model m;
            rec_model(r, &m);
            o->launches += 1;
            o->ms_total += ms;
            o->span_ms_total += span_ms(c, r);
            o->sites += r.sites * r.nrhs;
            o->flops += m.flops;
            o->bytes_compulsory += m.bytes_compulsory;
            o->bytes_paper += m.bytes_paper;
        }
        for (int q = 0; q < 3; ++q) {
            const int pr = q == 0 ? 8 : (q == 1 ? 4 : 2);
            if (prec_filter && pr != prec_filter) continue;
            const auto &t = c->tacc[q];
            o->launches += t.launches;
            o->sites += t.sites;
            o->ms_total += t.ms;
            o->span_ms_total += t.span_ms;
            o->flops += t.flops;
            o->bytes_compulsory += t.bytes_c;
            o->bytes_paper += t.bytes_p;
        }
    });
}

qudax_status qudax_halo_timeline(qudax_ctx *c, int enable, double *out7) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        if (out7) {
            QX_CHECK(c->tl_valid, QUDAX_ERR_STATE, "halo timeline: no split Dslash recorded");
            QX_CUDA(cudaStreamSynchronize(c->stream));
            QX_CUDA(cudaStreamSynchronize(c->comm_stream));
            for (int k = 1; k < 8; ++k) {
                float ms = 0;
                QX_CUDA(cudaEventElapsedTime(&ms, c->tl[0], c->tl[k]));
                out7[k - 1] = 1e3 * ms;
            }
        }
        if (enable && !c->tl[0])
            for (auto &e : c->tl) QX_CUDA(cudaEventCreate(&e));
        c->tl_on = enable != 0;
    });
}

qudax_status qudax_gauge_load(qudax_ctx *c, const double *host_gauge, const qudax_gauge_param *p) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] { gauge_load(c, host_gauge, p); });
}

size_t qudax_spinor_bytes(const qudax_ctx *c, int prec) {
    if (!c || (prec != 2 && prec != 4 && prec != 8)) return 0;
    return spinor_bytes(prec, c->g.stride);
}

static double *stage_buf(qudax_ctx *c) {
    if (!c->stage) c->stage = static_cast<double *>(dalloc(c, sizeof(double) * 24 * c->g.V));
    return c->stage;
}

qudax_status qudax_spinor_load(qudax_ctx *c, void *dst, int prec, int parity, const double *host_src) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(dst && host_src && (parity == 0 || parity == 1), QUDAX_ERR_ARG, "spinor_load: bad argument");
        double *st = stage_buf(c);
        h2d(c, st, host_src, sizeof(double) * 24 * c->g.V);
        launch_spinor_import(prec, c->g, parity, st, dst, c->stream);
        c->launches += 1;
        QX_CUDA(cudaStreamSynchronize(c->stream));
    });
}

qudax_status qudax_spinor_load_dev(qudax_ctx *c, void *dst, int prec, int parity, const double *dev_src) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(dst && dev_src && (parity == 0 || parity == 1), QUDAX_ERR_ARG, "spinor_load_dev: bad argument");
        launch_spinor_import(prec, c->g, parity, dev_src, dst, c->stream);
        c->launches += 1;
    });
}

qudax_status qudax_spinor_store(qudax_ctx *c, double *host_dst, const void *src, int prec, int parity) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(src && host_dst && (parity == 0 || parity == 1), QUDAX_ERR_ARG, "spinor_store: bad argument");
        double *st = stage_buf(c);
        const size_t n = sizeof(double) * 24 * c->g.V;
        h2d(c, st, host_dst, n);  // keep the other parity
        launch_spinor_export(prec, c->g, parity, src, st, c->stream);
        c->launches += 1;
        d2h(c, host_dst, st, n);
    });
}

qudax_status qudax_spinor_store_dev(qudax_ctx *c, double *dev_dst, const void *src, int prec, int parity) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(src && dev_dst && (parity == 0 || parity == 1), QUDAX_ERR_ARG, "spinor_store_dev: bad argument");
        launch_spinor_export(prec, c->g, parity, src, dev_dst, c->stream);
        c->launches += 1;
    });
}

qudax_status qudax_spinor_convert(qudax_ctx *c, void *dst, int dst_prec, const void *src, int src_prec) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(dst_prec);
        check_prec(src_prec);
        QX_CHECK(dst && src && dst != src, QUDAX_ERR_ARG, "spinor_convert: bad argument");
        convert_op(c, dst, dst_prec, src, src_prec);
    });
}

qudax_status qudax_dslash(qudax_ctx *c, void *out, const void *in, const void *x, int prec, int out_parity,
                          int dagger, int kind, double a) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] { dslash_op(c, out, in, x, prec, out_parity, dagger ? 1 : 0, kind, a); });
}

qudax_status qudax_dslash_multi(qudax_ctx *c, void *const *out, const void *const *in, const void *const *x,
                                int nrhs, int prec, int out_parity, int dagger, int kind, double a) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CHECK(out && in, QUDAX_ERR_ARG, "dslash_multi: null arrays");
        dslash_multi_op(c, out, in, x, nrhs, prec, out_parity, dagger ? 1 : 0, kind, a, 0);
    });
}

qudax_status qudax_matpc_multi(qudax_ctx *c, void *const *out, const void *const *in, int nrhs, int prec,
                               int dagger) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CHECK(out && in, QUDAX_ERR_ARG, "matpc_multi: null arrays");
        matpc_multi_op(c, out, in, nrhs, prec, dagger ? 1 : 0);
    });
}

qudax_status qudax_matpc(qudax_ctx *c, void *out, const void *in, int prec, int dagger) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CHECK(out && in && out != in, QUDAX_ERR_ARG, "matpc: bad fields");
        matpc_op(c, out, in, prec, dagger ? 1 : 0);
    });
}

qudax_status qudax_matpc_sym(qudax_ctx *c, void *out, const void *in, int prec, int dagger) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CHECK(out && in && out != in, QUDAX_ERR_ARG, "matpc_sym: bad fields");
        check_prec(prec);
        matpc_sym_op(c, out, in, prec, dagger ? 1 : 0, nullptr);
    });
}

qudax_status qudax_mdagm(qudax_ctx *c, void *out, const void *in, int prec) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        QX_CHECK(out && in && out != in, QUDAX_ERR_ARG, "mdagm: bad fields");
        check_prec(prec);
        void *t = tmp_even(c, prec);
        matpc_op(c, t, in, prec, 0);
        matpc_op(c, out, t, prec, 1);
    });
}

qudax_status qudax_norm2(qudax_ctx *c, const void *f, int prec, double *out) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(f && out, QUDAX_ERR_ARG, "norm2: null");
        void *fs[1] = {const_cast<void *>(f)};
        blas_op(c, OP_NORM2, prec, fs, nullptr, out);
    });
}

qudax_status qudax_cdot(qudax_ctx *c, const void *a, const void *b, int prec, double out[2]) {
    if (!c) return QUDAX_ERR_ARG;
    return guard(c, [&] {
        check_prec(prec);
        QX_CHECK(a && b && out, QUDAX_ERR_ARG, "cdot: null");
        void *fs[2] = {const_cast<void *>(a), const_cast<void *>(b)};
        blas_op(c, OP_CDOT, prec, fs, nullptr, out);
    });
}

}  // extern "C"

namespace {
using SolveFn = void (*)(qudax_ctx *, double *, const double *, const qudax_solve_param *, qudax_solve_stats *);

qudax_status solve_device_entry(SolveFn fn, qudax_ctx *c, double *x, const double *b, const qudax_solve_param *p,
                                qudax_solve_stats *st) {
    if (!c) return QUDAX_ERR_ARG;
    qudax_status s = guard(c, [&] {
        QX_CHECK(x && b && p && st, QUDAX_ERR_ARG, "solve: null argument");
        auto t0 = std::chrono::steady_clock::now();
        fn(c, x, b, p, st);
        st->secs = std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
        st->gflops = st->flops / st->secs * 1e-9;
    });
    if (s == QUDAX_OK && st && p && p->tol > 0 && st->true_res > p->tol * (1 + 1e-3)) return QUDAX_ERR_NOT_CONVERGED;
    return s;
}

// host buffers: H2D of b and D2H of x are inside the call (and its timing)
qudax_status solve_host_entry(SolveFn fn, qudax_ctx *c, double *host_x, const double *host_b,
                              const qudax_solve_param *p, qudax_solve_stats *st) {
    if (!c) return QUDAX_ERR_ARG;
    double *db = nullptr, *dx = nullptr;
    auto t0 = std::chrono::steady_clock::now();
    qudax_status s = guard(c, [&] {
        QX_CHECK(host_x && host_b && p && st, QUDAX_ERR_ARG, "solve: null argument");
        const size_t n = sizeof(double) * 24 * c->g.V;
        db = static_cast<double *>(dalloc(c, n));
        dx = static_cast<double *>(dalloc(c, n));
        h2d(c, db, host_b, n);
        fn(c, dx, db, p, st);
        d2h(c, host_x, dx, n);
        dfree(c, db);
        dfree(c, dx);
        db = dx = nullptr;
        st->secs = std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
        st->gflops = st->flops / st->secs * 1e-9;
    });
    if (db) { cudaStreamSynchronize(c->stream); dfree(c, db); }
    if (dx) dfree(c, dx);
    if (s == QUDAX_OK && p->tol > 0 && st->true_res > p->tol * (1 + 1e-3)) return QUDAX_ERR_NOT_CONVERGED;
    return s;
}
// batched solve: device slabs, or host slabs staged through the ctx (H2D / D2H inside)
qudax_status solve_multi_entry(qudax_ctx *c, double *const *x, const double *const *b, int nrhs,
                               const qudax_solve_param *p, qudax_solve_stats *st, bool host) {
    if (!c) return QUDAX_ERR_ARG;
    double *dbuf = nullptr;
    auto t0 = std::chrono::steady_clock::now();
    qudax_status s = guard(c, [&] {
        QX_CHECK(x && b && p && st && nrhs >= 1 && nrhs <= kMaxRhs, QUDAX_ERR_ARG, "solve_multi: bad argument");
        for (int j = 0; j < nrhs; ++j) QX_CHECK(x[j] && b[j], QUDAX_ERR_ARG, "solve_multi: null slab");
        double *dx[kMaxRhs];
        const double *db[kMaxRhs];
        const size_t n = sizeof(double) * 24 * c->g.V;
        if (host) {
            dbuf = static_cast<double *>(dalloc(c, 2 * n * nrhs));
            for (int j = 0; j < nrhs; ++j) {
                db[j] = dbuf + (size_t)2 * j * (n / sizeof(double));
                dx[j] = const_cast<double *>(db[j]) + n / sizeof(double);
                h2d(c, const_cast<double *>(db[j]), b[j], n);
            }
        } else {
            for (int j = 0; j < nrhs; ++j) {
                db[j] = b[j];
                dx[j] = x[j];
            }
        }
        solve_multi_dev(c, dx, db, nrhs, p, st);
        if (host) {
            for (int j = 0; j < nrhs; ++j) d2h(c, x[j], dx[j], n);
            dfree(c, dbuf);
            dbuf = nullptr;
        }
        const double secs = std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
        for (int j = 0; j < nrhs; ++j) {
            st[j].secs = secs;  // the batch's wall time
            st[j].gflops = st[j].flops / secs * 1e-9;
        }
    });
    if (dbuf) { cudaStreamSynchronize(c->stream); dfree(c, dbuf); }
    if (s == QUDAX_OK && p->tol > 0)
        for (int j = 0; j < nrhs; ++j)
            if (st[j].true_res > p->tol * (1 + 1e-3)) return QUDAX_ERR_NOT_CONVERGED;
    return s;
}
}  // namespace

extern "C" {

qudax_status qudax_solve_bicgstab_multi(qudax_ctx *c, double *const *host_x, const double *const *host_b, int nrhs,
                                        const qudax_solve_param *p, qudax_solve_stats *st) {
    return solve_multi_entry(c, host_x, host_b, nrhs, p, st, true);
}
qudax_status qudax_solve_bicgstab_multi_dev(qudax_ctx *c, double *const *x, const double *const *b, int nrhs,
                                            const qudax_solve_param *p, qudax_solve_stats *st) {
    return solve_multi_entry(c, x, b, nrhs, p, st, false);
}

qudax_status qudax_solve_bicgstab_dev(qudax_ctx *c, double *x, const double *b, const qudax_solve_param *p,
                                      qudax_solve_stats *st) {
    return solve_device_entry(solve_dev, c, x, b, p, st);
}
qudax_status qudax_solve_bicgstab(qudax_ctx *c, double *host_x, const double *host_b, const qudax_solve_param *p,
                                  qudax_solve_stats *st) {
    return solve_host_entry(solve_dev, c, host_x, host_b, p, st);
}
qudax_status qudax_solve_cgnr_dev(qudax_ctx *c, double *x, const double *b, const qudax_solve_param *p,
                                  qudax_solve_stats *st) {
    return solve_device_entry(cgnr_dev, c, x, b, p, st);
}
qudax_status qudax_solve_cgnr(qudax_ctx *c, double *host_x, const double *host_b, const qudax_solve_param *p,
                              qudax_solve_stats *st) {
    return solve_host_entry(cgnr_dev, c, host_x, host_b, p, st);
}

}  // extern "C"
