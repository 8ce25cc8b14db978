// blas.cu — fused BLAS-1 and reduction kernels for the BiCGstab driver ("kernel
// fusion wherever possible to reduce memory traffic"; P:721-725 global sums).  All vectors
// are parity fields (V_h sites) in the site-major SoA of one precision; arithmetic is in the
// storage precision's compute type (fp32 for half), every reduction accumulates in fp64 and
// is reduced deterministically (reduce.cuh: fixed per-CTA slots, the last CTA sums them in a
// fixed order — reading Q12), so results are bitwise reproducible run to run.
// Coefficients are either values or device scalars (CoefArg), so the solver iteration can run
// without host round trips.
#include <mutex>
#include <unordered_map>

#include "core.cuh"
#include "internal.h"
#include "reduce.cuh"

namespace qx {

constexpr int kBlasThreads = 256;
constexpr int kBlasMaxBlocks = 160 * 8;  // partials capacity: <= 8 resident 256-thread CTAs per SM

int blas_partial_blocks() { return kBlasMaxBlocks; }

// Exactly one full wave: SMs x resident CTAs per SM for this kernel (a fixed multiple of 148
// that does not fit one wave leaves a ragged second wave).  Cached per kernel; the grid is a
// property of the kernel and the device only, so the reductions stay deterministic.
template <typename K>
static int one_wave(K kernel) {
    static std::mutex mu;
    static std::unordered_map<const void *, int> cache;
    std::lock_guard<std::mutex> lk(mu);
    auto it = cache.find((const void *)kernel);
    if (it != cache.end()) return it->second;
    int dev = 0, sms = 0, per = 0;
    QX_CUDA(cudaGetDevice(&dev));
    QX_CUDA(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev));
    QX_CUDA(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, kernel, kBlasThreads, 0));
    int b = sms * (per > 0 ? per : 1);
    if (b > kBlasMaxBlocks) b = kBlasMaxBlocks;
    cache[(const void *)kernel] = b;
    return b;
}

template <int NRED>
__device__ __forceinline__ void block_reduce_store(double (&v)[NRED], const RedTail &t) {
    reduce_with_tail<NRED, kBlasThreads>(v, t);
}

// BiCGstab scalar recurrence after a multi-rank allreduce of S->red (single thread)
__global__ void k_coef(SolverScalars *S, int mode) {
    apply_coef(S, mode);
}
// first / last node of a batch graph (solver.cpp): the WHILE node's condition handle for the
// reduction tail that evaluates Algorithm R, and the batch's last iteration
__global__ void k_batch_begin(SolverScalars *S, unsigned long long cond, int n) {
    S->cond = cond;
    S->kstop = S->k + n;
}
__global__ void k_batch_end(SolverScalars *S) { S->cond = 0ull; }
// last node of the WHILE body: stop the loop after this iteration if the host must act
// (reliable update, convergence, maxiter: S->halt) or the batch is complete.  A kernel of its
// own so that the heavy kernels carry no conditional-handle call (ncu cannot profile kernels
// that can set a graph condition)
__global__ void k_batch_cond(const SolverScalars *S) {
    cudaGraphSetConditional((cudaGraphConditionalHandle)S->cond, (S->halt || S->k >= S->kstop) ? 0u : 1u);
}
void launch_batch_cond(const SolverScalars *S, cudaStream_t s) { k_batch_cond<<<1, 1, 0, s>>>(S); }
void launch_batch_begin(SolverScalars *S, unsigned long long cond, int n, cudaStream_t s) {
    k_batch_begin<<<1, 1, 0, s>>>(S, cond, n);
}
void launch_batch_end(SolverScalars *S, cudaStream_t s) { k_batch_end<<<1, 1, 0, s>>>(S); }
void launch_coef(SolverScalars *S, int mode, cudaStream_t s) {
    k_coef<<<1, 1, 0, s>>>(S, mode);
    QX_CUDA(cudaGetLastError());
}

// NCCL halo in tail mode (api.cpp dslash_op): after the exchange, one thread on the comm stream
// advances this rank's producer sequence number and raises the flags of every split dimension;
// the Dslash's boundary CTAs (RANGE_TAIL) acquire them (dslash.cuh p2p_wait).
__global__ void k_raise_flags(unsigned *flags, unsigned *seq, int mask) {
    const unsigned s = *seq + 1u;
    *seq = s;
    for (int m = 0; m < 4; ++m) {
        if (!(mask >> m & 1)) continue;
        asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(flags + 2 * m), "r"(s) : "memory");
        asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(flags + 2 * m + 1), "r"(s) : "memory");
    }
}
void launch_raise_flags(unsigned *flags, unsigned *seq, int mask, cudaStream_t s) {
    k_raise_flags<<<1, 1, 0, s>>>(flags, seq, mask);
    QX_CUDA(cudaGetLastError());
}

#define QX_GRID_LOOP(i) for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x)

// p <- r + beta (p - omega v)            (BiCGstab search direction)
template <int P>
__global__ void k_p_update(long Vh, long stride, const void *r, void *p, const void *v, CoefArg beta_, CoefArg omega_) {
    using R = typename Prec<P>::R;
    const double2 beta = coef_get(beta_), omega = coef_get(omega_);
    const Cx<R> b = cx((R)beta.x, (R)beta.y), w = cx((R)omega.x, (R)omega.y);
    QX_GRID_LOOP(i) {
        R rr[24], pp[24], vv[24];
        SpinorIO<P>::load(r, stride, i, rr);
        SpinorIO<P>::load(p, stride, i, pp);
        SpinorIO<P>::load(v, stride, i, vv);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            Cx<R> pk = cx(pp[2 * k], pp[2 * k + 1]), vk = cx(vv[2 * k], vv[2 * k + 1]);
            Cx<R> o = cx(rr[2 * k], rr[2 * k + 1]) + b * (pk - w * vk);
            pp[2 * k] = o.r;
            pp[2 * k + 1] = o.i;
        }
        SpinorIO<P>::store(p, stride, i, pp);
    }
}

// y <- y + c x   (c complex)
template <int P>
__global__ void k_caxpy(long Vh, long stride, CoefArg c_, const void *x, void *y, int rev) {
    using R = typename Prec<P>::R;
    const double2 c = coef_get(c_);
    const Cx<R> a = cx((R)c.x, (R)c.y);
    QX_GRID_LOOP(j) {
        const long i = rev ? Vh - 1 - j : j;  // (top-down: start where the previous kernel ended)
        R xx[24], yy[24];
        SpinorIO<P>::load(x, stride, i, xx);
        SpinorIO<P>::load(y, stride, i, yy);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            Cx<R> o = cx(yy[2 * k], yy[2 * k + 1]) + a * cx(xx[2 * k], xx[2 * k + 1]);
            yy[2 * k] = o.r;
            yy[2 * k + 1] = o.i;
        }
        SpinorIO<P>::store(y, stride, i, yy);
    }
}

// z <- x + a y  (real a); z may alias x or y
template <int P>
__global__ void k_xpay(long Vh, long stride, const void *x, double a, const void *y, void *z) {
    using R = typename Prec<P>::R;
    QX_GRID_LOOP(i) {
        R xx[24], yy[24];
        SpinorIO<P>::load(x, stride, i, xx);
        SpinorIO<P>::load(y, stride, i, yy);
#pragma unroll
        for (int k = 0; k < 24; ++k) xx[k] = xx[k] + (R)a * yy[k];
        SpinorIO<P>::store(z, stride, i, xx);
    }
}

// sum conj(a) b -> (re, im)
template <int P>
__global__ void k_cdot(long Vh, long stride, const void *a, const void *b, RedTail tail) {
    using R = typename Prec<P>::R;
    double acc[2] = {0, 0};
    QX_GRID_LOOP(i) {
        R aa[24], bb[24];
        SpinorIO<P>::load(a, stride, i, aa);
        SpinorIO<P>::load(b, stride, i, bb);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            acc[0] += (double)aa[2 * k] * bb[2 * k] + (double)aa[2 * k + 1] * bb[2 * k + 1];
            acc[1] += (double)aa[2 * k] * bb[2 * k + 1] - (double)aa[2 * k + 1] * bb[2 * k];
        }
    }
    block_reduce_store<2>(acc, tail);
}

// sum |a|^2
template <int P>
__global__ void k_norm2(long Vh, long stride, const void *a, RedTail tail) {
    using R = typename Prec<P>::R;
    double acc[1] = {0};
    QX_GRID_LOOP(i) {
        R aa[24];
        SpinorIO<P>::load(a, stride, i, aa);
#pragma unroll
        for (int k = 0; k < 24; ++k) acc[0] += (double)aa[k] * aa[k];
    }
    block_reduce_store<1>(acc, tail);
}

// (<t, s>, |t|^2)
template <int P>
__global__ void k_tdot(long Vh, long stride, const void *t, const void *s, RedTail tail) {
    using R = typename Prec<P>::R;
    double acc[3] = {0, 0, 0};
    QX_GRID_LOOP(i) {
        R tt[24], ss[24];
        SpinorIO<P>::load(t, stride, i, tt);
        SpinorIO<P>::load(s, stride, i, ss);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            acc[0] += (double)tt[2 * k] * ss[2 * k] + (double)tt[2 * k + 1] * ss[2 * k + 1];
            acc[1] += (double)tt[2 * k] * ss[2 * k + 1] - (double)tt[2 * k + 1] * ss[2 * k];
            acc[2] += (double)tt[2 * k] * tt[2 * k] + (double)tt[2 * k + 1] * tt[2 * k + 1];
        }
    }
    block_reduce_store<3>(acc, tail);
}

// x <- x + alpha p + omega s ; s <- s - omega t ; returns (|s|^2, <rhat, s>) of the new s
#ifndef QX_BICG_MINB
#define QX_BICG_MINB 1
#endif
template <int P>
__global__ void __launch_bounds__(kBlasThreads, P == 4 ? QX_BICG_MINB : 1)
k_bicg_final(long Vh, long stride, void *x, const void *p, void *s, const void *t, const void *rhat,
                             CoefArg alpha_, CoefArg omega_, RedTail tail) {
    using R = typename Prec<P>::R;
    const double2 alpha = coef_get(alpha_), omega = coef_get(omega_);
    const Cx<R> al = cx((R)alpha.x, (R)alpha.y), om = cx((R)omega.x, (R)omega.y);
    double acc[3] = {0, 0, 0};
    if constexpr (P == 4) {
        // fp32: one float4 block (two complex components) of all five fields at a time, in the
        // site's component order (so every value and every fp64 partial sum is bitwise the
        // whole-site version's): 54 instead of 72 registers, 4 instead of 3 resident 256-thread
        // CTAs per SM (-Xptxas -v), and the loads of the next block in flight while this one is
        // computed (the whole-site form was latency-bound at 0.78 of HBM,
        // profiles/r01k_ncu_blas.txt).  x and s are written by this kernel, so they are read
        // with plain (coherent) loads; only p, t and rhat take the read-only path.
        QX_GRID_LOOP(i) {
            float4 *X = reinterpret_cast<float4 *>(x);
            float4 *Sv = reinterpret_cast<float4 *>(s);
            const float4 *Pp = reinterpret_cast<const float4 *>(p), *T = reinterpret_cast<const float4 *>(t),
                         *H = reinterpret_cast<const float4 *>(rhat);
#pragma unroll
            for (int k = 0; k < 6; ++k) {
                const long j = (long)k * stride + i;
                const float4 xv = __ldcs(X + j), pv = __ldg(Pp + j), sv = __ldcs(Sv + j), tv = __ldg(T + j), hv = __ldg(H + j);
                const float xr[4] = {xv.x, xv.y, xv.z, xv.w}, pr[4] = {pv.x, pv.y, pv.z, pv.w};
                const float sr[4] = {sv.x, sv.y, sv.z, sv.w}, tr[4] = {tv.x, tv.y, tv.z, tv.w};
                const float hr[4] = {hv.x, hv.y, hv.z, hv.w};
                float xo[4], so[4];
#pragma unroll
                for (int c = 0; c < 2; ++c) {
                    const Cx<R> o = cx(xr[2 * c], xr[2 * c + 1]) + al * cx(pr[2 * c], pr[2 * c + 1]) +
                                    om * cx(sr[2 * c], sr[2 * c + 1]);
                    xo[2 * c] = o.r;
                    xo[2 * c + 1] = o.i;
                    const Cx<R> q = cx(sr[2 * c], sr[2 * c + 1]) - om * cx(tr[2 * c], tr[2 * c + 1]);
                    so[2 * c] = q.r;
                    so[2 * c + 1] = q.i;
                }
                X[j] = make_float4(xo[0], xo[1], xo[2], xo[3]);
                Sv[j] = make_float4(so[0], so[1], so[2], so[3]);
#pragma unroll
                for (int c = 0; c < 2; ++c) {
                    acc[0] += (double)so[2 * c] * so[2 * c] + (double)so[2 * c + 1] * so[2 * c + 1];
                    acc[1] += (double)hr[2 * c] * so[2 * c] + (double)hr[2 * c + 1] * so[2 * c + 1];
                    acc[2] += (double)hr[2 * c] * so[2 * c + 1] - (double)hr[2 * c + 1] * so[2 * c];
                }
            }
        }
        block_reduce_store<3>(acc, tail);
        return;
    }
    QX_GRID_LOOP(i) {
        R xx[24], pp[24], ss[24];
        SpinorIO<P>::load(x, stride, i, xx);
        SpinorIO<P>::load(p, stride, i, pp);
        SpinorIO<P>::load(s, stride, i, ss);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            Cx<R> o = cx(xx[2 * k], xx[2 * k + 1]) + al * cx(pp[2 * k], pp[2 * k + 1]) + om * cx(ss[2 * k], ss[2 * k + 1]);
            xx[2 * k] = o.r;
            xx[2 * k + 1] = o.i;
        }
        SpinorIO<P>::store(x, stride, i, xx);
        R tt[24];
        SpinorIO<P>::load(t, stride, i, tt);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            Cx<R> o = cx(ss[2 * k], ss[2 * k + 1]) - om * cx(tt[2 * k], tt[2 * k + 1]);
            ss[2 * k] = o.r;
            ss[2 * k + 1] = o.i;
        }
        SpinorIO<P>::store_requant(s, stride, i, ss);  // reduce exactly what was stored
        R rh[24];
        SpinorIO<P>::load(rhat, stride, i, rh);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            acc[0] += (double)ss[2 * k] * ss[2 * k] + (double)ss[2 * k + 1] * ss[2 * k + 1];
            acc[1] += (double)rh[2 * k] * ss[2 * k] + (double)rh[2 * k + 1] * ss[2 * k + 1];
            acc[2] += (double)rh[2 * k] * ss[2 * k + 1] - (double)rh[2 * k + 1] * ss[2 * k];
        }
    }
    block_reduce_store<3>(acc, tail);
}

// y(PD) <- y(PD) + x(PS)
template <int PD, int PS>
__global__ void k_xpy_mixed(long Vh, long stride, const void *x, void *y) {
    QX_GRID_LOOP(i) {
        typename Prec<PS>::R xx[24];
        typename Prec<PD>::R yy[24];
        SpinorIO<PS>::load(x, stride, i, xx);
        SpinorIO<PD>::load(y, stride, i, yy);
#pragma unroll
        for (int k = 0; k < 24; ++k) yy[k] += (typename Prec<PD>::R)xx[k];
        SpinorIO<PD>::store(y, stride, i, yy);
    }
}

// r <- b - r ; returns |r|^2
template <int P>
__global__ void k_bmr_norm(long Vh, long stride, const void *b, void *r, RedTail tail) {
    using R = typename Prec<P>::R;
    double acc[1] = {0};
    QX_GRID_LOOP(i) {
        R bb[24], rr[24];
        SpinorIO<P>::load(b, stride, i, bb);
        SpinorIO<P>::load(r, stride, i, rr);
#pragma unroll
        for (int k = 0; k < 24; ++k) rr[k] = bb[k] - rr[k];
        SpinorIO<P>::store_requant(r, stride, i, rr);
#pragma unroll
        for (int k = 0; k < 24; ++k) acc[0] += (double)rr[k] * rr[k];
    }
    block_reduce_store<1>(acc, tail);
}

// ---------------------------------------------------------------------------- dispatch
#define QX_PREC_SWITCH(prec, KCALL) \
    switch (prec) {                 \
        case 8: { constexpr int P = 8; KCALL; } break; \
        case 4: { constexpr int P = 4; KCALL; } break; \
        case 2: { constexpr int P = 2; KCALL; } break; \
        default: throw Error(QUDAX_ERR_ARG, "blas: bad precision"); \
    }

// one launch of kernel K on its one-wave grid; for reducing kernels the tail spans that grid
#define QX_LAUNCH(K, ...)                              \
    do {                                               \
        const int B_ = one_wave(K);                    \
        tail.total_blocks = B_;                        \
        tail.block_offset = 0;                         \
        K<<<B_, kBlasThreads, 0, s>>>(__VA_ARGS__);    \
    } while (0)

int blas_run(int op, int prec, const Geom &g, void *const *f, const CoefArg *co, RedTail tail,
             cudaStream_t s) {
    const long Vh = g.Vh, st = g.stride;
    int nred = 0;
    switch (op) {
        case OP_P_UPDATE:  // p = r + beta (p - omega v): r=f0, p=f1, v=f2
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_p_update<P>, Vh, st, f[0], f[1], f[2], co[0], co[1]));
            break;
        case OP_CAXPY:  // f1 += c f0
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_caxpy<P>, Vh, st, co[0], f[0], f[1], 0));
            break;
        case OP_CAXPY_REV:
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_caxpy<P>, Vh, st, co[0], f[0], f[1], 1));
            break;
        case OP_XPAY:  // f2 = f0 + a f1
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_xpay<P>, Vh, st, f[0], co[0].v.x, f[1], f[2]));
            break;
        case OP_CDOT:  // <f0, f1>
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_cdot<P>, Vh, st, f[0], f[1], tail));
            nred = 2;
            break;
        case OP_NORM2:
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_norm2<P>, Vh, st, f[0], tail));
            nred = 1;
            break;
        case OP_TDOT:  // (<f0, f1>, |f0|^2)
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_tdot<P>, Vh, st, f[0], f[1], tail));
            nred = 3;
            break;
        case OP_FINAL:  // x=f0, p=f1, s=f2, t=f3, rhat=f4
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_bicg_final<P>, Vh, st, f[0], f[1], f[2], f[3], f[4], co[0], co[1], tail));
            nred = 3;
            break;
        case OP_BMR_NORM:  // f1 = f0 - f1
            QX_PREC_SWITCH(prec, QX_LAUNCH(k_bmr_norm<P>, Vh, st, f[0], f[1], tail));
            nred = 1;
            break;
        default:
            throw Error(QUDAX_ERR_ARG, "blas: bad op");
    }
    QX_CUDA(cudaGetLastError());
    return nred;
}

void blas_xpy_mixed(int pd, int ps, const Geom &g, const void *x, void *y, cudaStream_t s) {
    const int T = kBlasThreads;
#define QX_XM(A, C) \
    if (pd == A && ps == C) { k_xpy_mixed<A, C><<<one_wave(k_xpy_mixed<A, C>), T, 0, s>>>(g.Vh, g.stride, x, y); QX_CUDA(cudaGetLastError()); return; }
    QX_XM(8, 8) QX_XM(8, 4) QX_XM(8, 2) QX_XM(4, 4) QX_XM(4, 2) QX_XM(2, 2) QX_XM(4, 8) QX_XM(2, 8) QX_XM(2, 4)
#undef QX_XM
    throw Error(QUDAX_ERR_ARG, "xpy_mixed: bad precision");
}

}  // namespace qx
