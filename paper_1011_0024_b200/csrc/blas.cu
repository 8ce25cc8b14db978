// blas.cu — fused BLAS-1 and reduction kernels for the BiCGstab driver ("kernel
// fusion wherever possible to reduce memory traffic"; P:721-725 global sums).  All vectors
// are parity fields (V_h sites) in the site-major SoA of one precision; arithmetic is in the
// storage precision's compute type (fp32 for half), every reduction accumulates in fp64 and
// is reduced deterministically: per-CTA partials in a fixed grid, then one CTA sums them in
// a fixed order (reading Q12), so results are bitwise reproducible run to run.
#include "core.cuh"
#include "dslash.cuh"
#include "internal.h"

namespace qx {

constexpr int kBlasThreads = 256;
constexpr int kBlasBlocks = 148 * 4;  // fixed grid: 4 CTAs per SM on 148 SMs

int blas_partial_blocks() { return kBlasBlocks; }

template <int NRED>
__device__ __forceinline__ void block_reduce_store(double (&v)[NRED], double *partials) {
    __shared__ double sm[kBlasThreads / 32][NRED > 0 ? NRED : 1];
#pragma unroll
    for (int k = 0; k < NRED; ++k)
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) v[k] += __shfl_xor_sync(0xffffffffu, v[k], o);
    const int w = threadIdx.x / 32, l = threadIdx.x % 32;
    if (l == 0)
#pragma unroll
        for (int k = 0; k < NRED; ++k) sm[w][k] = v[k];
    __syncthreads();
    if (threadIdx.x < NRED) {
        double s = 0;
        for (int ww = 0; ww < kBlasThreads / 32; ++ww) s += sm[ww][threadIdx.x];
        partials[blockIdx.x * NRED + threadIdx.x] = s;
    }
}

// single CTA: out[k] = sum_b partials[b * nred + k], fixed order
__global__ void k_reduce_final(const double *__restrict__ partials, int nblocks, int nred, double *out) {
    __shared__ double sm[kBlasThreads];
    for (int k = 0; k < nred; ++k) {
        double s = 0;
        for (int b = threadIdx.x; b < nblocks; b += blockDim.x) s += partials[b * nred + k];
        sm[threadIdx.x] = s;
        __syncthreads();
        for (int w = blockDim.x / 2; w > 0; w >>= 1) {
            if (threadIdx.x < w) sm[threadIdx.x] += sm[threadIdx.x + w];
            __syncthreads();
        }
        if (threadIdx.x == 0) out[k] = sm[0];
        __syncthreads();
    }
}

template <typename R>
using Sp = R[24];

// ---------------------------------------------------------------------------- kernels
// y = x + c * y ... each kernel documents its formula; c* are complex (re, im) as double2.

// p <- r + beta (p - omega v)            (BiCGstab search direction)
template <int P>
__global__ void k_p_update(long Vh, long stride, const void *r, void *p, const void *v, double2 beta, double2 omega) {
    using R = typename Prec<P>::R;
    const Cx<R> b = cx((R)beta.x, (R)beta.y), w = cx((R)omega.x, (R)omega.y);
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
__global__ void k_caxpy(long Vh, long stride, double2 c, const void *x, void *y) {
    using R = typename Prec<P>::R;
    const Cx<R> a = cx((R)c.x, (R)c.y);
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
__global__ void k_cdot(long Vh, long stride, const void *a, const void *b, double *partials) {
    using R = typename Prec<P>::R;
    double acc[2] = {0, 0};
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
        R aa[24], bb[24];
        SpinorIO<P>::load(a, stride, i, aa);
        SpinorIO<P>::load(b, stride, i, bb);
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            acc[0] += (double)aa[2 * k] * bb[2 * k] + (double)aa[2 * k + 1] * bb[2 * k + 1];
            acc[1] += (double)aa[2 * k] * bb[2 * k + 1] - (double)aa[2 * k + 1] * bb[2 * k];
        }
    }
    block_reduce_store<2>(acc, partials);
}

// sum |a|^2
template <int P>
__global__ void k_norm2(long Vh, long stride, const void *a, double *partials) {
    using R = typename Prec<P>::R;
    double acc[1] = {0};
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
        R aa[24];
        SpinorIO<P>::load(a, stride, i, aa);
#pragma unroll
        for (int k = 0; k < 24; ++k) acc[0] += (double)aa[k] * aa[k];
    }
    block_reduce_store<1>(acc, partials);
}

// (<t, s>, |t|^2)
template <int P>
__global__ void k_tdot(long Vh, long stride, const void *t, const void *s, double *partials) {
    using R = typename Prec<P>::R;
    double acc[3] = {0, 0, 0};
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
    block_reduce_store<3>(acc, partials);
}

// x <- x + alpha p + omega s ; s <- s - omega t ; returns (|s|^2, <rhat, s>) of the new s
template <int P>
__global__ void k_bicg_final(long Vh, long stride, void *x, const void *p, void *s, const void *t, const void *rhat,
                             double2 alpha, double2 omega, double *partials) {
    using R = typename Prec<P>::R;
    const Cx<R> al = cx((R)alpha.x, (R)alpha.y), om = cx((R)omega.x, (R)omega.y);
    double acc[3] = {0, 0, 0};
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
    block_reduce_store<3>(acc, partials);
}

// y(PD) <- y(PD) + x(PS)
template <int PD, int PS>
__global__ void k_xpy_mixed(long Vh, long stride, const void *x, void *y) {
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
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
__global__ void k_bmr_norm(long Vh, long stride, const void *b, void *r, double *partials) {
    using R = typename Prec<P>::R;
    double acc[1] = {0};
    for (long i = (long)blockIdx.x * blockDim.x + threadIdx.x; i < Vh; i += (long)gridDim.x * blockDim.x) {
        R bb[24], rr[24];
        SpinorIO<P>::load(b, stride, i, bb);
        SpinorIO<P>::load(r, stride, i, rr);
#pragma unroll
        for (int k = 0; k < 24; ++k) rr[k] = bb[k] - rr[k];
        SpinorIO<P>::store_requant(r, stride, i, rr);
#pragma unroll
        for (int k = 0; k < 24; ++k) acc[0] += (double)rr[k] * rr[k];
    }
    block_reduce_store<1>(acc, partials);
}

// ---------------------------------------------------------------------------- dispatch
#define QX_PREC_SWITCH(prec, KCALL) \
    switch (prec) {                 \
        case 8: { constexpr int P = 8; KCALL; } break; \
        case 4: { constexpr int P = 4; KCALL; } break; \
        case 2: { constexpr int P = 2; KCALL; } break; \
        default: throw Error(QUDAX_ERR_ARG, "blas: bad precision"); \
    }

static inline double2 d2(const double *c) { return make_double2(c[0], c[1]); }

// f: field pointers, coef: scalars, partials: device scratch (kBlasBlocks * 4 doubles),
// out: device result (up to 4 doubles).  Returns the number of reduced values (0 if none).
int blas_run(int op, int prec, const Geom &g, void *const *f, const double *coef, double *partials, double *out,
             cudaStream_t s) {
    const long Vh = g.Vh, st = g.stride;
    const int B = kBlasBlocks, T = kBlasThreads;
    int nred = 0;
    switch (op) {
        case 0:  // p_update(r=f0, p=f1, v=f2; beta=coef0,1, omega=coef2,3)
            QX_PREC_SWITCH(prec, (k_p_update<P><<<B, T, 0, s>>>(Vh, st, f[0], f[1], f[2], d2(coef), d2(coef + 2))));
            break;
        case 1:  // caxpy: f1 += c f0
            QX_PREC_SWITCH(prec, (k_caxpy<P><<<B, T, 0, s>>>(Vh, st, d2(coef), f[0], f[1])));
            break;
        case 2:  // xpay: f2 = f0 + a f1
            QX_PREC_SWITCH(prec, (k_xpay<P><<<B, T, 0, s>>>(Vh, st, f[0], coef[0], f[1], f[2])));
            break;
        case 3:  // cdot(f0, f1)
            QX_PREC_SWITCH(prec, (k_cdot<P><<<B, T, 0, s>>>(Vh, st, f[0], f[1], partials)));
            nred = 2;
            break;
        case 4:  // norm2(f0)
            QX_PREC_SWITCH(prec, (k_norm2<P><<<B, T, 0, s>>>(Vh, st, f[0], partials)));
            nred = 1;
            break;
        case 5:  // tdot(t=f0, s=f1)
            QX_PREC_SWITCH(prec, (k_tdot<P><<<B, T, 0, s>>>(Vh, st, f[0], f[1], partials)));
            nred = 3;
            break;
        case 6:  // final(x=f0, p=f1, s=f2, t=f3, rhat=f4; alpha=c0,1 omega=c2,3)
            QX_PREC_SWITCH(prec, (k_bicg_final<P><<<B, T, 0, s>>>(Vh, st, f[0], f[1], f[2], f[3], f[4], d2(coef), d2(coef + 2), partials)));
            nred = 3;
            break;
        case 7:  // bmr_norm: f1 = f0 - f1
            QX_PREC_SWITCH(prec, (k_bmr_norm<P><<<B, T, 0, s>>>(Vh, st, f[0], f[1], partials)));
            nred = 1;
            break;
        default:
            throw Error(QUDAX_ERR_ARG, "blas: bad op");
    }
    QX_CUDA(cudaGetLastError());
    if (nred) {
        k_reduce_final<<<1, kBlasThreads, 0, s>>>(partials, B, nred, out);
        QX_CUDA(cudaGetLastError());
    }
    return nred;
}

void blas_xpy_mixed(int pd, int ps, const Geom &g, const void *x, void *y, cudaStream_t s) {
    const int B = kBlasBlocks, T = kBlasThreads;
#define QX_XM(A, C) \
    if (pd == A && ps == C) { k_xpy_mixed<A, C><<<B, T, 0, s>>>(g.Vh, g.stride, x, y); QX_CUDA(cudaGetLastError()); return; }
    QX_XM(8, 8) QX_XM(8, 4) QX_XM(8, 2) QX_XM(4, 4) QX_XM(4, 2) QX_XM(2, 2) QX_XM(4, 8) QX_XM(2, 8) QX_XM(2, 4)
#undef QX_XM
    throw Error(QUDAX_ERR_ARG, "xpy_mixed: bad precision");
}

}  // namespace qx
