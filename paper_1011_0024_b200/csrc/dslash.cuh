// dslash.cuh — the Wilson-clover Dslash stencil (eq. (2); kernel structure
// P:384-395), one thread per output site of parity p.
//
// Per site x of parity p, for each of the 8 hops: load the link (reconstructing 12/8-real
// storage in registers), load the neighbour spinor of parity 1-p (24 reals for
// x, y, z; only the 12 reals selected by the diagonal temporal projector for t, eq. (6),
// P:504-506), spin-project to a half spinor (footnote 3), multiply by U or U^dag
// (the backward link U_mu(x-mu) is read at x-mu and conjugated by register relabeling,
// P:425-432), expand and accumulate.  The clover term is fused before the store.
//
// Spin basis: non-relativistic, psi_NR = S psi_DR with S = (1/sqrt2)[[1,1],[1,-1]] (2x2
// blocks of spin pairs), so 1 + gamma_4 = diag(2,2,0,0) and 1 - gamma_4 = diag(0,0,2,2).
// Projectors (1 + sigma gamma_mu), sigma = +-1, written as h = (h0, h1) and the
// reconstruction of rows 2, 3 (derived from gamma_mu^NR = S gamma_mu^DR S):
//   mu=x: h0 = p0 - s i p3, h1 = p1 - s i p2;   r2 =  s i h1, r3 =  s i h0
//   mu=y: h0 = p0 + s p3,   h1 = p1 - s p2;     r2 = -s h1,   r3 =  s h0
//   mu=z: h0 = p0 - s i p2, h1 = p1 + s i p3;   r2 =  s i h0, r3 = -s i h1
// Non-dagger: forward hop uses 1 - gamma (s = -1), backward 1 + gamma (s = +1) (eq. (2));
// the dagger flips s (D^dag = gamma5 D gamma5).
//
// Clover (72 reals = two Hermitian 6x6 chiral blocks C+, C-, each d[6] + lower triangle
// L[15]; stored already halved): with u = spins 0,1 and l = spins 2,3 of the NR spinor,
//   out_u = C+ (u + l) + C- (u - l),  out_l = C+ (u + l) - C- (u - l).
#pragma once
#include <cstdlib>
#include "core.cuh"
#include "internal.h"
#include "reduce.cuh"

namespace qx {

template <typename R>
__device__ __forceinline__ void su3_mul(const Cx<R> u[3][3], const Cx<R> v[3], Cx<R> out[3]) {
    if constexpr (sizeof(R) == 4) {  // 1 FMUL2 + 5 FFMA2 per row (fma_i: modifiers, no i v temporaries)
#pragma unroll
        for (int a = 0; a < 3; ++a) {
            float2 acc = __fmul2_rn(bc(u[a][0].r), f2(v[0]));
            acc = fma_i(acc, u[a][0].i, v[0]);
#pragma unroll
            for (int c = 1; c < 3; ++c) {
                acc = __ffma2_rn(bc(u[a][c].r), f2(v[c]), acc);
                acc = fma_i(acc, u[a][c].i, v[c]);
            }
            out[a] = cf(acc);
        }
    } else {
#pragma unroll
        for (int a = 0; a < 3; ++a) out[a] = u[a][0] * v[0] + u[a][1] * v[1] + u[a][2] * v[2];
    }
}
// U^dag v: out[a] = sum_c conj(u[c][a]) v[c]
template <typename R>
__device__ __forceinline__ void su3_dag_mul(const Cx<R> u[3][3], const Cx<R> v[3], Cx<R> out[3]) {
    if constexpr (sizeof(R) == 4) {
#pragma unroll
        for (int a = 0; a < 3; ++a) {
            float2 acc = __fmul2_rn(bc(u[0][a].r), f2(v[0]));
            acc = fma_mi(acc, u[0][a].i, v[0]);
#pragma unroll
            for (int c = 1; c < 3; ++c) {
                acc = __ffma2_rn(bc(u[c][a].r), f2(v[c]), acc);
                acc = fma_mi(acc, u[c][a].i, v[c]);
            }
            out[a] = cf(acc);
        }
    } else {
#pragma unroll
        for (int a = 0; a < 3; ++a)
            out[a] = conj_mul(u[0][a], v[0]) + conj_mul(u[1][a], v[1]) + conj_mul(u[2][a], v[2]);
    }
}

template <typename R>
__device__ __forceinline__ void unpack_spinor(const R *v, Cx<R> p[4][3]) {
#pragma unroll
    for (int s = 0; s < 4; ++s)
#pragma unroll
        for (int c = 0; c < 3; ++c) p[s][c] = cx(v[(s * 3 + c) * 2], v[(s * 3 + c) * 2 + 1]);
}

// spatial hop: project psi with (1 + sigma gamma_mu), multiply by U (or U^dag), accumulate
// (the projector formulas of the header, written with add_i(p, q) = p + S i q).  Split into the
// projection and the multiply-expand so a partitioned dimension's face pack projects with
// exactly this code and the receiving kernel finishes the hop with exactly this code.
template <int MU, int SIGMA, typename R>
__device__ __forceinline__ void spatial_project(const Cx<R> p[4][3], Cx<R> h0[3], Cx<R> h1[3]) {
#pragma unroll
    for (int c = 0; c < 3; ++c) {
        if constexpr (MU == 0) {  // h0 = p0 - s i p3, h1 = p1 - s i p2
            h0[c] = add_i<-SIGMA>(p[0][c], p[3][c]);
            h1[c] = add_i<-SIGMA>(p[1][c], p[2][c]);
        } else if constexpr (MU == 1) {  // h0 = p0 + s p3, h1 = p1 - s p2
            h0[c] = SIGMA > 0 ? p[0][c] + p[3][c] : p[0][c] - p[3][c];
            h1[c] = SIGMA > 0 ? p[1][c] - p[2][c] : p[1][c] + p[2][c];
        } else {  // h0 = p0 - s i p2, h1 = p1 + s i p3
            h0[c] = add_i<-SIGMA>(p[0][c], p[2][c]);
            h1[c] = add_i<SIGMA>(p[1][c], p[3][c]);
        }
    }
}
// Spin projection of a half-precision neighbour straight from its BIASED decode P = q + B
// (B = kHalfBias = 2^23 + 2^15, q the stored integer): every projected component is
// p_a + s q_b (lane signs s = +-1, q_b possibly the swapped pair) = P_a + s Q_b - (1 + s) B.
// t = P_a - (1 + s) B is an integer below 2^24 (exact), and t + s Q_b is the exact small
// integer p_a + s q_b rounded once by FFMA2 (exact) — bitwise the integers the unbiased
// decode + projection produce, with one FADD2 (none when both lanes subtract) + one FFMA2
// per complex component instead of the two bias FADD2s + one FFMA2.
#ifndef QX_BPROJ
#define QX_BPROJ 1
#endif
template <int SR, int SI>
__device__ __forceinline__ Cx<float> bproj(Cx<float> P, float2 Q) {
    float2 t = f2(P);
    if constexpr (SR > 0 || SI > 0) t = __fadd2_rn(t, make_float2(SR > 0 ? -2.f * kHalfBias : 0.f, SI > 0 ? -2.f * kHalfBias : 0.f));
    return cf(__ffma2_rn(Q, make_float2((float)SR, (float)SI), t));
}
__device__ __forceinline__ float2 swp(Cx<float> a) { return make_float2(a.i, a.r); }
template <int MU, int SIGMA>
__device__ __forceinline__ void spatial_project_b(const Cx<float> p[4][3], Cx<float> h0[3], Cx<float> h1[3]) {
#pragma unroll
    for (int c = 0; c < 3; ++c) {
        if constexpr (MU == 0) {  // h0 = p0 - s i p3, h1 = p1 - s i p2
            h0[c] = bproj<SIGMA, -SIGMA>(p[0][c], swp(p[3][c]));
            h1[c] = bproj<SIGMA, -SIGMA>(p[1][c], swp(p[2][c]));
        } else if constexpr (MU == 1) {  // h0 = p0 + s p3, h1 = p1 - s p2
            h0[c] = bproj<SIGMA, SIGMA>(p[0][c], f2(p[3][c]));
            h1[c] = bproj<-SIGMA, -SIGMA>(p[1][c], f2(p[2][c]));
        } else {  // h0 = p0 - s i p2, h1 = p1 + s i p3
            h0[c] = bproj<SIGMA, -SIGMA>(p[0][c], swp(p[2][c]));
            h1[c] = bproj<-SIGMA, SIGMA>(p[1][c], swp(p[3][c]));
        }
    }
}

// SC (deferred-scale half precision): h and u hold the stored integers, the hop result is
// c * (U h) — the scale rides on the expansion's FFMA2s instead of one FMUL2 per decoded pair
template <int MU, int SIGMA, bool ADJ, bool SC = false, typename R>
__device__ __forceinline__ void spatial_mult_expand(const Cx<R> h0[3], const Cx<R> h1[3], const Cx<R> u[3][3],
                                                    Cx<R> acc[4][3], R c = (R)1) {
    Cx<R> g0[3], g1[3];
    if constexpr (ADJ) {
        su3_dag_mul(u, h0, g0);
        su3_dag_mul(u, h1, g1);
    } else {
        su3_mul(u, h0, g0);
        su3_mul(u, h1, g1);
    }
    if constexpr (SC) {
        static_assert(sizeof(R) == 4, "deferred scale: fp32 arithmetic only");
        const float2 cc = bc(c), pc = make_float2(-c, c);  // acc + c g, acc + i c g
        const float2 ps = SIGMA > 0 ? pc : make_float2(c, -c);
#pragma unroll
        for (int k = 0; k < 3; ++k) {
            acc[0][k] = cf(__ffma2_rn(cc, f2(g0[k]), f2(acc[0][k])));
            acc[1][k] = cf(__ffma2_rn(cc, f2(g1[k]), f2(acc[1][k])));
            const float2 s0 = make_float2(g0[k].i, g0[k].r), s1 = make_float2(g1[k].i, g1[k].r);
            if constexpr (MU == 0) {  // r2 = s i h1, r3 = s i h0
                acc[2][k] = cf(__ffma2_rn(s1, ps, f2(acc[2][k])));
                acc[3][k] = cf(__ffma2_rn(s0, ps, f2(acc[3][k])));
            } else if constexpr (MU == 1) {  // r2 = -s h1, r3 = s h0
                acc[2][k] = cf(__ffma2_rn(bc(SIGMA > 0 ? -c : c), f2(g1[k]), f2(acc[2][k])));
                acc[3][k] = cf(__ffma2_rn(bc(SIGMA > 0 ? c : -c), f2(g0[k]), f2(acc[3][k])));
            } else {  // r2 = s i h0, r3 = -s i h1
                acc[2][k] = cf(__ffma2_rn(s0, ps, f2(acc[2][k])));
                acc[3][k] = cf(__ffma2_rn(s1, make_float2(-ps.x, -ps.y), f2(acc[3][k])));
            }
        }
        return;
    }
#pragma unroll
    for (int c = 0; c < 3; ++c) {
        acc[0][c] = acc[0][c] + g0[c];
        acc[1][c] = acc[1][c] + g1[c];
        if constexpr (MU == 0) {  // r2 = s i h1, r3 = s i h0
            acc[2][c] = add_i<SIGMA>(acc[2][c], g1[c]);
            acc[3][c] = add_i<SIGMA>(acc[3][c], g0[c]);
        } else if constexpr (MU == 1) {  // r2 = -s h1, r3 = s h0
            acc[2][c] = SIGMA > 0 ? acc[2][c] - g1[c] : acc[2][c] + g1[c];
            acc[3][c] = SIGMA > 0 ? acc[3][c] + g0[c] : acc[3][c] - g0[c];
        } else {  // r2 = s i h0, r3 = -s i h1
            acc[2][c] = add_i<SIGMA>(acc[2][c], g0[c]);
            acc[3][c] = add_i<-SIGMA>(acc[3][c], g1[c]);
        }
    }
}
template <int MU, int SIGMA, bool ADJ, bool SC = false, typename R>
__device__ __forceinline__ void spatial_hop(const Cx<R> p[4][3], const Cx<R> u[3][3], Cx<R> acc[4][3], R c = (R)1) {
    Cx<R> h0[3], h1[3];
    spatial_project<MU, SIGMA>(p, h0, h1);
    spatial_mult_expand<MU, SIGMA, ADJ, SC>(h0, h1, u, acc, c);
}

// Decoding with or without the deferred scale (DF): returns the factor the values carry
template <bool DF, int P, int N>
__device__ __forceinline__ typename Prec<P>::R dec_vec(const RawVec<P, N> &r, typename Prec<P>::R *out) {
    if constexpr (DF) {
        r.decode_q(out);
        return r.scale();
    } else {
        r.decode(out);
        return (typename Prec<P>::R)1;
    }
}
template <bool DF, int P, int RECON>
__device__ __forceinline__ typename Prec<P>::R dec_link(const RawLink<P, RECON> &l, Cx<typename Prec<P>::R> u[3][3]) {
    if constexpr (DF) {
        l.decode_q(u);
        return kHalfInv;
    } else {
        l.decode(u);
        return (typename Prec<P>::R)1;
    }
}
// whether the half-precision Dslash defers the decode scale (recon 8 reconstructs through
// sqrt/sincos of the true values, so it keeps the scaled decode).  QX_NO_DEFER: A/B builds.
template <int P, int RECON>
__host__ __device__ constexpr bool dslash_defer() {
#ifdef QX_NO_DEFER
    return false;
#else
    return P == 2 && RECON != 8;
#endif
}

// Faces of a partitioned X / Y / Z: the projected half spinor (h0, h1), 12 reals in the
// arithmetic precision R, site-major blocks of 16-byte vectors (fs = padded face sites)
template <typename R>
struct SFace {
    static constexpr int NB = (sizeof(R) == 8) ? 6 : 3;
    static __device__ __forceinline__ void load(const void *base, long fs, long f, Cx<R> h0[3], Cx<R> h1[3]) {
        R v[12];
        if constexpr (sizeof(R) == 8) {
            const double2 *p = reinterpret_cast<const double2 *>(base);
#pragma unroll
            for (int k = 0; k < 6; ++k) {
                const double2 d = __ldg(p + k * fs + f);
                v[2 * k] = d.x;
                v[2 * k + 1] = d.y;
            }
        } else {
            const float4 *p = reinterpret_cast<const float4 *>(base);
#pragma unroll
            for (int k = 0; k < 3; ++k) {
                const float4 d = __ldg(p + k * fs + f);
                v[4 * k] = d.x; v[4 * k + 1] = d.y; v[4 * k + 2] = d.z; v[4 * k + 3] = d.w;
            }
        }
#pragma unroll
        for (int c = 0; c < 3; ++c) {
            h0[c] = cx(v[2 * c], v[2 * c + 1]);
            h1[c] = cx(v[6 + 2 * c], v[6 + 2 * c + 1]);
        }
    }
    static __device__ __forceinline__ void store(void *base, long fs, long f, const Cx<R> h0[3], const Cx<R> h1[3]) {
        R v[12];
#pragma unroll
        for (int c = 0; c < 3; ++c) {
            v[2 * c] = h0[c].r; v[2 * c + 1] = h0[c].i;
            v[6 + 2 * c] = h1[c].r; v[6 + 2 * c + 1] = h1[c].i;
        }
        if constexpr (sizeof(R) == 8) {
            double2 *p = reinterpret_cast<double2 *>(base);
#pragma unroll
            for (int k = 0; k < 6; ++k) p[k * fs + f] = make_double2(v[2 * k], v[2 * k + 1]);
        } else {
            float4 *p = reinterpret_cast<float4 *>(base);
#pragma unroll
            for (int k = 0; k < 3; ++k) p[k * fs + f] = make_float4(v[4 * k], v[4 * k + 1], v[4 * k + 2], v[4 * k + 3]);
        }
    }
};
// A partitioned X / Y / Z face as the receiving Dslash reads it.  fp64 / fp32: the sender's
// spin projection (SFace).  Half: the sender's raw 16-bit record (same layout as a half spinor
// field with stride fs, norm included; 52 B per site, less than a projected fp32 face) projected
// here from exactly the values the unpartitioned kernel decodes.
template <int P, int MU, int SIGMA, bool DF>
__device__ __forceinline__ typename Prec<P>::R ghost_half(const void *base, long fs, long f, Cx<typename Prec<P>::R> h0[3],
                                                          Cx<typename Prec<P>::R> h1[3]) {
    using R = typename Prec<P>::R;
    if constexpr (P == 2) {
        RawVec<2, 24> sv;
        sv.template load_spinor<0>(base, fs, f);
        R v[24];
        Cx<R> ps[4][3];
        const R sc = dec_vec<DF>(sv, v);
        unpack_spinor(v, ps);
        spatial_project<MU, SIGMA>(ps, h0, h1);
        return sc;
    } else {
        SFace<R>::load(base, fs, f, h0, h1);
        return (R)1;
    }
}
// index of a site in the face of dimension mu (lexicographic over the other three local
// coordinates, halved: the sites of one parity on a face pair up along the fastest of them)
template <int MU>
__device__ __forceinline__ int face_index(int x, int y, int z, int t, int X, int Y, int Z) {
    if constexpr (MU == 0) return ((t * Z + z) * Y + y) >> 1;
    else if constexpr (MU == 1) return ((t * Z + z) * X + x) >> 1;
    else return ((t * Y + y) * X + x) >> 1;
}

// temporal hop: h = the 12 selected reals (upper half if UPPER); result 2 U h into the same half
template <bool UPPER, bool ADJ, typename R>
__device__ __forceinline__ void temporal_hop(const R *hv, const Cx<R> u[3][3], R coef, Cx<R> acc[4][3]) {
    Cx<R> h0[3], h1[3], g0[3], g1[3];
#pragma unroll
    for (int c = 0; c < 3; ++c) {
        h0[c] = cx(hv[c * 2], hv[c * 2 + 1]);
        h1[c] = cx(hv[6 + c * 2], hv[6 + c * 2 + 1]);
    }
    if constexpr (ADJ) {
        su3_dag_mul(u, h0, g0);
        su3_dag_mul(u, h1, g1);
    } else {
        su3_mul(u, h0, g0);
        su3_mul(u, h1, g1);
    }
    constexpr int s0 = UPPER ? 0 : 2;
#pragma unroll
    for (int c = 0; c < 3; ++c) {
        acc[s0][c] = axpy(coef, g0[c], acc[s0][c]);
        acc[s0 + 1][c] = axpy(coef, g1[c], acc[s0 + 1][c]);
    }
}

// Hermitian 6x6 (d[6], lower triangle L[15]) times v
template <typename R>
__device__ __forceinline__ void herm6_mul(const R *m, const Cx<R> v[6], Cx<R> out[6]) {
    if constexpr (sizeof(R) == 4) {  // out_i += L v_j and out_j += conj(L) v_i: 2 FFMA2 each
        float2 o[6];
#pragma unroll
        for (int i = 0; i < 6; ++i) o[i] = __fmul2_rn(bc(m[i]), f2(v[i]));
#pragma unroll
        for (int i = 1; i < 6; ++i)
#pragma unroll
            for (int j = 0; j < i; ++j) {
                const int k = i * (i - 1) / 2 + j;
                const float Lr = m[6 + 2 * k], Li = m[6 + 2 * k + 1];
                o[i] = __ffma2_rn(bc(Lr), f2(v[j]), o[i]);
                o[i] = fma_i(o[i], Li, v[j]);
                o[j] = __ffma2_rn(bc(Lr), f2(v[i]), o[j]);
                o[j] = fma_mi(o[j], Li, v[i]);
            }
#pragma unroll
        for (int i = 0; i < 6; ++i) out[i] = cf(o[i]);
    } else {
#pragma unroll
        for (int i = 0; i < 6; ++i) out[i] = m[i] * v[i];
#pragma unroll
        for (int i = 1; i < 6; ++i)
#pragma unroll
            for (int j = 0; j < i; ++j) {
                const int k = i * (i - 1) / 2 + j;
                Cx<R> L = cx(m[6 + 2 * k], m[6 + 2 * k + 1]);
                out[i] = out[i] + L * v[j];
                out[j] = out[j] + conj_mul(L, v[i]);
            }
    }
}

template <int P>
struct CloverIO {
    using R = typename Prec<P>::R;
    // chiral block b (0: C+, 1: C-) of site i: 36 reals.  DF (half): the stored integers, the
    // returned block scale to be applied to the product (deferred-scale decode)
    template <bool DF = false>
    static __device__ __forceinline__ R load(const void *base, long stride, long i, int b, R *m) {
        if constexpr (P == 8) {
            Blocks<8, 18, true>::load(base, stride, i, 18 * b, m);
        } else if constexpr (P == 4) {
            Blocks<4, 9, true>::load(base, stride, i, 9 * b, m);
        } else {
            static_assert(P == 2 || !DF, "deferred clover scale: half only");
            // 9 uint4 regions (reals 8k..8k+7); chiral block b = reals 36b..36b+35, so region 4
            // is split: its low 8 bytes end C+, its high 8 bytes start C-
            const float2 nn = ld_stream(reinterpret_cast<const float2 *>(cptr(base, (size_t)144 * stride)) + i);
            const float scale = (b ? nn.y : nn.x) * kHalfInv;
            uint32_t q[18];
            const int r0 = b ? 5 : 0;
#pragma unroll
            for (int k = 0; k < 4; ++k) {
                const uint4 w = ld_stream_u4(reinterpret_cast<const uint4 *>(cptr(base, (size_t)16 * (r0 + k) * stride)) + i);
                const int o = b ? 2 + 4 * k : 4 * k;
                q[o] = w.x; q[o + 1] = w.y; q[o + 2] = w.z; q[o + 3] = w.w;
            }
            const uint2 mid = ld_stream_u2(reinterpret_cast<const uint2 *>(cptr(base, (size_t)64 * stride + 8 * b)) + 2 * i);
            q[b ? 0 : 16] = mid.x;
            q[b ? 1 : 17] = mid.y;
#pragma unroll
            for (int k = 0; k < 18; ++k) {
                const float2 d = DF ? dq2_q(q[k]) : dq2(q[k], scale);
                m[2 * k] = d.x;
                m[2 * k + 1] = d.y;
            }
            return DF ? scale : 1.f;
        }
        return (R)1;
    }
};

template <int P>
__device__ __forceinline__ void apply_clover(const void *cl, long stride, long i, const Cx<typename Prec<P>::R> in[4][3],
                                             Cx<typename Prec<P>::R> out[4][3]) {
    using R = typename Prec<P>::R;
    Cx<R> va[6], vb[6], wa[6], wb[6];
#pragma unroll
    for (int s = 0; s < 2; ++s)
#pragma unroll
        for (int c = 0; c < 3; ++c) {
            va[s * 3 + c] = in[s][c] + in[s + 2][c];
            vb[s * 3 + c] = in[s][c] - in[s + 2][c];
        }
    constexpr bool DF = (P == 2) && dslash_defer<2, 12>();
    {
        R m[36];
        const R sc = CloverIO<P>::template load<DF>(cl, stride, i, 0, m);
        if constexpr (DF) {
#pragma unroll
            for (int k = 0; k < 6; ++k) va[k] = sc * va[k];
        }
        herm6_mul(m, va, wa);
    }
    {
        R m[36];
        const R sc = CloverIO<P>::template load<DF>(cl, stride, i, 1, m);
        if constexpr (DF) {
#pragma unroll
            for (int k = 0; k < 6; ++k) vb[k] = sc * vb[k];
        }
        herm6_mul(m, vb, wb);
    }
#pragma unroll
    for (int s = 0; s < 2; ++s)
#pragma unroll
        for (int c = 0; c < 3; ++c) {
            out[s][c] = wa[s * 3 + c] + wb[s * 3 + c];
            out[s + 2][c] = wa[s * 3 + c] - wb[s * 3 + c];
        }
}

// Whether a direction issues both hops' loads before computing either (measured,
// profiles/r01_variants.log): fp64 yes (+4%), fp32 no (spills at the 80-register cap), half
// yes except recon-12 (within 3%).  QX_PAIR_MASK overrides: bit 0 half, 1 fp32, 2 fp64.
template <int P, int RECON>
__host__ __device__ constexpr bool dslash_pair() {
#ifdef QX_PAIR_MASK
    return (QX_PAIR_MASK >> (P == 2 ? 0 : (P == 4 ? 1 : 2))) & 1;
#else
    return P == 8 || (P == 2 && RECON != 12);
#endif
}
#ifndef QX_DSLASH_THREADS
#define QX_DSLASH_THREADS 128
#endif
// Minimum resident CTAs per SM (register cap).  Measured on B200 at 32^3x64
// (profiles/r01_variants.log, profiles/r02y_*): fp32 needs >= 6 x 128 threads in flight per SM
// to cover HBM latency (80 regs; 7 x 128 = 72 regs spills and loses up to 3 % on the xpay); half
// runs 7 x 128 (72 regs: since the i-multiplications became operand modifiers its few spills
// cost less than the extra warps gain, -3 % per kernel, r02y; round 1 measured 6 better); fp64
// must not be capped (152 regs; capping spills and loses 20 %).
template <int P> struct DslashMinBlocks { static constexpr int value = (P == 8) ? 1 : (P == 2 ? 7 : 6); };
#ifdef QX_DSLASH_MINB
#define QX_MINB_OF(P) QX_DSLASH_MINB
#else
#define QX_MINB_OF(P) DslashMinBlocks<P>::value
#endif
// eight-parameter links (sincos / sqrt reconstruction): half recon-8 needs the registers of
// 6 CTAs per SM (at 7 it spills 156 B: 125.2 vs 121.4 us clover-inverse, r02aj); fp32 recon-8
// stays at 6 (5 CTAs: 143.9 vs 141.7 us)
#ifndef QX_R8_MINB_F32
#define QX_R8_MINB_F32 6
#endif
#ifndef QX_R8_MINB_F16
#define QX_R8_MINB_F16 6
#endif
// half recon-18 (both hops' raw operands in flight, dslash_pair) spills 150-180 B at 7 CTAs
#ifndef QX_R18_MINB_F16
#define QX_R18_MINB_F16 6
#endif
#ifdef QX_DSLASH_MINB
#define QX_MINB_OF2(P, RECON) QX_DSLASH_MINB
#else
#define QX_MINB_OF2(P, RECON)                                                               \
    ((RECON) == 8 && (P) == 4                                                               \
         ? QX_R8_MINB_F32                                                                   \
         : ((RECON) == 8 && (P) == 2 ? QX_R8_MINB_F16                                       \
                                     : ((RECON) == 18 && (P) == 2 ? QX_R18_MINB_F16 : DslashMinBlocks<P>::value)))
#endif
// L1 prefetch (QX_RED_PF: the fused reduction's second operand, see dslash_site)
__device__ __forceinline__ void pf_l1(const void *p) { asm volatile("prefetch.global.L1 [%0];" ::"l"(p)); }
#ifndef QX_RED_PF
#define QX_RED_PF 1
#endif
template <int P>
__device__ __forceinline__ void pf_spinor_l1(const void *base, long stride, long j) {
    if constexpr (P == 2) {
        for (int h = 0; h < 2; ++h) {
            pf_l1(cptr(base, h_spinor_u(stride, h) + 16 * j));
            pf_l1(cptr(base, h_spinor_v(stride, h) + 8 * j));
        }
        pf_l1(cptr(base, (size_t)48 * stride + 4 * j));
    } else {
        constexpr int NB = (P == 8) ? 12 : 6;
#pragma unroll
        for (int k = 0; k < NB; ++k) pf_l1(cptr(base, (size_t)16 * (k * stride + j)));
    }
}
// The fused reductions' per-site partials (reading R5: the 24-term sums in the kernel's
// arithmetic precision, accumulated over sites in fp64): (<out, w>, |out|^2) for RED_XDOT_NORM
// (w = x), <w, out> for RED_RHAT_DOT (w = rhat0).  fp32: three packed lane-wise sums
// A = sum o (.) w, B = sum o (.) swap(w), C = sum o (.) o (one FFMA2 each per complex value;
// the swap is an operand modifier), combined at the end: Re = A.x + A.y, Im = B.x - B.y
// (resp. B.y - B.x), |o|^2 = C.x + C.y.  Shared by the single- and multi-RHS kernels so that
// a batched solve stays bitwise its independent solves.
template <typename R>
__device__ __forceinline__ void site_partials(const R *o, const R *w, int red_kind, double *red) {
#ifndef QX_RED_SITE_F64
    if constexpr (sizeof(R) == 4) {
        float2 A = __fmul2_rn(make_float2(o[0], o[1]), make_float2(w[0], w[1]));
        float2 B = __fmul2_rn(make_float2(o[0], o[1]), make_float2(w[1], w[0]));
#pragma unroll
        for (int k = 1; k < 12; ++k) {
            A = __ffma2_rn(make_float2(o[2 * k], o[2 * k + 1]), make_float2(w[2 * k], w[2 * k + 1]), A);
            B = __ffma2_rn(make_float2(o[2 * k], o[2 * k + 1]), make_float2(w[2 * k + 1], w[2 * k]), B);
        }
        if (red_kind == RED_XDOT_NORM) {
            float2 C = __fmul2_rn(make_float2(o[0], o[1]), make_float2(o[0], o[1]));
#pragma unroll
            for (int k = 1; k < 12; ++k)
                C = __ffma2_rn(make_float2(o[2 * k], o[2 * k + 1]), make_float2(o[2 * k], o[2 * k + 1]), C);
            red[0] += (double)(A.x + A.y);
            red[1] += (double)(B.x - B.y);
            red[2] += (double)(C.x + C.y);
        } else {
            red[0] += (double)(A.x + A.y);
            red[1] += (double)(B.y - B.x);
        }
        return;
    }
    using RA = R;
#else
    using RA = double;
#endif
    RA s0 = 0, s1 = 0, s2 = 0;
#pragma unroll
    for (int k = 0; k < 12; ++k) {
        const RA orr = o[2 * k], oi = o[2 * k + 1], wr = w[2 * k], wi = w[2 * k + 1];
        if (red_kind == RED_XDOT_NORM) {  // (<out, x>, |out|^2)
            s0 += orr * wr + oi * wi;
            s1 += orr * wi - oi * wr;
            s2 += orr * orr + oi * oi;
        } else {                          // <rhat, out>
            s0 += wr * orr + wi * oi;
            s1 += wr * oi - wi * orr;
        }
    }
    red[0] += (double)s0;
    red[1] += (double)s1;
    red[2] += (double)s2;
}

// one output site; red[] receives this site's contribution to the optional fused reduction
// INMODE: load mode of the neighbour spinors (0 read-only path; 2 L2-coherent, for inputs
// written by other CTAs earlier in the same launch — the fused Mhat kernel)
// SS: the variant for contexts with a partitioned X, Y or Z (ghost-aware spatial hops); kept a
// separate instantiation so the unpartitioned kernels keep their register allocation
template <int P, int RECON, bool DAG, int KIND, int INMODE = 0, bool SS = false>
__device__ __forceinline__ void dslash_site(const DslashArgs &a, const void *fin, void *fout, const void *fx, int tid,
                                            double red[3], long goff = 0, int sbit = 0) {
    using R = typename Prec<P>::R;
    if (a.reverse) tid = a.nthreads - 1 - tid;
    const int X = a.X, Y = a.Y, Z = a.Z, Xh = a.Xh;
    int i, xh, y, z, t;
    // the boundary sites of a multi-dimensional split follow the interior box in one RANGE_TAIL
    // launch (kernel-initiated halo)
    const bool ss_box = SS && (a.range == RANGE_INTERIOR || (a.range == RANGE_TAIL && tid < a.tail_ni));
    if (SS && a.range == RANGE_TAIL && !ss_box) tid -= a.tail_ni;
    if (ss_box) {  // the interior box of a multi-dimensional split
        int r = tid;
        xh = r % a.bn[0] + a.blo[0];
        r /= a.bn[0];
        y = r % a.bn[1] + a.blo[1];
        r /= a.bn[1];
        z = r % a.bn[2] + a.blo[2];
        t = r / a.bn[2] + a.blo[3];
        i = ((t * Z + z) * Y + y) * Xh + xh;
    } else {
        if (a.range == RANGE_ALL) i = tid;
        else if (a.range == RANGE_INTERIOR) i = a.F + tid;  // T-only split: t in [1, T_loc-2]
        else if (SS) i = __ldg(a.blist + tid);  // complement of the interior box (BOUNDARY / TAIL)
        else if (a.range == RANGE_TAIL) {
            const int ni = (a.T_loc - 2) * a.F;
            const int j = tid - ni;
            i = (tid < ni) ? a.F + tid : ((j < a.F) ? j : (a.T_loc - 1) * a.F + (j - a.F));
        } else i = (tid < a.F) ? tid : (a.T_loc - 1) * a.F + (tid - a.F);
        int r = fdiv(i, a.dXh);
        xh = i - r * Xh;
        const int r2 = fdiv(r, a.dY);
        y = r - r2 * Y;
        t = fdiv(r2, a.dZ);
        z = r2 - t * Z;
    }
    const int x = 2 * xh + ((a.parity + y + z + t) & 1);
    const int p = a.parity, op = 1 - p;
    const int XY = X * Y;
    const int XYZ = XY * Z;
    const int lex = ((t * Z + z) * Y + y) * X + x;

    constexpr int SF = DAG ? +1 : -1;  // sigma of the forward hop
    constexpr int SB = -SF;

    Cx<R> acc[4][3];
    // xpay: out = T x + a D in.  The site-local T x is computed FIRST and carried in the
    // accumulator as (1/a) T x, so its loads (x, clover) overlap the stencil's instead of
    // adding a dependent memory round trip after it; out = a * acc at the end.
    const bool xpay_early = (KIND == QUDAX_CLOVER_XPAY) && (a.a != 0.0);
    if (xpay_early) {
        R v[24];
        Cx<R> xs[4][3];
        SpinorIO<P>::load(fx, a.stride, i, v);
        unpack_spinor(v, xs);
        apply_clover<P>(a.clover, a.stride, i, xs, acc);
        const R inv_a = (R)(1.0 / a.a);
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) acc[s][c] = inv_a * acc[s][c];
    } else {
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) acc[s][c] = cx((R)0, (R)0);
    }

    // Each direction loads raw (undecoded) neighbour spinors and links.  With PAIR the loads
    // of the backward hop are issued before the forward hop is computed: twice the bytes in
    // flight per thread (dslash_pair).
    constexpr bool PAIR = dslash_pair<P, RECON>();
    constexpr bool DF = dslash_defer<P, RECON>();
    auto spatial = [&](auto mu_c, int coord, int Lmu, int nf, int nb) {
        constexpr int MU = decltype(mu_c)::value;
        // operand sources of the two hops: the input field, or (partitioned X) the neighbour's
        // raw face records — a per-lane pointer select, so the warps (every one of which holds
        // x = 0 / x = X-1 sites) do not diverge
        const void *fsrc = fin, *bsrc = fin, *lbsrc = a.gauge[MU][op];
        long fstr = a.stride, bstr = a.stride, lbstr = a.stride;
        int lbi = nb;
        if constexpr (SS && MU == 0) {
            if (a.smask & 1) {
                const int f = face_index<0>(x, y, z, t, X, Y, Z);
                if (coord == Lmu - 1) { fsrc = cptr(a.sghost_fwd[0], sbit ? a.sp2p_pdist[0] : 0); fstr = a.sfs[0]; nf = f; }
                if (coord == 0) {
                    bsrc = cptr(a.sghost_back[0], sbit ? a.sp2p_pdist[0] : 0); bstr = a.sfs[0]; nb = f;
                    lbsrc = a.gauge_sghost[0]; lbstr = a.sfs[0]; lbi = f;
                }
            }
        }
        if (SS && MU > 0 && ((a.smask >> MU) & 1)) {
            // partitioned Y / Z: a hop off the local box reads the neighbour's projected face
            // (whole rows / planes: no divergence)
            const bool gf = (coord == Lmu - 1), gb = (coord == 0);
            if (gf || gb) {
                const int f = face_index<MU>(x, y, z, t, X, Y, Z);
                Cx<R> h0[3], h1[3], u[3][3];
                R sc;
                if (gf) {
                    sc = ghost_half<P, MU, SF, DF>(cptr(a.sghost_fwd[MU], sbit ? a.sp2p_pdist[MU] : 0), a.sfs[MU], f, h0, h1);
                } else {
                    RawVec<P, 24> sv;
                    sv.template load_spinor<INMODE>(fin, a.stride, nf);
                    R v[24];
                    Cx<R> ps[4][3];
                    sc = dec_vec<DF>(sv, v);
                    unpack_spinor(v, ps);
                    spatial_project<MU, SF>(ps, h0, h1);
                }
                {
                    RawLink<P, RECON> l;
                    l.load(a.gauge[MU][p], a.stride, i);
                    sc *= dec_link<DF>(l, u);
                }
                spatial_mult_expand<MU, SF, false, DF>(h0, h1, u, acc, sc);
                if (gb) {
                    sc = ghost_half<P, MU, SB, DF>(cptr(a.sghost_back[MU], sbit ? a.sp2p_pdist[MU] : 0), a.sfs[MU], f, h0, h1);
                    RawLink<P, RECON> l;
                    l.load(a.gauge_sghost[MU], a.sfs[MU], f);
                    sc *= dec_link<DF>(l, u);
                } else {
                    RawVec<P, 24> sv;
                    sv.template load_spinor<INMODE>(fin, a.stride, nb);
                    R v[24];
                    Cx<R> ps[4][3];
                    sc = dec_vec<DF>(sv, v);
                    unpack_spinor(v, ps);
                    spatial_project<MU, SB>(ps, h0, h1);
                    RawLink<P, RECON> l;
                    l.load(a.gauge[MU][op], a.stride, nb);
                    sc *= dec_link<DF>(l, u);
                }
                spatial_mult_expand<MU, SB, true, DF>(h0, h1, u, acc, sc);
                return;
            }
        }
        RawVec<P, 24> sf, sb;
        RawLink<P, RECON> lf, lb;
        sf.template load_spinor<INMODE>(fsrc, fstr, nf);
        lf.load(a.gauge[MU][p], a.stride, i);
        if constexpr (PAIR) {
            sb.template load_spinor<INMODE>(bsrc, bstr, nb);
            lb.load(lbsrc, lbstr, lbi);
        }
        if constexpr (DF && QX_BPROJ) {
            R v[24];
            Cx<R> ps[4][3], u[3][3], h0[3], h1[3];
            sf.decode_b(v);
            unpack_spinor(v, ps);
            spatial_project_b<MU, SF>(ps, h0, h1);
            const R sc = sf.scale() * dec_link<DF>(lf, u);
            spatial_mult_expand<MU, SF, false, DF>(h0, h1, u, acc, sc);
        } else {
            R v[24];
            Cx<R> ps[4][3], u[3][3];
            R sc = dec_vec<DF>(sf, v);
            unpack_spinor(v, ps);
            sc *= dec_link<DF>(lf, u);
            spatial_hop<MU, SF, false, DF>(ps, u, acc, sc);
        }
        if constexpr (!PAIR) {
            sb.template load_spinor<INMODE>(bsrc, bstr, nb);
            lb.load(lbsrc, lbstr, lbi);
        }
        if constexpr (DF && QX_BPROJ) {
            R v[24];
            Cx<R> ps[4][3], u[3][3], h0[3], h1[3];
            sb.decode_b(v);
            unpack_spinor(v, ps);
            spatial_project_b<MU, SB>(ps, h0, h1);
            const R sc = sb.scale() * dec_link<DF>(lb, u);
            spatial_mult_expand<MU, SB, true, DF>(h0, h1, u, acc, sc);
        } else {
            R v[24];
            Cx<R> ps[4][3], u[3][3];
            R sc = dec_vec<DF>(sb, v);
            unpack_spinor(v, ps);
            sc *= dec_link<DF>(lb, u);
            spatial_hop<MU, SB, true, DF>(ps, u, acc, sc);
        }
    };
    // (neighbour indices computed at each call: holding all six live across the hops costs
    // registers at the 80-register cap — measured up to 13 % on fp32 recon-8, r02m)
    spatial(std::integral_constant<int, 0>{}, x, X, (x == X - 1 ? lex - (X - 1) : lex + 1) >> 1,
            (x == 0 ? lex + (X - 1) : lex - 1) >> 1);
    spatial(std::integral_constant<int, 1>{}, y, Y, (y == Y - 1 ? lex - (Y - 1) * X : lex + X) >> 1,
            (y == 0 ? lex + (Y - 1) * X : lex - X) >> 1);
    spatial(std::integral_constant<int, 2>{}, z, Z, (z == Z - 1 ? lex - (Z - 1) * XY : lex + XY) >> 1,
            (z == 0 ? lex + (Z - 1) * XY : lex - XY) >> 1);

    // ---- t direction: diagonal projectors, 12 reals per neighbour (eq. (6))
    {
        // forward: (1 + SF gamma_4): SF = -1 -> lower spins, SF = +1 -> upper spins;
        // backward: (1 + SB gamma_4)
        constexpr bool FWD_UPPER = (SF > 0);
        constexpr bool BWD_UPPER = (SB > 0);
        const int T_loc = a.T_loc;
        // operand addresses first (ghost face / periodic wrap / interior), then one load each
        const bool fwd_ghost = (t == T_loc - 1) && a.ghosted;
        const bool bwd_ghost = (t == 0) && a.ghosted;
        const R cf = (t == T_loc - 1) ? (R)(2.0 * a.bc_fwd) : (R)2;
        const R cb = (t == 0) ? (R)(2.0 * a.bc_back) : (R)2;
        const int nfw = (t == T_loc - 1 ? lex - (T_loc - 1) * XYZ : lex + XYZ) >> 1;
        const int nbw = (t == 0 ? lex + (T_loc - 1) * XYZ : lex - XYZ) >> 1;
        RawVec<P, 12> hf, hb;
        RawLink<P, RECON> lf, lb;
        auto load_f = [&] {
            if (fwd_ghost) hf.load_face(static_cast<const char *>(a.ghost_fwd) + goff, a.fstride, i - t * a.F);
            else hf.template load_half<INMODE>(fin, a.stride, nfw, FWD_UPPER ? 0 : 1);
            lf.load(a.gauge[3][p], a.stride, i);
        };
        auto load_b = [&] {
            if (bwd_ghost) {
                hb.load_face(static_cast<const char *>(a.ghost_back) + goff, a.fstride, i);
                lb.load(a.gauge_ghost, a.fstride, i);
            } else {
                hb.template load_half<INMODE>(fin, a.stride, nbw, BWD_UPPER ? 0 : 1);
                lb.load(a.gauge[3][op], a.stride, nbw);
            }
        };
        load_f();
        if constexpr (PAIR) load_b();
#if QX_RED_PF
        // the fused reduction's second operand (x or rhat0) is read right after the store: pull
        // its lines into L1 while the last hops are computed (a dependent L2 round trip at the
        // very end of every thread otherwise)
        if (a.red_kind != RED_NONE) {
            const void *w = a.red_kind == RED_XDOT_NORM ? fx : (a.nrhs > 1 ? a.rhat_m[blockIdx.x % a.nrhs] : a.rhat);
            pf_spinor_l1<P>(w, a.stride, i);
        }
#endif
        {
            R h[12];
            Cx<R> u[3][3];
            R sc = dec_vec<DF>(hf, h);
            sc *= dec_link<DF>(lf, u);
            temporal_hop<FWD_UPPER, false>(h, u, DF ? cf * sc : cf, acc);
        }
        if constexpr (!PAIR) load_b();
        {
            R h[12];
            Cx<R> u[3][3];
            R sc = dec_vec<DF>(hb, h);
            sc *= dec_link<DF>(lb, u);
            temporal_hop<BWD_UPPER, true>(h, u, DF ? cb * sc : cb, acc);
        }
    }

    // ---- epilogue: fused clover
    Cx<R> res[4][3];
    if constexpr (KIND == QUDAX_HOP) {
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) res[s][c] = acc[s][c];
    } else if constexpr (KIND == QUDAX_CLOVER_INV) {
        apply_clover<P>(a.clover, a.stride, i, acc, res);
    } else if constexpr (KIND == QUDAX_CLOVER_INV_XPAY) {  // symmetric Schur: out = x + a T^{-1} D in
        Cx<R> ti[4][3], xs[4][3];
        apply_clover<P>(a.clover, a.stride, i, acc, ti);
        R v[24];
        SpinorIO<P>::load(fx, a.stride, i, v);
        unpack_spinor(v, xs);
        const R co = (R)a.a;
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) res[s][c] = axpy(co, ti[s][c], xs[s][c]);
    } else if (xpay_early) {
        const R co = (R)a.a;
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) res[s][c] = co * acc[s][c];
    } else {  // a == 0: out = T x
        R v[24];
        Cx<R> xs[4][3];
        SpinorIO<P>::load(fx, a.stride, i, v);
        unpack_spinor(v, xs);
        apply_clover<P>(a.clover, a.stride, i, xs, res);
    }
    R o[24];
#pragma unroll
    for (int s = 0; s < 4; ++s)
#pragma unroll
        for (int c = 0; c < 3; ++c) {
            o[(s * 3 + c) * 2] = res[s][c].r;
            o[(s * 3 + c) * 2 + 1] = res[s][c].i;
        }
    if (a.red_kind == RED_NONE) {
        SpinorIO<P>::store(fout, a.stride, i, o);
        return;
    }
    // fused BiCGstab reductions over what was stored (half: the requantised values)
    SpinorIO<P>::store_requant(fout, a.stride, i, o);
    R w[24];
    // (multi-RHS launch: this CTA's right-hand side, recomputed here rather than kept live)
    const void *rh = a.nrhs > 1 ? a.rhat_m[blockIdx.x % a.nrhs] : a.rhat;
    SpinorIO<P>::load(a.red_kind == RED_XDOT_NORM ? fx : rh, a.stride, i, w);
    site_partials<R>(o, w, a.red_kind, red);
}

// Kernel-initiated halo (QUDAX_HALO_P2P): one thread per CTA acquires the two flags the
// neighbours raise after storing this sequence number's faces into our ghosts.  The wait is
// bounded (a stalled neighbour must not hang the GPU): on timeout the CTA raises the context's
// device error word, which the host checks at its next synchronisation and reports as
// QUDAX_ERR_COMM instead of returning an operator applied to stale ghosts.  Returns the ghost
// byte offset of the sequence parity.
__device__ __forceinline__ unsigned ld_acquire_sys(const unsigned *p) {
    unsigned v;
    asm volatile("ld.acquire.sys.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ int p2p_wait(const DslashArgs &a) {
    __shared__ unsigned s_seq;
    if (threadIdx.x == 0) {
        const unsigned s = *reinterpret_cast<const volatile unsigned *>(a.p2p_cseq) + 1u;
        bool ok = false;
        for (long spin = 0; spin < (1L << 24) && !ok; ++spin) {  // >= 2 s of 128 ns sleeps
            ok = true;
            for (int m = 0; m < 4 && ok; ++m)
                if (a.p2p_mask >> m & 1)
                    ok = (int)(ld_acquire_sys(a.p2p_flags + 2 * m) - s) >= 0 &&
                         (int)(ld_acquire_sys(a.p2p_flags + 2 * m + 1) - s) >= 0;
            if (!ok) __nanosleep(128);
        }
        if (!ok && a.err) atomicExch(a.err, 1);
        s_seq = s;
    }
    __syncthreads();
    return (int)(s_seq & 1u);
}

// Kernel-timing span (kernel timing on: a.span != nullptr): the first CTA to arrive stamps
// %globaltimer into span[0], the last CTA to finish into span[1] and resets the arrival counters
// (span[2]: two 32-bit counters), so a launch slot can be replayed in a CUDA graph.  The span is
// the kernel's own execution time, without the launch bubbles the event-record nodes around it
// add in graph replay.  Not inlined: inlined, they cost the clover-inverse kernel 16 B of spills.
__device__ __forceinline__ unsigned long long globaltimer_ns() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}
static __device__ __noinline__ void span_begin(unsigned long long *span) {
    if (span && threadIdx.x == 0 && atomicAdd(reinterpret_cast<unsigned *>(span + 2), 1u) == 0u)
        span[0] = globaltimer_ns();
}
static __device__ __noinline__ void span_end(unsigned long long *span) {
    if (!span) return;
    // (thread 0's own end stands for its CTA's: no barrier, which would keep values live)
    if (threadIdx.x == 0) {
        if (atomicAdd(reinterpret_cast<unsigned *>(span + 2) + 1, 1u) == gridDim.x - 1) {
            span[1] = globaltimer_ns();
            span[2] = 0ull;  // both counters
        }
    }
}

template <int P, int RECON, bool DAG, int KIND, bool SS>
__device__ __forceinline__ void dslash_body(const DslashArgs &a);
template <int P, int RECON, bool DAG, int KIND, bool SS>
__global__ void __launch_bounds__(QX_DSLASH_THREADS, QX_MINB_OF2(P, RECON)) dslash_kernel(const __grid_constant__ DslashArgs a) {
#ifndef QX_SPAN
#define QX_SPAN 1
#endif
    // (the test is on the parameter, outside the calls: no call at all unless kernel timing runs
    // in span mode)
    if (QX_SPAN && a.span) span_begin(a.span);
    dslash_body<P, RECON, DAG, KIND, SS>(a);
    if (QX_SPAN && a.span) span_end(a.span);
}
template <int P, int RECON, bool DAG, int KIND, bool SS>
__device__ __forceinline__ void dslash_body(const DslashArgs &a) {
    // one thread per output site (a one-wave grid-stride variant measured 8-25% slower: the
    // hardware CTA scheduler balances the memory-latency-bound CTAs better than a fixed wave)
    // multi-RHS (a.nrhs > 1): consecutive CTAs take the same sites for different right-hand
    // sides, so the links and clover they stream are served from L2 after the first of them
    // (no solver-batch gate: a batch's remaining iterations after a reliable-update request are
    // not launched at all — the WHILE node of the batch graph stops, solver.cpp)
    int blk = blockIdx.x, rhs = 0;
    if (a.nrhs > 1) {
        rhs = blk % a.nrhs;
        blk /= a.nrhs;
    }
    const int tid = blk * blockDim.x + threadIdx.x;
    double red[3] = {0.0, 0.0, 0.0};
    const void *fin = a.nrhs > 1 ? a.in_m[rhs] : a.in;
    void *fout = a.nrhs > 1 ? a.out_m[rhs] : a.out;
    const void *fx = a.nrhs > 1 ? a.x_m[rhs] : a.x;
    long goff = (long)rhs * a.ghost_rhs_bytes;  // multi-RHS halo: this RHS's ghost faces
    int sbit = 0;                               // kernel-initiated halo: sequence parity of the ghosts
    // RANGE_TAIL: only CTAs holding boundary sites (the grid's last ones) wait for the halo
    if (a.p2p_flags && (a.range != RANGE_TAIL || (blk + 1) * (int)blockDim.x > a.tail_ni)) {
        sbit = p2p_wait(a);
        goff = sbit ? a.p2p_pdist : 0L;
    }
    if (tid < a.nthreads) dslash_site<P, RECON, DAG, KIND, 0, SS>(a, fin, fout, fx, tid, red, goff, sbit);
    if (a.p2p_flags) {  // the last CTA to finish advances the consumed-halo counter
        __syncthreads();
        if (threadIdx.x == 0 && atomicAdd(a.p2p_ccount, 1u) == gridDim.x - 1) {
            *a.p2p_ccount = 0u;
            *a.p2p_cseq += 1u;
        }
    }
    if (a.red_kind != RED_NONE) {
        if (a.nrhs > 1) reduce_with_tail<3, QX_DSLASH_THREADS>(red, a.tail_m[blockIdx.x % a.nrhs], blockIdx.x / a.nrhs);
        else reduce_with_tail<3, QX_DSLASH_THREADS>(red, a.tail);
    }
}

template <int P, int RC, bool DG, int KD>
int dslash_blocks(int nthreads) {
    return (nthreads + QX_DSLASH_THREADS - 1) / QX_DSLASH_THREADS;
}

template <int P>
int dslash_blocks_prec(int recon, int dagger, int kind, int nthreads) {
#define QX_DB(RC, DG, KD) \
    if (recon == RC && dagger == DG && kind == KD) return dslash_blocks<P, RC, DG, KD>(nthreads);
#define QX_DB_K(RC, DG) QX_DB(RC, DG, 0) QX_DB(RC, DG, 1) QX_DB(RC, DG, 2) QX_DB(RC, DG, 3)
#define QX_DB_D(RC) QX_DB_K(RC, false) QX_DB_K(RC, true)
    QX_DB_D(18) QX_DB_D(12) QX_DB_D(8)
#undef QX_DB_D
#undef QX_DB_K
#undef QX_DB
    throw Error(QUDAX_ERR_ARG, "dslash: unsupported recon/kind");
}

// several right-hand sides per thread (dslash_mr.cuh, instantiated in dslash_f{32,16}_mr.cu so
// the two kernel families compile in parallel)
bool launch_dslash_mr_f32(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
bool launch_dslash_mr_f16(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);

template <int P, bool SS = false>
void launch_dslash_prec(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    const int threads = QX_DSLASH_THREADS;
    if (a.nthreads <= 0) return;
    if constexpr (P != 8 && !SS) {  // several right-hand sides per thread (dslash_mr.cuh)
        if (a.nrhs > 1 && !(a.variant & kVariantOneRhsPerThread) &&
            (P == 4 ? launch_dslash_mr_f32(recon, dagger, kind, a, s) : launch_dslash_mr_f16(recon, dagger, kind, a, s)))
            return;
    }
#define QX_DS(RC, DG, KD)                                                                       \
    if (recon == RC && dagger == DG && kind == KD) {                                            \
        dslash_kernel<P, RC, DG, KD, SS><<<dslash_blocks<P, RC, DG, KD>(a.nthreads) * (a.nrhs > 1 ? a.nrhs : 1), \
                                       threads, 0, s>>>(a);                                     \
        return;                                                                                 \
    }
#define QX_DS_K(RC, DG) QX_DS(RC, DG, 0) QX_DS(RC, DG, 1) QX_DS(RC, DG, 2) QX_DS(RC, DG, 3)
#define QX_DS_D(RC) QX_DS_K(RC, false) QX_DS_K(RC, true)
    QX_DS_D(18) QX_DS_D(12) QX_DS_D(8)
#undef QX_DS_D
#undef QX_DS_K
#undef QX_DS
    throw Error(QUDAX_ERR_ARG, "dslash: unsupported recon/kind");
}

}  // namespace qx
