// dslash_mr.cuh — multi-RHS Dslash with NR right-hand sides per thread.
//
// The single-RHS-per-thread multi-RHS launch (dslash.cuh, a.nrhs > 1) streams each link and
// clover block from HBM about once, but every (site, RHS) thread still loads, decodes and
// reconstructs the 8 links and the clover itself (from L2): at 8 RHS the kernel runs at the
// FMA-pipe / latency floor of the per-site work, not at the byte bound.  Here one thread owns a
// site for NR right-hand sides: each link is loaded and reconstructed once and applied to the
// NR neighbour spinors, each clover block once for the NR vectors.  Same arithmetic per RHS as
// dslash_site (same helpers, same operation order), so the result is bitwise the single-RHS
// one.  Unpartitioned lattices, or T-partitioned ones with the multi-RHS halo (interior /
// boundary ranges, one ghost face per RHS); an odd last group repeats its last RHS and skips its
// stores.
#pragma once
#include "dslash.cuh"

namespace qx {

#ifdef QX_MR_MINB
template <int P, int NR> struct DslashMrMinBlocks { static constexpr int value = QX_MR_MINB; };
#else
template <int P, int NR> struct DslashMrMinBlocks { static constexpr int value = NR == 1 ? 6 : 4; };
#endif

#ifndef QX_MR_NR
#define QX_MR_NR 2
#endif

template <int P, int NR>
__device__ __forceinline__ void apply_clover_mr(const void *cl, long stride, long i, const Cx<typename Prec<P>::R> (*in)[4][3],
                                                Cx<typename Prec<P>::R> (*out)[4][3]) {
    using R = typename Prec<P>::R;
    constexpr bool DF = (P == 2) && dslash_defer<2, 12>();
    Cx<R> wa[NR][6];
#pragma unroll
    for (int b = 0; b < 2; ++b) {
        R m[36];
        const R sc = CloverIO<P>::template load<DF>(cl, stride, i, b, m);
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            Cx<R> v[6], w[6];
#pragma unroll
            for (int s = 0; s < 2; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c)
                    v[s * 3 + c] = b == 0 ? in[r][s][c] + in[r][s + 2][c] : in[r][s][c] - in[r][s + 2][c];
            if constexpr (DF) {
#pragma unroll
                for (int k = 0; k < 6; ++k) v[k] = sc * v[k];
            }
            herm6_mul(m, v, w);
            if (b == 0) {
#pragma unroll
                for (int k = 0; k < 6; ++k) wa[r][k] = w[k];
            } else {
#pragma unroll
                for (int s = 0; s < 2; ++s)
#pragma unroll
                    for (int c = 0; c < 3; ++c) {
                        out[r][s][c] = wa[r][s * 3 + c] + w[s * 3 + c];
                        out[r][s + 2][c] = wa[r][s * 3 + c] - w[s * 3 + c];
                    }
            }
        }
    }
}

template <int P, int RECON, bool DAG, int KIND, int NR>
__device__ __forceinline__ void dslash_site_mr(const DslashArgs &a, int tid, int r0, const void *const *fin,
                                               void *const *fout, const void *const *fx, const void *const *frh,
                                               bool last_valid, double (*red)[3]) {
    using R = typename Prec<P>::R;
    if (a.reverse) tid = a.nthreads - 1 - tid;
    // T-partitioned contexts (multi-RHS halo): interior sites t in [1, T_loc-2], or the 2F
    // boundary sites (t = 0 and t = T_loc-1), as in dslash_site
    const int i = a.range == RANGE_ALL ? tid
                  : (a.range == RANGE_INTERIOR ? a.F + tid : (tid < a.F ? tid : (a.T_loc - 1) * a.F + (tid - a.F)));
    const int X = a.X, Y = a.Y, Z = a.Z, Xh = a.Xh;
    int xh, y, z, t;
    {
        const int r = fdiv(i, a.dXh);
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
    constexpr int SF = DAG ? +1 : -1;
    constexpr int SB = -SF;
    constexpr bool DF = dslash_defer<P, RECON>();

    Cx<R> acc[NR][4][3];
    const bool xpay_early = (KIND == QUDAX_CLOVER_XPAY) && (a.a != 0.0);
    if (xpay_early) {
        Cx<R> xs[NR][4][3];
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            R v[24];
            SpinorIO<P>::load(fx[r], a.stride, i, v);
            unpack_spinor(v, xs[r]);
        }
        apply_clover_mr<P, NR>(a.clover, a.stride, i, xs, acc);
        const R inv_a = (R)(1.0 / a.a);
#pragma unroll
        for (int r = 0; r < NR; ++r)
#pragma unroll
            for (int s = 0; s < 4; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c) acc[r][s][c] = inv_a * acc[r][s][c];
    } else {
#pragma unroll
        for (int r = 0; r < NR; ++r)
#pragma unroll
            for (int s = 0; s < 4; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c) acc[r][s][c] = cx((R)0, (R)0);
    }

    // one spatial hop for the NR right-hand sides: the link is loaded and reconstructed once
    auto hop = [&](auto mu_c, auto sg_c, auto adj_c, const void *lbase, int li, int n) {
        constexpr int MU = decltype(mu_c)::value;
        constexpr int SG = decltype(sg_c)::value;
        constexpr bool ADJ = decltype(adj_c)::value;
        RawLink<P, RECON> l;
        l.load(lbase, a.stride, li);
        RawVec<P, 24> sv;
        sv.template load_spinor<0>(fin[0], a.stride, n);
        Cx<R> u[3][3];
        const R usc = dec_link<DF>(l, u);
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            RawVec<P, 24> cur = sv;
            if (r + 1 < NR) sv.template load_spinor<0>(fin[r + 1], a.stride, n);  // next RHS in flight
            R v[24];
            Cx<R> ps[4][3], h0[3], h1[3];
            R sc;
            if constexpr (DF && QX_BPROJ) {
                cur.decode_b(v);
                unpack_spinor(v, ps);
                spatial_project_b<MU, SG>(ps, h0, h1);
                sc = cur.scale() * usc;
            } else {
                sc = dec_vec<DF>(cur, v);
                unpack_spinor(v, ps);
                spatial_project<MU, SG>(ps, h0, h1);
                sc *= usc;
            }
            spatial_mult_expand<MU, SG, ADJ, DF>(h0, h1, u, acc[r], sc);
        }
    };
    using I0 = std::integral_constant<int, 0>;
    using I1 = std::integral_constant<int, 1>;
    using I2 = std::integral_constant<int, 2>;
    using PF = std::integral_constant<int, SF>;
    using PB = std::integral_constant<int, SB>;
    using NA = std::integral_constant<bool, false>;
    using AD = std::integral_constant<bool, true>;
    {
        const int nf = (x == X - 1 ? lex - (X - 1) : lex + 1) >> 1, nb = (x == 0 ? lex + (X - 1) : lex - 1) >> 1;
        hop(I0{}, PF{}, NA{}, a.gauge[0][p], i, nf);
        hop(I0{}, PB{}, AD{}, a.gauge[0][op], nb, nb);
    }
    {
        const int nf = (y == Y - 1 ? lex - (Y - 1) * X : lex + X) >> 1, nb = (y == 0 ? lex + (Y - 1) * X : lex - X) >> 1;
        hop(I1{}, PF{}, NA{}, a.gauge[1][p], i, nf);
        hop(I1{}, PB{}, AD{}, a.gauge[1][op], nb, nb);
    }
    {
        const int nf = (z == Z - 1 ? lex - (Z - 1) * XY : lex + XY) >> 1, nb = (z == 0 ? lex + (Z - 1) * XY : lex - XY) >> 1;
        hop(I2{}, PF{}, NA{}, a.gauge[2][p], i, nf);
        hop(I2{}, PB{}, AD{}, a.gauge[2][op], nb, nb);
    }
    // t direction: diagonal projectors, 12 reals per neighbour (eq. (6)); periodic wrap with the
    // boundary sign on the local edge, or (T-partitioned, a.ghosted) the neighbours' faces: one
    // halo carries every right-hand side, RHS k's face at k * a.ghost_rhs_bytes
    {
        constexpr bool FWD_UPPER = (SF > 0);
        constexpr bool BWD_UPPER = (SB > 0);
        const int T_loc = a.T_loc;
        const R cf = (t == T_loc - 1) ? (R)(2.0 * a.bc_fwd) : (R)2;
        const R cb = (t == 0) ? (R)(2.0 * a.bc_back) : (R)2;
        const int nfw = (t == T_loc - 1 ? lex - (T_loc - 1) * XYZ : lex + XYZ) >> 1;
        const int nbw = (t == 0 ? lex + (T_loc - 1) * XYZ : lex - XYZ) >> 1;
        const bool fwd_ghost = (t == T_loc - 1) && a.ghosted;
        const bool bwd_ghost = (t == 0) && a.ghosted;
        auto thop = [&](auto up_c, auto adj_c, bool ghost, const void *gbase, long gf, const void *lbase, long lstr,
                        int li, int n, R coef) {
            constexpr bool UP = decltype(up_c)::value;
            constexpr bool ADJ = decltype(adj_c)::value;
            RawLink<P, RECON> l;
            l.load(lbase, lstr, li);
            auto ld = [&](RawVec<P, 12> &hv, int r) {
                if (ghost) hv.load_face(static_cast<const char *>(gbase) + (long)(r0 + r) * a.ghost_rhs_bytes, a.fstride, gf);
                else hv.template load_half<0>(fin[r], a.stride, n, UP ? 0 : 1);
            };
            RawVec<P, 12> hv;
            ld(hv, 0);
            Cx<R> u[3][3];
            const R usc = dec_link<DF>(l, u);
#pragma unroll
            for (int r = 0; r < NR; ++r) {
                RawVec<P, 12> cur = hv;
                if (r + 1 < NR) ld(hv, r + 1);
                R h[12];
                R sc = dec_vec<DF>(cur, h);
                sc *= usc;
                temporal_hop<UP, ADJ>(h, u, DF ? coef * sc : coef, acc[r]);
            }
        };
        thop(std::integral_constant<bool, FWD_UPPER>{}, NA{}, fwd_ghost, a.ghost_fwd, (long)(i - t * a.F),
             a.gauge[3][p], a.stride, i, nfw, cf);
        if (bwd_ghost)
            thop(std::integral_constant<bool, BWD_UPPER>{}, AD{}, true, a.ghost_back, (long)i, a.gauge_ghost, a.fstride,
                 i, nbw, cb);
        else
            thop(std::integral_constant<bool, BWD_UPPER>{}, AD{}, false, a.ghost_back, (long)i, a.gauge[3][op], a.stride,
                 nbw, nbw, cb);
    }

    // epilogue: fused clover, store, optional per-RHS reductions
    Cx<R> res[NR][4][3];
    if constexpr (KIND == QUDAX_HOP) {
#pragma unroll
        for (int r = 0; r < NR; ++r)
#pragma unroll
            for (int s = 0; s < 4; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c) res[r][s][c] = acc[r][s][c];
    } else if constexpr (KIND == QUDAX_CLOVER_INV) {
        apply_clover_mr<P, NR>(a.clover, a.stride, i, acc, res);
    } else if constexpr (KIND == QUDAX_CLOVER_INV_XPAY) {
        Cx<R> ti[NR][4][3];
        apply_clover_mr<P, NR>(a.clover, a.stride, i, acc, ti);
        const R co = (R)a.a;
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            R v[24];
            Cx<R> xs[4][3];
            SpinorIO<P>::load(fx[r], a.stride, i, v);
            unpack_spinor(v, xs);
#pragma unroll
            for (int s = 0; s < 4; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c) res[r][s][c] = axpy(co, ti[r][s][c], xs[s][c]);
        }
    } else if (xpay_early) {
        const R co = (R)a.a;
#pragma unroll
        for (int r = 0; r < NR; ++r)
#pragma unroll
            for (int s = 0; s < 4; ++s)
#pragma unroll
                for (int c = 0; c < 3; ++c) res[r][s][c] = co * acc[r][s][c];
    } else {  // a == 0: out = T x
        Cx<R> xs[NR][4][3];
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            R v[24];
            SpinorIO<P>::load(fx[r], a.stride, i, v);
            unpack_spinor(v, xs[r]);
        }
        apply_clover_mr<P, NR>(a.clover, a.stride, i, xs, res);
    }
#pragma unroll
    for (int r = 0; r < NR; ++r) {
        if (r == NR - 1 && !last_valid) break;
        R o[24];
#pragma unroll
        for (int s = 0; s < 4; ++s)
#pragma unroll
            for (int c = 0; c < 3; ++c) {
                o[(s * 3 + c) * 2] = res[r][s][c].r;
                o[(s * 3 + c) * 2 + 1] = res[r][s][c].i;
            }
        if (a.red_kind == RED_NONE) {
            SpinorIO<P>::store(fout[r], a.stride, i, o);
            continue;
        }
        SpinorIO<P>::store_requant(fout[r], a.stride, i, o);
        R w[24];
        SpinorIO<P>::load(a.red_kind == RED_XDOT_NORM ? fx[r] : frh[r], a.stride, i, w);
        site_partials<R>(o, w, a.red_kind, red[r]);
    }
}

// grid: (site blocks) x (RHS groups of NR), consecutive CTAs = the groups of one site block
template <int P, int RECON, bool DAG, int KIND, int NR>
__device__ __forceinline__ void dslash_mr_body(const DslashArgs &a);
template <int P, int RECON, bool DAG, int KIND, int NR>
__global__ void __launch_bounds__(QX_DSLASH_THREADS, DslashMrMinBlocks<P, NR>::value) dslash_mr_kernel(const __grid_constant__ DslashArgs a) {
    if (a.span) span_begin(a.span);
    dslash_mr_body<P, RECON, DAG, KIND, NR>(a);
    if (a.span) span_end(a.span);
}
template <int P, int RECON, bool DAG, int KIND, int NR>
__device__ __forceinline__ void dslash_mr_body(const DslashArgs &a) {
    const int ng = (a.nrhs + NR - 1) / NR;
    const int grp = blockIdx.x % ng, blk = blockIdx.x / ng;
    const int r0 = grp * NR;
    const bool last_valid = r0 + NR - 1 < a.nrhs;
    const void *fin[NR];
    void *fout[NR];
    const void *fx[NR], *frh[NR];
#pragma unroll
    for (int r = 0; r < NR; ++r) {
        const int k = min(r0 + r, a.nrhs - 1);
        fin[r] = a.in_m[k];
        fout[r] = a.out_m[k];
        fx[r] = a.x_m[k];
        frh[r] = a.rhat_m[k];
    }
    const int tid = blk * blockDim.x + threadIdx.x;
    double red[NR][3] = {};
    if (tid < a.nthreads) dslash_site_mr<P, RECON, DAG, KIND, NR>(a, tid, r0, fin, fout, fx, frh, last_valid, red);
    if (a.red_kind != RED_NONE) {
#pragma unroll
        for (int r = 0; r < NR; ++r) {
            // reduce_with_tail's shared scratch is reused by the next call: the CTA that finishes
            // a reduction has thread 0 still reading it after the other threads return
            if (r > 0) __syncthreads();
            if (r0 + r < a.nrhs) reduce_with_tail<3, QX_DSLASH_THREADS>(red[r], a.tail_m[r0 + r], blk);
        }
    }
}

template <int P>
bool launch_dslash_mr_prec(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    constexpr int NR = QX_MR_NR;
    if (a.nrhs < 2 || a.smask || a.range == RANGE_TAIL || a.p2p_flags) return false;
    const int grid = ((a.nthreads + QX_DSLASH_THREADS - 1) / QX_DSLASH_THREADS) * ((a.nrhs + NR - 1) / NR);
#define QX_MR(RC, DG, KD)                                                                             \
    if (recon == RC && dagger == DG && kind == KD) {                                                  \
        dslash_mr_kernel<P, RC, DG, KD, NR><<<grid, QX_DSLASH_THREADS, 0, s>>>(a);                    \
        return true;                                                                                  \
    }
#define QX_MR_K(RC, DG) QX_MR(RC, DG, 0) QX_MR(RC, DG, 1) QX_MR(RC, DG, 2) QX_MR(RC, DG, 3)
#define QX_MR_D(RC) QX_MR_K(RC, false) QX_MR_K(RC, true)
    QX_MR_D(18) QX_MR_D(12) QX_MR_D(8)
#undef QX_MR_D
#undef QX_MR_K
#undef QX_MR
    return false;
}

}  // namespace qx
