// layout.cu — field reordering and setup kernels (all on the device):
//  * spinor import/export: host-order DeGrand-Rossi AoS fp64 <-> non-relativistic-basis
//    site-major SoA in fp64 / fp32 / half (eqs. (3)-(4); eq. (6) basis change,
//    P:479-506; half-precision encoding, reading Q7), one parity at a time;
//  * gauge pack: fp64 links -> per-direction, per-parity SoA with 18/12/8-real storage
//    (reading Q6), plus the backward temporal ghost link face;
//  * clover build + invert: four-leaf field strength -> T = 1 + 2 kappa A and T^{-1} as two
//    Hermitian 6x6 chiral blocks per site, fp64 (reading Q1);
//  * face pack for the T-direction halo.
#include "core.cuh"
#include "dslash.cuh"
#include "internal.h"

namespace qx {

__host__ __device__ constexpr double kInvSqrt2 = 0.70710678118654752440;

// coordinates of cb site i of parity p (local; t0 is even so local parity = global parity)
struct Coord {
    int x, y, z, t, lex;
};
__device__ __forceinline__ Coord cb_coord(int i, int p, int X, int Y, int Z) {
    const int Xh = X / 2;
    Coord c;
    int xh = i % Xh;
    int r = i / Xh;
    c.y = r % Y;
    r /= Y;
    c.z = r % Z;
    c.t = r / Z;
    c.x = 2 * xh + ((p + c.y + c.z + c.t) & 1);
    c.lex = ((c.t * Z + c.z) * Y + c.y) * X + c.x;
    return c;
}

// ============================================================================ spinors
// The host-order slab holds one 192-byte DR record per site, sites of the two parities
// interleaved; a parity field visits every other record.  Both directions stage a CTA's 128
// records in shared memory so the global side moves whole records with consecutive 16-byte
// accesses (one record per 12 lanes) — round 1's per-thread access of its own record (24 scalar
// loads or stores 384 bytes apart across a warp) ran the export at ~1.1 TB/s (half-sector
// writes; gpurun r01k launch list: 270 us per export at 32^3x64).
constexpr int kXferThreads = 128;
template <int P>
__global__ void __launch_bounds__(kXferThreads) k_spinor_import(int X, int Y, int Z, int Vh, long stride, int parity,
                                                                const double *__restrict__ src, void *__restrict__ dst) {
    using R = typename Prec<P>::R;
    __shared__ double st[kXferThreads * 24];
    __shared__ int lexs[kXferThreads];
    const int i0 = blockIdx.x * kXferThreads;
    const int i = i0 + threadIdx.x;
    const int nsite = min(kXferThreads, Vh - i0);
    if (i < Vh) lexs[threadIdx.x] = cb_coord(i, parity, X, Y, Z).lex;
    __syncthreads();
    for (int q = threadIdx.x; q < nsite * 12; q += kXferThreads) {
        const int sidx = q / 12, ch = q - 12 * (q / 12);
        const double2 v = __ldg(reinterpret_cast<const double2 *>(src + (size_t)lexs[sidx] * 24) + ch);
        st[sidx * 24 + 2 * ch] = v.x;
        st[sidx * 24 + 2 * ch + 1] = v.y;
    }
    __syncthreads();
    if (i >= Vh) return;
    const double *d = st + threadIdx.x * 24;
    // psi_NR = S psi_DR: NR0 = (DR0 + DR2)/sqrt2, NR1 = (DR1 + DR3)/sqrt2,
    //                    NR2 = (DR0 - DR2)/sqrt2, NR3 = (DR1 - DR3)/sqrt2
    R o[24];
#pragma unroll
    for (int k = 0; k < 12; ++k) {  // k runs over (spin in {0,1}) x colour x re/im
        const double up = d[k], lo = d[k + 12];
        o[k] = (R)((up + lo) * kInvSqrt2);
        o[k + 12] = (R)((up - lo) * kInvSqrt2);
    }
    SpinorIO<P>::store(dst, stride, i, o);
}

template <int P>
__global__ void __launch_bounds__(kXferThreads) k_spinor_export(int X, int Y, int Z, int Vh, long stride, int parity,
                                                                const void *__restrict__ src, double *__restrict__ dst) {
    using R = typename Prec<P>::R;
    __shared__ double st[kXferThreads * 24];
    __shared__ int lexs[kXferThreads];
    const int i0 = blockIdx.x * kXferThreads;
    const int i = i0 + threadIdx.x;
    const int nsite = min(kXferThreads, Vh - i0);
    if (i < Vh) {
        lexs[threadIdx.x] = cb_coord(i, parity, X, Y, Z).lex;
        R v[24];
        SpinorIO<P>::load(src, stride, i, v);
        double *d = st + threadIdx.x * 24;
#pragma unroll
        for (int k = 0; k < 12; ++k) {
            const double up = (double)v[k], lo = (double)v[k + 12];
            d[k] = (up + lo) * kInvSqrt2;
            d[k + 12] = (up - lo) * kInvSqrt2;
        }
    }
    __syncthreads();
    for (int q = threadIdx.x; q < nsite * 12; q += kXferThreads) {
        const int sidx = q / 12, ch = q - 12 * (q / 12);
        reinterpret_cast<double2 *>(dst + (size_t)lexs[sidx] * 24)[ch] =
            make_double2(st[sidx * 24 + 2 * ch], st[sidx * 24 + 2 * ch + 1]);
    }
}

template <int PD, int PS>
__global__ void k_spinor_convert(int Vh, long stride, void *__restrict__ dst, const void *__restrict__ src) {
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= Vh) return;
    typename Prec<PS>::R v[24];
    SpinorIO<PS>::load(src, stride, i, v);
    typename Prec<PD>::R o[24];
#pragma unroll
    for (int k = 0; k < 24; ++k) o[k] = (typename Prec<PD>::R)v[k];
    SpinorIO<PD>::store(dst, stride, i, o);
}

static inline int nblk(long n, int t) { return (int)((n + t - 1) / t); }

void launch_spinor_import(int prec, const Geom &g, int parity, const double *src, void *dst, cudaStream_t s) {
    const int T = kXferThreads;
    if (prec == 8) k_spinor_import<8><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    else if (prec == 4) k_spinor_import<4><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    else k_spinor_import<2><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    QX_CUDA(cudaGetLastError());
}
void launch_spinor_export(int prec, const Geom &g, int parity, const void *src, double *dst, cudaStream_t s) {
    const int T = kXferThreads;
    if (prec == 8) k_spinor_export<8><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    else if (prec == 4) k_spinor_export<4><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    else k_spinor_export<2><<<nblk(g.Vh, T), T, 0, s>>>(g.X, g.Y, g.Z, (int)g.Vh, g.stride, parity, src, dst);
    QX_CUDA(cudaGetLastError());
}
void launch_spinor_convert(int pd, int ps, const Geom &g, void *dst, const void *src, cudaStream_t s) {
    const int T = 128;
    const int b = nblk(g.Vh, T);
    const int n = (int)g.Vh;
#define QX_CV(A, B) \
    if (pd == A && ps == B) { k_spinor_convert<A, B><<<b, T, 0, s>>>(n, g.stride, dst, src); QX_CUDA(cudaGetLastError()); return; }
    QX_CV(8, 8) QX_CV(8, 4) QX_CV(8, 2) QX_CV(4, 8) QX_CV(4, 4) QX_CV(4, 2) QX_CV(2, 8) QX_CV(2, 4) QX_CV(2, 2)
#undef QX_CV
    throw Error(QUDAX_ERR_ARG, "convert: bad precision");
}

// ============================================================================ gauge
// ext: fp64 site-major AoS [Et][Ez][Ey][Ex][4][3][3] complex; E_mu = L_mu + 2 on split
// dimensions (ext index 0 = local -1, L_mu + 1 = local L_mu), else L_mu (periodic wrap in-kernel).
struct ExtGeom {
    int L[4], E[4], s[4];  // local extents, ext extents, 1 if split
};
static ExtGeom ext_geom(const Geom &g) {
    ExtGeom e;
    for (int m = 0; m < 4; ++m) {
        e.L[m] = g.L[m];
        e.s[m] = (g.split >> m) & 1;
        e.E[m] = g.L[m] + 2 * e.s[m];
    }
    return e;
}
// link U_mu at local coordinates c (each in [-1, L] on split dims, any integer elsewhere: wrapped)
__device__ __forceinline__ const double *ext_link(const double *ext, const ExtGeom &e, const int c[4], int mu) {
    long idx = 0;
    for (int d = 3; d >= 0; --d) {
        const int v = e.s[d] ? c[d] + 1 : ((c[d] % e.L[d]) + e.L[d]) % e.L[d];
        idx = idx * e.E[d] + v;
    }
    return ext + (idx * 4 + mu) * 18;
}

// host-order box [4][T][Z][Y][X][18] -> ext interior; one thread per (mu, site)
__global__ void k_ext_fill(ExtGeom e, const double *__restrict__ box, double *__restrict__ ext) {
    const long V = (long)e.L[0] * e.L[1] * e.L[2] * e.L[3];
    const long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (k >= 4 * V) return;
    const int mu = (int)(k / V);
    long lex = k % V;
    int c[4];
    for (int d = 0; d < 4; ++d) {
        c[d] = (int)(lex % e.L[d]);
        lex /= e.L[d];
    }
    const double *src = box + k * 18;
    double *dst = const_cast<double *>(ext_link(ext, e, c, mu));
#pragma unroll
    for (int j = 0; j < 18; ++j) dst[j] = src[j];
}

void launch_ext_fill(const Geom &g, const double *box, double *ext, cudaStream_t s) {
    const int T = 128;
    k_ext_fill<<<(int)((4 * g.V + T - 1) / T), T, 0, s>>>(ext_geom(g), box, ext);
    QX_CUDA(cudaGetLastError());
}

long ext_slice_doubles(const Geom &g, int mu) { return ext_sites(g) / ext_extent(g, mu) * 72; }

// the ext cross-section at ext index idx along mu (every ext index of the other dimensions,
// so the halos received along earlier dimensions travel on: corners) <-> contiguous buffer
__global__ void k_ext_slice(ExtGeom e, double *ext, int mu, int idx, double *buf, int to_buf) {
    long n = 72;
    for (int d = 0; d < 4; ++d)
        if (d != mu) n *= e.E[d];
    const long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (k >= n) return;
    const int j = (int)(k % 72);
    long r = k / 72;
    long site = 0, mul = 1;
    for (int d = 0; d < 4; ++d) {
        long v;
        if (d == mu) {
            v = idx;
        } else {
            v = r % e.E[d];
            r /= e.E[d];
        }
        site += v * mul;
        mul *= e.E[d];
    }
    double *p = ext + site * 72 + j;
    if (to_buf) buf[k] = *p;
    else *p = buf[k];
}

void launch_ext_slice(const Geom &g, double *ext, int mu, int e, double *buf, bool to_buf, cudaStream_t s) {
    const long n = ext_slice_doubles(g, mu);
    const int T = 256;
    k_ext_slice<<<(int)((n + T - 1) / T), T, 0, s>>>(ext_geom(g), ext, mu, e, buf, to_buf ? 1 : 0);
    QX_CUDA(cudaGetLastError());
}

template <int P, int RECON>
__device__ void encode_store_link(const double *l /*18*/, void *base, long stride, long i, int *bad) {
    double raw[18];
    int n = 0;
    if constexpr (RECON == 18) {
        for (int k = 0; k < 18; ++k) raw[n++] = l[k];
    } else if constexpr (RECON == 12) {
        for (int k = 0; k < 12; ++k) raw[n++] = l[k];
    } else {
        double th0 = atan2(l[1], l[0]);     // arg u00
        double th2 = atan2(l[13], l[12]);   // arg u20
        if constexpr (P == 2) {
            th0 /= 3.14159265358979323846;
            th2 /= 3.14159265358979323846;
        }
        raw[n++] = th0;
        raw[n++] = th2;
        raw[n++] = l[2]; raw[n++] = l[3];   // u01
        raw[n++] = l[4]; raw[n++] = l[5];   // u02
        raw[n++] = l[6]; raw[n++] = l[7];   // u10
        double nn = l[2] * l[2] + l[3] * l[3] + l[4] * l[4] + l[5] * l[5];
        if (nn < 1e-6) atomicAdd(bad, 1);
    }
    if constexpr (P == 8) {
        double2 *p = reinterpret_cast<double2 *>(base);
        for (int k = 0; k < RECON / 2; ++k) p[k * stride + i] = make_double2(raw[2 * k], raw[2 * k + 1]);
    } else if constexpr (P == 4) {
        float4 *p = reinterpret_cast<float4 *>(base);
        constexpr int NB = RECON / 4;
        for (int k = 0; k < NB; ++k)
            p[k * stride + i] = make_float4((float)raw[4 * k], (float)raw[4 * k + 1], (float)raw[4 * k + 2], (float)raw[4 * k + 3]);
        if constexpr (RECON % 4) {
            float2 *q = reinterpret_cast<float2 *>(reinterpret_cast<char *>(base) + (size_t)NB * 16 * stride);
            q[i] = make_float2((float)raw[RECON - 2], (float)raw[RECON - 1]);
        }
    } else {
        // HLink layout (core.cuh): RECON/8 uint4 regions, then uint2 (RECON%8 == 4), then uint32
        auto q16 = [](double v) { return (uint32_t)(uint16_t)h16_code(__double2int_rn(v * 32767.0)); };
        auto w2 = [&](int k) { return q16(raw[k]) | (q16(raw[k + 1]) << 16); };
        constexpr int N16 = RECON / 8;
        for (int k = 0; k < N16; ++k)
            reinterpret_cast<uint4 *>(mptr(base, (size_t)16 * k * stride))[i] = make_uint4(w2(8 * k), w2(8 * k + 2), w2(8 * k + 4), w2(8 * k + 6));
        size_t off = (size_t)16 * N16 * stride;
        if constexpr (RECON % 8 >= 4) {
            reinterpret_cast<uint2 *>(mptr(base, off))[i] = make_uint2(w2(8 * N16), w2(8 * N16 + 2));
            off += (size_t)8 * stride;
        }
        if constexpr (RECON % 4 == 2) reinterpret_cast<uint32_t *>(mptr(base, off))[i] = w2(RECON - 2);
    }
}

struct GaugeDst {
    void *d[4][2];
    void *ghost[4][2];
    long Fd[4], fsd[4];
};

// coordinates of face site f (parity q) of dimension mu at x_mu = xm: the inverse of
// dslash.cuh face_index (lexicographic over the other three coordinates, halved)
__device__ __forceinline__ void face_site(int mu, long f, int xm, int q, const int L[4], int c[4]) {
    c[mu] = xm;
    const int a = (mu == 0) ? 1 : 0;             // the fastest of the other dimensions (paired)
    const int b = (mu <= 1) ? 2 : 1, d = (mu <= 2) ? 3 : 2;
    const int ah = L[a] / 2;
    int ch = (int)(f % ah);
    long r = f / ah;
    c[b] = (int)(r % L[b]);
    c[d] = (int)(r / L[b]);
    c[a] = 2 * ch + ((q + xm + c[b] + c[d]) & 1);
}

template <int P, int RECON>
__global__ void k_gauge_pack(ExtGeom e, long Vh, long stride, const double *__restrict__ ext, GaugeDst dst, int *bad) {
    const long n_bulk = 8 * Vh;  // (mu, parity, i)
    long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (k < n_bulk) {
        const int mu = (int)(k / (2 * Vh));
        const int p = (int)((k / Vh) % 2);
        const int i = (int)(k % Vh);
        Coord c = cb_coord(i, p, e.L[0], e.L[1], e.L[2]);
        const int cc[4] = {c.x, c.y, c.z, c.t};
        encode_store_link<P, RECON>(ext_link(ext, e, cc, mu), dst.d[mu][p], stride, i, bad);
        return;
    }
    k -= n_bulk;
    // backward ghost links U_mu(x - mu) at local x_mu = -1 of every split dimension, per site
    // parity q, face layout
    for (int mu = 0; mu < 4; ++mu) {
        if (!e.s[mu]) continue;
        if (k < 2 * dst.Fd[mu]) {
            const int q = (int)(k / dst.Fd[mu]);
            const long f = k % dst.Fd[mu];
            int c[4];
            face_site(mu, f, -1, q, e.L, c);
            encode_store_link<P, RECON>(ext_link(ext, e, c, mu), dst.ghost[mu][q], dst.fsd[mu], f, bad);
            return;
        }
        k -= 2 * dst.Fd[mu];
    }
}

void launch_gauge_pack2(int prec, int recon, const Geom &g, const double *ext, void *const dst[4][2],
                        void *const ghost[4][2], int *bad, cudaStream_t s) {
    GaugeDst d;
    long n = 8 * g.Vh;
    for (int m = 0; m < 4; ++m) {
        for (int p = 0; p < 2; ++p) {
            d.d[m][p] = dst[m][p];
            d.ghost[m][p] = ghost[m][p];
        }
        d.Fd[m] = g.Fd[m];
        d.fsd[m] = g.fsd[m];
        if (g.split >> m & 1) n += 2 * g.Fd[m];
    }
    const int T = 128;
    const int b = nblk(n, T);
    const ExtGeom e = ext_geom(g);
#define QX_GP(PP, RR)                                                               \
    if (prec == PP && recon == RR) {                                                \
        k_gauge_pack<PP, RR><<<b, T, 0, s>>>(e, g.Vh, g.stride, ext, d, bad);       \
        QX_CUDA(cudaGetLastError());                                                \
        return;                                                                     \
    }
    QX_GP(8, 18) QX_GP(8, 12) QX_GP(8, 8) QX_GP(4, 18) QX_GP(4, 12) QX_GP(4, 8) QX_GP(2, 18) QX_GP(2, 12) QX_GP(2, 8)
#undef QX_GP
    throw Error(QUDAX_ERR_ARG, "gauge pack: bad precision/reconstruct");
}

// ============================================================================ clover
// DeGrand-Rossi gamma matrices (gamma_4 reproduces eq. (6) left side),
// entries (re, im).  Product's own copy, written from the convention, not shared.
__constant__ double c_gamma[4][4][4][2] = {
    {{{0, 0}, {0, 0}, {0, 0}, {0, 1}}, {{0, 0}, {0, 0}, {0, 1}, {0, 0}}, {{0, 0}, {0, -1}, {0, 0}, {0, 0}}, {{0, -1}, {0, 0}, {0, 0}, {0, 0}}},
    {{{0, 0}, {0, 0}, {0, 0}, {-1, 0}}, {{0, 0}, {0, 0}, {1, 0}, {0, 0}}, {{0, 0}, {1, 0}, {0, 0}, {0, 0}}, {{-1, 0}, {0, 0}, {0, 0}, {0, 0}}},
    {{{0, 0}, {0, 0}, {0, 1}, {0, 0}}, {{0, 0}, {0, 0}, {0, 0}, {0, -1}}, {{0, -1}, {0, 0}, {0, 0}, {0, 0}}, {{0, 0}, {0, 1}, {0, 0}, {0, 0}}},
    {{{0, 0}, {0, 0}, {1, 0}, {0, 0}}, {{0, 0}, {0, 0}, {0, 0}, {1, 0}}, {{1, 0}, {0, 0}, {0, 0}, {0, 0}}, {{0, 0}, {1, 0}, {0, 0}, {0, 0}}},
};

using Cd = Cx<double>;
struct M3 {
    Cd m[3][3];
};
__device__ __forceinline__ M3 load_m3(const double *l) {
    M3 r;
    for (int a = 0; a < 3; ++a)
        for (int b = 0; b < 3; ++b) r.m[a][b] = cx(l[(a * 3 + b) * 2], l[(a * 3 + b) * 2 + 1]);
    return r;
}
__device__ __forceinline__ M3 mul(const M3 &A, const M3 &B) {
    M3 r;
    for (int a = 0; a < 3; ++a)
        for (int b = 0; b < 3; ++b) r.m[a][b] = A.m[a][0] * B.m[0][b] + A.m[a][1] * B.m[1][b] + A.m[a][2] * B.m[2][b];
    return r;
}
__device__ __forceinline__ M3 dagm(const M3 &A) {
    M3 r;
    for (int a = 0; a < 3; ++a)
        for (int b = 0; b < 3; ++b) r.m[a][b] = conj(A.m[b][a]);
    return r;
}

// Gauss-Jordan inversion of a 6x6 complex matrix with partial pivoting; returns 0 if singular
__device__ int invert6(Cd a[6][6], Cd inv[6][6]) {
    for (int i = 0; i < 6; ++i)
        for (int j = 0; j < 6; ++j) inv[i][j] = cx(i == j ? 1.0 : 0.0, 0.0);
    for (int c = 0; c < 6; ++c) {
        int piv = c;
        double best = norm2(a[c][c]);
        for (int r = c + 1; r < 6; ++r)
            if (norm2(a[r][c]) > best) { best = norm2(a[r][c]); piv = r; }
        if (best < 1e-300) return 0;
        if (piv != c)
            for (int j = 0; j < 6; ++j) {
                Cd t = a[c][j]; a[c][j] = a[piv][j]; a[piv][j] = t;
                t = inv[c][j]; inv[c][j] = inv[piv][j]; inv[piv][j] = t;
            }
        const double dn = 1.0 / norm2(a[c][c]);
        const Cd ip = cx(a[c][c].r * dn, -a[c][c].i * dn);
        for (int j = 0; j < 6; ++j) { a[c][j] = ip * a[c][j]; inv[c][j] = ip * inv[c][j]; }
        for (int r = 0; r < 6; ++r) {
            if (r == c) continue;
            const Cd f = a[r][c];
            for (int j = 0; j < 6; ++j) { a[r][j] = a[r][j] - f * a[c][j]; inv[r][j] = inv[r][j] - f * inv[c][j]; }
        }
    }
    return 1;
}

// store Hermitian 6x6 (halved) as d[6], lower-triangle L[15] (re, im)
__device__ void store_herm6_half(const Cd m[6][6], double *out) {
    for (int i = 0; i < 6; ++i) out[i] = 0.5 * m[i][i].r;
    for (int i = 1; i < 6; ++i)
        for (int j = 0; j < i; ++j) {
            const int k = i * (i - 1) / 2 + j;
            // symmetrise against rounding: average of m[i][j] and conj(m[j][i])
            out[6 + 2 * k] = 0.25 * (m[i][j].r + m[j][i].r);
            out[6 + 2 * k + 1] = 0.25 * (m[i][j].i - m[j][i].i);
        }
}

// one thread per local site (both parities); T[p], Tinv[p]: fp64 [Vh][72]
__global__ void k_clover_build(ExtGeom e, double kappa, double csw, const double *__restrict__ ext,
                               double *T0, double *T1, double *I0, double *I1, int *bad) {
    const int X = e.L[0], Y = e.L[1];
    const long Vs = (long)X * Y * e.L[2];
    const long V = Vs * e.L[3];
    const long lexl = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (lexl >= V) return;
    int c[4];
    c[0] = (int)(lexl % X);
    c[1] = (int)((lexl / X) % Y);
    c[2] = (int)((lexl / ((long)X * Y)) % e.L[2]);
    c[3] = (int)(lexl / Vs);
    const int parity = (c[0] + c[1] + c[2] + c[3]) & 1;
    const long cb = lexl >> 1;
    // link U_mu at (site + shifts): halo of split dimensions, periodic wrap of the others
    auto L = [&](int mu, int dm, int dmv, int nu, int dn) -> M3 {
        int s[4] = {c[0], c[1], c[2], c[3]};
        s[dmv] += dm;
        s[nu] += dn;
        return load_m3(ext_link(ext, e, s, mu));
    };
    // block-diagonal chiral pieces of sum_{mu<nu} gamma_mu gamma_nu (x) F_munu
    Cd Bup[6][6], Blo[6][6];
    for (int i = 0; i < 6; ++i)
        for (int j = 0; j < 6; ++j) { Bup[i][j] = cx(0.0, 0.0); Blo[i][j] = cx(0.0, 0.0); }
    for (int mu = 0; mu < 4; ++mu)
        for (int nu = mu + 1; nu < 4; ++nu) {
            // leaves (counter-clockwise in the mu-nu plane, starting and ending at x)
            M3 l1 = mul(mul(mul(L(mu, 0, mu, nu, 0), L(nu, 1, mu, nu, 0)), dagm(L(mu, 0, mu, nu, 1))), dagm(L(nu, 0, mu, nu, 0)));
            M3 l2 = mul(mul(mul(L(nu, 0, mu, nu, 0), dagm(L(mu, -1, mu, nu, 1))), dagm(L(nu, -1, mu, nu, 0))), L(mu, -1, mu, nu, 0));
            M3 l3 = mul(mul(mul(dagm(L(mu, -1, mu, nu, 0)), dagm(L(nu, -1, mu, nu, -1))), L(mu, -1, mu, nu, -1)), L(nu, 0, mu, nu, -1));
            M3 l4 = mul(mul(mul(dagm(L(nu, 0, mu, nu, -1)), L(mu, 0, mu, nu, -1)), L(nu, 1, mu, nu, -1)), dagm(L(mu, 0, mu, nu, 0)));
            Cd F[3][3];
            for (int a = 0; a < 3; ++a)
                for (int b = 0; b < 3; ++b) {
                    Cd q = l1.m[a][b] + l2.m[a][b] + l3.m[a][b] + l4.m[a][b];
                    Cd qd = conj(l1.m[b][a] + l2.m[b][a] + l3.m[b][a] + l4.m[b][a]);
                    F[a][b] = 0.125 * (q - qd);
                }
            // gamma_mu gamma_nu
            Cd gg[4][4];
            for (int r = 0; r < 4; ++r)
                for (int s = 0; s < 4; ++s) {
                    Cd v = cx(0.0, 0.0);
                    for (int k = 0; k < 4; ++k)
                        v = v + cx(c_gamma[mu][r][k][0], c_gamma[mu][r][k][1]) * cx(c_gamma[nu][k][s][0], c_gamma[nu][k][s][1]);
                    gg[r][s] = v;
                }
            for (int r = 0; r < 2; ++r)
                for (int s = 0; s < 2; ++s)
                    for (int a = 0; a < 3; ++a)
                        for (int b = 0; b < 3; ++b) {
                            Bup[r * 3 + a][s * 3 + b] = Bup[r * 3 + a][s * 3 + b] + gg[r][s] * F[a][b];
                            Blo[r * 3 + a][s * 3 + b] = Blo[r * 3 + a][s * 3 + b] + gg[r + 2][s + 2] * F[a][b];
                        }
        }
    // T = 1 + 2 kappa A, A = -(csw/2) sum gamma gamma F  ->  T = 1 - kappa csw sum(...)
    const double coef = -kappa * csw;
    for (int i = 0; i < 6; ++i)
        for (int j = 0; j < 6; ++j) {
            Bup[i][j] = coef * Bup[i][j];
            Blo[i][j] = coef * Blo[i][j];
            if (i == j) {
                Bup[i][j].r += 1.0;
                Blo[i][j].r += 1.0;
            }
        }
    double *To = parity ? T1 : T0;
    double *Io = parity ? I1 : I0;
    store_herm6_half(Bup, To + cb * 72);
    store_herm6_half(Blo, To + cb * 72 + 36);
    Cd inv[6][6];
    if (!invert6(Bup, inv)) atomicAdd(bad, 1);
    store_herm6_half(inv, Io + cb * 72);
    if (!invert6(Blo, inv)) atomicAdd(bad, 1);
    store_herm6_half(inv, Io + cb * 72 + 36);
}

void launch_clover_build(const Geom &g, const double *ext, double kappa, double csw, double *T[2], double *Tinv[2],
                         int *bad, cudaStream_t s) {
    const int TB = 64;
    k_clover_build<<<nblk(g.V, TB), TB, 0, s>>>(ext_geom(g), kappa, csw, ext, T[0], T[1], Tinv[0], Tinv[1], bad);
    QX_CUDA(cudaGetLastError());
}

// fp64 AoS [Vh][72] -> SoA in prec (half: per-chiral-block float norms)
template <int P>
__global__ void k_clover_pack(long Vh, long stride, const double *__restrict__ src, void *__restrict__ dst) {
    const long i = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= Vh) return;
    const double *s = src + i * 72;
    if constexpr (P == 8) {
        double2 *p = reinterpret_cast<double2 *>(dst);
        for (int k = 0; k < 36; ++k) p[k * stride + i] = make_double2(s[2 * k], s[2 * k + 1]);
    } else if constexpr (P == 4) {
        float4 *p = reinterpret_cast<float4 *>(dst);
        for (int k = 0; k < 18; ++k)
            p[k * stride + i] = make_float4((float)s[4 * k], (float)s[4 * k + 1], (float)s[4 * k + 2], (float)s[4 * k + 3]);
    } else {
        // 9 uint4 regions of 8 reals; C+ = reals 0..35 (scale n.x), C- = 36..71 (scale n.y)
        float2 *nrm = reinterpret_cast<float2 *>(mptr(dst, (size_t)144 * stride));
        float n[2], inv[2];
        for (int b = 0; b < 2; ++b) {
            double m = 0;
            for (int k = 0; k < 36; ++k) m = fmax(m, fabs(s[36 * b + k]));
            n[b] = (float)m;
            inv[b] = m > 0 ? kHalfMax / (float)m : 0.f;
        }
        auto q16 = [&](int k) {
            return (uint32_t)(uint16_t)h16_code(__float2int_rn((float)s[k] * inv[k >= 36 ? 1 : 0]));
        };
        auto w2 = [&](int k) { return q16(k) | (q16(k + 1) << 16); };
        for (int r = 0; r < 9; ++r)
            reinterpret_cast<uint4 *>(mptr(dst, (size_t)16 * r * stride))[i] =
                make_uint4(w2(8 * r), w2(8 * r + 2), w2(8 * r + 4), w2(8 * r + 6));
        nrm[i] = make_float2(n[0], n[1]);
    }
}

void launch_clover_pack(int prec, const Geom &g, const double *src, void *dst, cudaStream_t s) {
    const int T = 128;
    if (prec == 8) k_clover_pack<8><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, src, dst);
    else if (prec == 4) k_clover_pack<4><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, src, dst);
    else k_clover_pack<2><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, src, dst);
    QX_CUDA(cudaGetLastError());
}

// site-local clover multiply out = C in (C = T or T^{-1} of the field's parity)
template <int P>
__global__ void k_clover_apply(long Vh, long stride, const void *__restrict__ cl, const void *__restrict__ in,
                               void *__restrict__ out) {
    using R = typename Prec<P>::R;
    const long i = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= Vh) return;
    R v[24];
    SpinorIO<P>::load(in, stride, i, v);
    Cx<R> ps[4][3], o[4][3];
    unpack_spinor(v, ps);
    apply_clover<P>(cl, stride, i, ps, o);
    for (int s = 0; s < 4; ++s)
        for (int c = 0; c < 3; ++c) {
            v[(s * 3 + c) * 2] = o[s][c].r;
            v[(s * 3 + c) * 2 + 1] = o[s][c].i;
        }
    SpinorIO<P>::store(out, stride, i, v);
}

void launch_clover_apply(int prec, const Geom &g, const void *cl, const void *in, void *out, cudaStream_t s) {
    const int T = 128;
    if (prec == 8) k_clover_apply<8><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, cl, in, out);
    else if (prec == 4) k_clover_apply<4><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, cl, in, out);
    else k_clover_apply<2><<<nblk(g.Vh, T), T, 0, s>>>(g.Vh, g.stride, cl, in, out);
    QX_CUDA(cudaGetLastError());
}

// ============================================================================ faces
// Raw copy of one 12-real half (3 float4 / 6 double2 / one H12 record + the site norm): bits only,
// so a partitioned Dslash reads exactly what the unpartitioned one reads.
template <int P>
__device__ __forceinline__ void k_pack_faces_body(long F, long T_loc, long stride, long fstride, int half_back,
                                                  int half_fwd, const void *__restrict__ in, void *__restrict__ sb,
                                                  void *__restrict__ sf) {
    long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (k >= 2 * F) return;
    const bool fwd = k >= F;
    const long f = fwd ? k - F : k;
    const long i = fwd ? (T_loc - 1) * F + f : f;
    void *dst = fwd ? sf : sb;
    const int half = fwd ? half_fwd : half_back;
    if constexpr (P == 8) {
        const double2 *s = reinterpret_cast<const double2 *>(in);
        double2 *d = reinterpret_cast<double2 *>(dst);
        for (int b = 0; b < 6; ++b) d[b * fstride + f] = s[(6 * half + b) * stride + i];
    } else if constexpr (P == 4) {
        const float4 *s = reinterpret_cast<const float4 *>(in);
        float4 *d = reinterpret_cast<float4 *>(dst);
        for (int b = 0; b < 3; ++b) d[b * fstride + f] = s[(3 * half + b) * stride + i];
    } else {
        reinterpret_cast<uint4 *>(dst)[f] = reinterpret_cast<const uint4 *>(cptr(in, h_spinor_u(stride, half)))[i];
        reinterpret_cast<uint2 *>(mptr(dst, (size_t)16 * fstride))[f] =
            reinterpret_cast<const uint2 *>(cptr(in, h_spinor_v(stride, half)))[i];
        FaceIO<2>::norms(dst, fstride)[f] = SpinorIO<2>::norms(in, stride)[i];
    }
}
template <int P>
__global__ void k_pack_faces(long F, long T_loc, long stride, long fstride, int half_back, int half_fwd,
                             const void *__restrict__ in, void *__restrict__ sb, void *__restrict__ sf) {
    k_pack_faces_body<P>(F, T_loc, stride, fstride, half_back, half_fwd, in, sb, sf);
}

// system-scope release store of a flag (the kernel-initiated halo's sequence numbers): each CTA's
// ghost stores are ordered before its arrival on the pack counter by bar.sync + one system-scope
// fence (cumulative, as in a grid barrier), and the last CTA's fence + release orders all of
// them before the flags
__device__ __forceinline__ void st_release_sys(unsigned *p, unsigned v) {
    asm volatile("st.release.sys.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// Faces of the partitioned X / Y / Z: the x_mu = 0 face goes backward and
// feeds the receiver's FORWARD hop, so it is projected with (1 + SF gamma_mu); the x_mu = L-1
// face goes forward and feeds the backward hop (1 + SB gamma_mu).  Projection by the Dslash's
// own spatial_project on the values the Dslash would decode: the receiver finishes the hop
// bit-identically to the unpartitioned kernel.  Half precision ships the raw 16-bit record and
// its norm instead (52 B per site vs 48 B projected in fp32); the receiver projects it
// (dslash.cuh ghost_half) — measured: a projected half face differed from the unsplit kernel
// by one half-precision quantum on ~4% of the Y-face sites.  X faces are raw in every precision:
// the receiver reads them through the ordinary hop with a per-lane pointer select (x = 0 and
// x = X-1 sites sit in every warp, so a separate ghost branch would diverge everywhere).
struct SPackArgs {
    int L[4];
    int mask;       // split spatial dims
    int q;          // parity of the packed (input) field
    long Fd[3], fsd[3], stride;
    void *sb[3], *sf[3];
};
// one face site of a partitioned X / Y / Z (face index f of dimension mu, fwd: the x_mu = L-1
// face) -> dst (face layout, fs padded sites)
template <int P, bool DAG>
__device__ __forceinline__ void pack_spatial_one(int mu, long f, bool fwd, const int L[4], int q, long stride,
                                                 const void *__restrict__ in, void *dst, long fs) {
    using R = typename Prec<P>::R;
    int c[4];
    face_site(mu, f, fwd ? L[mu] - 1 : 0, q, L, c);
    const long i = (((long)(c[3] * L[2] + c[2]) * L[1] + c[1]) * L[0] + c[0]) >> 1;
    if (sface_raw(P, mu)) {  // the raw record (+ half norm): bits only, the receiver projects
        if constexpr (P == 2) {
            for (int hf = 0; hf < 2; ++hf) {
                reinterpret_cast<uint4 *>(mptr(dst, h_spinor_u(fs, hf)))[f] =
                    reinterpret_cast<const uint4 *>(cptr(in, h_spinor_u(stride, hf)))[i];
                reinterpret_cast<uint2 *>(mptr(dst, h_spinor_v(fs, hf)))[f] =
                    reinterpret_cast<const uint2 *>(cptr(in, h_spinor_v(stride, hf)))[i];
            }
            SpinorIO<2>::norms(dst, fs)[f] = SpinorIO<2>::norms(in, stride)[i];
        } else {
            using V = typename StoreVec<P>::V;
            constexpr int NB = (P == 8) ? 12 : 6;
            for (int b = 0; b < NB; ++b)
                reinterpret_cast<V *>(dst)[b * fs + f] = reinterpret_cast<const V *>(in)[b * stride + i];
        }
        return;
    }
    RawVec<P, 24> raw;
    raw.template load_spinor<0>(in, stride, i);
    R v[24];
    Cx<R> ps[4][3], h0[3], h1[3];
    raw.decode(v);
    unpack_spinor(v, ps);
    constexpr int SF = DAG ? +1 : -1, SB = -SF;
    if (mu == 0) {
        if (fwd) spatial_project<0, SB>(ps, h0, h1); else spatial_project<0, SF>(ps, h0, h1);
    } else if (mu == 1) {
        if (fwd) spatial_project<1, SB>(ps, h0, h1); else spatial_project<1, SF>(ps, h0, h1);
    } else {
        if (fwd) spatial_project<2, SB>(ps, h0, h1); else spatial_project<2, SF>(ps, h0, h1);
    }
    SFace<R>::store(dst, fs, f, h0, h1);
}

template <int P, bool DAG>
__global__ void k_pack_spatial(const __grid_constant__ SPackArgs a, const void *__restrict__ in) {
    long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    int mu = 0;
    for (; mu < 3; ++mu) {
        if (!(a.mask >> mu & 1)) continue;
        if (k < 2 * a.Fd[mu]) break;
        k -= 2 * a.Fd[mu];
    }
    if (mu == 3) return;
    const bool fwd = k >= a.Fd[mu];
    const long f = fwd ? k - a.Fd[mu] : k;
    pack_spatial_one<P, DAG>(mu, f, fwd, a.L, a.q, a.stride, in, fwd ? a.sf[mu] : a.sb[mu], a.fsd[mu]);
}

// Kernel-initiated halo of a general process grid (QUDAX_HALO_P2P): every
// split dimension's two faces (T: the diagonal-projector halves, bits only; X / Y / Z: as
// k_pack_spatial) stored straight into the neighbours' ghost buffers (peer memory), then the
// last CTA raises, in each neighbour, the flag of the ghost it filled (system-scope release of
// the sequence number).  One launch for all dimensions: one producer counter.
template <int P, bool DAG>
__global__ void k_pack_p2p(const __grid_constant__ P2PPackArgs a, const void *__restrict__ in) {
    __shared__ bool last;
    const unsigned s = *reinterpret_cast<volatile unsigned *>(a.seq) + 1u;
    const bool odd = (s & 1u) != 0;
    long k = (long)blockIdx.x * blockDim.x + threadIdx.x;
    int mu = 0;
    for (; mu < 4; ++mu) {
        if (!(a.mask >> mu & 1)) continue;
        if (k < 2 * a.Fd[mu]) break;
        k -= 2 * a.Fd[mu];
    }
    if (mu < 4) {
        const bool fwd = k >= a.Fd[mu];
        const long f = fwd ? k - a.Fd[mu] : k;
        char *dst = (fwd ? a.dst_f[mu] : a.dst_b[mu]) + (odd ? a.pdist[mu] : 0);
        if (mu == 3) {
            const long i = fwd ? (a.L[3] - 1) * a.Fd[3] + f : f;
            const int half = fwd ? a.half_fwd : a.half_back;
            if constexpr (P == 8) {
                const double2 *sp = reinterpret_cast<const double2 *>(in);
                double2 *d = reinterpret_cast<double2 *>(dst);
                for (int b = 0; b < 6; ++b) d[b * a.fsd[3] + f] = sp[(6 * half + b) * a.stride + i];
            } else if constexpr (P == 4) {
                const float4 *sp = reinterpret_cast<const float4 *>(in);
                float4 *d = reinterpret_cast<float4 *>(dst);
                for (int b = 0; b < 3; ++b) d[b * a.fsd[3] + f] = sp[(3 * half + b) * a.stride + i];
            } else {
                reinterpret_cast<uint4 *>(dst)[f] = reinterpret_cast<const uint4 *>(cptr(in, h_spinor_u(a.stride, half)))[i];
                reinterpret_cast<uint2 *>(mptr(dst, (size_t)16 * a.fsd[3]))[f] =
                    reinterpret_cast<const uint2 *>(cptr(in, h_spinor_v(a.stride, half)))[i];
                FaceIO<2>::norms(dst, a.fsd[3])[f] = SpinorIO<2>::norms(in, a.stride)[i];
            }
        } else {
            pack_spatial_one<P, DAG>(mu, f, fwd, a.L, a.q, a.stride, in, dst, a.fsd[mu]);
        }
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence_system();
        last = (atomicAdd(a.count, 1u) == gridDim.x - 1);
    }
    __syncthreads();
    if (last && threadIdx.x == 0) {
        *a.count = 0u;
        *a.seq = s;
        __threadfence_system();
        for (int m = 0; m < 4; ++m) {
            if (!(a.mask >> m & 1)) continue;
            st_release_sys(a.flag_b[m], s);  // the backward neighbour's "forward ghost filled"
            st_release_sys(a.flag_f[m], s);  // the forward neighbour's "backward ghost filled"
        }
    }
}

void launch_pack_p2p(int prec, int dagger, const P2PPackArgs &a, const void *in, cudaStream_t s) {
    long n = 0;
    for (int m = 0; m < 4; ++m)
        if (a.mask >> m & 1) n += 2 * a.Fd[m];
    const int T = 128;
    const int b = n > 0 ? nblk(n, T) : 1;
#define QX_PP2(PP)                                                                  \
    if (prec == PP) {                                                               \
        if (dagger) k_pack_p2p<PP, true><<<b, T, 0, s>>>(a, in);                     \
        else k_pack_p2p<PP, false><<<b, T, 0, s>>>(a, in);                           \
        QX_CUDA(cudaGetLastError());                                                 \
        return;                                                                      \
    }
    QX_PP2(8) QX_PP2(4) QX_PP2(2)
#undef QX_PP2
    throw Error(QUDAX_ERR_ARG, "pack p2p: bad precision");
}

size_t sface_bytes(int prec, int mu, long fs) { return sface_raw(prec, mu) ? spinor_bytes(prec, fs) : (size_t)12 * prec * fs; }

void launch_pack_spatial(int prec, int dagger, const Geom &g, int in_parity, const void *in, void *const sb[3],
                         void *const sf[3], cudaStream_t s) {
    SPackArgs a{};
    long n = 0;
    for (int m = 0; m < 4; ++m) a.L[m] = g.L[m];
    a.mask = spatial_split(g);
    a.q = in_parity;
    a.stride = g.stride;
    for (int m = 0; m < 3; ++m) {
        a.Fd[m] = g.Fd[m];
        a.fsd[m] = g.fsd[m];
        a.sb[m] = sb[m];
        a.sf[m] = sf[m];
        if (a.mask >> m & 1) n += 2 * g.Fd[m];
    }
    if (!n) return;
    const int T = 128;
    const int b = nblk(n, T);
#define QX_PS(PP)                                                                  \
    if (prec == PP) {                                                              \
        if (dagger) k_pack_spatial<PP, true><<<b, T, 0, s>>>(a, in);               \
        else k_pack_spatial<PP, false><<<b, T, 0, s>>>(a, in);                     \
        QX_CUDA(cudaGetLastError());                                               \
        return;                                                                    \
    }
    QX_PS(8) QX_PS(4) QX_PS(2)
#undef QX_PS
    throw Error(QUDAX_ERR_ARG, "pack spatial: bad precision");
}

void launch_pack_faces(int prec, int dagger, const Geom &g, const void *in, void *send_back, void *send_fwd,
                       cudaStream_t s) {
    // non-dagger: the receiver's forward hop (1 - gamma_4) needs LOWER spins of our t=0 slice
    // (sent backward); its backward hop (1 + gamma_4) needs UPPER spins of our t=T_loc-1 slice
    // (sent forward).  The dagger swaps the halves (reading Q15).
    const int half_back = dagger ? 0 : 1;
    const int half_fwd = dagger ? 1 : 0;
    const int T = 128;
    const int b = nblk(2 * g.F, T);
    if (prec == 8) k_pack_faces<8><<<b, T, 0, s>>>(g.F, g.T_loc, g.stride, g.fstride, half_back, half_fwd, in, send_back, send_fwd);
    else if (prec == 4) k_pack_faces<4><<<b, T, 0, s>>>(g.F, g.T_loc, g.stride, g.fstride, half_back, half_fwd, in, send_back, send_fwd);
    else k_pack_faces<2><<<b, T, 0, s>>>(g.F, g.T_loc, g.stride, g.fstride, half_back, half_fwd, in, send_back, send_fwd);
    QX_CUDA(cudaGetLastError());
}

}  // namespace qx
