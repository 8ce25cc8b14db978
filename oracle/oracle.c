/*
 * oracle.c — TEST INFRASTRUCTURE ONLY.  A plain, slow, obviously-correct fp64 CPU
 * implementation of the Wilson-clover operator of arXiv:1011.0024, used to
 * check the CUDA path.  Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference leg may load it.  It shares no code, header, table or constant with
 * paper_1011_0024_b200/ (the product) and never imports it.
 *
 * Conventions (all readings listed in DESIGN.md §Readings):
 *   - site index lex = ((t*Z + z)*Y + y)*X + x, x fastest; dims = {X, Y, Z, T}
 *   - spinor psi[lex][spin][colour] complex double, DeGrand-Rossi chiral basis
 *   - gauge  U[mu][lex][row][col] complex double, mu = 0..3 <-> x, y, z, t
 *   - 12x12 site matrices M[lex][s*3+a][s'*3+b]
 *
 * No projection tricks, no basis change, no link compression, no even-odd layout:
 * full 4x4 gamma matrices times full 3x3 links, exactly as eq. (2) is written.
 *
 * Functions and the passages they follow:
 *   oracle_gamma        gamma_mu in the DeGrand-Rossi basis (eq. (6) left side,
 *                       P:484-490, fixes 1 +/- gamma_4)
 *   oracle_dslash       D of eq. (2), P:152-162:
 *                         (D psi)(x) = sum_mu [ P^{-mu} U_mu(x) psi(x+mu)
 *                                              + P^{+mu} U_mu(x-mu)^dag psi(x-mu) ]
 *                       with P^{+-mu} = 1 +- gamma_mu; dagger=1 gives the explicit
 *                       adjoint D^dag (hops with 1+gamma forward, 1-gamma backward).
 *                       Temporal hops crossing the GLOBAL boundary carry t_bc
 *                       ("boundary conditions"; reading Q5).
 *   oracle_clover       A_x of eq. (2) (footnote 1 P:183-184), read as the
 *                       Sheikholeslami-Wohlert term [6]: four-leaf
 *                       F_munu = (Q_munu - Q_munu^dag)/8,
 *                       A = -(csw/2) sum_{mu<nu} gamma_mu gamma_nu (x) F_munu,
 *                       returned as T = 1 + 2 kappa A (reading Q1, Q4).
 *   oracle_invert12     T^{-1}: 12x12 complex Gauss-Jordan with partial pivoting.
 *   oracle_site_mult    out(x) = M(x) in(x).
 */
#include <complex.h>
#include <math.h>
#include <stdlib.h>
#include <string.h>

typedef double complex cplx;

/* DeGrand-Rossi gamma matrices, gamma[mu][row][col], mu = 0..3 (x, y, z, t). */
static const cplx GAMMA[4][4][4] = {
    {{0, 0, 0, I}, {0, 0, I, 0}, {0, -I, 0, 0}, {-I, 0, 0, 0}},
    {{0, 0, 0, -1}, {0, 0, 1, 0}, {0, 1, 0, 0}, {-1, 0, 0, 0}},
    {{0, 0, I, 0}, {0, 0, 0, -I}, {-I, 0, 0, 0}, {0, I, 0, 0}},
    {{0, 0, 1, 0}, {0, 0, 0, 1}, {1, 0, 0, 0}, {0, 1, 0, 0}},
};

void oracle_gamma(int mu, double *out /* [4][4][2] */) {
    for (int r = 0; r < 4; ++r)
        for (int c = 0; c < 4; ++c) {
            out[(r * 4 + c) * 2] = creal(GAMMA[mu][r][c]);
            out[(r * 4 + c) * 2 + 1] = cimag(GAMMA[mu][r][c]);
        }
}

static inline long lex_of(long x, long y, long z, long t, const int d[4]) {
    return ((t * d[2] + z) * d[1] + y) * d[0] + x;
}

/* neighbour of site (c[0..3]) in direction mu, step +-1, periodic on the given array. */
static inline long neighbour(const long c[4], int mu, int step, const int d[4]) {
    long n[4] = {c[0], c[1], c[2], c[3]};
    n[mu] = (n[mu] + step + d[mu]) % d[mu];
    return lex_of(n[0], n[1], n[2], n[3], d);
}

/*
 * out = D in  (dagger = 0)   or   out = D^dag in  (dagger = 1), every site of the array.
 * The array is treated as periodic in all four directions.  t_global_offset / T_global
 * place the array on the global lattice (array timeslice t is global timeslice
 * (t + t_global_offset) mod T_global) so that the boundary factor t_bc is applied to the
 * forward hop out of global t = T_global-1 and the backward hop out of global t = 0.
 * For the plain global lattice: t_global_offset = 0, T_global = dims[3].
 */
/* (D in)(x) or (D^dag in)(x) at the single site s, written to out[12] */
static void dslash_one(cplx *out, long s, const cplx *U, const cplx *in, const int dims[4], long V, double t_bc,
                       int dagger, int t_global_offset, int T_global) {
    /* non-dagger: forward hop (x+mu) uses (1 - gamma_mu), backward (x-mu) uses (1 + gamma_mu);
       the explicit adjoint swaps them. */
    const double sf = dagger ? +1.0 : -1.0;
    const double sb = -sf;
    {
        long c[4];
        c[0] = s % dims[0];
        c[1] = (s / dims[0]) % dims[1];
        c[2] = (s / ((long)dims[0] * dims[1])) % dims[2];
        c[3] = s / ((long)dims[0] * dims[1] * dims[2]);
        long tg = ((c[3] + t_global_offset) % T_global + T_global) % T_global;
        cplx acc[4][3];
        memset(acc, 0, sizeof(acc));
        for (int mu = 0; mu < 4; ++mu) {
            /* forward: P U_mu(x) psi(x+mu) */
            {
                long xf = neighbour(c, mu, +1, dims);
                double bc = (mu == 3 && tg == T_global - 1) ? t_bc : 1.0;
                const cplx *u = U + ((long)mu * V + s) * 9;
                const cplx *p = in + xf * 12;
                cplx chi[4][3];
                for (int sp = 0; sp < 4; ++sp)
                    for (int a = 0; a < 3; ++a) {
                        cplx v = 0;
                        for (int b = 0; b < 3; ++b) v += u[a * 3 + b] * p[sp * 3 + b];
                        chi[sp][a] = bc * v;
                    }
                for (int r = 0; r < 4; ++r)
                    for (int a = 0; a < 3; ++a) {
                        cplx v = chi[r][a];
                        for (int k = 0; k < 4; ++k) v += sf * GAMMA[mu][r][k] * chi[k][a];
                        acc[r][a] += v;
                    }
            }
            /* backward: P U_mu(x-mu)^dag psi(x-mu) */
            {
                long xb = neighbour(c, mu, -1, dims);
                double bc = (mu == 3 && tg == 0) ? t_bc : 1.0;
                const cplx *u = U + ((long)mu * V + xb) * 9;
                const cplx *p = in + xb * 12;
                cplx chi[4][3];
                for (int sp = 0; sp < 4; ++sp)
                    for (int a = 0; a < 3; ++a) {
                        cplx v = 0;
                        for (int b = 0; b < 3; ++b) v += conj(u[b * 3 + a]) * p[sp * 3 + b];
                        chi[sp][a] = bc * v;
                    }
                for (int r = 0; r < 4; ++r)
                    for (int a = 0; a < 3; ++a) {
                        cplx v = chi[r][a];
                        for (int k = 0; k < 4; ++k) v += sb * GAMMA[mu][r][k] * chi[k][a];
                        acc[r][a] += v;
                    }
            }
        }
        memcpy(out, acc, sizeof(acc));
    }
}

void oracle_dslash(double *out_, const double *U_, const double *in_, const int dims[4],
                   double t_bc, int dagger, int t_global_offset, int T_global) {
    cplx *out = (cplx *)out_;
    const long V = (long)dims[0] * dims[1] * dims[2] * dims[3];
#pragma omp parallel for schedule(static)
    for (long s = 0; s < V; ++s)
        dslash_one(out + s * 12, s, (const cplx *)U_, (const cplx *)in_, dims, V, t_bc, dagger, t_global_offset,
                   T_global);
}

/* The same operator evaluated only at the listed sites: out[k] = (D in)(sites[k]).  Used to
 * check full-size GPU results on a sample of output sites. */
void oracle_dslash_sites(double *out_, const double *U_, const double *in_, const int dims[4], double t_bc,
                         int dagger, const long *sites, long nsites) {
    cplx *out = (cplx *)out_;
    const long V = (long)dims[0] * dims[1] * dims[2] * dims[3];
#pragma omp parallel for schedule(static)
    for (long k = 0; k < nsites; ++k)
        dslash_one(out + k * 12, sites[k], (const cplx *)U_, (const cplx *)in_, dims, V, t_bc, dagger, 0, dims[3]);
}

/* 3x3 helpers */
static void mm(cplx r[9], const cplx a[9], const cplx b[9]) {
    for (int i = 0; i < 3; ++i)
        for (int j = 0; j < 3; ++j) {
            cplx v = 0;
            for (int k = 0; k < 3; ++k) v += a[i * 3 + k] * b[k * 3 + j];
            r[i * 3 + j] = v;
        }
}
static void dag(cplx r[9], const cplx a[9]) {
    for (int i = 0; i < 3; ++i)
        for (int j = 0; j < 3; ++j) r[i * 3 + j] = conj(a[j * 3 + i]);
}
static const cplx *link(const cplx *U, int mu, long site, long V) { return U + ((long)mu * V + site) * 9; }

/* site offset by (dmu along mu) and (dnu along nu) */
static long shift2(const long c[4], int mu, int dmu, int nu, int dnu, const int d[4]) {
    long n[4] = {c[0], c[1], c[2], c[3]};
    n[mu] = (n[mu] + dmu + 2 * d[mu]) % d[mu];
    n[nu] = (n[nu] + dnu + 2 * d[nu]) % d[nu];
    return lex_of(n[0], n[1], n[2], n[3], d);
}

/*
 * T(x) = 1 + 2 kappa A(x) with A = -(csw/2) sum_{mu<nu} gamma_mu gamma_nu (x) F_munu(x),
 * F_munu = (Q_munu - Q_munu^dag)/8, Q_munu = sum of the four leaves (oriented
 * plaquettes starting and ending at x, counter-clockwise in the mu-nu plane):
 *   L1 = U_mu(x) U_nu(x+mu) U_mu(x+nu)^dag U_nu(x)^dag
 *   L2 = U_nu(x) U_mu(x+nu-mu)^dag U_nu(x-mu)^dag U_mu(x-mu)
 *   L3 = U_mu(x-mu)^dag U_nu(x-mu-nu)^dag U_mu(x-mu-nu) U_nu(x-nu)
 *   L4 = U_nu(x-nu)^dag U_mu(x-nu) U_nu(x-nu+mu) U_mu(x)^dag
 * Array treated periodic (gauge links carry no fermion boundary phase).
 * Out: Tout[lex][12][12] complex.
 */
static void clover_one(cplx *Tout, long s, const cplx *U, const int dims[4], long V, double kappa, double csw) {
    {
        long c[4];
        c[0] = s % dims[0];
        c[1] = (s / dims[0]) % dims[1];
        c[2] = (s / ((long)dims[0] * dims[1])) % dims[2];
        c[3] = s / ((long)dims[0] * dims[1] * dims[2]);
        cplx T[12][12];
        memset(T, 0, sizeof(T));
        for (int i = 0; i < 12; ++i) T[i][i] = 1.0;
        for (int mu = 0; mu < 4; ++mu)
            for (int nu = mu + 1; nu < 4; ++nu) {
                cplx Q[9] = {0}, t1[9], t2[9], t3[9], d1[9], d2[9];
                long x = s;
                long xpm = shift2(c, mu, +1, nu, 0, dims);
                long xpn = shift2(c, mu, 0, nu, +1, dims);
                long xmm = shift2(c, mu, -1, nu, 0, dims);
                long xmn = shift2(c, mu, 0, nu, -1, dims);
                long xpn_mm = shift2(c, mu, -1, nu, +1, dims);
                long xmm_mn = shift2(c, mu, -1, nu, -1, dims);
                long xmn_pm = shift2(c, mu, +1, nu, -1, dims);
                /* L1 */
                mm(t1, link(U, mu, x, V), link(U, nu, xpm, V));
                dag(d1, link(U, mu, xpn, V));
                mm(t2, t1, d1);
                dag(d2, link(U, nu, x, V));
                mm(t3, t2, d2);
                for (int k = 0; k < 9; ++k) Q[k] += t3[k];
                /* L2 */
                dag(d1, link(U, mu, xpn_mm, V));
                mm(t1, link(U, nu, x, V), d1);
                dag(d2, link(U, nu, xmm, V));
                mm(t2, t1, d2);
                mm(t3, t2, link(U, mu, xmm, V));
                for (int k = 0; k < 9; ++k) Q[k] += t3[k];
                /* L3 */
                dag(d1, link(U, mu, xmm, V));
                dag(d2, link(U, nu, xmm_mn, V));
                mm(t1, d1, d2);
                mm(t2, t1, link(U, mu, xmm_mn, V));
                mm(t3, t2, link(U, nu, xmn, V));
                for (int k = 0; k < 9; ++k) Q[k] += t3[k];
                /* L4 */
                dag(d1, link(U, nu, xmn, V));
                mm(t1, d1, link(U, mu, xmn, V));
                mm(t2, t1, link(U, nu, xmn_pm, V));
                dag(d2, link(U, mu, x, V));
                mm(t3, t2, d2);
                for (int k = 0; k < 9; ++k) Q[k] += t3[k];
                cplx F[9];
                for (int i = 0; i < 3; ++i)
                    for (int j = 0; j < 3; ++j) F[i * 3 + j] = (Q[i * 3 + j] - conj(Q[j * 3 + i])) / 8.0;
                /* gamma_mu gamma_nu */
                cplx gg[4][4];
                for (int r = 0; r < 4; ++r)
                    for (int q = 0; q < 4; ++q) {
                        cplx v = 0;
                        for (int k = 0; k < 4; ++k) v += GAMMA[mu][r][k] * GAMMA[nu][k][q];
                        gg[r][q] = v;
                    }
                const double coef = 2.0 * kappa * (-0.5 * csw);
                for (int r = 0; r < 4; ++r)
                    for (int q = 0; q < 4; ++q)
                        for (int a = 0; a < 3; ++a)
                            for (int b = 0; b < 3; ++b) T[r * 3 + a][q * 3 + b] += coef * gg[r][q] * F[a * 3 + b];
            }
        memcpy(Tout, T, sizeof(T));
    }
}

void oracle_clover(double *Tout_, const double *U_, const int dims[4], double kappa, double csw) {
    cplx *Tout = (cplx *)Tout_;
    const long V = (long)dims[0] * dims[1] * dims[2] * dims[3];
#pragma omp parallel for schedule(static)
    for (long s = 0; s < V; ++s) clover_one(Tout + s * 144, s, (const cplx *)U_, dims, V, kappa, csw);
}

/* T at the listed sites only: Tout[k] = T(sites[k]). */
void oracle_clover_sites(double *Tout_, const double *U_, const int dims[4], double kappa, double csw,
                         const long *sites, long nsites) {
    cplx *Tout = (cplx *)Tout_;
    const long V = (long)dims[0] * dims[1] * dims[2] * dims[3];
#pragma omp parallel for schedule(static)
    for (long k = 0; k < nsites; ++k) clover_one(Tout + k * 144, sites[k], (const cplx *)U_, dims, V, kappa, csw);
}

/* Tinv(x) = T(x)^{-1} by Gauss-Jordan elimination with partial pivoting.
 * Returns the number of sites whose pivot magnitude fell below 1e-300 (singular). */
int oracle_invert12(double *out_, const double *in_, long V) {
    cplx *out = (cplx *)out_;
    const cplx *in = (const cplx *)in_;
    int bad = 0;
#pragma omp parallel for schedule(static) reduction(+ : bad)
    for (long s = 0; s < V; ++s) {
        cplx a[12][24];
        for (int i = 0; i < 12; ++i)
            for (int j = 0; j < 12; ++j) {
                a[i][j] = in[s * 144 + i * 12 + j];
                a[i][12 + j] = (i == j) ? 1.0 : 0.0;
            }
        for (int col = 0; col < 12; ++col) {
            int piv = col;
            double best = cabs(a[col][col]);
            for (int r = col + 1; r < 12; ++r)
                if (cabs(a[r][col]) > best) { best = cabs(a[r][col]); piv = r; }
            if (best < 1e-300) { bad++; break; }
            if (piv != col)
                for (int j = 0; j < 24; ++j) { cplx t = a[col][j]; a[col][j] = a[piv][j]; a[piv][j] = t; }
            cplx inv = 1.0 / a[col][col];
            for (int j = 0; j < 24; ++j) a[col][j] *= inv;
            for (int r = 0; r < 12; ++r) {
                if (r == col) continue;
                cplx f = a[r][col];
                if (f == 0) continue;
                for (int j = 0; j < 24; ++j) a[r][j] -= f * a[col][j];
            }
        }
        for (int i = 0; i < 12; ++i)
            for (int j = 0; j < 12; ++j) out[s * 144 + i * 12 + j] = a[i][12 + j];
    }
    return bad;
}

/* out(x) = M(x) in(x), M[lex][12][12], in/out [lex][12] */
void oracle_site_mult(double *out_, const double *M_, const double *in_, long V) {
    cplx *out = (cplx *)out_;
    const cplx *M = (const cplx *)M_;
    const cplx *in = (const cplx *)in_;
#pragma omp parallel for schedule(static)
    for (long s = 0; s < V; ++s) {
        cplx r[12];
        for (int i = 0; i < 12; ++i) {
            cplx v = 0;
            for (int j = 0; j < 12; ++j) v += M[s * 144 + i * 12 + j] * in[s * 12 + j];
            r[i] = v;
        }
        memcpy(out + s * 12, r, sizeof(r));
    }
}
