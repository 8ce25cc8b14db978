/*
 * qgen.c — seeded, counter-based synthetic inputs shared by the oracle side and the
 * CUDA side (tests, bench, smoke).  This module holds NONE of the method's
 * arithmetic: no Dirac operator, no clover, no projection, no reconstruction.  It only
 * draws random numbers and builds the SU(3) / spinor INPUT fields the paper's
 * experiments use:
 *
 *   - weak-field gauge configurations, PAPER.md P:765-769 (Sec. VII-A): "starting with
 *     all link matrices set to the identity, mixing in a small amount of random noise,
 *     and re-unitarizing the links to bring the links back to the SU(3) manifold";
 *   - Haar-random SU(3) links (the eps < 0 case: no identity component);
 *   - Gaussian colour-spinor fields (random right-hand sides / test vectors).
 *
 * Counter-based (Philox4x32-10): the value at global site (x,y,z,t), direction mu,
 * draw d depends only on (seed, t, z, y, x, mu, d), never on how the lattice is sliced
 * across ranks, so every rank can generate its own T-slab (plus halo timeslices)
 * without communication and the global field is identical for every rank count
 * (SURVEY.md §8(c) item 7).
 *
 * Layouts (host, AoS, lexicographic, x fastest):
 *   gauge : double[4][nt][Z][Y][X][3][3][2]   (mu, t, z, y, x, row, col, re/im)
 *   spinor: double[nt][Z][Y][X][4][3][2]      (t, z, y, x, spin, colour, re/im)
 * The timeslices written are t_global = (t_begin + k) mod T, k = 0..nt-1.
 */
#include <math.h>
#include <stdint.h>
#include <string.h>

#define PHILOX_M0 0xD2511F53u
#define PHILOX_M1 0xCD9E8D57u
#define PHILOX_W0 0x9E3779B9u
#define PHILOX_W1 0xBB67AE85u

static void philox4x32_10(const uint32_t ctr_in[4], const uint32_t key_in[2], uint32_t out[4]) {
    uint32_t c0 = ctr_in[0], c1 = ctr_in[1], c2 = ctr_in[2], c3 = ctr_in[3];
    uint32_t k0 = key_in[0], k1 = key_in[1];
    for (int r = 0; r < 10; ++r) {
        uint64_t p0 = (uint64_t)PHILOX_M0 * c0;
        uint64_t p1 = (uint64_t)PHILOX_M1 * c2;
        uint32_t hi0 = (uint32_t)(p0 >> 32), lo0 = (uint32_t)p0;
        uint32_t hi1 = (uint32_t)(p1 >> 32), lo1 = (uint32_t)p1;
        c0 = hi1 ^ c1 ^ k0;
        c1 = lo1;
        c2 = hi0 ^ c3 ^ k1;
        c3 = lo0;
        k0 += PHILOX_W0;
        k1 += PHILOX_W1;
    }
    out[0] = c0; out[1] = c1; out[2] = c2; out[3] = c3;
}

/* 4 standard normals from one Philox block (Box-Muller on two uniform pairs). */
static void normals4(uint64_t seed, uint32_t stream, uint64_t site, uint32_t mu, uint32_t draw,
                     double g[4]) {
    uint32_t key[2] = {(uint32_t)seed, (uint32_t)(seed >> 32) ^ (stream * 0x85EBCA6Bu)};
    uint32_t ctr[4] = {(uint32_t)site, (uint32_t)(site >> 32), mu, draw};
    uint32_t u[4];
    philox4x32_10(ctr, key, u);
    const double inv = 1.0 / 4294967296.0;
    for (int k = 0; k < 2; ++k) {
        double u1 = ((double)u[2 * k] + 0.5) * inv;
        double u2 = ((double)u[2 * k + 1] + 0.5) * inv;
        double r = sqrt(-2.0 * log(u1));
        g[2 * k] = r * cos(2.0 * M_PI * u2);
        g[2 * k + 1] = r * sin(2.0 * M_PI * u2);
    }
}

/* One SU(3) link into m[3][3][2].  eps >= 0: rows 0,1 = e_row + eps*G (weak field);
 * eps < 0: rows 0,1 = G (Haar).  Then Gram-Schmidt of rows 0,1 and row 2 chosen as
 * the unique unit vector orthogonal to both with det = +1, i.e. conj(row0 x row1). */
static void su3_link(uint64_t seed, uint64_t site, uint32_t mu, double eps, double m[3][3][2]) {
    double g[12];
    normals4(seed, 1u, site, mu, 0u, g);
    normals4(seed, 1u, site, mu, 1u, g + 4);
    normals4(seed, 1u, site, mu, 2u, g + 8);
    double a[2][3][2];
    for (int r = 0; r < 2; ++r)
        for (int c = 0; c < 3; ++c) {
            double re = g[(r * 3 + c) * 2], im = g[(r * 3 + c) * 2 + 1];
            if (eps >= 0.0) {
                re = eps * re + (r == c ? 1.0 : 0.0);
                im = eps * im;
            }
            a[r][c][0] = re;
            a[r][c][1] = im;
        }
    /* normalise row 0 */
    double n0 = 0;
    for (int c = 0; c < 3; ++c) n0 += a[0][c][0] * a[0][c][0] + a[0][c][1] * a[0][c][1];
    n0 = 1.0 / sqrt(n0);
    for (int c = 0; c < 3; ++c) { a[0][c][0] *= n0; a[0][c][1] *= n0; }
    /* row1 -= <row0,row1> row0, <a,b> = sum conj(a) b */
    double pr = 0, pi = 0;
    for (int c = 0; c < 3; ++c) {
        pr += a[0][c][0] * a[1][c][0] + a[0][c][1] * a[1][c][1];
        pi += a[0][c][0] * a[1][c][1] - a[0][c][1] * a[1][c][0];
    }
    for (int c = 0; c < 3; ++c) {
        a[1][c][0] -= pr * a[0][c][0] - pi * a[0][c][1];
        a[1][c][1] -= pr * a[0][c][1] + pi * a[0][c][0];
    }
    double n1 = 0;
    for (int c = 0; c < 3; ++c) n1 += a[1][c][0] * a[1][c][0] + a[1][c][1] * a[1][c][1];
    n1 = 1.0 / sqrt(n1);
    for (int c = 0; c < 3; ++c) { a[1][c][0] *= n1; a[1][c][1] *= n1; }
    for (int r = 0; r < 2; ++r)
        for (int c = 0; c < 3; ++c) { m[r][c][0] = a[r][c][0]; m[r][c][1] = a[r][c][1]; }
    /* row2 = conj(row0 x row1) */
    for (int c = 0; c < 3; ++c) {
        int c1 = (c + 1) % 3, c2 = (c + 2) % 3;
        /* (a0[c1]*a1[c2] - a0[c2]*a1[c1]) */
        double xr = a[0][c1][0] * a[1][c2][0] - a[0][c1][1] * a[1][c2][1]
                  - (a[0][c2][0] * a[1][c1][0] - a[0][c2][1] * a[1][c1][1]);
        double xi = a[0][c1][0] * a[1][c2][1] + a[0][c1][1] * a[1][c2][0]
                  - (a[0][c2][0] * a[1][c1][1] + a[0][c2][1] * a[1][c1][0]);
        m[2][c][0] = xr;
        m[2][c][1] = -xi;
    }
}

static inline long tmod(long t, long T) { long r = t % T; return r < 0 ? r + T : r; }

/* gauge: double[4][nt][Z][Y][X][3][3][2]; eps < 0 => Haar. */
void qgen_gauge(double *out, const int dims[4], int t_begin, int nt, uint64_t seed, double eps) {
    const long X = dims[0], Y = dims[1], Z = dims[2], T = dims[3];
    const long Vs = X * Y * Z;
    const long Vloc = Vs * nt;
#pragma omp parallel for schedule(static)
    for (long k = 0; k < 4 * Vloc; ++k) {
        long mu = k / Vloc, rem = k % Vloc;
        long tl = rem / Vs, s = rem % Vs;
        long tg = tmod(t_begin + tl, T);
        uint64_t site = (uint64_t)(tg * Vs + s);
        double m[3][3][2];
        su3_link(seed, site, (uint32_t)mu, eps, m);
        memcpy(out + k * 18, m, sizeof(m));
    }
}

/* spinor: double[nt][Z][Y][X][4][3][2], unit-variance Gaussian per real component. */
void qgen_spinor(double *out, const int dims[4], int t_begin, int nt, uint64_t seed) {
    const long X = dims[0], Y = dims[1], Z = dims[2], T = dims[3];
    const long Vs = X * Y * Z;
    const long Vloc = Vs * nt;
#pragma omp parallel for schedule(static)
    for (long k = 0; k < Vloc; ++k) {
        long tl = k / Vs, s = k % Vs;
        long tg = tmod(t_begin + tl, T);
        uint64_t site = (uint64_t)(tg * Vs + s);
        for (uint32_t d = 0; d < 6; ++d) normals4(seed, 2u, site, 0u, d, out + k * 24 + 4 * d);
    }
}

/* Gaussian SU(3)-valued gauge transformation G(x) (Haar), one matrix per site:
 * double[nt][Z][Y][X][3][3][2].  Used only by covariance tests. */
void qgen_gauge_transform(double *out, const int dims[4], int t_begin, int nt, uint64_t seed) {
    const long X = dims[0], Y = dims[1], Z = dims[2], T = dims[3];
    const long Vs = X * Y * Z;
    const long Vloc = Vs * nt;
#pragma omp parallel for schedule(static)
    for (long k = 0; k < Vloc; ++k) {
        long tl = k / Vs, s = k % Vs;
        long tg = tmod(t_begin + tl, T);
        double m[3][3][2];
        su3_link(seed ^ 0x5bd1e995ull, (uint64_t)(tg * Vs + s), 7u, -1.0, m);
        memcpy(out + k * 18, m, sizeof(m));
    }
}

/* Sub-box generators (multi-dimensional partitioning): the same per-site counters as above on the
 * box origin[mu] .. origin[mu] + ext[mu] - 1 of the global lattice (wrapped), so every rank of any
 * process grid draws exactly its part of the one global field.
 * gauge: double[4][et][ez][ey][ex][3][3][2]; spinor: double[et][ez][ey][ex][4][3][2]. */
static inline uint64_t box_site(const int dims[4], const int o[4], long xl, long yl, long zl, long tl) {
    const long X = dims[0], Y = dims[1], Z = dims[2], T = dims[3];
    long xg = tmod(o[0] + xl, X), yg = tmod(o[1] + yl, Y), zg = tmod(o[2] + zl, Z), tg = tmod(o[3] + tl, T);
    return (uint64_t)(((tg * Z + zg) * Y + yg) * X + xg);
}
void qgen_gauge_box(double *out, const int dims[4], const int o[4], const int e[4], uint64_t seed, double eps) {
    const long V = (long)e[0] * e[1] * e[2] * e[3];
#pragma omp parallel for schedule(static)
    for (long k = 0; k < 4 * V; ++k) {
        long mu = k / V, r = k % V;
        long xl = r % e[0]; r /= e[0];
        long yl = r % e[1]; r /= e[1];
        long zl = r % e[2];
        long tl = r / e[2];
        double m[3][3][2];
        su3_link(seed, box_site(dims, o, xl, yl, zl, tl), (uint32_t)mu, eps, m);
        memcpy(out + k * 18, m, sizeof(m));
    }
}
void qgen_spinor_box(double *out, const int dims[4], const int o[4], const int e[4], uint64_t seed) {
    const long V = (long)e[0] * e[1] * e[2] * e[3];
#pragma omp parallel for schedule(static)
    for (long k = 0; k < V; ++k) {
        long r = k;
        long xl = r % e[0]; r /= e[0];
        long yl = r % e[1]; r /= e[1];
        long zl = r % e[2];
        long tl = r / e[2];
        const uint64_t site = box_site(dims, o, xl, yl, zl, tl);
        for (uint32_t d = 0; d < 6; ++d) normals4(seed, 2u, site, 0u, d, out + k * 24 + 4 * d);
    }
}
