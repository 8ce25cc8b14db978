// internal.h — host-side declarations shared by the C++ runtime and the CUDA kernels.
// Not part of the ABI (see include/qudax.h).
#pragma once

#include <cuda_runtime.h>

#include <cstddef>
#include <cstdint>
#include <stdexcept>
#include <string>

#include "qudax.h"

namespace qx {

// ----------------------------------------------------------------------------- errors
struct Error : std::runtime_error {
    qudax_status status;
    Error(qudax_status s, const std::string &m) : std::runtime_error(m), status(s) {}
};

#define QX_CUDA(call)                                                                        \
    do {                                                                                     \
        cudaError_t e_ = (call);                                                             \
        if (e_ != cudaSuccess)                                                               \
            throw ::qx::Error(e_ == cudaErrorMemoryAllocation ? QUDAX_ERR_OOM : QUDAX_ERR_CUDA, \
                              std::string(#call) + ": " + cudaGetErrorString(e_));          \
    } while (0)

#define QX_CHECK(cond, status, msg)                          \
    do {                                                     \
        if (!(cond)) throw ::qx::Error((status), (msg));     \
    } while (0)

// ----------------------------------------------------------------------------- layouts
// Site-major SoA (eq. (4)): a field with N reals per site is stored as blocks of
// 16-byte (fp64, fp32) or 8-byte (half) vectors; block b, site i lives at
// base + (b * stride + i) * vec_bytes.  stride = number of sites padded to 64.
inline long pad64(long n) { return (n + 63) / 64 * 64; }

// bytes of one "N-real" site-major array with `stride` sites in precision prec.
// fp64: N/2 double2; fp32: N/4 float4 (+1 float2 if N%4==2); half: N/4 short4 (+1 short2).
inline size_t soa_bytes(int prec, int nreal, long stride) {
    if (prec == 8) return (size_t)(nreal / 2) * 16 * stride;
    if (prec == 4) return ((size_t)(nreal / 4) * 16 + (nreal % 4 ? 8 : 0)) * stride;
    return ((size_t)(nreal / 4) * 8 + (nreal % 4 ? 4 : 0)) * stride;
}
// spinor (24 reals) + half norm (one float per site)
inline size_t spinor_bytes(int prec, long stride) {
    return soa_bytes(prec, 24, stride) + (prec == 2 ? (size_t)4 * stride : 0);
}
// projected face (12 reals) + half norm
inline size_t face_bytes(int prec, long fstride) {
    return soa_bytes(prec, 12, fstride) + (prec == 2 ? (size_t)4 * fstride : 0);
}
// clover: 72 reals = two 6x6 Hermitian chiral blocks; half adds 2 floats (one per block)
inline size_t clover_bytes(int prec, long stride) {
    return soa_bytes(prec, 72, stride) + (prec == 2 ? (size_t)8 * stride : 0);
}

// ----------------------------------------------------------------------------- geometry
struct Geom {
    int X, Y, Z, T;        // LOCAL extents X_loc, Y_loc, Z_loc and the global T
    int T_loc, t0, rank, nranks;
    int Xh;                // X/2
    long Vs, V, Vh, F;     // X*Y*Z, local volume, V/2, T-face sites = Vs/2
    long stride, fstride;  // padded Vh, padded F
    // process grid: rank = ((ct*Pz + cz)*Py + cy)*Px + cx
    int G[4];              // global dims
    int L[4];              // local dims (X, Y, Z, T_loc)
    int P[4], c[4], o[4];  // grid, coordinates, origin
    int nbf[4], nbb[4];    // neighbour ranks per dimension
    int split;             // bit mu: dimension mu has ghost zones
    long Fd[4], fsd[4];    // per-parity face sites along mu (V / L_mu / 2) and padded
    // interior box in (xh, y, z, t) coordinates (sites whose hops never touch a ghost) and its size
    int blo[4], bn[4];
    long n_int;            // interior sites; Vh - n_int boundary sites
};
// bit mu of the dimensions whose ghosts are NOT the T face (X, Y, Z)
inline int spatial_split(const Geom &g) { return g.split & 7; }

// ----------------------------------------------------------------------------- reductions
// device-resident BiCGstab scalars (Algorithm R), advanced by apply_coef after each reduction
// The iteration's update rule (Algorithm R, solver.cpp) is evaluated on the device right after
// the |r|^2 reduction (COEF_RHO with decide != 0): the host reads the scalars once per batch of
// up to `poll_every` iterations instead of after every iteration.  A batch is a CUDA graph whose
// WHILE node repeats one iteration while the condition `cond` holds; the iteration's last
// kernel (k_batch_cond) clears it when the tail that evaluates the rule asked for a reliable
// update (`halt`: also convergence and maxiter) or the batch is complete (k == kstop) — so no further kernel of the batch is launched at all, and
// the iterates are exactly those of a host decision taken after every iteration.
constexpr int kHistRing = 64;  // per-iteration |r| of the current batch (poll_every <= kHistRing)
struct SolverScalars {
    double2 rho, rho_new, alpha, malpha, omega, beta;
    double r2;
    double red[3];
    // Algorithm R state advanced on the device (decide != 0)
    double rNorm, r0Norm, maxrr, maxrx;
    double delta, stop;          // update threshold, tol * ||bhat||
    int k, maxiter;              // iterations done in this solve, cap
    int decide;                  // evaluate the update rule after COEF_RHO
    int halt;                    // an iteration of this batch asked for a reliable update
    int updX, blown;             // its flags (reading R3 for blown)
    int kstop;                   // the batch's last iteration (WHILE-graph batches)
    unsigned long long cond;     // cudaGraphConditionalHandle of the running batch graph, 0: none
    double hist[kHistRing];      // |r_k| (iterated) at ring slot (k - 1) % kHistRing
};
enum CoefMode { COEF_NONE = 0, COEF_ALPHA = 1, COEF_OMEGA = 2, COEF_RHO = 3 };
// Kernel-side global sum over peer memory (QUDAX_HALO_P2P mode: the
// solver's per-iteration sums fused with their allreduce): every rank owns one
// IPC-exported slot area [kArChannels][2][kMaxPeers] of {3 sums, sequence}.  The CTA that
// finishes a reduction stores its rank's totals into slot [chan][seq & 1][rank] of EVERY rank
// (peer stores over NVLink, then a system-scope release of the sequence word), acquires the
// nranks slots of its own area for this sequence, and adds them in rank order — so every rank
// gets bitwise the same sums with no host involvement and no NCCL launch.  Channel = the
// reduction stream (0: single-RHS, 1 + k: right-hand side k of a multi-RHS launch, whose tails
// finish in any order); two sequence parities suffice because no rank can start sequence s + 2
// of a channel before every rank has finished reading s (it needs their s + 1 totals first).
constexpr int kMaxPeers = 8;
constexpr int kArChannels = 1 + 8;  // 1 + kMaxRhs
struct DevAllreduce {
    double *slots[kMaxPeers];  // each rank's slot area (this rank's own at [rank]), peer-mapped
    unsigned *seq;             // [kArChannels] this rank's per-channel sequence counters
    int nranks, rank;
    int *err;                  // device error word (wait timeout)
};
// a grid reduction with a last-CTA tail (reduce.cuh)
struct RedTail {
    double *partials;      // [total_blocks][nred] per-CTA sums
    unsigned *counter;     // zero on entry, reset to zero by the last CTA
    int total_blocks;      // CTAs contributing (all launches of this reduction)
    int block_offset;      // this launch's first slot
    double *out;           // totals (S->red when coef_mode != COEF_NONE)
    SolverScalars *S;
    int coef_mode;
    const DevAllreduce *dar = nullptr;  // kernel-side global sum (device pointer), nullptr: local only
    int chan = 0;                       // its channel
};

// ----------------------------------------------------------------------------- kernels
// RANGE_TAIL: every site, interior first and the 2F boundary sites in the LAST CTAs of the
// grid, which alone wait for the kernel-initiated halo (one launch: the interior overlaps the
// peers' face stores, the boundary fills the grid's tail)
enum SiteRange { RANGE_ALL = 0, RANGE_INTERIOR = 1, RANGE_BOUNDARY = 2, RANGE_TAIL = 3 };
constexpr int kMaxRhs = 8;
constexpr int kGroupHost = 64;  // = reduce.cuh kGroup (slots per tail group)

// Division by a run-time constant d >= 1 for 0 <= n < 2^31 without the integer-division
// emulation (I2F/MUFU/F2I + ~20 ALU/FMA instructions): q = umulhi(n, m) >> sh with
// l = ceil(log2 d), m = floor(2^(31+l)/d) + 1, sh = l - 1 (Granlund-Montgomery; m*d - 2^(31+l)
// is in (0, d] <= 2^l, so n*(m*d - 2^(31+l)) < 2^(31+l) and the quotient is exact).  d = 1:
// m = 0 marks the identity.
struct FastDiv {
    unsigned m;
    int sh, d;
};
inline FastDiv make_fastdiv(int d) {
    FastDiv f{0u, 0, d};
    if (d <= 1) return f;
    int l = 0;
    while ((1LL << l) < d) ++l;
    f.m = (unsigned)(((1ULL << (31 + l)) / (unsigned long long)d) + 1ULL);
    f.sh = l - 1;
    return f;
}
#ifdef __CUDACC__
__device__ __forceinline__ int fdiv(int n, const FastDiv &f) {
    return f.m ? (int)(__umulhi((unsigned)n, f.m) >> f.sh) : n;
}
#endif

struct DslashArgs {
    // geometry
    int X, Y, Z, T_loc, Xh;
    int Vh, F;
    FastDiv dXh, dY, dZ;   // site index -> (xh, y, z, t) without integer division
    long stride, fstride;
    // partitioned X / Y / Z: bit mu of smask set -> hops off the local box
    // in mu read spin-projected half spinors (arithmetic precision) from sghost_{back,fwd}[mu]
    // (face layout, sfs[mu] padded sites) and the backward link from gauge_sghost[mu]
    int smask;
    long sfs[3];
    const void *sghost_back[3], *sghost_fwd[3];
    const void *gauge_sghost[3];
    // RANGE_INTERIOR: the interior box (xh, y, z, t) = blo + [0, bn); RANGE_BOUNDARY with
    // blist != nullptr: sites blist[0 .. nthreads) (the complement of the box)
    int blo[4], bn[4];
    const int *blist;
    int parity;            // output parity p
    int range;             // SiteRange
    int ghosted;           // 1: t-hops off the slab read ghost buffers; 0: periodic wrap
    int nthreads;          // sites this launch covers
    double bc_fwd, bc_back; // sign on the t-hop out of local t=T_loc-1 (fwd) / t=0 (back)
    double a;              // xpay coefficient
    const void *in;        // parity 1-p spinor
    void *out;             // parity p spinor
    const void *x;         // parity p spinor (xpay)
    const void *gauge[4][2];
    const void *gauge_ghost; // U_t at global t0-1, parity 1-p, face layout (F sites)
    const void *clover;    // parity p: T (xpay) or T^{-1} (clover_inv)
    const void *ghost_back; // upper (non-dagger) half-spinors from rank-1, face layout
    const void *ghost_fwd;  // lower (non-dagger) half-spinors from rank+1
    long ghost_rhs_bytes;   // multi-RHS halo: RHS k's ghost faces sit k * ghost_rhs_bytes further on
    // kernel-initiated halo: this launch consumes halo number s = *p2p_cseq + 1: before reading
    // ghosts its boundary CTAs wait until p2p_flags[2 mu], p2p_flags[2 mu + 1] >= s for every
    // split dimension mu of p2p_mask (system-scope acquire); ghosts of odd s sit p2p_pdist (T)
    // / sp2p_pdist[mu] (X, Y, Z) bytes on.  RANGE_TAIL: the first tail_ni sites are interior
    // (no ghost reads), the CTAs beyond them wait.  The launch's last CTA (counter
    // p2p_ccount) advances *p2p_cseq.  The pack kernel keeps its own producer counter, so the
    // two may run concurrently.
    unsigned *p2p_cseq;
    unsigned *p2p_ccount;
    const unsigned *p2p_flags;
    long p2p_pdist;
    long sp2p_pdist[3];
    int p2p_mask;
    int tail_ni;
    // optional fused reduction over the output (BiCGstab, P:542-558 kernel fusion)
    int red_kind;          // RED_NONE, RED_XDOT_NORM: (<out,x>, |out|^2), RED_RHAT_DOT: <rhat,out>
    RedTail tail;          // 3 sums per CTA; block_offset set per launch (split launches)
    const void *rhat;
    int reverse;           // 1: map CTAs to sites from the top of the range down (L2 reuse, see matpc)
    int *err;              // device error word (kernel-initiated halo wait timeout -> QUDAX_ERR_COMM)
    int variant;           // kVariant* bits (init flags: test / comparison instantiations)
    unsigned long long *span; // kernel timing on: {first-CTA start, last-CTA end, counters} (ns)
    // multi-RHS launch: nrhs > 1 uses in_m / out_m / x_m instead of in/out/x
    int nrhs;
    const void *in_m[kMaxRhs];
    void *out_m[kMaxRhs];
    const void *x_m[kMaxRhs];
    // fused reductions of a multi-RHS launch: one tail per right-hand side (the CTAs of one RHS
    // form their own deterministic reduction; block index = site block)
    const void *rhat_m[kMaxRhs];
    RedTail tail_m[kMaxRhs];
};
enum DslashRed { RED_NONE = 0, RED_XDOT_NORM = 1, RED_RHAT_DOT = 2 };
enum DslashVariant { kVariantForceSS = 1, kVariantOneRhsPerThread = 2 };


void launch_dslash_f64(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
void launch_dslash_f32(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
void launch_dslash_f16(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
// CTAs a launch of `nthreads` sites uses (one resident wave at most)
int dslash_blocks_f64(int recon, int dagger, int kind, int nthreads);
int dslash_blocks_f32(int recon, int dagger, int kind, int nthreads);
int dslash_blocks_f16(int recon, int dagger, int kind, int nthreads);

// face pack of the partitioned X / Y / Z dimensions (bit mu of g.split, mu < 3): for each, the
// x_mu = 0 face projected with the receiver's forward-hop projector -> sb[mu], the x_mu = L-1
// face with its backward-hop projector -> sf[mu]; 12 reals per site in the arithmetic precision
void launch_pack_spatial(int prec, int dagger, const Geom &g, int in_parity, const void *in, void *const sb[3],
                         void *const sf[3], cudaStream_t s);
// whether the faces along mu carry raw spinor records (half everywhere; X in every precision)
// instead of spin-projected half spinors in the arithmetic precision
__host__ __device__ inline bool sface_raw(int prec, int mu) { return prec == 2 || mu == 0; }
// bytes of one spatial face buffer along mu
size_t sface_bytes(int prec, int mu, long fs);
// face pack: t_loc = 0 slice half (lower if !dagger) -> send_back; t_loc = T_loc-1 half
// (upper if !dagger) -> send_fwd.  `in` is the Dslash input field (parity 1-p).
void launch_pack_faces(int prec, int dagger, const Geom &g, const void *in, void *send_back,
                       void *send_fwd, cudaStream_t s);

// kernel-initiated halo of any process grid (QUDAX_HALO_P2P): all split dimensions' faces
// stored into the neighbours' ghosts (peer memory), then their flags raised (layout.cu)
struct P2PPackArgs {
    int L[4];
    int mask;               // split dimensions
    int q;                  // parity of the packed (input) field
    long Fd[4], fsd[4];     // per-parity face sites along mu, padded
    long stride;
    char *dst_b[4];         // backward neighbour's forward-ghost buffer (sequence parity 0)
    char *dst_f[4];         // forward neighbour's backward-ghost buffer
    long pdist[4];          // bytes to the sequence-parity-1 buffer
    unsigned *flag_b[4];    // backward neighbour's "forward ghost filled" flag of mu
    unsigned *flag_f[4];    // forward neighbour's "backward ghost filled" flag of mu
    unsigned *seq, *count;  // this rank's producer sequence and CTA counter
    int half_back, half_fwd; // T faces: spin halves sent backward / forward (reading Q15)
};
void launch_pack_p2p(int prec, int dagger, const P2PPackArgs &a, const void *in, cudaStream_t s);

// layout conversion (DR AoS fp64 <-> NR SoA prec), one parity
void launch_spinor_import(int prec, const Geom &g, int parity, const double *src, void *dst, cudaStream_t s);
void launch_spinor_export(int prec, const Geom &g, int parity, const void *src, double *dst, cudaStream_t s);
void launch_spinor_convert(int dst_prec, int src_prec, const Geom &g, void *dst, const void *src, cudaStream_t s);

// gauge: extended fp64 site-major AoS ext[Et][Ez][Ey][Ex][4][3][3] complex, E_mu = L_mu + 2 for
// split dimensions (ext index 0 = local -1, L_mu + 1 = local L_mu), L_mu otherwise.
inline long ext_extent(const Geom &g, int mu) { return g.L[mu] + ((g.split >> mu & 1) ? 2 : 0); }
inline long ext_sites(const Geom &g) { return ext_extent(g, 0) * ext_extent(g, 1) * ext_extent(g, 2) * ext_extent(g, 3); }
// host-order box [4][T_loc][Z][Y][X][18] (device) -> ext interior
void launch_ext_fill(const Geom &g, const double *box, double *ext, cudaStream_t s);
// ext cross-section at ext index e along mu (all ext extents of the other dims) <-> buf
void launch_ext_slice(const Geom &g, double *ext, int mu, int e, double *buf, bool to_buf, cudaStream_t s);
long ext_slice_doubles(const Geom &g, int mu);
// ext -> per-mu, per-parity SoA (prec, recon) plus the backward ghost links U_mu(x - mu) at
// x_mu = 0 of every split dimension, per site parity, in face layout (ghost[mu][parity]).
// *bad counts links with |u01|^2+|u02|^2 < 1e-6 (recon 8).
void launch_gauge_pack2(int prec, int recon, const Geom &g, const double *ext, void *const dst[4][2],
                        void *const ghost[4][2], int *bad, cudaStream_t s);
// clover: from the extended fp64 gauge, T = 1 + 2 kappa A and T^{-1} as two 6x6 Hermitian
// chiral blocks per site (fp64 [Vh][72], halved for the NR rotation), both parities.
void launch_clover_build(const Geom &g, const double *ext, double kappa, double csw, double *T[2],
                         double *Tinv[2], int *bad_sites, cudaStream_t s);
void launch_clover_pack(int prec, const Geom &g, const double *src, void *dst, cudaStream_t s);
void launch_clover_apply(int prec, const Geom &g, const void *cl, const void *in, void *out, cudaStream_t s);

// BLAS / reductions (blas.cu).  ops: 0 p_update, 1 caxpy, 2 xpay, 3 cdot, 4 norm2, 5 tdot,
// 6 bicgstab final update, 7 r = b - r with |r|^2.  Returns the number of reduced doubles
// written to `out` (device).
// OP_CAXPY_REV: OP_CAXPY walking the sites top-down (the solver's L2-aware kernel order)
enum BlasOp { OP_P_UPDATE = 0, OP_CAXPY, OP_XPAY, OP_CDOT, OP_NORM2, OP_TDOT, OP_FINAL, OP_BMR_NORM, OP_CAXPY_REV };
// a BLAS coefficient: the value v, or (d != nullptr) a device scalar read by the kernel
struct CoefArg {
    double2 v;
    const double2 *d;
};
#ifdef __CUDACC__
__device__ __forceinline__ double2 coef_get(const CoefArg &c) { return c.d ? *c.d : c.v; }
#endif
// `tail` describes the reduction of reducing ops (partials/counter/out/S/coef_mode; the
// block fields are filled in here).  Returns the number of reduced doubles (0 if none).
int blas_run(int op, int prec, const Geom &g, void *const *f, const CoefArg *co, RedTail tail,
             cudaStream_t s);
void launch_coef(SolverScalars *S, int mode, cudaStream_t s);
void launch_batch_begin(SolverScalars *S, unsigned long long cond, int n, cudaStream_t s);
void launch_batch_end(SolverScalars *S, cudaStream_t s);
void launch_batch_cond(const SolverScalars *S, cudaStream_t s);
// flags[2 mu], flags[2 mu + 1] = ++*seq for every mu in mask (NCCL halo tail mode)
void launch_raise_flags(unsigned *flags, unsigned *seq, int mask, cudaStream_t s);
void blas_xpy_mixed(int pd, int ps, const Geom &g, const void *x, void *y, cudaStream_t s);
int blas_partial_blocks();

}  // namespace qx
