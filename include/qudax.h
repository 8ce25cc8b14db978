/*
 * qudax.h — C ABI of the B200-native even-odd Wilson-clover Dslash / halo / mixed-precision
 * BiCGstab library (the hot path of arXiv:1011.0024, "Parallelizing the QUDA Library for
 * Multi-GPU Calculations in Lattice QCD"; PAPER.md line numbers cited as P:a-b).
 *
 * The paper's library exposes "a simple C interface to allow for easy integration with LQCD
 * application software": the only large transfers are "the initial upload of the
 * source vector to the GPU and the final download of the solution, aside from occasional
 * small messages needed to complete global sums".  This header is that
 * boundary.  Plain pointers and sizes only; no C++ or torch types.
 *
 * ---------------------------------------------------------------------------------------
 * Conventions (all readings of the paper are listed in DESIGN.md "Readings")
 * ---------------------------------------------------------------------------------------
 * Lattice  global X x Y x Z x T (x fastest, t slowest), split over a process grid
 *          Px x Py x Pz x Pt = nranks (the paper splits T only and names
 *          further dimensions as future work, P:572-578 — SURVEY 8(f) item 4).  Default grid
 *          (proc_grid all 0): 1 x 1 x 1 x nranks.  Rank r has grid coordinates
 *          r = ((ct*Pz + cz)*Py + cy)*Px + cx (x fastest) and owns the box
 *          [c_mu*L_mu, (c_mu+1)*L_mu) with L_mu = dims_mu / P_mu ("local dims").  Requires X_loc
 *          even and, in every partitioned dimension, an even local extent >= 2 (so local and
 *          global parity agree); a partitioned X needs Y_loc even too.  Site parity =
 *          (x + y + z + t) mod 2 in global coordinates.
 * Host gauge  const double[4][T_loc][Z_loc][Y_loc][X_loc][3][3][2]: the rank's box, U_mu(x) stored at x
 *          (P:425-432), row-major 3x3 complex, mu = 0..3 <-> x, y, z, t.  Borrowed for the
 *          duration of the call only.
 * Host spinor double[T_loc][Z_loc][Y_loc][X_loc][4][3][2] in the DeGrand-Rossi chiral basis (the
 *          "conventional chiral basis" of eq. (6)).  Borrowed per call.
 * Operator M_kappa = 2 kappa M(eq. (2)) = T - kappa D with T = 1 + 2 kappa A (clover A of
 *          eq. (2); kappa = 1/(2(4+m))).  Even-odd: the solver works
 *          on the asymmetric Schur complement on even sites
 *              Mhat = T_ee - kappa^2 D_eo T_oo^{-1} D_oe,   Mhat^dag = gamma5 Mhat gamma5.
 * Device spinor fields ("parity fields") are plain device buffers owned by the CALLER, of
 *          qudax_spinor_bytes(ctx, prec) bytes, holding the V_h = V_loc/2 sites of one parity
 *          in the library's site-major SoA layout (eq. (4): N_int/N_vec blocks of
 *          V_h 16-byte short vectors; non-relativistic spin basis, eq. (6)).  Half precision
 *          appends one float norm per site (value = norm * q / 32767, norm = the
 *          site's largest |component|; a site whose norm is <= 1e-30 is stored as zero,
 *          DESIGN.md reading R6).  The layout is opaque to callers:
 *          move data in and out with qudax_spinor_load/store.  Reductions never see ghost
 *          zones: ghosts live in separate library-owned buffers.
 *
 * Precision / reconstruct: prec = bytes per stored real
 *          (2 = 16-bit fixed point "half", 4 = fp32, 8 = fp64); recon = reals stored per link
 *          (18 full, 12 two-row with row3 = conj(row1 x row2), 8 = two phases + u01,u02,u10).
 *
 * Ownership: the ctx owns every internal device allocation (through the dev_alloc/dev_free
 *          hooks when given — the Python binding passes PyTorch's caching allocator — else
 *          cudaMalloc) and its comm stream.  Host pointers are borrowed per call.
 * Ordering: qudax_dslash / qudax_matpc / qudax_mdagm / qudax_spinor_load_dev are
 *          stream-ordered on the ctx compute stream and return before the GPU finishes.
 *          qudax_gauge_load, qudax_spinor_load/store (host), reductions and the solvers are
 *          synchronous.
 * Errors:  every call returns a qudax_status; no C++ exception crosses the ABI.  CUDA and NCCL
 *          failures are sticky (the ctx must be finalized); qudax_last_error() explains.
 * Threads: a ctx is not thread-safe.  With nranks > 1 every rank must make the same sequence
 *          of calls (collective ordering rule).
 */
#ifndef QUDAX_H
#define QUDAX_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define QUDAX_ABI_VERSION 5

typedef enum {
    QUDAX_OK = 0,
    QUDAX_ERR_ARG = 1,           /* bad dims, parity, precision, null pointer, state mismatch */
    QUDAX_ERR_STATE = 2,         /* call out of order (e.g. dslash before gauge_load) or sticky error */
    QUDAX_ERR_CUDA = 3,          /* CUDA runtime failure (sticky) */
    QUDAX_ERR_NCCL = 4,          /* NCCL failure (sticky) */
    QUDAX_ERR_UNSUPPORTED = 5,   /* e.g. 8-reconstruct on near-singular links (reading Q6) */
    QUDAX_ERR_NOT_CONVERGED = 6, /* solver hit maxiter; x holds the last iterate */
    QUDAX_ERR_OOM = 7,           /* device allocation failed */
    QUDAX_ERR_COMM = 8           /* host transport hook returned non-zero, or a kernel-initiated halo
                                    wait timed out (a neighbour stalled: the result is not returned) */
} qudax_status;

typedef enum { QUDAX_HALF = 2, QUDAX_SINGLE = 4, QUDAX_DOUBLE = 8 } qudax_prec;
typedef enum { QUDAX_RECON_18 = 18, QUDAX_RECON_12 = 12, QUDAX_RECON_8 = 8 } qudax_recon;
typedef enum { QUDAX_EVEN = 0, QUDAX_ODD = 1 } qudax_parity;

/* What a single Dslash kernel computes on the output parity p (input field of parity 1-p):
 *   HOP         out = D_{p,1-p} in                                   (1320 flops/site)
 *   CLOVER_INV  out = T_pp^{-1} D_{p,1-p} in                         (+504, clover fused,
 *                                                                      P:390-395)
 *   CLOVER_XPAY out = T_pp x + a * D_{p,1-p} in                     (+504 +48)
 *   CLOVER_INV_XPAY out = x + a * T_pp^{-1} D_{p,1-p} in            (+504 +48)
 * Mhat = [kernel CLOVER_INV on odd] then [kernel CLOVER_XPAY on even, a = -kappa^2];
 * the symmetric form T_ee^{-1} Mhat ends with CLOVER_INV_XPAY instead. */
typedef enum { QUDAX_HOP = 0, QUDAX_CLOVER_INV = 1, QUDAX_CLOVER_XPAY = 2, QUDAX_CLOVER_INV_XPAY = 3 } qudax_dslash_kind;

/* Halo transport:
 *   NONE  nranks must be 1; the Dslash wraps every dimension periodically inside one kernel.
 *   NCCL  ncclSend/ncclRecv of spin-projected faces on a comm stream, overlapped with the
 *         interior kernel; ncclAllReduce for global sums.  With
 *         nranks == 1 this is the loopback test mode: faces go through NCCL to self and every
 *         global sum through ncclAllReduce on the one-rank communicator, so the N > 1 code
 *         path (including its CUDA-graph capture) runs on one GPU.
 *   Faces: T faces carry the 12 reals the diagonal temporal projector keeps, in the storage
 *         precision (bits only, half with its norm; eq. (6)).  Faces of a partitioned
 *         X, Y or Z carry the spin-projected half spinor (1 -+ gamma_mu) psi (footnote 3,
 *         P:665-670), 12 reals in the kernel's arithmetic precision (fp64 for double, fp32 for
 *         single and half), computed by the pack kernel with the Dslash's own projection code,
 *         so a partitioned Dslash is bitwise equal to the unpartitioned one.
 *   HOST  faces staged through pinned host memory and exchanged by the caller's hooks
 *         (the paper's non-overlapped strategy); used to run several ranks on
 *         one GPU in tests. */
typedef enum { QUDAX_COMM_NONE = 0, QUDAX_COMM_NCCL = 1, QUDAX_COMM_HOST = 2 } qudax_comm_kind;

/* Spinor halo path of the Dslash when the lattice is split (or in loopback):
 *   COMM  faces packed into local buffers and moved by the `comm` transport above.
 *   P2P   kernel-initiated over peer memory (the paper's wish to share
 *         memory between CUDA and message passing).  The face-pack kernel stores
 *         the spin-projected faces straight into the T-neighbours' ghost buffers (CUDA IPC
 *         mappings of their device memory: NVLink/NVSwitch on a multi-GPU node) and then
 *         raises a sequence flag in the neighbour's memory with a system-scope release; the
 *         boundary kernel acquires both of its own flags before reading its ghosts.  Nothing is
 *         enqueued by the host between the kernels and no face is copied twice.  Ghosts are
 *         double-buffered by sequence parity (a rank can run at most one halo ahead of its
 *         neighbours, because each boundary kernel waits for both of them).  The IPC handles
 *         are swapped once at init over `comm` (host_exchange hook or NCCL); gauge-ghost setup
 *         and global sums keep using `comm`.  With nranks == 1 (comm NONE allowed) the
 *         neighbour is the rank itself: the loopback test of the kernel path.  P2P supports a
 *         T-only split (split_mask = T); other grids return QUDAX_ERR_UNSUPPORTED at init. */
typedef enum { QUDAX_HALO_COMM = 0, QUDAX_HALO_P2P = 1 } qudax_halo_kind;

/* Behaviour flags of qudax_init_param.flags (0 = the defaults every measurement uses).  Test and
 * comparison switches only; none changes a result beyond its documented rounding. */
typedef enum {
    QUDAX_FLAG_NO_GRAPHS = 1,          /* solver iterations enqueued eagerly, not replayed as CUDA graphs */
    QUDAX_FLAG_DEBUG_SOLVER = 2,       /* per-iteration solver scalars to stderr */
    QUDAX_FLAG_FORCE_SS = 4,           /* the partitioned-X/Y/Z kernel instantiation on every lattice (test) */
    QUDAX_FLAG_ONE_RHS_PER_THREAD = 8, /* multi-RHS launches with one right-hand side per thread (comparison) */
    QUDAX_FLAG_TIMING_BREAKDOWN = 16   /* per-(precision, kind, reduction) Dslash times to stderr at finalize */
} qudax_init_flag;

typedef struct qudax_ctx qudax_ctx;

/* Host transport hooks for QUDAX_COMM_HOST.  exchange: send send_fwd (bytes) to rank_fwd and
 * send_back to rank_back, receive from rank_back into recv_back and from rank_fwd into recv_fwd
 * (the two neighbours of this rank along one partitioned dimension; they may be the same rank,
 * or this rank itself in loopback).  Messages between one pair of ranks must be matched in
 * call order: send_fwd pairs with the peer's recv_back.  allreduce: in-place sum of n doubles
 * over ranks.  Return 0 on success. */
typedef int (*qudax_exchange_fn)(int rank_fwd, int rank_back, const void *send_fwd, const void *send_back,
                                 void *recv_back, void *recv_fwd, size_t bytes, void *user);
typedef int (*qudax_allreduce_fn)(double *vals, int n, void *user);
typedef void *(*qudax_alloc_fn)(size_t bytes, void *user);
typedef void (*qudax_free_fn)(void *ptr, void *user);

typedef struct {
    int global_dims[4];          /* X, Y, Z, T */
    int nranks, rank, device;    /* device = CUDA ordinal this rank drives */
    int comm;                    /* qudax_comm_kind */
    int overlap;                 /* NCCL: 1 = interior kernel overlaps the halo,
                                    0 = exchange first then one kernel */
    const void *nccl_id;         /* QUDAX_COMM_NCCL: 128-byte ncclUniqueId from qudax_nccl_unique_id
                                    on rank 0, broadcast by the caller */
    uintptr_t stream;            /* compute cudaStream_t (e.g. torch current stream), 0 = own */
    qudax_alloc_fn dev_alloc;    /* optional device allocator hooks (NULL = cudaMalloc) */
    qudax_free_fn dev_free;
    void *alloc_user;
    qudax_exchange_fn host_exchange; /* QUDAX_COMM_HOST hooks */
    qudax_allreduce_fn host_allreduce;
    void *comm_user;
    int halo;                    /* qudax_halo_kind (0 = COMM) */
    int proc_grid[4];            /* Px, Py, Pz, Pt with product nranks; all 0 = (1, 1, 1, nranks) */
    int split_mask;              /* bit mu set: dimension mu uses ghost zones (halo exchange).  0 =
                                    default: every dimension with P_mu > 1, and T alone when
                                    nranks == 1 with a transport (loopback).  A non-zero mask must
                                    contain every dimension with P_mu > 1; extra bits are loopback
                                    dimensions (the rank is its own neighbour) for tests. */
    int flags;                   /* qudax_init_flag bits (0 = defaults) */
    int copy_threads;            /* host threads of the pageable host<->device copies (0 = min(8, cores));
                                    process-wide, fixed by the first context that copies */
} qudax_init_param;

typedef struct {
    int prec, recon;             /* outer ("high") precision copy of gauge + clover */
    int prec_sloppy, recon_sloppy; /* inner ("sloppy") copy for reliable updates */
    int t_boundary;              /* +1 periodic, -1 antiperiodic in T (reading Q5) */
    double kappa, csw;           /* M_kappa = T - kappa D, T = 1 + 2 kappa A(csw) (readings Q1, Q4) */
} qudax_gauge_param;

typedef struct {
    double tol;                  /* stop when the TRUE residual ||b - M x|| / ||b|| <= tol (Q9) */
    double delta;                /* reliable-update threshold (Algorithm R) */
    int maxiter;                 /* iteration cap; tol = 0 with maxiter = k runs exactly k iterations */
    int prec_sloppy;             /* precision of the Krylov iteration (must have a gauge copy) */
    int prec;                    /* outer precision of x, r and the reliable-update residual */
    int use_schur;               /* 1: solve the full system M x = b via prepare/Mhat/reconstruct with the
                                    asymmetric Schur form; 2: the same with the symmetric form
                                    (qudax_matpc_sym); 0: solve Mhat x_e = b_e only */
    double *res_history;         /* optional host array: ||r_k|| / ||bhat|| after iteration k (the
                                    iterated residual, replaced by the true one at reliable updates) */
    int history_cap;             /* capacity of res_history (0 = none) */
    int poll_every;              /* BiCGstab: at most this many iterations between host reads of the
                                    device-side scalars, 1..64 (0 = 16).  A batch is one CUDA graph whose
                                    WHILE node repeats the iteration on the device; Algorithm R's update
                                    rule is evaluated on the device after every iteration, and an
                                    iteration that calls for a reliable update (or converges) ends the
                                    batch, so the iterates do not depend on poll_every. */
} qudax_solve_param;

typedef struct {
    int iters, reliable_updates;
    double true_res;             /* fp64 ||b - M x|| / ||b|| of the returned x (full system if use_schur) */
    double true_res_schur;       /* fp64 ||bhat - Mhat x_e|| / ||bhat|| */
    double secs;                 /* wall time of the call (includes H2D / D2H for the host entry) */
    double flops;                /* effective flops (P:755-758 convention, reading Q16) */
    double gflops;
    int restarts;                /* Krylov restarts after a (near) breakdown of the sloppy recurrences */
    int host_polls;              /* host reads of the device-side solver scalars (BiCGstab: batches) */
    int device_batches;          /* of those, batches the device looped over in one WHILE-node graph */
} qudax_solve_stats;

/* Per-site work and traffic model, for reporting and tests. */
typedef struct {
    double flops;                /* effective flops per output site (reconstruction not counted) */
    double bytes_paper;          /* paper model: every neighbour gather is memory traffic */
    double bytes_compulsory;     /* each link / clover / spinor read once, output written once */
} qudax_site_model;

typedef struct {
    int T_loc, t0;               /* local T extent and first global timeslice */
    int rank_fwd, rank_back;     /* T-direction neighbours */
    long V_loc, V_h, V_s, face_sites; /* local volume, per-parity volume, X_loc*Y_loc*Z_loc, V_s/2 */
    int applies_bc_fwd, applies_bc_back; /* this rank owns global t=T-1 / t=0 */
    size_t face_bytes[3];        /* one T face (12 reals per site) in half/single/double,
                                    half including its per-site norms */
    int proc_grid[4];            /* process grid */
    int coords[4];               /* this rank's grid coordinates */
    int local_dims[4];           /* X_loc, Y_loc, Z_loc, T_loc */
    int origin[4];               /* global coordinates of local site (0,0,0,0) */
    int nb_fwd[4], nb_back[4];   /* neighbour ranks along each dimension (self if P_mu = 1) */
    int split_mask;              /* dimensions with ghost zones (see qudax_init_param) */
    long face_sites_dim[4];      /* per-parity face sites V_loc / L_mu / 2 along each dimension */
} qudax_partition;

/* Accumulated CUDA-event timing of the Dslash kernel launches since qudax_kernel_timing(ctx, 1). */
typedef struct {
    long long launches;          /* Dslash kernel launches recorded (interior + boundary count separately) */
    long long sites;             /* output sites processed by them */
    double ms_total;             /* sum of per-launch durations (events on the launching stream) */
    double flops;                /* effective flops of those launches (qudax_model per kind) */
    double bytes_compulsory;     /* algorithmic bytes (compulsory model) of those launches */
    double bytes_paper;          /* paper-model bytes */
    double span_ms_total;        /* sum of the launches' in-kernel spans: %globaltimer of the first CTA
                                    to start to that of the last CTA to finish (the kernel's own
                                    execution time, without the launch bubble of the events) */
} qudax_kernel_stats;

/* ---- host-only helpers (no GPU needed) ---- */
int qudax_abi_version(void);
const char *qudax_status_string(int status);
/* Partition bookkeeping of rank `rank` of `nranks`.  proc_grid may be
 * NULL (T only); split_mask as in qudax_init_param (0 = default). */
qudax_status qudax_partition_info(const int global_dims[4], const int proc_grid[4], int nranks, int rank,
                                  int split_mask, qudax_partition *out);
/* Site model for one Dslash kernel of `kind` (flops: 1320 + 504 clover + 48 xpay, Q16), or for
 * the whole Mhat when kind = -1 (3696 flops / 2976 bytes at fp32 recon 12), or for
 * the single-launch (fused) Mhat when kind = -2 (compulsory bytes: links once, T and T^{-1},
 * input, output and the intermediate written once). */
qudax_status qudax_model(int prec, int recon, int kind, qudax_site_model *out);
/* ncclGetUniqueId into out[128] (rank 0 calls, caller broadcasts). */
qudax_status qudax_nccl_unique_id(void *out128);

/* ---- context ---- */
qudax_status qudax_init(qudax_ctx **ctx, const qudax_init_param *p);
qudax_status qudax_finalize(qudax_ctx *ctx);
const char *qudax_last_error(const qudax_ctx *ctx);
qudax_status qudax_sync(qudax_ctx *ctx);
/* Number of library kernels launched by this ctx so far (for launch accounting). */
long long qudax_launch_count(const qudax_ctx *ctx);
qudax_status qudax_get_partition(const qudax_ctx *ctx, qudax_partition *out);
/* Per-launch timing of the Dslash kernels; clears the records.  enable: 0 off; 1 CUDA events
 * around every launch on the launching stream; 2 events plus the in-kernel span (first CTA's
 * start to last CTA's end by %globaltimer, qudax_kernel_stats.span_ms_total), which costs the
 * kernels a few microseconds of their own. */
qudax_status qudax_kernel_timing(qudax_ctx *ctx, int enable);
/* Synchronise and sum the recorded Dslash launches of precision prec_filter (0 = all). */
qudax_status qudax_get_kernel_stats(qudax_ctx *ctx, int prec_filter, qudax_kernel_stats *out);
/* Diagnostic timeline of the halo overlap on the NCCL path.  enable = 1: every
 * subsequent eagerly launched split Dslash records CUDA events on both streams; out7 (may be
 * NULL) receives, for the last recorded call, the microseconds from its start (compute stream)
 * to: pack start, exchange start, exchange end (comm stream), interior kernel start, interior
 * end, boundary kernel start, boundary end (compute stream).  Without an interior/boundary split
 * (overlap off) the three "interior" marks coincide with the boundary start.  enable = 0 stops
 * recording.  QUDAX_ERR_STATE if nothing was recorded. */
qudax_status qudax_halo_timeline(qudax_ctx *ctx, int enable, double *out7);

/* ---- gauge field and clover (setup) ----
 * Uploads the host box, exchanges a one-site gauge halo (with corners: one dimension after the
 * other, each message including the halos already received) with the neighbours of every
 * partitioned dimension (once), builds A and T^{-1} in fp64 on the device and stores gauge + clover in
 * the outer and sloppy (precision, reconstruct) formats.  Returns QUDAX_ERR_UNSUPPORTED for
 * reconstruct 8 when some link has |u01|^2 + |u02|^2 < 1e-6. */
qudax_status qudax_gauge_load(qudax_ctx *ctx, const double *host_gauge, const qudax_gauge_param *p);

/* ---- spinor fields ---- */
size_t qudax_spinor_bytes(const qudax_ctx *ctx, int prec);
/* Host full local slab (DeGrand-Rossi, fp64) -> one parity of a device field in `prec`.
 * Basis change to the non-relativistic basis, parity split and precision conversion run in a
 * device kernel; only the H2D copy is done by the host. */
qudax_status qudax_spinor_load(qudax_ctx *ctx, void *dst, int prec, int parity, const double *host_src);
/* Same, source already on the device (double[T_loc][Z][Y][X][4][3][2]). */
qudax_status qudax_spinor_load_dev(qudax_ctx *ctx, void *dst, int prec, int parity, const double *dev_src);
/* Device field (one parity) -> the sites of that parity of a host full local slab (DR basis,
 * fp64).  Sites of the other parity are left untouched. */
qudax_status qudax_spinor_store(qudax_ctx *ctx, double *host_dst, const void *src, int prec, int parity);
qudax_status qudax_spinor_store_dev(qudax_ctx *ctx, double *dev_dst, const void *src, int prec, int parity);
/* Precision conversion between two device parity fields (re-quantises half). */
qudax_status qudax_spinor_convert(qudax_ctx *ctx, void *dst, int dst_prec, const void *src, int src_prec);

/* ---- operator (stream-ordered) ---- */
/* One Dslash kernel (with its halo exchange when partitioned): see qudax_dslash_kind.
 * x is read only for CLOVER_XPAY (same parity as out). dagger: D -> D^dag = gamma5 D gamma5. */
qudax_status qudax_dslash(qudax_ctx *ctx, void *out, const void *in, const void *x, int prec,
                          int out_parity, int dagger, int kind, double a);
/* out_e = Mhat in_e (dagger = 0) or Mhat^dag in_e (dagger = 1); 2 Dslash kernels + 2 halos. */
qudax_status qudax_matpc(qudax_ctx *ctx, void *out, const void *in, int prec, int dagger);
/* Symmetric Schur form: out_e = in_e - kappa^2 T_ee^{-1} D_eo T_oo^{-1} D_oe in_e
 * = T_ee^{-1} Mhat in_e — kernels CLOVER_INV then CLOVER_INV_XPAY; dagger = 1 applies the explicit
 * adjoint in_e - kappa^2 (D^dag)_eo T_oo^{-1} (D^dag)_oe T_ee^{-1} in_e (clover apply, CLOVER_INV,
 * HOP and an xpay: it is not gamma5-Hermitian, so no dagger-by-flag shortcut). */
qudax_status qudax_matpc_sym(qudax_ctx *ctx, void *out, const void *in, int prec, int dagger);
/* Multi-RHS forms (the paper's production calls the solver for many
 * right-hand sides per configuration): nrhs (1..8) independent fields
 * in one launch that streams the links and clover from HBM about once for all of them.
 * Arrays of nrhs device field pointers; x may be NULL unless kind = CLOVER_XPAY.  Results are
 * bitwise those of nrhs single calls.  Partitioned contexts apply the single-RHS path per field. */
qudax_status qudax_dslash_multi(qudax_ctx *ctx, void *const *out, const void *const *in, const void *const *x,
                                int nrhs, int prec, int out_parity, int dagger, int kind, double a);
qudax_status qudax_matpc_multi(qudax_ctx *ctx, void *const *out, const void *const *in, int nrhs, int prec,
                               int dagger);
/* out_e = Mhat^dag Mhat in_e (the CGNR normal operator). */
qudax_status qudax_mdagm(qudax_ctx *ctx, void *out, const void *in, int prec);

/* ---- global reductions over the even (parity) field, fp64 accumulation, all ranks ---- */
qudax_status qudax_norm2(qudax_ctx *ctx, const void *f, int prec, double *out);
qudax_status qudax_cdot(qudax_ctx *ctx, const void *a, const void *b, int prec, double out_re_im[2]);

/* ---- solver: mixed-precision reliable-update BiCGstab ---- */
/* Host buffers: full local slabs (DR basis, fp64).  H2D of b and D2H of x are inside. */
qudax_status qudax_solve_bicgstab(qudax_ctx *ctx, double *host_x, const double *host_b,
                                  const qudax_solve_param *p, qudax_solve_stats *st);
/* Same with device-resident fp64 full local slabs. */
qudax_status qudax_solve_bicgstab_dev(qudax_ctx *ctx, double *dev_x, const double *dev_b,
                                      const qudax_solve_param *p, qudax_solve_stats *st);

/* Batched mixed-precision BiCGstab for nrhs (1..8) sources on the same gauge field (SURVEY 8(f)
 * item 2; the paper solves 6 sources per configuration).  Every system runs its own
 * Algorithm R — iterates, reliable updates and the returned x are exactly those of nrhs calls of
 * qudax_solve_bicgstab on an unpartitioned context — but each iteration applies Mhat to all
 * still-active systems with one multi-RHS kernel pair, the <rhat0, v> and (<t, s>, |t|^2)
 * reductions fused per system into its epilogue.  use_schur 0 or 1 (asymmetric form); the
 * residual history, if requested, is that of system 0.  host_x / host_b: arrays of nrhs full
 * local slabs (as qudax_solve_bicgstab); st: nrhs stats (secs = the batch's wall time).
 * Returns QUDAX_ERR_NOT_CONVERGED if any system missed tol. */
qudax_status qudax_solve_bicgstab_multi(qudax_ctx *ctx, double *const *host_x, const double *const *host_b, int nrhs,
                                        const qudax_solve_param *p, qudax_solve_stats *st);
qudax_status qudax_solve_bicgstab_multi_dev(qudax_ctx *ctx, double *const *dev_x, const double *const *dev_b,
                                            int nrhs, const qudax_solve_param *p, qudax_solve_stats *st);

/* CGNR ("Conjugate Gradients [7] on the normal equations"): CG on
 * Mhat^dag Mhat x_e = Mhat^dag bhat in precision p->prec (prec_sloppy and delta ignored), with
 * the same Schur prepare / reconstruct and the same TRUE-residual stopping test as BiCGstab. */
qudax_status qudax_solve_cgnr(qudax_ctx *ctx, double *host_x, const double *host_b,
                              const qudax_solve_param *p, qudax_solve_stats *st);
qudax_status qudax_solve_cgnr_dev(qudax_ctx *ctx, double *dev_x, const double *dev_b,
                                  const qudax_solve_param *p, qudax_solve_stats *st);

#ifdef __cplusplus
}
#endif
#endif /* QUDAX_H */
