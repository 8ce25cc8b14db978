// reduce.cuh — deterministic grid reductions with "last CTA finishes" tails, and the
// device-side BiCGstab scalar recurrences (Algorithm R, csrc/solver.cpp).
//
// Every CTA writes its fp64 partial sums to a fixed slot.  Two-level tail: CTAs form groups
// of kGroup consecutive slots; the last CTA of a group to arrive sums that group's slots in
// index order into a group slot; the last group to finish sums the group slots in index
// order, writes the totals, optionally advances the solver scalars, and resets the counters.
// The result never depends on arrival order (bitwise reproducible, reading Q12), and no CTA
// reads more than max(kGroup, n_groups) partials — a single-CTA sweep over the 8192 partials
// of a Dslash launch measured 10+ us of serial tail.
#pragma once
#include "internal.h"

namespace qx {

constexpr int kGroup = 64;
static_assert(kGroup == kGroupHost, "host-side slot sizing (internal.h) must match");

__device__ __forceinline__ double2 cdiv(double2 a, double2 b) {
    const double d = b.x * b.x + b.y * b.y;
    return make_double2((a.x * b.x + a.y * b.y) / d, (a.y * b.x - a.x * b.y) / d);
}
__device__ __forceinline__ double2 cmul(double2 a, double2 b) {
    return make_double2(a.x * b.x - a.y * b.y, a.x * b.y + a.y * b.x);
}

// BiCGstab recurrences from the globally summed S->red (complex numbers stored (re, im))
__device__ __forceinline__ void apply_coef(SolverScalars *S, int mode) {
    const double *r = S->red;
    if (mode == COEF_ALPHA) {          // alpha = rho' / <rhat0, v>
        S->alpha = cdiv(S->rho_new, make_double2(r[0], r[1]));
        S->malpha = make_double2(-S->alpha.x, -S->alpha.y);
    } else if (mode == COEF_OMEGA) {   // omega = <t, s> / |t|^2
        S->omega = make_double2(r[0] / r[2], r[1] / r[2]);
    } else if (mode == COEF_RHO) {     // |r|^2, rho' = <rhat0, r>, beta = (rho'/rho)(alpha/omega)
        S->r2 = r[0];
        S->rho = S->rho_new;
        S->rho_new = make_double2(r[1], r[2]);
        S->beta = cmul(cdiv(S->rho_new, S->rho), cdiv(S->alpha, S->omega));
        if (S->decide) {
            // Algorithm R's update rule (solver.cpp header), the same comparisons in the same
            // order as the host-side version it replaces
            const double rn = sqrt(S->r2);
            S->k += 1;
            S->hist[(S->k - 1) % kHistRing] = rn;
            S->rNorm = rn;
            const bool blown = !isfinite(rn) || rn > 1e2 * S->maxrr;  // reading R3
            if (!blown) {
                if (rn > S->maxrx) S->maxrx = rn;
                if (rn > S->maxrr) S->maxrr = rn;
            }
            const bool updX = !blown && (rn < S->delta * S->r0Norm) && (S->r0Norm <= S->maxrx);
            const bool updR = blown || ((rn < S->delta * S->maxrr) && (S->r0Norm <= S->maxrr)) || updX ||
                              (rn <= S->stop) || (S->k >= S->maxiter);
            if (updR) {
                S->updX = updX;
                S->blown = blown;
                S->halt = 1;
            }
        }
    }
}

// Publishing a partial: a release atomic orders this thread's earlier slot stores before the
// counter update (MEMBAR.ALL.GPU + ATOM) — __threadfence() + atomicAdd is a sequentially
// consistent fence that also invalidates the SM's L1 (CCTL.IVALL) in every CTA, dropping the
// neighbour spinors the other resident CTAs are reusing.  Only the CTA that finishes a group
// acquires (and invalidates) before reading the other CTAs' slots.
__device__ __forceinline__ unsigned atomic_add_release(unsigned *p, unsigned v) {
    unsigned prev;
    asm volatile("atom.add.release.gpu.global.u32 %0, [%1], %2;" : "=r"(prev) : "l"(p), "r"(v) : "memory");
    return prev;
}
__device__ __forceinline__ void fence_acquire() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }

// CTA-wide fixed-order sum of slots [b0, b1) of `src` (NRED values per slot) -> thread 0's out
template <int NRED, int NT>
__device__ __forceinline__ void cta_sum_slots(const double *src, int b0, int b1, double (&res)[NRED],
                                              double (&sm)[NT / 32][NRED]) {
    double acc[NRED];
#pragma unroll
    for (int k = 0; k < NRED; ++k) acc[k] = 0.0;
    for (int b = b0 + (int)threadIdx.x; b < b1; b += NT)
#pragma unroll
        for (int k = 0; k < NRED; ++k) acc[k] += __ldcg(src + (size_t)b * NRED + k);
#pragma unroll
    for (int k = 0; k < NRED; ++k)
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) acc[k] += __shfl_xor_sync(0xffffffffu, acc[k], o);
    __syncthreads();
    if ((threadIdx.x & 31) == 0)
#pragma unroll
        for (int k = 0; k < NRED; ++k) sm[threadIdx.x >> 5][k] = acc[k];
    __syncthreads();
    if (threadIdx.x == 0)
        for (int k = 0; k < NRED; ++k) {
            double s = 0.0;
            for (int w = 0; w < NT / 32; ++w) s += sm[w][k];
            res[k] = s;
        }
}

// Kernel-side global sum (DevAllreduce, internal.h) of the NRED totals in v, by one thread.
__device__ __forceinline__ unsigned long long ld_acquire_sys_u64(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_release_sys_u64(unsigned long long *p, unsigned long long v) {
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
template <int NRED>
__device__ __forceinline__ void dev_allreduce(const DevAllreduce &d, int chan, double (&v)[NRED]) {
    static_assert(NRED <= 3, "slot holds 3 sums");
    const unsigned s = d.seq[chan] + 1u;
    d.seq[chan] = s;
    const size_t base = ((size_t)chan * 2 + (s & 1u)) * kMaxPeers;
    for (int r = 0; r < d.nranks; ++r) {  // this rank's totals into slot [rank] of every rank
        double *dst = d.slots[r] + (base + d.rank) * 4;
        for (int k = 0; k < NRED; ++k) dst[k] = v[k];
        st_release_sys_u64(reinterpret_cast<unsigned long long *>(dst + 3), (unsigned long long)s);
    }
    double tot[NRED];
    for (int k = 0; k < NRED; ++k) tot[k] = 0.0;
    const double *own = d.slots[d.rank];
    for (int r = 0; r < d.nranks; ++r) {  // fixed rank order: bitwise identical on every rank
        const double *src = own + (base + r) * 4;
        const unsigned long long *sq = reinterpret_cast<const unsigned long long *>(src + 3);
        bool ok = false;
        for (long spin = 0; spin < (1L << 24) && !ok; ++spin) {
            ok = ld_acquire_sys_u64(sq) == (unsigned long long)s;
            if (!ok) __nanosleep(64);
        }
        if (!ok && d.err) atomicExch(d.err, 2);
        for (int k = 0; k < NRED; ++k) tot[k] += *reinterpret_cast<const volatile double *>(src + k);
    }
    for (int k = 0; k < NRED; ++k) v[k] = tot[k];
}

// v[] -> this CTA's partial; the last CTA of the whole reduction produces t.out[0..NRED).
// Layout: t.partials[0 .. total) CTA slots, then ceil(total/kGroup) group slots.
// Counters: t.counter[0] groups done, t.counter[1 + g] CTAs done in group g (all zero on entry).
// blk: this CTA's index within the reduction (-1: blockIdx.x)
// Callers that run it twice in one kernel need a __syncthreads() between the calls: in the CTA
// that finishes a reduction, thread 0 is still reading the shared scratch when the others return.
template <int NRED, int NT>
__device__ __forceinline__ void reduce_with_tail(double (&v)[NRED], const RedTail &t, int blk = -1) {
    __shared__ double sm[NT / 32][NRED];
    __shared__ int stage;  // 0: not last in group; 1: last in group; 2: last overall
    const int gb = t.block_offset + (blk < 0 ? (int)blockIdx.x : blk);
    const int ngroups = (t.total_blocks + kGroup - 1) / kGroup;
    const int grp = gb / kGroup;
    double *gslots = t.partials + (size_t)t.total_blocks * NRED;
#pragma unroll
    for (int k = 0; k < NRED; ++k)
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) v[k] += __shfl_xor_sync(0xffffffffu, v[k], o);
    if ((threadIdx.x & 31) == 0)
#pragma unroll
        for (int k = 0; k < NRED; ++k) sm[threadIdx.x >> 5][k] = v[k];
    __syncthreads();
    if (threadIdx.x == 0) {
        for (int k = 0; k < NRED; ++k) {
            double s = 0.0;
            for (int w = 0; w < NT / 32; ++w) s += sm[w][k];
            t.partials[(size_t)gb * NRED + k] = s;
        }
        const int gsize = min(kGroup, t.total_blocks - grp * kGroup);
        const unsigned prev = atomic_add_release(t.counter + 1 + grp, 1u);
        stage = (prev == (unsigned)gsize - 1u) ? 1 : 0;
    }
    __syncthreads();
    if (stage == 0) return;
    fence_acquire();
    double res[NRED];
    cta_sum_slots<NRED, NT>(t.partials, grp * kGroup, min(t.total_blocks, (grp + 1) * kGroup), res, sm);
    if (threadIdx.x == 0) {
        for (int k = 0; k < NRED; ++k) gslots[(size_t)grp * NRED + k] = res[k];
        t.counter[1 + grp] = 0u;
        const unsigned prev = atomic_add_release(t.counter, 1u);
        stage = (prev == (unsigned)ngroups - 1u) ? 2 : 0;
    }
    __syncthreads();
    if (stage != 2) return;
    fence_acquire();
    cta_sum_slots<NRED, NT>(gslots, 0, ngroups, res, sm);
    if (threadIdx.x == 0) {
        if (t.dar) dev_allreduce<NRED>(*t.dar, t.chan, res);  // the global sum, in-kernel
        for (int k = 0; k < NRED; ++k) t.out[k] = res[k];
        if (t.coef_mode != COEF_NONE) apply_coef(t.S, t.coef_mode);
        t.counter[0] = 0u;  // ready for the next stream-ordered reduction
    }
}

}  // namespace qx
