// matpc_fused.cuh — Mhat = T_ee - kappa^2 D_eo T_oo^{-1} D_oe as ONE persistent
// kernel that keeps the intermediate T_oo^{-1} D_oe x and the links in the 126 MB L2.
//
// The two Dslash kernels of Mhat each stream the whole gauge field (384 of the 1824
// compulsory bytes per site in fp32-12) and the second re-reads the first one's output.  Here
// both phases run in a single launch as a wavefront in T: work items are (phase, timeslice,
// chunk of 128 sites), dispensed in a fixed order by an atomic counter —
//   A(t): tmp_o(t) = T_oo^{-1} D_oe x_e        on the odd sites of timeslice t
//   B(t): out_e(t) = T_ee x_e - kappa^2 D_eo tmp_o  on the even sites of timeslice t
// with B(t) issued LAG timeslices behind A, so the links and tmp_o it needs (timeslices
// t-1, t, t+1) were touched moments earlier and are still in L2.  B(t) waits (per-timeslice
// completion counters) until A(t-1), A(t), A(t+1) are done.  Deadlock-free for any number of
// resident CTAs: an item only ever waits for items dispensed before it, and those are held
// by running CTAs that never wait on later items.  Single-GPU (unpartitioned) only: a
// partitioned Mhat needs a halo exchange of tmp_o between the phases and uses the two-kernel
// path.  Per-site arithmetic is dslash_site, so results are bitwise those of the two kernels.
#pragma once
#include "dslash.cuh"

#ifndef QX_FUSED_INMODE
#define QX_FUSED_INMODE 0
#endif

namespace qx {

__device__ __forceinline__ unsigned ld_acquire_u32(const unsigned *p) {
    unsigned v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}

template <int P, int RECON, bool DAG>
__global__ void __launch_bounds__(QX_DSLASH_THREADS, QX_MINB_OF(P)) matpc_fused_kernel(const __grid_constant__ FusedArgs f) {
    __shared__ int s_item;
    double red[3] = {0.0, 0.0, 0.0};
    const int T = f.A.T_loc, F = f.A.F, chunks = f.chunks;
    // the next item is requested one round ahead so the atomic's latency overlaps the work
    // (still deadlock-free: the smallest unfinished item is always some CTA's current item)
    if (threadIdx.x == 0) s_item = (int)atomicAdd(f.work, 1u);
    for (;;) {
        __syncthreads();
        const int item = s_item;
        __syncthreads();  // s_item is rewritten below
        if (item >= f.total_items) break;
        if (threadIdx.x == 0) s_item = (int)atomicAdd(f.work, 1u);
        const int stage = f.stages[item / chunks];
        const int chunk = item % chunks;
        const bool phaseB = stage >= T;
        const int t = phaseB ? stage - T : stage;
        const int j = chunk * QX_DSLASH_THREADS + (int)threadIdx.x;
        const int site = t * F + j;
        if (!phaseB) {
            if (j < F) dslash_site<P, RECON, DAG, QUDAX_CLOVER_INV, 0>(f.A, f.A.in, f.A.out, nullptr, site, red);
            __threadfence();
            __syncthreads();
            if (threadIdx.x == 0) atomicAdd(f.doneA + t, 1u);
        } else {
            if (threadIdx.x == 0) {
                const int tm = t == 0 ? T - 1 : t - 1, tp = t == T - 1 ? 0 : t + 1;
                // bounded: a broken dependency order must surface as a wrong result, never a hang
                for (long spin = 0; spin < (1L << 26); ++spin) {
                    if (ld_acquire_u32(f.doneA + tm) >= (unsigned)chunks && ld_acquire_u32(f.doneA + t) >= (unsigned)chunks &&
                        ld_acquire_u32(f.doneA + tp) >= (unsigned)chunks)
                        break;
                    __nanosleep(64);
                }
            }
            __syncthreads();
            // tmp_o lines are final before any CTA reads them (B waits for A), so even the
            // non-coherent read-only path can never see stale data (QX_FUSED_INMODE=2: L2-only)
            if (j < F) dslash_site<P, RECON, DAG, QUDAX_CLOVER_XPAY, QX_FUSED_INMODE>(f.B, f.B.in, f.B.out, f.B.x, site, red);
        }
    }
    if (f.B.red_kind != RED_NONE) reduce_with_tail<3, QX_DSLASH_THREADS>(red, f.B.tail);
}

template <int P>
int matpc_fused_wave(int recon, int dagger) {
    static int cache[2][3] = {{0, 0, 0}, {0, 0, 0}};
    const int ri = recon == 18 ? 0 : (recon == 12 ? 1 : 2);
    int &w = cache[dagger ? 1 : 0][ri];
    if (w) return w;
    int dev = 0, sms = 0, per = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
#define QX_FW(RC, DG) \
    if (recon == RC && (bool)dagger == DG) \
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, matpc_fused_kernel<P, RC, DG>, QX_DSLASH_THREADS, 0);
    QX_FW(18, false) QX_FW(18, true) QX_FW(12, false) QX_FW(12, true) QX_FW(8, false) QX_FW(8, true)
#undef QX_FW
    w = sms * (per > 0 ? per : 1);
    return w;
}

template <int P>
void launch_matpc_fused_prec(int recon, int dagger, const FusedArgs &f, int grid, cudaStream_t s) {
#define QX_FL(RC, DG)                                                                        \
    if (recon == RC && (bool)dagger == DG) {                                                 \
        matpc_fused_kernel<P, RC, DG><<<grid, QX_DSLASH_THREADS, 0, s>>>(f);                 \
        return;                                                                              \
    }
    QX_FL(18, false) QX_FL(18, true) QX_FL(12, false) QX_FL(12, true) QX_FL(8, false) QX_FL(8, true)
#undef QX_FL
    throw Error(QUDAX_ERR_ARG, "fused matpc: unsupported recon");
}

}  // namespace qx
