// dslash_f32.cu — instantiation of the Dslash kernel family for storage precision 4 bytes/real
// (split per precision so the 18 variants per precision compile in parallel).
#include <cstdlib>

#include "dslash.cuh"
#include "matpc_fused.cuh"

namespace qx {
void launch_dslash_f32_ss(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
void launch_dslash_f32(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    static const bool force_ss = std::getenv("QUDAX_FORCE_SS") != nullptr;  // debug: SS variant everywhere
    if (a.smask || force_ss) launch_dslash_f32_ss(recon, dagger, kind, a, s);  // partitioned X / Y / Z
    else launch_dslash_prec<4>(recon, dagger, kind, a, s);
}
int dslash_threads() { return QX_DSLASH_THREADS; }
int dslash_blocks_f32(int recon, int dagger, int kind, int nthreads) {
    return dslash_blocks_prec<4>(recon, dagger, kind, nthreads);
}
void launch_matpc_fused_f32(int recon, int dagger, const FusedArgs &f, int grid, cudaStream_t s) {
    launch_matpc_fused_prec<4>(recon, dagger, f, grid, s);
}
int matpc_fused_wave_f32(int recon, int dagger) { return matpc_fused_wave<4>(recon, dagger); }
}  // namespace qx
