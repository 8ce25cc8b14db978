// dslash_f16.cu — instantiation of the Dslash kernel family for storage precision 2 bytes/real
// (split per precision so the 18 variants per precision compile in parallel).
#include "dslash.cuh"

namespace qx {
void launch_dslash_f16_ss(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s);
void launch_dslash_f16(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    // partitioned X / Y / Z, or the test flag that runs that instantiation everywhere
    if (a.smask || (a.variant & kVariantForceSS)) launch_dslash_f16_ss(recon, dagger, kind, a, s);  // partitioned X / Y / Z
    else launch_dslash_prec<2>(recon, dagger, kind, a, s);
}
int dslash_blocks_f16(int recon, int dagger, int kind, int nthreads) {
    return dslash_blocks_prec<2>(recon, dagger, kind, nthreads);
}
}  // namespace qx
