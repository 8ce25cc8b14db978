// dslash_f32_ss.cu — the Dslash kernel family for storage precision 4 bytes/real in its
// partitioned-X/Y/Z variant (ghost-aware spatial hops), compiled apart so
// the unpartitioned kernels keep their register allocation and both compile in parallel.
#include "dslash.cuh"

namespace qx {
void launch_dslash_f32_ss(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    launch_dslash_prec<4, true>(recon, dagger, kind, a, s);
}
}  // namespace qx
