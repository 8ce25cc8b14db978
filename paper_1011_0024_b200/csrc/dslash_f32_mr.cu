// dslash_f32_mr.cu — the multi-RHS (several right-hand sides per thread) Dslash family for
// storage precision 4 bytes/real (dslash_mr.cuh), compiled apart from dslash_f32.cu.
#include "dslash_mr.cuh"

namespace qx {
bool launch_dslash_mr_f32(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    return launch_dslash_mr_prec<4>(recon, dagger, kind, a, s);
}
}  // namespace qx
