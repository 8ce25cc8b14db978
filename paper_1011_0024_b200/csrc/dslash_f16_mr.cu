// dslash_f16_mr.cu — the multi-RHS (several right-hand sides per thread) Dslash family for
// storage precision 2 bytes/real (dslash_mr.cuh), compiled apart from dslash_f16.cu.
#include "dslash_mr.cuh"

namespace qx {
bool launch_dslash_mr_f16(int recon, int dagger, int kind, const DslashArgs &a, cudaStream_t s) {
    return launch_dslash_mr_prec<2>(recon, dagger, kind, a, s);
}
}  // namespace qx
