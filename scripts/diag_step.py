"""Break the bench step down: Mhat alone vs solver iterations with / without reliable updates."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402

dims = (32, 32, 32, 64)
U = qgen.gauge(dims, 1005, eps=0.1)
b = qgen.spinor(dims, 2005)
ctx = qudax.Context(dims)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
bd = torch.from_numpy(b.view(np.float64)).cuda()
xd = torch.zeros_like(bd)
torch.cuda.synchronize()


def timed(fn, n=3):
    fn()
    ctx.sync()
    t = time.perf_counter()
    for _ in range(n):
        fn()
    ctx.sync()
    return (time.perf_counter() - t) / n


fi, fo = ctx.new_field(4), ctx.new_field(4)
ctx.spinor_load_dev(fi, 4, 0, bd)
m = timed(lambda: [ctx.matpc(fo, fi, 4) for _ in range(100)])
print(f"100 Mhat fp32-12: {m*1e3:.2f} ms  ({m*1e4:.1f} us each)")
for label, kw in [("delta=0.1 mixed", dict(delta=0.1, prec=8, prec_sloppy=4)),
                  ("delta=0 mixed (1 update)", dict(delta=0.0, prec=8, prec_sloppy=4)),
                  ("delta=0 uniform fp32", dict(delta=0.0, prec=4, prec_sloppy=4))]:
    st = {}

    def run():
        st.update(ctx.solve_dev(xd, bd, tol=0.0, maxiter=100, allow_not_converged=True, **kw))
    t = timed(run)
    print(f"solve 100 it {label}: {t*1e3:.2f} ms  updates {st['reliable_updates']}  per-iter {t*1e4:.1f} us")
ctx.kernel_timing(True)
ctx.solve_dev(xd, bd, tol=0.0, maxiter=100, delta=0.0, prec=4, prec_sloppy=4, allow_not_converged=True)
ks = ctx.kernel_stats()
print("dslash in solve:", ks["launches"], "launches", ks["ms_total"] / ks["launches"] * 1e3, "us avg")
ctx.kernel_timing(False)
