import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import qgen
from paper_1011_0024_b200 import qudax
dims = tuple(int(v) for v in (sys.argv[1] if len(sys.argv) > 1 else "24,24,24,128").split(","))
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
b = qgen.point_source(dims, 0, 0)
for name, P, R, Ps, delta, tol in [("double-single", 8, 18, 4, 0.1, 1e-14), ("double-half", 8, 18, 2, 1e-2, 1e-14),
                                   ("single-half", 4, 12, 2, 0.1, 1e-7), ("double-half d=0.1", 8, 18, 2, 0.1, 1e-14)]:
    ctx.gauge_load(U, 0.124, 1.0, prec=P, recon=R, prec_sloppy=Ps, recon_sloppy=12)
    h = np.zeros(3000)
    x, st = ctx.solve(b, tol=tol, delta=delta, maxiter=3000, prec=P, prec_sloppy=Ps, allow_not_converged=True, history=h)
    n = st["iters"]
    print(name, {k: st[k] for k in ("iters", "reliable_updates", "true_res", "secs")})
    print("   hist[::20]", np.array2string(h[:n:20][:40], precision=1))
