"""Reliable-update threshold delta for the fp64-outer solves (paper gives no value for
double-single; reading Q11): iterations, updates, time and true residual of the 6
config-3 point sources (24^3x128, tol 1e-14) per delta, device buffers."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
for ps in (4, 2):
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=ps, recon_sloppy=12, t_boundary=-1)
    srcs = [torch.from_numpy(qgen.point_source(dims, s, c).view(np.float64).reshape(-1)).cuda() for c in range(3) for s in range(2)]
    x = torch.zeros_like(srcs[0])
    ctx.solve_dev(x, srcs[0], tol=0, delta=0.1, maxiter=3, prec=8, prec_sloppy=ps, allow_not_converged=True)
    for delta in (0.1, 0.03, 0.01, 0.003, 0.001):
        its, ups, tr, ts = [], [], [], []
        for b in srcs:
            torch.cuda.synchronize(); t = time.perf_counter()
            st = ctx.solve_dev(x, b, tol=1e-14, delta=delta, maxiter=4000, prec=8, prec_sloppy=ps, allow_not_converged=True)
            torch.cuda.synchronize(); ts.append(time.perf_counter() - t)
            its.append(st["iters"]); ups.append(st["reliable_updates"]); tr.append(st["true_res"])
        print(f"sloppy {ps} delta {delta}: iters {its} updates {ups} max true res {max(tr):.2e} mean time {np.mean(ts)*1e3:.1f} ms", flush=True)
ctx.close()
