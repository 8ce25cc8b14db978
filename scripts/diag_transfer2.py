"""Host-buffer solve overhead split: fresh output array (first-touch page faults inside the
call) vs a reused, already-touched output array; QUDAX_COPY_THREADS varied by the caller."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12, t_boundary=-1)
b = qgen.point_source(dims, 0, 0)
kw = dict(tol=1e-14, delta=1e-2, maxiter=20000, prec=8, prec_sloppy=2)
ctx.solve(b, tol=0, delta=1e-2, maxiter=3, prec=8, prec_sloppy=2, allow_not_converged=True)
for _ in range(2):
    _, st = ctx.solve(b, **kw)
    print("fresh out   :", round(st["secs"] * 1e3, 1), "ms", flush=True)
out = np.ones_like(b)
for _ in range(2):
    _, st = ctx.solve(b, out=out, **kw)
    print("reused out  :", round(st["secs"] * 1e3, 1), "ms", flush=True)
bd = torch.from_numpy(b.view(np.float64).reshape(-1)).cuda()
xd = torch.zeros_like(bd)
for _ in range(2):
    torch.cuda.synchronize(); t = time.perf_counter()
    ctx.solve_dev(xd, bd, **kw); torch.cuda.synchronize()
    print("device bufs :", round((time.perf_counter() - t) * 1e3, 1), "ms", flush=True)
ctx.close()
