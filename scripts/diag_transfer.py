"""Where the config-3 host-buffer solve time goes: pageable vs pinned H2D/D2H of one 24^3x128
fp64 slab, and solve (host buffers) vs solve_dev (device buffers) for one point source."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
n = 24 * 24 * 24 * 128 * 24
host = np.random.default_rng(0).standard_normal(n)
pin = torch.empty(n, dtype=torch.float64).pin_memory()
dev = torch.empty(n, dtype=torch.float64, device="cuda")
for label, src in (("pageable", torch.from_numpy(host)), ("pinned", pin)):
    for _ in range(2):
        torch.cuda.synchronize(); t = time.perf_counter(); dev.copy_(src); torch.cuda.synchronize()
        h2d = time.perf_counter() - t
        t = time.perf_counter(); src.copy_(dev); torch.cuda.synchronize()
        d2h = time.perf_counter() - t
    print(f"{label}: H2D {h2d*1e3:.1f} ms ({n*8/h2d/1e9:.1f} GB/s), D2H {d2h*1e3:.1f} ms ({n*8/d2h/1e9:.1f} GB/s)", flush=True)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12, t_boundary=-1)
b = qgen.point_source(dims, 0, 0)
ctx.solve(b, tol=0, delta=0.1, maxiter=3, prec=8, prec_sloppy=4, allow_not_converged=True)
for _ in range(2):
    _, st = ctx.solve(b, tol=1e-14, delta=0.1, maxiter=20000, prec=8, prec_sloppy=4)
    print("solve (host buffers):", round(st["secs"], 4), st["iters"], flush=True)
bd = torch.from_numpy(b.view(np.float64).reshape(-1)).cuda()
xd = torch.zeros_like(bd)
for _ in range(2):
    torch.cuda.synchronize(); t = time.perf_counter()
    st = ctx.solve_dev(xd, bd, tol=1e-14, delta=0.1, maxiter=20000, prec=8, prec_sloppy=4)
    torch.cuda.synchronize()
    print("solve_dev:", round(time.perf_counter() - t, 4), st["iters"], flush=True)
ctx.close()
