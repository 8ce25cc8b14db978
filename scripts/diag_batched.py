"""Debug: steady-state time of a batched solve vs single solves (fixed iteration count, device
slabs, so host copies and convergence schedules do not enter)."""
import sys
import time
sys.path.insert(0, ".")
import torch
import qgen
from paper_1011_0024_b200 import qudax

dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
ps = int(sys.argv[1]) if len(sys.argv) > 1 else 4
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=ps, recon_sloppy=12)
n = 6
bs = [torch.from_numpy(qgen.point_source(dims, s, c).view("float64")).cuda() for c in range(3) for s in range(2)]
xs = [torch.zeros_like(b) for b in bs]
for iters in (10, 110):
    for rep in range(2):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        sts = ctx.solve_multi_dev(xs, bs, tol=0, delta=0.1, maxiter=iters, prec=8, prec_sloppy=ps, allow_not_converged=True)
        tm = time.perf_counter() - t0
        t0 = time.perf_counter()
        for x, b in zip(xs, bs):
            ctx.solve_dev(x, b, tol=0, delta=0.1, maxiter=iters, prec=8, prec_sloppy=ps, allow_not_converged=True)
        torch.cuda.synchronize()
        t1 = time.perf_counter() - t0
        print(f"iters {iters} rep {rep}: batched {tm*1e3:.1f} ms, 6 singles {t1*1e3:.1f} ms, updates {[s['reliable_updates'] for s in sts]}")
