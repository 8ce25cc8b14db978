"""Multi-RHS (two per thread) vs single-RHS Dslash at a large lattice, bitwise, every kind;
then the batched vs independent double-half solve of the config-3 sources (iterations)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = tuple(int(v) for v in os.environ.get("DIMS", "24,24,24,128").split(","))
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
for prec in (2, 4):
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=prec, recon_sloppy=12, t_boundary=-1)
    n = 3
    psis = [qgen.spinor(dims, 50 + k) for k in range(n)]
    ins = [ctx.new_field(prec) for _ in range(n)]
    xs = [ctx.new_field(prec) for _ in range(n)]
    for k in range(n):
        ctx.spinor_load(ins[k], prec, 1, psis[k])
        ctx.spinor_load(xs[k], prec, 0, psis[(k + 1) % n])
    for kind, a in ((0, -0.3), (1, -0.3), (2, -0.015376), (3, -0.3)):
        outs = [ctx.new_field(prec) for _ in range(n)]
        ctx.dslash_multi(outs, ins, prec, 0, dagger=False, kind=kind, xs=xs, a=a)
        bad = []
        for k in range(n):
            single = ctx.new_field(prec)
            ctx.dslash(single, ins[k], prec, 0, dagger=False, kind=kind, x=xs[k], a=a)
            ctx.sync()
            if not bool((single == outs[k]).all()):
                bad.append((k, int((single != outs[k]).sum())))
        print("prec", prec, "kind", kind, "mismatches", bad, flush=True)
srcs = [qgen.point_source(dims, s, c) for c in range(3) for s in range(2)]
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12, t_boundary=-1)
_, sts = ctx.solve_multi(srcs, tol=1e-14, delta=1e-2, maxiter=4000, prec=8, prec_sloppy=2)
ind = [ctx.solve(b, tol=1e-14, delta=1e-2, maxiter=4000, prec=8, prec_sloppy=2)[1] for b in srcs]
print("batched iters", [s["iters"] for s in sts], "independent", [s["iters"] for s in ind], flush=True)
ctx.close()
