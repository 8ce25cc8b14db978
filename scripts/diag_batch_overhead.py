"""Where the solver step's time outside the kernels goes: per-iteration time of the bench
workload (32^3x64, double-single) from solves of 100 and 200 iterations, for several batch sizes
(poll_every), against eager launches — the difference of the two lengths removes the fixed
per-solve work (Schur prepare / reconstruct, import / export, final residual).

    python scripts/diag_batch_overhead.py
"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
os.environ.setdefault("NCCL_GRAPH_MIXING_SUPPORT", "0")

import numpy as np  # noqa: E402
import torch  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402


def main():
    dims = (32, 32, 32, 64)
    U = qgen.gauge(dims, 1005, eps=0.1)
    b_host = qgen.spinor(dims, 2005)
    for flags in (0, qudax.FLAG_NO_GRAPHS):
        ctx = qudax.Context(dims, flags=flags)
        ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12, t_boundary=-1)
        with torch.cuda.stream(ctx.stream):
            b = torch.from_numpy(b_host.view(np.float64).reshape(-1)).cuda()
            x = torch.zeros_like(b)
        ctx.stream.synchronize()
        for poll in ((4, 16, 64) if flags == 0 else (16,)):
            res = {}
            for iters in (100, 200):
                kw = dict(tol=0.0, delta=1e-3, maxiter=iters, prec=8, prec_sloppy=4, allow_not_converged=True,
                          poll_every=poll)
                for _ in range(2):
                    ctx.solve_dev(x, b, **kw)
                ts = []
                for _ in range(5):
                    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    e0.record(ctx.stream)
                    st = ctx.solve_dev(x, b, **kw)
                    e1.record(ctx.stream)
                    e1.synchronize()
                    ts.append(e0.elapsed_time(e1))
                res[iters] = (sorted(ts)[2], st)
            per_it = (res[200][0] - res[100][0]) / 100.0
            # kernel time per iteration: the same 100 extra iterations with per-launch events
            ctx.kernel_timing(True)
            ctx.solve_dev(x, b, tol=0.0, delta=1e-3, maxiter=100, prec=8, prec_sloppy=4, allow_not_converged=True,
                          poll_every=poll)
            ks = ctx.kernel_stats()
            ctx.kernel_timing(False)
            print(json.dumps({"flags": flags, "poll_every": poll, "ms_100": res[100][0], "ms_200": res[200][0],
                              "ms_per_iteration": per_it, "updates_100": res[100][1]["reliable_updates"],
                              "updates_200": res[200][1]["reliable_updates"],
                              "host_polls_100": res[100][1]["host_polls"],
                              "dslash_ms_per_100_iters_events": ks["ms_total"],
                              "dslash_launches": ks["launches"]}), flush=True)
        ctx.close()


if __name__ == "__main__":
    main()
