#!/bin/bash
# Round-2 pass AB: which graph node of the NCCL-loopback iteration keeps it out of a WHILE body.
TAG=${1:-r02ab}
OUT=gpurun_out/$TAG
mkdir -p $OUT
cat > /tmp/lb.py <<'PY'
import qgen
from paper_1011_0024_b200 import qudax
dims = (16, 16, 16, 32)
U = qgen.gauge(dims, 1003, eps=0.1)
b = qgen.point_source(dims, 0, 0)
for ov in (False, True):
    ctx = qudax.Context(dims, comm=qudax.COMM_NCCL, overlap=ov, nccl_id=qudax.nccl_unique_id())
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    for _ in range(2):
        x, st = ctx.solve(b, tol=1e-12, delta=1e-3, maxiter=2000, prec=8, prec_sloppy=4)
    print("overlap", ov, {k: st[k] for k in ("iters", "host_polls", "device_batches", "secs")}, flush=True)
    ctx.close()
PY
PYTHONPATH=$PWD timeout 300 python /tmp/lb.py > $OUT/default.txt 2>&1
NCCL_GRAPH_MIXING_SUPPORT=0 PYTHONPATH=$PWD timeout 300 python /tmp/lb.py > $OUT/nomixing.txt 2>&1
ls -la $OUT
