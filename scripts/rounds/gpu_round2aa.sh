#!/bin/bash
# Round-2 pass AA: L2-aware kernel directions in the BiCGstab iteration (head, QX_SOLVER_ORDER 1)
# vs the previous order (lib_var/order0), alternating on one box; solver tests; NCCL-loopback
# solve statistics (does its iteration fit a WHILE node?).
TAG=${1:-r02aa}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py tests/gpu/test_multirhs.py -x -q > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
for r in 1 2 3; do
  for L in default order0; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.$r.json 2> $OUT/step_$L.$r.err
  done
done
unset QUDAX_LIB
timeout 300 python - > $OUT/loopback_stats.txt 2>&1 <<'PY'
import qgen
from paper_1011_0024_b200 import qudax
dims = (16, 16, 16, 32)
U = qgen.gauge(dims, 1003, eps=0.1)
b = qgen.point_source(dims, 0, 0)
for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
    for ov in (False, True):
        ctx = qudax.Context(dims, comm=comm, overlap=ov, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        for _ in range(2):
            x, st = ctx.solve(b, tol=1e-12, delta=1e-3, maxiter=2000, prec=8, prec_sloppy=4)
        print("comm", comm, "overlap", ov, {k: st[k] for k in ("iters", "reliable_updates", "host_polls", "device_batches", "true_res", "secs")})
        ctx.close()
PY
ls -la $OUT
