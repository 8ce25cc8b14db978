"""Mixed-precision reliable-update BiCGstab through the C-ABI,
checked against the fp64 oracle: the oracle's own true residual of the GPU solution, the
GPU-reported residual vs the oracle's (|diff| <= 1e-9), and the solution vs the oracle solve."""
import numpy as np
import pytest

import oracle
import qgen
from paper_1011_0024_b200 import qudax

pytestmark = pytest.mark.gpu

DIMS = (8, 8, 8, 16)
KAPPA, CSW = 0.124, 1.0


@pytest.fixture(scope="module")
def system():
    U = qgen.gauge(DIMS, 1003, eps=0.1)  # weak field
    wc = oracle.WilsonClover(U, KAPPA, CSW, -1.0)
    return U, wc


@pytest.mark.parametrize("mode", [
    # (prec, recon, prec_sloppy, recon_sloppy, delta, tol)
    (8, 18, 4, 12, 0.1, 1e-12),   # double-single (reading Q11)
    (8, 18, 2, 12, 1e-2, 1e-12),  # double-half (P:787-790 delta = 1e-2)
    (8, 12, 8, 12, 1e-5, 1e-12),  # uniform double (delta = 1e-5)
    (4, 12, 2, 12, 0.1, 1e-6),    # single-half (delta = 1e-1), tol near fp32 floor
])
def test_solver_vs_oracle(torch_cuda, system, mode):
    U, wc = system
    prec, recon, ps, rs, delta, tol = mode
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=prec, recon=recon, prec_sloppy=ps, recon_sloppy=rs, t_boundary=-1)
    for spin, colour in ((0, 0), (1, 2)):
        b = qgen.point_source(DIMS, spin, colour)
        x, st = ctx.solve(b, tol=tol, delta=delta, maxiter=5000, prec=prec, prec_sloppy=ps)
        res_oracle = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
        print(mode, st["iters"], st["reliable_updates"], st["true_res"], res_oracle)
        if prec == 8:
            assert res_oracle <= tol * (1 + 1e-3) + 1e-15
            assert abs(st["true_res"] - res_oracle) <= 1e-9
        else:
            assert res_oracle <= tol * 1.5
        # solution vs oracle BiCGstab on the Schur system
        bh = wc.prepare(b)
        xe, _ = oracle.bicgstab(wc.matpc, bh, tol=1e-13, maxiter=5000)
        xo = wc.reconstruct(xe, b)
        assert np.linalg.norm(x - xo) / np.linalg.norm(xo) < (1e-9 if prec == 8 else 1e-4)
    ctx.close()


def test_uniform_double_tracks_oracle_history(torch_cuda, system):
    """Uniform fp64 with delta = 0 (no intermediate reliable updates) must follow the oracle's
    textbook BiCGstab residual history: pins the alpha / beta / omega recurrences."""
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18)
    b = qgen.point_source(DIMS, 0, 0)
    h = np.zeros(200)
    ctx.solve(b, tol=1e-12, delta=0.0, maxiter=200, prec=8, prec_sloppy=8, history=h)
    _, hist = oracle.bicgstab(wc.matpc, wc.prepare(b), tol=1e-12, maxiter=200)
    hist = np.array(hist)
    assert np.all(np.abs(h[:10] - hist[:10]) <= 1e-8 * hist[:10])
    ctx.close()


def test_solver_fixed_iterations_and_device_entry(torch_cuda, system):
    import torch
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    b = qgen.spinor(DIMS, 77)
    bd = torch.from_numpy(b.view(np.float64).copy()).cuda()
    xd = torch.zeros_like(bd)
    st = ctx.solve_dev(xd, bd, tol=0.0, delta=0.1, maxiter=7, prec=8, prec_sloppy=4, allow_not_converged=True)
    assert st["iters"] == 7
    x = xd.cpu().numpy().view(np.complex128).reshape(b.shape)
    res = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
    assert abs(res - st["true_res"]) < 1e-9
    ctx.close()


def test_loopback_solve_matches_unsplit(torch_cuda, system):
    """The solver through the split halo path (NCCL loopback at N=1, CUDA-graph replay with the
    NCCL p2p inside) reproduces the unsplit solve: the exchange moves bits only; only the
    grouping of the fused reductions' partial sums differs (interior/boundary CTAs)."""
    U, wc = system
    b = qgen.point_source(DIMS, 1, 0)
    xs = []
    for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
        ctx = qudax.Context(DIMS, comm=comm, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        x, st = ctx.solve(b, tol=1e-10, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4)
        xs.append((x, st["iters"]))
        ctx.close()
    assert abs(xs[0][1] - xs[1][1]) <= 1
    assert np.linalg.norm(xs[0][0] - xs[1][0]) / np.linalg.norm(xs[0][0]) < 1e-8


@pytest.mark.parametrize("prec,recon,tol", [(8, 18, 1e-12), (4, 12, 1e-5)])
def test_cgnr_vs_oracle(torch_cuda, system, prec, recon, tol):
    """CGNR on the normal equations: the oracle's fp64 true
    residual of the solution meets tol; the solution agrees with the oracle's BiCGstab one."""
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=prec, recon=recon, t_boundary=-1)
    b = qgen.point_source(DIMS, 0, 2)
    x, st = ctx.solve_cgnr(b, tol=tol, maxiter=5000, prec=prec)
    res = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
    print("cgnr", prec, st["iters"], st["true_res"], res)
    assert res <= tol * (1.5 if prec == 4 else 1.001)
    if prec == 8:
        assert abs(res - st["true_res"]) <= 1e-9
    ctx.close()


@pytest.mark.parametrize("mode", [(8, 18, 4, 12, 0.1), (8, 18, 2, 12, 0.1)])
def test_symmetric_schur_bicgstab_vs_oracle(torch_cuda, system, mode):
    """use_schur = 2: the symmetric form T_ee^{-1} Mhat.  The solver stops on
    the symmetric system's true residual; the full-system residual of the reconstructed x is
    reported and checked by the oracle (it differs from the Schur one by O(|T_ee|))."""
    U, wc = system
    prec, recon, ps, rs, delta = mode
    tol = 1e-12
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=prec, recon=recon, prec_sloppy=ps, recon_sloppy=rs, t_boundary=-1)
    its = {}
    for schur in (1, 2):
        b = qgen.point_source(DIMS, 0, 1)
        x, st = ctx.solve(b, tol=tol, delta=delta, maxiter=5000, prec=prec, prec_sloppy=ps, use_schur=schur)
        res_oracle = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
        print("schur", schur, mode, st["iters"], st["true_res"], res_oracle)
        assert res_oracle <= 10 * tol
        assert abs(st["true_res"] - res_oracle) <= 1e-9
        its[schur] = st["iters"]
    assert its[2] <= 1.2 * its[1] + 5
    ctx.close()


def test_symmetric_uniform_double_tracks_oracle_history(torch_cuda, system):
    """delta = 0 fp64 on the symmetric system follows the oracle's BiCGstab on
    (matpc_sym, prepare_sym) for its first 10 iterations."""
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18)
    b = qgen.point_source(DIMS, 1, 1)
    h = np.zeros(200)
    ctx.solve(b, tol=1e-12, delta=0.0, maxiter=200, prec=8, prec_sloppy=8, history=h, use_schur=2)
    _, hist = oracle.bicgstab(wc.matpc_sym, wc.prepare_sym(b), tol=1e-12, maxiter=200)
    hist = np.array(hist)
    assert np.all(np.abs(h[:10] - hist[:10]) <= 1e-8 * hist[:10])
    ctx.close()


def test_symmetric_cgnr_vs_oracle(torch_cuda, system):
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, t_boundary=-1)
    b = qgen.point_source(DIMS, 1, 2)
    x, st = ctx.solve_cgnr(b, tol=1e-12, maxiter=5000, prec=8, use_schur=2)
    res = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
    print("cgnr sym", st["iters"], st["true_res"], res)
    assert res <= 1e-11
    assert abs(res - st["true_res"]) <= 1e-9
    ctx.close()


@pytest.mark.parametrize("mode", [(4, 12, 0.1), (2, 12, 0.1)])
def test_batched_solve_equals_independent_solves(torch_cuda, system, mode):
    """Batched BiCGstab (6 sources per configuration): one
    multi-RHS Mhat kernel pair per iteration with per-system fused reductions.  Every system's
    iterations, reliable updates and solution are BITWISE those of its own single solve (same
    per-site code, same per-CTA reduction slots), and the oracle confirms each true residual."""
    U, wc = system
    ps, rs, delta = mode
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=ps, recon_sloppy=rs, t_boundary=-1)
    srcs = [qgen.point_source(DIMS, s, c) for s in (0, 1) for c in (0, 1, 2)]
    xs, sts = ctx.solve_multi(srcs, tol=1e-12, delta=delta, maxiter=5000, prec=8, prec_sloppy=ps)
    for b, x, st in zip(srcs, xs, sts):
        x1, st1 = ctx.solve(b, tol=1e-12, delta=delta, maxiter=5000, prec=8, prec_sloppy=ps)
        assert (st["iters"], st["reliable_updates"]) == (st1["iters"], st1["reliable_updates"])
        assert np.array_equal(x, x1)
        res_oracle = np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b)
        assert res_oracle <= 1e-12 * (1 + 1e-3) + 1e-15
        assert abs(st["true_res"] - res_oracle) <= 1e-9
    ctx.close()


def test_batched_solve_mixed_convergence(torch_cuda, system):
    """Systems that converge at different iterations leave the batch (the multi-RHS launches
    shrink); a zero source converges at once; maxiter caps are reported per system."""
    U, wc = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12, t_boundary=-1)
    b0 = qgen.point_source(DIMS, 0, 0)
    b1 = qgen.spinor(DIMS, 4242)          # a Gaussian source: more iterations than a point source
    bz = np.zeros_like(b0)
    xs, sts = ctx.solve_multi([b0, b1, bz], tol=1e-10, delta=0.1, maxiter=5000, prec=8, prec_sloppy=4)
    assert sts[2]["iters"] == 0 and not np.any(xs[2])
    assert sts[0]["iters"] != sts[1]["iters"]
    for b, x in zip((b0, b1), xs[:2]):
        assert np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b) <= 1e-10 * (1 + 1e-3)
    _, sts = ctx.solve_multi([b0, b1], tol=1e-14, delta=0.1, maxiter=7, prec=8, prec_sloppy=4,
                             allow_not_converged=True)
    assert all(s["iters"] == 7 for s in sts)
    ctx.close()


def test_half_sloppy_small_delta_stagnation_restart(torch_cuda):
    """Double-half with a small reliable-update threshold (delta 3e-3) on a config-3 source
    (24^3x128 weak field, colour 1 spin 0) whose residual decays by > 30 orders of magnitude
    across the lattice: half-precision sites with norms below ~1e-34 made 32767/norm overflow,
    the requantised values the fused reductions use turned into NaN (0 * inf), and every
    iteration broke down and restarted (true residual stuck at 2.5e-3 after 4000 iterations,
    scripts/diag_stall.py).  Such sites are now stored as zero (core.cuh kHalfTinyNorm)."""
    import torch
    dims = (24, 24, 24, 128)
    U = qgen.gauge(dims, 1003, eps=0.1)
    ctx = qudax.Context(dims)
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12, t_boundary=-1)
    b = torch.from_numpy(qgen.point_source(dims, 0, 1).view(np.float64).reshape(-1)).cuda()
    x = torch.zeros_like(b)
    st = ctx.solve_dev(x, b, tol=1e-14, delta=3e-3, maxiter=1500, prec=8, prec_sloppy=2, allow_not_converged=True)
    assert st["true_res"] <= 1e-14 * (1 + 1e-3), st
    assert st["iters"] < 600, st
    ctx.close()


def test_batched_equals_independent_at_config3_size(torch_cuda):
    """Batched double-half solve of the six config-3 point sources (24^3x128) takes exactly the
    iterations of the six independent solves.  Regression: the two-RHS-per-thread kernel ran
    two fused reductions back to back, and the CTA finishing the first one still read the shared
    scratch the second one was writing (rare, timing-dependent: a wrong global sum, then a
    different Krylov sequence — iterations 150-163 instead of 141 for source 0)."""
    dims = (24, 24, 24, 128)
    U = qgen.gauge(dims, 1003, eps=0.1)
    ctx = qudax.Context(dims)
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12, t_boundary=-1)
    srcs = [qgen.point_source(dims, s, c) for c in range(3) for s in range(2)]
    _, sts = ctx.solve_multi(srcs, tol=1e-14, delta=1e-2, maxiter=1000, prec=8, prec_sloppy=2)
    for b, st in zip(srcs, sts):
        _, one = ctx.solve(b, tol=1e-14, delta=1e-2, maxiter=1000, prec=8, prec_sloppy=2)
        assert (st["iters"], st["reliable_updates"]) == (one["iters"], one["reliable_updates"])
        assert st["true_res"] <= 1e-14 * (1 + 1e-3)
    ctx.close()


def test_poll_every_and_eager_are_bitwise_identical(torch_cuda, system):
    """Algorithm R's update rule runs on the device after every iteration; the host reads the
    scalars once per batch of up to poll_every iterations (one replay of a graph whose WHILE node
    loops over the iteration on the device), and an iteration that asks for a reliable update
    ends its batch.  The iterates must therefore not depend on the batch size or on graph replay:
    bitwise equal x, the same iteration count, updates and residual history for poll_every
    1 / 3 / 4 / 16 and with graphs disabled — and the batches must really run on the device
    (device_batches, host_polls)."""
    U, wc = system
    b = qgen.point_source(DIMS, 0, 1)
    runs = []
    for flags, poll in ((0, 1), (0, 3), (0, 4), (0, 16), (qudax.FLAG_NO_GRAPHS, 4)):
        ctx = qudax.Context(DIMS, flags=flags)
        ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        h = np.zeros(400)
        x, st = ctx.solve(b, tol=1e-12, delta=1e-2, maxiter=400, prec=8, prec_sloppy=4, history=h, poll_every=poll)
        runs.append((x, st, h))
        ctx.close()
        if flags & qudax.FLAG_NO_GRAPHS:
            assert st["device_batches"] == 0 and st["host_polls"] == st["iters"], st
        elif poll > 1:
            assert st["device_batches"] >= 1, st
            assert st["host_polls"] <= st["iters"] // poll + st["reliable_updates"] + 3, st
    x0, st0, h0 = runs[0]
    assert st0["reliable_updates"] >= 2
    for x, st, h in runs[1:]:
        assert st["iters"] == st0["iters"] and st["reliable_updates"] == st0["reliable_updates"]
        assert np.array_equal(x, x0)
        assert np.array_equal(h, h0)
    res = np.linalg.norm(wc.M(x0) - b) / np.linalg.norm(b)
    assert res <= 1e-12 * (1 + 1e-3)


def test_loopback_nccl_solve_bitwise_with_allreduce_in_graph(torch_cuda, system):
    """The N > 1 code path on one GPU: NCCL loopback without overlap (pack -> ncclSend/Recv to
    self -> one whole-lattice kernel, so the fused reductions keep the unsplit CTA grouping), the
    three per-iteration sums through ncclAllReduce on the one-rank communicator followed by the
    coefficient kernel, all captured in the cached iteration graph.  Must be bitwise equal to the
    unsplit solve (the exchange and the one-rank allreduce move bits only)."""
    U, wc = system
    b = qgen.point_source(DIMS, 1, 1)
    out = []
    for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
        ctx = qudax.Context(DIMS, comm=comm, overlap=False, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        h = np.zeros(400)
        for _ in range(2):  # the second solve replays the cached graph
            x, st = ctx.solve(b, tol=1e-11, delta=1e-2, maxiter=400, prec=8, prec_sloppy=4, history=h)
        out.append((x, st, h.copy()))
        ctx.close()
    assert out[0][1]["iters"] == out[1][1]["iters"]
    assert np.array_equal(out[0][2], out[1][2])
    assert np.array_equal(out[0][0], out[1][0])


def test_binding_rejects_bad_buffers(torch_cuda, system):
    """The binding validates every pointer it hands to the library: a CUDA tensor
    on a host entry point, float32 or undersized buffers, a host array on a device entry point."""
    import torch
    U, _ = system
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    b = qgen.point_source(DIMS, 0, 0)
    bd = torch.from_numpy(b.view(np.float64).copy()).cuda()
    with pytest.raises(ValueError):
        ctx.solve(bd)                                   # device tensor to the host entry
    with pytest.raises(ValueError):
        ctx.solve(b, out=np.zeros(10, dtype=np.complex128))
    with pytest.raises(ValueError):
        ctx.solve_dev(torch.zeros_like(bd).float(), bd)  # float32 x
    with pytest.raises(ValueError):
        ctx.solve_dev(torch.zeros(100, dtype=torch.float64, device="cuda"), bd)
    with pytest.raises(ValueError):
        ctx.solve_dev(torch.zeros_like(bd).cpu(), bd)
    f = ctx.new_field(4)
    with pytest.raises(ValueError):
        ctx.matpc(f, f[:100], 4)
    with pytest.raises(ValueError):
        ctx.matpc(ctx.new_field(2), ctx.new_field(2), 4)  # half-sized buffers for an fp32 operator
    ctx.close()


_WHILE_NCCL_CHILD = r"""
import hashlib, json, sys
import numpy as np
sys.path.insert(0, sys.argv[1])
import qgen
from paper_1011_0024_b200 import qudax
dims = (8, 8, 8, 16)
U = qgen.gauge(dims, 1003, eps=0.1)
b = qgen.point_source(dims, 1, 2)
out = {}
for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
    for ov in ((False,) if comm == qudax.COMM_NONE else (False, True)):
        ctx = qudax.Context(dims, comm=comm, overlap=ov, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        for _ in range(2):  # the second solve replays the cached batch graph
            x, st = ctx.solve(b, tol=1e-11, delta=1e-2, maxiter=400, prec=8, prec_sloppy=4)
        out[f"{comm}-{int(ov)}"] = {"x": hashlib.sha256(x.tobytes()).hexdigest(), "iters": st["iters"],
                                     "device_batches": st["device_batches"], "host_polls": st["host_polls"],
                                     "true_res": st["true_res"]}
        ctx.close()
print(json.dumps(out))
"""


def test_nccl_loopback_iterations_in_while_node(torch_cuda, tmp_path):
    """The N > 1 solver path with the device-side batch loop: with NCCL's graph-mixing support off
    (it adds event-wait nodes a conditional graph body cannot hold; bench.py switches it off),
    the NCCL-loopback iteration — halo send/recv and the allreduce of the fused sums, with and
    without the overlapped tail launch — runs inside the WHILE node (device_batches > 0, far
    fewer host polls than iterations); without overlap (one whole-lattice kernel, the unsplit
    reduction grouping) it is bitwise the unsplit solve, with overlap within the tolerance.  A
    child process, so the NCCL environment is set before NCCL initialises."""
    import json
    import os
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
    env = dict(os.environ, NCCL_GRAPH_MIXING_SUPPORT="0")
    r = subprocess.run([sys.executable, "-c", _WHILE_NCCL_CHILD, root], env=env, capture_output=True, text=True,
                       timeout=600)
    assert r.returncode == 0, r.stderr[-2000:]
    out = json.loads(r.stdout.strip().splitlines()[-1])
    ref = out["0-0"]
    assert ref["device_batches"] > 0
    for key in ("1-0", "1-1"):
        st = out[key]
        assert st["device_batches"] > 0, (key, st, r.stderr[-1000:])
        assert st["host_polls"] < st["iters"], (key, st)
        assert st["true_res"] <= 1e-11 * (1 + 1e-3), (key, st)
    st = out["1-0"]
    assert st["iters"] == ref["iters"] and st["x"] == ref["x"] and st["true_res"] == ref["true_res"], (st, ref)
