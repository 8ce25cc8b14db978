"""world_size > 1 tests of the multi-rank host logic on CPU (gloo, 127.0.0.1):
partition bookkeeping of libqudax (qudax_partition_info), the host face transport the binding
hands to the library (make_gloo_transport), and the T-slab decomposition itself checked at the
level of the operator: each rank applies the oracle's D to its slab plus one ghost timeslice
per side received from its neighbours, and the gathered result equals the global D."""
import ctypes
import os
import socket

import numpy as np
import pytest
import torch.distributed as dist
import torch.multiprocessing as mp


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _init(rank, n, port):
    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=n)


def _w_partition(rank, n, port, q):
    _init(rank, n, port)
    from paper_1011_0024_b200 import qudax
    dims = (8, 4, 4, 16)
    p = qudax.partition_info(dims, n, rank)
    allp = [None] * n
    dist.all_gather_object(allp, p)
    if rank == 0:
        ok = sorted(x["t0"] for x in allp) == [r * (16 // n) for r in range(n)]
        ok &= all(x["T_loc"] * n == 16 for x in allp)
        ok &= all(allp[x["rank_fwd"]]["rank_back"] == r for r, x in enumerate(allp))
        ok &= sum(x["applies_bc_fwd"] for x in allp) == 1 and sum(x["applies_bc_back"] for x in allp) == 1
        ok &= allp[n - 1]["applies_bc_fwd"] == 1 and allp[0]["applies_bc_back"] == 1
        q.put(bool(ok))
    dist.destroy_process_group()


def _w_transport(rank, n, port, q):
    _init(rank, n, port)
    from paper_1011_0024_b200 import qudax
    ex, ar = qudax.make_gloo_transport()
    nb = 4096
    sf = np.full(nb, rank * 2 + 1, dtype=np.uint8)   # goes forward to rank+1
    sb = np.full(nb, rank * 2 + 2, dtype=np.uint8)   # goes backward to rank-1
    rb, rf = np.zeros(nb, np.uint8), np.zeros(nb, np.uint8)
    back, fwd = (rank - 1) % n, (rank + 1) % n
    rc = ex(fwd, back, sf.ctypes.data, sb.ctypes.data, rb.ctypes.data, rf.ctypes.data, nb, None)
    ok = rc == 0 and np.all(rb == back * 2 + 1) and np.all(rf == fwd * 2 + 2)
    vals = np.array([rank + 1.0, 2.0 * rank], dtype=np.float64)
    rc2 = ar(vals.ctypes.data_as(ctypes.POINTER(ctypes.c_double)), 2, None)
    ok &= rc2 == 0 and vals[0] == n * (n + 1) / 2 and vals[1] == n * (n - 1)
    oks = [None] * n
    dist.all_gather_object(oks, bool(ok))
    if rank == 0:
        q.put(all(oks))
    dist.destroy_process_group()


def _w_slab_operator(rank, n, port, q):
    """Rank r owns global t in [r T_loc, (r+1) T_loc); ghost timeslices come from the ring
    neighbours by point-to-point messages, never from the generator."""
    _init(rank, n, port)
    import torch

    import oracle
    import qgen
    dims = (4, 4, 2, 8)
    T_loc = dims[3] // n
    t0 = rank * T_loc
    U = qgen.gauge(dims, 7, t_begin=t0, nt=T_loc)
    psi = qgen.spinor(dims, 8, t_begin=t0, nt=T_loc)
    fwd, back = (rank + 1) % n, (rank - 1) % n
    # spinor ghosts: last slice -> forward neighbour, first slice -> backward neighbour;
    # gauge ghost: the backward neighbour's last-timeslice links
    def xchg(send_fwd, send_back):
        rb, rf = np.empty_like(send_fwd), np.empty_like(send_back)
        T = lambda a: torch.from_numpy(a.view(np.float64))
        ops = [dist.P2POp(dist.isend, T(send_fwd), fwd, tag=0), dist.P2POp(dist.irecv, T(rb), back, tag=0),
               dist.P2POp(dist.isend, T(send_back), back, tag=1), dist.P2POp(dist.irecv, T(rf), fwd, tag=1)]
        for r in dist.batch_isend_irecv(ops):
            r.wait()
        return rb, rf
    gb, gf = xchg(np.ascontiguousarray(psi[-1]), np.ascontiguousarray(psi[0]))
    ub, uf = xchg(np.ascontiguousarray(U[:, -1]), np.ascontiguousarray(U[:, 0]))
    Uext = np.concatenate([ub[:, None], U, uf[:, None]], axis=1)
    pext = np.concatenate([gb[None], psi, gf[None]], axis=0)
    out = oracle.dslash(Uext, pext, -1.0, t_global_offset=t0 - 1, T_global=dims[3])[1:-1]
    allout = [None] * n
    dist.all_gather_object(allout, out)
    if rank == 0:
        full = oracle.dslash(qgen.gauge(dims, 7), qgen.spinor(dims, 8), -1.0)
        q.put(bool(np.array_equal(np.concatenate(allout, axis=0), full)))
    dist.destroy_process_group()


def _spawn(fn, n):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=fn, args=(r, n, PORT[0], q)) for r in range(n)]
    for p in procs:
        p.start()
    res = q.get(timeout=300)
    for p in procs:
        p.join(timeout=120)
    return res


PORT = [0]


@pytest.fixture(autouse=True)
def _fresh_port():
    PORT[0] = _port()


@pytest.mark.parametrize("n", [2, 4])
def test_partition_bookkeeping_world(n):
    assert _spawn(_w_partition, n)


@pytest.mark.parametrize("n", [2, 3])
def test_host_transport_world(n):
    assert _spawn(_w_transport, n)


@pytest.mark.parametrize("n", [2, 4])
def test_slab_decomposition_matches_global_operator(n):
    assert _spawn(_w_slab_operator, n)
