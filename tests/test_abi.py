"""CPU-side checks of the C-ABI library: it loads, exports every symbol include/qudax.h
declares, and its host-only bookkeeping (partition, work/traffic model) matches the paper."""
import ctypes
import os
import re

import pytest

from paper_1011_0024_b200 import qudax
from qtest_util import ROOT, read_golden


def header_symbols():
    src = open(os.path.join(ROOT, "include", "qudax.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(qudax_[a-z0-9_]+)\s*\(", src)) - {"qudax_exchange_fn", "qudax_allreduce_fn",
                                                                          "qudax_alloc_fn", "qudax_free_fn"})


def test_library_exports_every_header_symbol():
    L = qudax.lib()
    syms = header_symbols()
    assert len(syms) >= 25
    missing = [s for s in syms if not hasattr(L, s)]
    assert not missing, missing
    # the binding declares a signature for each of them
    assert set(syms) == set(qudax.SIGNATURES), set(syms) ^ set(qudax.SIGNATURES)


def test_abi_version_and_status_strings():
    assert qudax.lib().qudax_abi_version() == 5
    assert qudax.status_string(0) == "ok"
    assert "unsupported" in qudax.status_string(5)


def test_site_model_reproduces_paper_counts():
    """Mhat costs 3696 flops per 2976 bytes in single precision (fp32, 2-row links)."""
    _, kv = read_golden("paper_counts.txt")
    m = qudax.site_model(4, 12, -1)
    assert m["flops"] == kv["flops_per_site_matpc_fp32"]
    assert m["bytes_paper"] == kv["bytes_per_site_matpc_fp32"]
    # SURVEY 8(d) byte table (compulsory bytes per Dslash output site, clover fused)
    expect = {(8, 18): 2112, (8, 12): 1728, (8, 8): 1472, (4, 18): 1056, (4, 12): 864, (4, 8): 736,
              (2, 18): 544, (2, 12): 448, (2, 8): 384}
    for (p, r), b in expect.items():
        assert qudax.site_model(p, r, qudax.CLOVER_INV)["bytes_compulsory"] == b, (p, r)
    assert qudax.site_model(4, 12, qudax.HOP)["flops"] == 1320
    assert qudax.site_model(4, 12, qudax.CLOVER_INV)["flops"] == 1824
    assert qudax.site_model(4, 12, qudax.CLOVER_XPAY)["flops"] == 1872


def test_partition_info():
    p = qudax.partition_info((32, 32, 32, 256), 8, 3)
    assert p["T_loc"] == 32 and p["t0"] == 96
    assert p["rank_fwd"] == 4 and p["rank_back"] == 2
    assert p["V_s"] == 32 ** 3 and p["V_h"] == 32 ** 3 * 16 and p["face_sites"] == 32 ** 3 // 2
    assert not p["applies_bc_fwd"] and not p["applies_bc_back"]
    # face message sizes at 32^3 — 786,432 B fp32, 458,752 B half, 1,572,864 B fp64
    assert p["face_bytes"] == {"single": 786432, "half": 458752, "double": 1572864}
    p0 = qudax.partition_info((4, 4, 4, 8), 2, 0)
    p1 = qudax.partition_info((4, 4, 4, 8), 2, 1)
    assert p0["applies_bc_back"] and not p0["applies_bc_fwd"]
    assert p1["applies_bc_fwd"] and not p1["applies_bc_back"]
    one = qudax.partition_info((4, 4, 4, 8), 1, 0)
    assert one["applies_bc_fwd"] and one["applies_bc_back"] and one["rank_fwd"] == 0
    for bad in [((3, 4, 4, 8), 1, 0), ((4, 4, 4, 8), 3, 0), ((4, 4, 4, 6), 2, 0), ((4, 4, 4, 8), 8, 0),
                ((4, 4, 4, 8), 2, 2)]:
        with pytest.raises(qudax.QudaxError):
            qudax.partition_info(*bad)


def test_partition_grid():
    """Process grids: rank = ((ct Pz + cz) Py + cy) Px + cx, local boxes
    tile the global lattice, neighbours are mutual, faces are V_loc / L_mu / 2 sites."""
    dims, grid = (8, 4, 8, 16), (2, 1, 2, 2)
    n = 8
    parts = [qudax.partition_info(dims, n, r, proc_grid=grid) for r in range(n)]
    seen = set()
    for r, p in enumerate(parts):
        assert p["proc_grid"] == grid and p["local_dims"] == (4, 4, 4, 8)
        cx, cy, cz, ct = p["coords"]
        assert r == ((ct * grid[2] + cz) * grid[1] + cy) * grid[0] + cx
        assert p["origin"] == tuple(c * l for c, l in zip(p["coords"], p["local_dims"]))
        seen.add(p["origin"])
        assert p["split_mask"] == 0b1101  # x, z, t split; y not
        for mu in range(4):
            assert parts[p["nb_fwd"][mu]]["nb_back"][mu] == r
            q = parts[p["nb_fwd"][mu]]
            for nu in range(4):  # the forward neighbour differs in coordinate mu only
                want = (p["coords"][nu] + (nu == mu)) % grid[nu]
                assert q["coords"][nu] == want
            assert p["face_sites_dim"][mu] == 4 * 4 * 4 * 8 // p["local_dims"][mu] // 2
        assert p["T_loc"] == 8 and p["t0"] == ct * 8
        assert p["applies_bc_fwd"] == (ct == 1) and p["applies_bc_back"] == (ct == 0)
    assert len(seen) == n
    # default grid = T slabs; loopback mask on one rank; bad grids
    assert qudax.partition_info((4, 4, 4, 8), 2, 1)["proc_grid"] == (1, 1, 1, 2)
    assert qudax.partition_info((4, 4, 4, 8), 1, 0, split_mask=0b0100)["split_mask"] == 0b0100
    for args, kw in [(((4, 4, 4, 8), 4, 0), {"proc_grid": (1, 1, 2, 1)}),     # product != nranks
                     (((4, 4, 6, 8), 2, 0), {"proc_grid": (1, 1, 2, 1)}),     # Z_loc = 3 odd
                     (((4, 4, 4, 8), 2, 0), {"proc_grid": (1, 1, 2, 1), "split_mask": 8}),  # misses z
                     (((4, 3, 4, 8), 2, 0), {"proc_grid": (2, 1, 1, 1)}),     # X split needs Y even
                     (((4, 4, 4, 8), 1, 0), {"split_mask": 16})]:
        with pytest.raises(qudax.QudaxError):
            qudax.partition_info(*args, **kw)


def test_init_without_gpu_fails_loudly():
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    p = qudax.InitParam()
    p.global_dims = (ctypes.c_int * 4)(4, 4, 4, 4)
    p.nranks, p.rank, p.device, p.comm = 1, 0, 0, qudax.COMM_NONE
    h = ctypes.c_void_p()
    st = qudax.lib().qudax_init(ctypes.byref(h), ctypes.byref(p))
    assert st == 3  # QUDAX_ERR_CUDA: no silent CPU fallback
    assert not h.value


def test_binding_struct_layouts_match_header(tmp_path):
    """The ctypes mirrors of the header's structs have the C compiler's sizes and field offsets
    (a field added to the header but not to the binding would silently shift every later one)."""
    import subprocess
    structs = {"qudax_init_param": qudax.InitParam, "qudax_gauge_param": qudax.GaugeParam,
               "qudax_solve_param": qudax.SolveParam, "qudax_solve_stats": qudax.SolveStats,
               "qudax_site_model": qudax.SiteModel, "qudax_kernel_stats": qudax.KernelStats,
               "qudax_partition": qudax.Partition}
    lines = ['#include <stdio.h>', '#include <stddef.h>', '#include "qudax.h"', "int main(void) {"]
    for cname, py in structs.items():
        lines.append(f'printf("{cname} size %zu\\n", sizeof({cname}));')
        for f, _ in py._fields_:
            lines.append(f'printf("{cname} {f} %zu\\n", offsetof({cname}, {f}));')
    lines += ["return 0;", "}"]
    src = tmp_path / "layout.c"
    src.write_text("\n".join(lines))
    exe = tmp_path / "layout"
    subprocess.run(["gcc", "-std=c11", "-I", os.path.join(ROOT, "include"), str(src), "-o", str(exe)], check=True)
    got = {}
    for ln in subprocess.run([str(exe)], capture_output=True, text=True, check=True).stdout.splitlines():
        c, f, v = ln.split()
        got[(c, f)] = int(v)
    for cname, py in structs.items():
        assert got[(cname, "size")] == ctypes.sizeof(py), cname
        for f, _ in py._fields_:
            assert got[(cname, f)] == getattr(py, f).offset, (cname, f)
