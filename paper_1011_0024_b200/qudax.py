"""Thin Python binding of libqudax (include/qudax.h) — argument marshalling only.

Every step of the hot path runs in the library's CUDA kernels; this module only converts
numpy / torch objects to plain pointers and sizes.  PyTorch is used for device memory (the
caching allocator backs both the caller's fields and, through the dev_alloc hooks, the
library's internal buffers), for streams, and for torch.distributed (rank bookkeeping, the
NCCL unique-id broadcast, and the gloo-backed host transport used in tests).

There is no CPU fallback: if libqudax.so is missing or no CUDA device is present, the
operations raise.
"""
import ctypes
import os

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("QUDAX_LIB") or os.path.join(_HERE, "lib", "libqudax.so")  # override: experiments only

HALF, SINGLE, DOUBLE = 2, 4, 8
EVEN, ODD = 0, 1
HOP, CLOVER_INV, CLOVER_XPAY, CLOVER_INV_XPAY = 0, 1, 2, 3
COMM_NONE, COMM_NCCL, COMM_HOST = 0, 1, 2
HALO_COMM, HALO_P2P = 0, 1
# qudax_init_flag bits (include/qudax.h): test / comparison switches, 0 = defaults
FLAG_NO_GRAPHS, FLAG_DEBUG_SOLVER, FLAG_FORCE_SS, FLAG_ONE_RHS_PER_THREAD, FLAG_TIMING_BREAKDOWN = 1, 2, 4, 8, 16
PREC_NAMES = {"half": 2, "single": 4, "double": 8, "f16": 2, "f32": 4, "f64": 8}

STATUS = {0: "QUDAX_OK", 1: "QUDAX_ERR_ARG", 2: "QUDAX_ERR_STATE", 3: "QUDAX_ERR_CUDA", 4: "QUDAX_ERR_NCCL",
          5: "QUDAX_ERR_UNSUPPORTED", 6: "QUDAX_ERR_NOT_CONVERGED", 7: "QUDAX_ERR_OOM", 8: "QUDAX_ERR_COMM"}


class QudaxError(RuntimeError):
    def __init__(self, status, msg):
        super().__init__(f"{STATUS.get(status, status)}: {msg}")
        self.status = status


# ----------------------------------------------------------------------------- ctypes structs
EXCHANGE_FN = ctypes.CFUNCTYPE(ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_void_p, ctypes.c_void_p,
                               ctypes.c_void_p, ctypes.c_void_p, ctypes.c_size_t, ctypes.c_void_p)
ALLREDUCE_FN = ctypes.CFUNCTYPE(ctypes.c_int, ctypes.POINTER(ctypes.c_double), ctypes.c_int, ctypes.c_void_p)
ALLOC_FN = ctypes.CFUNCTYPE(ctypes.c_void_p, ctypes.c_size_t, ctypes.c_void_p)
FREE_FN = ctypes.CFUNCTYPE(None, ctypes.c_void_p, ctypes.c_void_p)


class InitParam(ctypes.Structure):
    _fields_ = [("global_dims", ctypes.c_int * 4), ("nranks", ctypes.c_int), ("rank", ctypes.c_int),
                ("device", ctypes.c_int), ("comm", ctypes.c_int), ("overlap", ctypes.c_int),
                ("nccl_id", ctypes.c_void_p), ("stream", ctypes.c_size_t),
                ("dev_alloc", ALLOC_FN), ("dev_free", FREE_FN), ("alloc_user", ctypes.c_void_p),
                ("host_exchange", EXCHANGE_FN), ("host_allreduce", ALLREDUCE_FN), ("comm_user", ctypes.c_void_p),
                ("halo", ctypes.c_int), ("proc_grid", ctypes.c_int * 4), ("split_mask", ctypes.c_int),
                ("flags", ctypes.c_int), ("copy_threads", ctypes.c_int)]


class GaugeParam(ctypes.Structure):
    _fields_ = [("prec", ctypes.c_int), ("recon", ctypes.c_int), ("prec_sloppy", ctypes.c_int),
                ("recon_sloppy", ctypes.c_int), ("t_boundary", ctypes.c_int), ("kappa", ctypes.c_double),
                ("csw", ctypes.c_double)]


class SolveParam(ctypes.Structure):
    _fields_ = [("tol", ctypes.c_double), ("delta", ctypes.c_double), ("maxiter", ctypes.c_int),
                ("prec_sloppy", ctypes.c_int), ("prec", ctypes.c_int), ("use_schur", ctypes.c_int),
                ("res_history", ctypes.POINTER(ctypes.c_double)), ("history_cap", ctypes.c_int),
                ("poll_every", ctypes.c_int)]


class SolveStats(ctypes.Structure):
    _fields_ = [("iters", ctypes.c_int), ("reliable_updates", ctypes.c_int), ("true_res", ctypes.c_double),
                ("true_res_schur", ctypes.c_double), ("secs", ctypes.c_double), ("flops", ctypes.c_double),
                ("gflops", ctypes.c_double), ("restarts", ctypes.c_int),
                ("host_polls", ctypes.c_int), ("device_batches", ctypes.c_int)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


class SiteModel(ctypes.Structure):
    _fields_ = [("flops", ctypes.c_double), ("bytes_paper", ctypes.c_double), ("bytes_compulsory", ctypes.c_double)]


class KernelStats(ctypes.Structure):
    _fields_ = [("launches", ctypes.c_longlong), ("sites", ctypes.c_longlong), ("ms_total", ctypes.c_double),
                ("flops", ctypes.c_double), ("bytes_compulsory", ctypes.c_double), ("bytes_paper", ctypes.c_double),
                ("span_ms_total", ctypes.c_double)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


class Partition(ctypes.Structure):
    _fields_ = [("T_loc", ctypes.c_int), ("t0", ctypes.c_int), ("rank_fwd", ctypes.c_int),
                ("rank_back", ctypes.c_int), ("V_loc", ctypes.c_long), ("V_h", ctypes.c_long),
                ("V_s", ctypes.c_long), ("face_sites", ctypes.c_long), ("applies_bc_fwd", ctypes.c_int),
                ("applies_bc_back", ctypes.c_int), ("face_bytes", ctypes.c_size_t * 3),
                ("proc_grid", ctypes.c_int * 4), ("coords", ctypes.c_int * 4), ("local_dims", ctypes.c_int * 4),
                ("origin", ctypes.c_int * 4), ("nb_fwd", ctypes.c_int * 4), ("nb_back", ctypes.c_int * 4),
                ("split_mask", ctypes.c_int), ("face_sites_dim", ctypes.c_long * 4)]

    def as_dict(self):
        d = {}
        for k, _ in self._fields_:
            v = getattr(self, k)
            d[k] = tuple(v) if k not in ("face_bytes",) and hasattr(v, "__len__") else v
        d["face_bytes"] = {"half": self.face_bytes[0], "single": self.face_bytes[1], "double": self.face_bytes[2]}
        return d


_lib = None

# every symbol include/qudax.h declares, with its ctypes signature
_P, _I, _D, _Z = ctypes.c_void_p, ctypes.c_int, ctypes.c_double, ctypes.c_size_t
_DP = ctypes.POINTER(ctypes.c_double)
SIGNATURES = {
    "qudax_abi_version": ([], _I),
    "qudax_status_string": ([_I], ctypes.c_char_p),
    "qudax_partition_info": ([ctypes.POINTER(ctypes.c_int), ctypes.POINTER(ctypes.c_int), _I, _I, _I,
                              ctypes.POINTER(Partition)], _I),
    "qudax_model": ([_I, _I, _I, ctypes.POINTER(SiteModel)], _I),
    "qudax_nccl_unique_id": ([_P], _I),
    "qudax_init": ([ctypes.POINTER(_P), ctypes.POINTER(InitParam)], _I),
    "qudax_finalize": ([_P], _I),
    "qudax_last_error": ([_P], ctypes.c_char_p),
    "qudax_sync": ([_P], _I),
    "qudax_launch_count": ([_P], ctypes.c_longlong),
    "qudax_get_partition": ([_P, ctypes.POINTER(Partition)], _I),
    "qudax_kernel_timing": ([_P, _I], _I),
    "qudax_get_kernel_stats": ([_P, _I, ctypes.POINTER(KernelStats)], _I),
    "qudax_halo_timeline": ([_P, _I, _DP], _I),
    "qudax_gauge_load": ([_P, _DP, ctypes.POINTER(GaugeParam)], _I),
    "qudax_spinor_bytes": ([_P, _I], _Z),
    "qudax_spinor_load": ([_P, _P, _I, _I, _DP], _I),
    "qudax_spinor_load_dev": ([_P, _P, _I, _I, _P], _I),
    "qudax_spinor_store": ([_P, _DP, _P, _I, _I], _I),
    "qudax_spinor_store_dev": ([_P, _P, _P, _I, _I], _I),
    "qudax_spinor_convert": ([_P, _P, _I, _P, _I], _I),
    "qudax_dslash": ([_P, _P, _P, _P, _I, _I, _I, _I, _D], _I),
    "qudax_matpc": ([_P, _P, _P, _I, _I], _I),
    "qudax_matpc_sym": ([_P, _P, _P, _I, _I], _I),
    "qudax_dslash_multi": ([_P, ctypes.POINTER(_P), ctypes.POINTER(_P), ctypes.POINTER(_P), _I, _I, _I, _I, _I, _D], _I),
    "qudax_matpc_multi": ([_P, ctypes.POINTER(_P), ctypes.POINTER(_P), _I, _I, _I], _I),
    "qudax_mdagm": ([_P, _P, _P, _I], _I),
    "qudax_norm2": ([_P, _P, _I, _DP], _I),
    "qudax_cdot": ([_P, _P, _P, _I, _DP], _I),
    "qudax_solve_bicgstab": ([_P, _DP, _DP, ctypes.POINTER(SolveParam), ctypes.POINTER(SolveStats)], _I),
    "qudax_solve_bicgstab_dev": ([_P, _P, _P, ctypes.POINTER(SolveParam), ctypes.POINTER(SolveStats)], _I),
    "qudax_solve_bicgstab_multi": ([_P, ctypes.POINTER(_P), ctypes.POINTER(_P), _I, ctypes.POINTER(SolveParam),
                                    ctypes.POINTER(SolveStats)], _I),
    "qudax_solve_bicgstab_multi_dev": ([_P, ctypes.POINTER(_P), ctypes.POINTER(_P), _I, ctypes.POINTER(SolveParam),
                                        ctypes.POINTER(SolveStats)], _I),
    "qudax_solve_cgnr": ([_P, _DP, _DP, ctypes.POINTER(SolveParam), ctypes.POINTER(SolveStats)], _I),
    "qudax_solve_cgnr_dev": ([_P, _P, _P, ctypes.POINTER(SolveParam), ctypes.POINTER(SolveStats)], _I),
}


def lib():
    """Load libqudax.so (fails loudly when it has not been built — no fallback)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} not built: run `python -m paper_1011_0024_b200.build` "
                              "(there is no CPU fallback)")
        L = ctypes.CDLL(LIB_PATH)
        for name, (args, res) in SIGNATURES.items():
            fn = getattr(L, name)
            fn.argtypes = args
            fn.restype = res
        _lib = L
    return _lib


def status_string(s):
    return lib().qudax_status_string(int(s)).decode()


def partition_info(global_dims, nranks, rank, proc_grid=None, split_mask=0):
    """Rank bookkeeping of a process grid (default 1 x 1 x 1 x nranks: T slabs)."""
    out = Partition()
    dims = (ctypes.c_int * 4)(*global_dims)
    grid = (ctypes.c_int * 4)(*proc_grid) if proc_grid is not None else None
    st = lib().qudax_partition_info(dims, grid, int(nranks), int(rank), int(split_mask), ctypes.byref(out))
    if st:
        raise QudaxError(st, "partition_info")
    return out.as_dict()


def site_model(prec, recon, kind):
    """Per-site flops / bytes of one Dslash kernel (kind 0-2) or of Mhat (kind -1)."""
    out = SiteModel()
    st = lib().qudax_model(int(prec), int(recon), int(kind), ctypes.byref(out))
    if st:
        raise QudaxError(st, "model")
    return {"flops": out.flops, "bytes_paper": out.bytes_paper, "bytes_compulsory": out.bytes_compulsory}


def nccl_unique_id():
    buf = ctypes.create_string_buffer(128)
    st = lib().qudax_nccl_unique_id(buf)
    if st:
        raise QudaxError(st, "ncclGetUniqueId")
    return bytes(buf.raw)


def _dptr(a):
    assert a.dtype == np.complex128 and a.flags.c_contiguous
    return a.ctypes.data_as(_DP)


# ----------------------------------------------------------------------------- host transport
def make_gloo_transport(group=None):
    """Host-staged face exchange and allreduce over torch.distributed (gloo), for
    QUDAX_COMM_HOST: the paper's non-overlapped strategy with message passing
    between processes.  Returns (exchange_fn, allreduce_fn) Python callables with the raw
    pointer signature of qudax_exchange_fn / qudax_allreduce_fn."""
    import torch
    import torch.distributed as dist

    def as_tensor(ptr, n):
        arr = np.ctypeslib.as_array((ctypes.c_uint8 * n).from_address(ptr))
        return torch.from_numpy(arr)

    def exchange(fwd, back, send_fwd, send_back, recv_back, recv_fwd, nbytes, _user):
        try:
            sf, sb = as_tensor(send_fwd, nbytes), as_tensor(send_back, nbytes)
            rb, rf = as_tensor(recv_back, nbytes), as_tensor(recv_fwd, nbytes)
            ops = [dist.P2POp(dist.isend, sf, fwd, group, tag=0), dist.P2POp(dist.irecv, rb, back, group, tag=0),
                   dist.P2POp(dist.isend, sb, back, group, tag=1), dist.P2POp(dist.irecv, rf, fwd, group, tag=1)]
            for req in dist.batch_isend_irecv(ops):
                req.wait()
            return 0
        except Exception:  # noqa: BLE001 - reported to the library as a status
            import traceback
            traceback.print_exc()
            return 1

    def allreduce(vals, n, _user):
        try:
            arr = np.ctypeslib.as_array(vals, shape=(n,))
            t = torch.from_numpy(arr)
            dist.all_reduce(t, group=group)
            return 0
        except Exception:  # noqa: BLE001
            import traceback
            traceback.print_exc()
            return 1

    return exchange, allreduce


# ----------------------------------------------------------------------------- context
class Context:
    """One rank's qudax context (one GPU).  Fields are torch uint8 CUDA tensors of
    spinor_bytes(prec) bytes holding one parity in the library's layout."""

    def __init__(self, global_dims, nranks=1, rank=0, device=0, comm=COMM_NONE, overlap=True, nccl_id=None,
                 stream=None, torch_allocator=True, transport=None, halo=HALO_COMM, proc_grid=None, split_mask=0,
                 flags=0, copy_threads=0):
        import torch
        self._torch = torch
        self.global_dims = tuple(int(d) for d in global_dims)
        self.device = int(device)
        torch.cuda.set_device(self.device)
        # the library's compute stream: a dedicated torch stream unless the caller passes one;
        # record events / order torch work against ctx.stream
        self.stream = stream if stream is not None else torch.cuda.Stream(self.device)
        p = InitParam()
        p.global_dims = (ctypes.c_int * 4)(*self.global_dims)
        p.nranks, p.rank, p.device, p.comm, p.overlap = int(nranks), int(rank), self.device, int(comm), int(bool(overlap))
        p.halo = int(halo)
        if proc_grid is not None:
            p.proc_grid = (ctypes.c_int * 4)(*proc_grid)
        p.split_mask = int(split_mask)
        p.flags, p.copy_threads = int(flags), int(copy_threads)
        self._id = None
        if comm == COMM_NCCL:
            self._id = ctypes.create_string_buffer(bytes(nccl_id), 128)
            p.nccl_id = ctypes.cast(self._id, ctypes.c_void_p)
        p.stream = int(self.stream.cuda_stream)
        self._live = {}
        if torch_allocator:
            dev, strm = self.device, self.stream

            def _alloc(nbytes, _u):
                try:
                    return int(torch.cuda.caching_allocator_alloc(int(nbytes), dev, strm))
                except Exception:  # noqa: BLE001 - OOM is reported by the library
                    return None

            def _free(ptr, _u):
                try:
                    torch.cuda.caching_allocator_delete(int(ptr))
                except Exception:  # noqa: BLE001 - interpreter shutdown: the process frees it
                    pass

            self._alloc_cb, self._free_cb = ALLOC_FN(_alloc), FREE_FN(_free)
            p.dev_alloc, p.dev_free = self._alloc_cb, self._free_cb
        if comm == COMM_HOST:
            ex, ar = transport if transport is not None else make_gloo_transport()
            self._ex_cb, self._ar_cb = EXCHANGE_FN(ex), ALLREDUCE_FN(ar)
            p.host_exchange, p.host_allreduce = self._ex_cb, self._ar_cb
        self._h = ctypes.c_void_p()
        self._check(lib().qudax_init(ctypes.byref(self._h), ctypes.byref(p)), ctx=False)
        part = Partition()
        self._check(lib().qudax_get_partition(self._h, ctypes.byref(part)))
        self.partition = part.as_dict()
        self.local_dims = tuple(self.partition["local_dims"])

    # -- argument validation (every pointer handed to the library is checked first: a CUDA tensor
    # given to a host entry point, a float32 or undersized buffer would otherwise be read or
    # written out of bounds by the C side)
    @property
    def _slab_reals(self):
        X, Y, Z, T_loc = self.local_dims
        return 24 * X * Y * Z * T_loc

    def _host_slab(self, a, name, writable=False):
        """A full local slab in host memory: numpy complex128 [T_loc, Z, Y, X, 4, 3] or a CPU
        float64 / complex128 torch tensor with the same number of reals; returns a double*."""
        X, Y, Z, T_loc = self.local_dims
        if hasattr(a, "data_ptr"):
            torch = self._torch
            if a.device.type != "cpu":
                raise ValueError(f"{name}: host entry point needs a CPU tensor, got {a.device}")
            if a.dtype not in (torch.float64, torch.complex128) or not a.is_contiguous():
                raise ValueError(f"{name}: need a contiguous float64/complex128 tensor, got {a.dtype}")
            reals = a.numel() * (2 if a.dtype == torch.complex128 else 1)
            if reals != self._slab_reals:
                raise ValueError(f"{name}: {reals} reals, the local slab has {self._slab_reals}")
            return ctypes.cast(a.data_ptr(), _DP)
        if not isinstance(a, np.ndarray) or a.dtype != np.complex128 or not a.flags.c_contiguous:
            raise ValueError(f"{name}: need a C-contiguous complex128 numpy array")
        if a.shape != (T_loc, Z, Y, X, 4, 3):
            raise ValueError(f"{name}: shape {a.shape}, expected {(T_loc, Z, Y, X, 4, 3)}")
        if writable and not a.flags.writeable:
            raise ValueError(f"{name}: array is read-only")
        return a.ctypes.data_as(_DP)

    def _dev_slab(self, t, name):
        """A full local slab on this context's GPU: contiguous float64 (or complex128) tensor."""
        torch = self._torch
        if not hasattr(t, "data_ptr") or t.device.type != "cuda" or t.device.index != self.device:
            raise ValueError(f"{name}: need a CUDA tensor on cuda:{self.device}")
        if t.dtype not in (torch.float64, torch.complex128) or not t.is_contiguous():
            raise ValueError(f"{name}: need a contiguous float64/complex128 CUDA tensor, got {t.dtype}")
        reals = t.numel() * (2 if t.dtype == torch.complex128 else 1)
        if reals != self._slab_reals:
            raise ValueError(f"{name}: {reals} reals, the local slab has {self._slab_reals}")
        return t.data_ptr()

    def _field(self, f, prec, name="field"):
        """A parity field: a CUDA uint8 tensor of at least spinor_bytes(prec) bytes on this GPU."""
        if f is None:
            return None
        if not hasattr(f, "data_ptr") or f.device.type != "cuda" or f.device.index != self.device:
            raise ValueError(f"{name}: need a CUDA tensor on cuda:{self.device}")
        if not f.is_contiguous() or f.numel() * f.element_size() < self.spinor_bytes(prec):
            raise ValueError(f"{name}: need a contiguous buffer of >= {self.spinor_bytes(prec)} bytes")
        return f.data_ptr()

    # -- plumbing
    def _check(self, st, ctx=True):
        if st:
            msg = lib().qudax_last_error(self._h).decode() if ctx and self._h else ""
            raise QudaxError(st, msg)

    def close(self):
        if getattr(self, "_h", None) and self._h.value:
            lib().qudax_finalize(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:  # noqa: BLE001
            pass

    @property
    def handle(self):
        return self._h

    def launch_count(self):
        return int(lib().qudax_launch_count(self._h))

    def sync(self):
        self._check(lib().qudax_sync(self._h))

    def kernel_timing(self, enable=True, span=False):
        """Per-launch CUDA-event timing of the Dslash kernels (span=True: also the in-kernel
        %globaltimer span, which costs the kernels a few microseconds)."""
        self._check(lib().qudax_kernel_timing(self._h, 2 if (enable and span) else int(bool(enable))))

    def halo_timeline(self, enable=True, read=False):
        """Diagnostic halo-overlap timeline (NCCL path): enable recording; with read=True return
        the last recorded call's marks (µs from its start): pack start, exchange start, exchange
        end, interior start, interior end, boundary start, boundary end."""
        out = (ctypes.c_double * 7)() if read else None
        self._check(lib().qudax_halo_timeline(self._h, int(bool(enable)), out))
        if read:
            keys = ("pack_start", "exchange_start", "exchange_end", "interior_start", "interior_end",
                    "boundary_start", "boundary_end")
            return dict(zip(keys, list(out)))
        return None

    def kernel_stats(self, prec=0):
        out = KernelStats()
        self._check(lib().qudax_get_kernel_stats(self._h, int(prec), ctypes.byref(out)))
        return out.as_dict()

    # -- gauge
    def gauge_load(self, U, kappa, csw, prec=SINGLE, recon=12, prec_sloppy=None, recon_sloppy=None, t_boundary=-1):
        U = np.ascontiguousarray(U, dtype=np.complex128)
        X, Y, Z, T_loc = self.local_dims
        assert U.shape == (4, T_loc, Z, Y, X, 3, 3), U.shape
        g = GaugeParam(int(prec), int(recon), int(prec if prec_sloppy is None else prec_sloppy),
                       int(recon if recon_sloppy is None else recon_sloppy), int(t_boundary), float(kappa), float(csw))
        self._check(lib().qudax_gauge_load(self._h, _dptr(U), ctypes.byref(g)))
        self.kappa, self.csw = float(kappa), float(csw)

    # -- fields
    def spinor_bytes(self, prec):
        return int(lib().qudax_spinor_bytes(self._h, int(prec)))

    def new_field(self, prec):
        """A zeroed parity field, allocated and cleared on the library stream."""
        with self._torch.cuda.stream(self.stream):
            return self._torch.zeros(self.spinor_bytes(prec), dtype=self._torch.uint8, device=f"cuda:{self.device}")

    def spinor_load(self, field, prec, parity, psi):
        psi = np.ascontiguousarray(psi, dtype=np.complex128)
        X, Y, Z, T_loc = self.local_dims
        assert psi.shape == (T_loc, Z, Y, X, 4, 3), psi.shape
        self._check(lib().qudax_spinor_load(self._h, self._field(field, prec), int(prec), int(parity), _dptr(psi)))

    def spinor_load_dev(self, field, prec, parity, src):
        self._check(lib().qudax_spinor_load_dev(self._h, self._field(field, prec), int(prec), int(parity),
                                                self._dev_slab(src, "src")))

    def spinor_store(self, field, prec, parity, out=None):
        X, Y, Z, T_loc = self.local_dims
        if out is None:
            out = np.zeros((T_loc, Z, Y, X, 4, 3), dtype=np.complex128)
        op = self._host_slab(out, "out", writable=True)
        self._check(lib().qudax_spinor_store(self._h, op, self._field(field, prec), int(prec), int(parity)))
        return out

    def spinor_store_dev(self, dst, field, prec, parity):
        self._check(lib().qudax_spinor_store_dev(self._h, self._dev_slab(dst, "dst"), self._field(field, prec), int(prec),
                                                 int(parity)))

    def convert(self, dst, dst_prec, src, src_prec):
        self._check(lib().qudax_spinor_convert(self._h, self._field(dst, dst_prec, "dst"), int(dst_prec),
                                               self._field(src, src_prec, "src"), int(src_prec)))

    # -- operator
    def dslash(self, out, inp, prec, out_parity, dagger=False, kind=HOP, x=None, a=0.0):
        xp = self._field(x, prec, "x")
        self._check(lib().qudax_dslash(self._h, self._field(out, prec, "out"), self._field(inp, prec, "in"), xp,
                                       int(prec), int(out_parity),
                                       int(bool(dagger)), int(kind), float(a)))

    def matpc(self, out, inp, prec, dagger=False):
        self._check(lib().qudax_matpc(self._h, self._field(out, prec, "out"), self._field(inp, prec, "in"), int(prec),
                                      int(bool(dagger))))

    def matpc_sym(self, out, inp, prec, dagger=False):
        """Symmetric Schur form T_ee^{-1} Mhat (or its explicit adjoint)."""
        self._check(lib().qudax_matpc_sym(self._h, self._field(out, prec, "out"), self._field(inp, prec, "in"),
                                          int(prec), int(bool(dagger))))

    def _ptrs(self, fields, prec):
        return (_P * len(fields))(*[self._field(f, prec) for f in fields])

    def dslash_multi(self, outs, ins, prec, out_parity, dagger=False, kind=HOP, xs=None, a=0.0):
        if len(outs) != len(ins) or (xs is not None and len(xs) != len(ins)):
            raise ValueError("dslash_multi: outs / ins / xs lengths differ")
        xp = self._ptrs(xs, prec) if xs is not None else None
        self._check(lib().qudax_dslash_multi(self._h, self._ptrs(outs, prec), self._ptrs(ins, prec), xp, len(ins), int(prec),
                                             int(out_parity), int(bool(dagger)), int(kind), float(a)))

    def matpc_multi(self, outs, ins, prec, dagger=False):
        if len(outs) != len(ins):
            raise ValueError("matpc_multi: outs / ins lengths differ")
        self._check(lib().qudax_matpc_multi(self._h, self._ptrs(outs, prec), self._ptrs(ins, prec), len(ins), int(prec),
                                            int(bool(dagger))))

    def mdagm(self, out, inp, prec):
        self._check(lib().qudax_mdagm(self._h, self._field(out, prec, "out"), self._field(inp, prec, "in"), int(prec)))

    def norm2(self, f, prec):
        r = ctypes.c_double()
        self._check(lib().qudax_norm2(self._h, self._field(f, prec), int(prec), ctypes.byref(r)))
        return r.value

    def cdot(self, a, b, prec):
        r = (ctypes.c_double * 2)()
        self._check(lib().qudax_cdot(self._h, self._field(a, prec, "a"), self._field(b, prec, "b"), int(prec), r))
        return complex(r[0], r[1])

    # -- solver
    def _solve_param(self, tol, delta, maxiter, prec, prec_sloppy, use_schur, history=None, poll_every=0):
        # use_schur: True/1 asymmetric Schur form, 2 (or "sym") symmetric, False/0 even system only
        us = 2 if use_schur in (2, "sym") else int(bool(use_schur))
        sp = SolveParam(float(tol), float(delta), int(maxiter), int(prec_sloppy), int(prec), us)
        if history is not None:
            if not isinstance(history, np.ndarray) or history.dtype != np.float64 or not history.flags.c_contiguous:
                raise ValueError("history: need a C-contiguous float64 numpy array")
            sp.res_history = history.ctypes.data_as(_DP)
            sp.history_cap = int(history.size)
        sp.poll_every = int(poll_every)
        return sp

    def _finish(self, rc, allow_not_converged):
        if rc and not (allow_not_converged and rc == 6):
            self._check(rc)

    def solve_cgnr(self, b, tol=1e-10, maxiter=10000, prec=DOUBLE, use_schur=True, allow_not_converged=False,
                   history=None):
        """CGNR on Mhat^dag Mhat in one precision; host arrays as in solve()."""
        b = np.ascontiguousarray(b, dtype=np.complex128)
        x = np.zeros_like(b)
        bp, xp = self._host_slab(b, "b"), self._host_slab(x, "x", writable=True)
        sp = self._solve_param(tol, 0.0, maxiter, prec, prec, use_schur, history)
        st = SolveStats()
        self._finish(lib().qudax_solve_cgnr(self._h, xp, bp, ctypes.byref(sp), ctypes.byref(st)), allow_not_converged)
        return x, st.as_dict()

    def solve(self, b, tol=1e-10, delta=0.1, maxiter=10000, prec=DOUBLE, prec_sloppy=SINGLE, use_schur=True,
              allow_not_converged=False, history=None, out=None, poll_every=0):
        """x = M^{-1} b (host arrays, full local slab, DR basis); returns (x, stats dict).
        b: numpy complex128 [T_loc, Z, Y, X, 4, 3] or a CPU float64 torch tensor of the same size
        (e.g. a pinned buffer; then `out` may be a preallocated one).  history: optional float64
        numpy array receiving ||r_k||/||bhat|| per iteration."""
        if hasattr(b, "data_ptr"):
            x = out if out is not None else self._torch.zeros_like(b)
        else:
            b = np.ascontiguousarray(b, dtype=np.complex128)
            x = np.zeros_like(b) if out is None else out
        bp, xp = self._host_slab(b, "b"), self._host_slab(x, "out", writable=True)
        sp = self._solve_param(tol, delta, maxiter, prec, prec_sloppy, use_schur, history, poll_every)
        st = SolveStats()
        self._finish(lib().qudax_solve_bicgstab(self._h, xp, bp, ctypes.byref(sp), ctypes.byref(st)),
                     allow_not_converged)
        return x, st.as_dict()

    def solve_multi(self, bs, tol=1e-10, delta=0.1, maxiter=10000, prec=DOUBLE, prec_sloppy=SINGLE, use_schur=True,
                    allow_not_converged=False, history=None, outs=None):
        """Batched solve of len(bs) <= 8 sources (host arrays, full local slabs): one multi-RHS
        Mhat kernel pair per iteration for all still-active systems.  Returns (xs, [stats])."""
        bs = [np.ascontiguousarray(b, dtype=np.complex128) for b in bs]
        xs = outs if outs is not None else [np.zeros_like(b) for b in bs]
        if len(xs) != len(bs):
            raise ValueError("solve_multi: outs / bs lengths differ")
        n = len(bs)
        bp = (_P * n)(*[ctypes.cast(self._host_slab(b, f"bs[{j}]"), _P).value for j, b in enumerate(bs)])
        xp = (_P * n)(*[ctypes.cast(self._host_slab(x, f"outs[{j}]", writable=True), _P).value for j, x in enumerate(xs)])
        sp = self._solve_param(tol, delta, maxiter, prec, prec_sloppy, use_schur, history)
        st = (SolveStats * n)()
        self._finish(lib().qudax_solve_bicgstab_multi(self._h, xp, bp, n, ctypes.byref(sp), st), allow_not_converged)
        return xs, [s.as_dict() for s in st]

    def solve_multi_dev(self, xs, bs, tol=1e-10, delta=0.1, maxiter=10000, prec=DOUBLE, prec_sloppy=SINGLE,
                        use_schur=True, allow_not_converged=False):
        """Device-resident batched solve: lists of float64 CUDA tensors (full local slabs)."""
        if len(xs) != len(bs):
            raise ValueError("solve_multi_dev: xs / bs lengths differ")
        n = len(bs)
        bp = (_P * n)(*[self._dev_slab(b, f"bs[{j}]") for j, b in enumerate(bs)])
        xp = (_P * n)(*[self._dev_slab(x, f"xs[{j}]") for j, x in enumerate(xs)])
        sp = self._solve_param(tol, delta, maxiter, prec, prec_sloppy, use_schur)
        st = (SolveStats * n)()
        self._finish(lib().qudax_solve_bicgstab_multi_dev(self._h, xp, bp, n, ctypes.byref(sp), st),
                     allow_not_converged)
        return [s.as_dict() for s in st]

    def solve_dev(self, x, b, tol=1e-10, delta=0.1, maxiter=10000, prec=DOUBLE, prec_sloppy=SINGLE, use_schur=True,
                  allow_not_converged=False, history=None, poll_every=0):
        """Device-resident variant: x, b are float64 CUDA tensors holding the full local slab
        (T_loc, Z, Y, X, 4, 3, 2)."""
        xp, bp = self._dev_slab(x, "x"), self._dev_slab(b, "b")
        sp = self._solve_param(tol, delta, maxiter, prec, prec_sloppy, use_schur, history, poll_every)
        st = SolveStats()
        self._finish(lib().qudax_solve_bicgstab_dev(self._h, xp, bp, ctypes.byref(sp), ctypes.byref(st)),
                     allow_not_converged)
        return st.as_dict()

    def solve_cgnr_dev(self, x, b, tol=1e-10, maxiter=10000, prec=DOUBLE, use_schur=True, allow_not_converged=False):
        """Device-resident CGNR (x, b as in solve_dev)."""
        xp, bp = self._dev_slab(x, "x"), self._dev_slab(b, "b")
        sp = self._solve_param(tol, 0.0, maxiter, prec, prec, use_schur)
        st = SolveStats()
        self._finish(lib().qudax_solve_cgnr_dev(self._h, xp, bp, ctypes.byref(sp), ctypes.byref(st)),
                     allow_not_converged)
        return st.as_dict()
