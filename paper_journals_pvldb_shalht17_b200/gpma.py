"""Thin ctypes binding of include/gpma.h (argument marshalling only).

Every entry point forwards to the sm_100a library ``lib/libgpma.so``; there is no
Python or CPU fallback -- importing this module on a machine without the built
library raises, and the calls fail loudly without a CUDA device.

Arrays may be torch tensors (CUDA or CPU; CPU tensors are passed as host pointers
and staged by the library) or numpy arrays (host).  Keys are int64 tensors holding
the u64 bits ``src << 32 | dst``; values int32 holding u32 bits.
"""
from __future__ import annotations

import ctypes as C
import os

import numpy as np

from .buildlib import LIB

INSERT, DELETE = 0, 1
DELETE_LAZY, DELETE_REBALANCE = 0, 1
OK = 0
STATUS = {0: "ok", 1: "invalid argument", 2: "vertex id out of range", 3: "reserved key or value",
          4: "out of device memory", 5: "CUDA error", 6: "poisoned handle"}


class GpmaError(RuntimeError):
    def __init__(self, status: int, msg: str = ""):
        super().__init__(f"gpma status {status} ({STATUS.get(status, '?')}): {msg}")
        self.status = status


ALLOC_FN = C.CFUNCTYPE(C.c_void_p, C.c_size_t, C.c_void_p, C.c_void_p)
FREE_FN = C.CFUNCTYPE(None, C.c_void_p, C.c_void_p, C.c_void_p)


class gpma_config(C.Structure):
    _fields_ = [("struct_size", C.c_uint32), ("leaf_slots", C.c_uint32), ("initial_capacity", C.c_uint64),
                ("rho_leaf_bp", C.c_uint16), ("rho_root_bp", C.c_uint16), ("tau_leaf_bp", C.c_uint16),
                ("tau_root_bp", C.c_uint16), ("init_density_bp", C.c_uint16), ("algorithm", C.c_uint16),
                ("delete_mode", C.c_uint32), ("row_begin", C.c_uint32), ("row_end", C.c_uint32),
                ("alloc", ALLOC_FN), ("free", FREE_FN), ("alloc_ctx", C.c_void_p)]


def torch_allocator_hooks():
    """gpma_config.alloc / free through PyTorch's caching allocator (SURVEY §8(b) "Ownership":
    the store's memory then shows up in torch.cuda.memory_allocated and is reused by torch)."""
    import torch

    def _alloc(nbytes, stream, ctx):
        try:
            return torch.cuda.caching_allocator_alloc(int(nbytes), stream=int(stream or 0))
        except Exception:
            return None          # -> GPMA_ERR_OOM

    def _free(ptr, stream, ctx):
        if ptr:
            torch.cuda.caching_allocator_delete(int(ptr))

    return ALLOC_FN(_alloc), FREE_FN(_free)


class gpma_stats_t(C.Structure):
    _fields_ = [("num_vertices", C.c_uint32), ("leaf_slots", C.c_uint32), ("capacity", C.c_uint64),
                ("height", C.c_uint32), ("delete_mode", C.c_uint32), ("live_edges", C.c_uint64),
                ("tombstones", C.c_uint64), ("resizes", C.c_uint64), ("last_unique", C.c_uint64),
                ("last_pending", C.c_uint64), ("last_slots_rewritten", C.c_uint64),
                ("last_windows_rewritten", C.c_uint64), ("last_top_level", C.c_uint32),
                ("last_resized", C.c_uint32), ("last_rounds", C.c_uint64), ("last_level0_windows", C.c_uint64),
                ("total_batches", C.c_uint64), ("total_insert_keys", C.c_uint64), ("total_delete_keys", C.c_uint64),
                ("total_slots_rewritten", C.c_uint64), ("total_windows_rewritten", C.c_uint64),
                ("last_pending_level1", C.c_uint64), ("last_levels_skipped", C.c_uint64),
                ("last_big_head_windows", C.c_uint64)]


_lib = None


def lib() -> C.CDLL:
    """Load libgpma.so (built by __graft_entry__.build()); raise if it is missing."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB):
            raise ImportError(f"libgpma.so not built at {LIB}: run __graft_entry__.build()")
        L = C.CDLL(LIB)
        P, u64, u32, i32, st = C.c_void_p, C.c_uint64, C.c_uint32, C.c_int, C.c_int
        sig = {
            "gpma_config_default": (None, [P]),
            "gpma_create": (st, [u32, P, P, u64, P, P, P]),
            "gpma_create_raw": (st, [u32, u64, u32, P, P, P, P, P]),
            "gpma_destroy": (st, [P]),
            "gpma_update_batch": (st, [P, P, P, u64, i32, P]),
            "gpma_bfs": (st, [P, u32, P, P]),
            "gpma_cc": (st, [P, P, P]),
            "gpma_pagerank": (st, [P, P, i32, C.c_double, C.c_double, i32, P, P]),
            "gpma_pagerank_f32": (st, [P, P, i32, C.c_float, C.c_float, i32, P, P]),
            "gpma_export_csr": (st, [P, P, P, P, u64, P, P]),
            "gpma_stats": (st, [P, P]),
            "gpma_stats_host": (st, [P, P]),
            "gpma_debug_dump": (st, [P, P, P, P, P, P, P]),
            "gpma_debug_set_trace": (st, [P, i32]),
            "gpma_debug_dump_aux": (st, [P, P, P, P, P]),
            "gpma_dist_unique_id": (st, [P]),
            "gpma_dist_create": (st, [P, i32, i32, u32, P, P, u64, P, P, P]),
            "gpma_dist_info": (st, [P, P, P, P, P]),
            "gpma_debug_trace": (st, [P, P, u64, P]),
            "gpma_kernel_launches": (u64, [P]),
            "gpma_route": (st, [P, P, P, u64, u32, P, P, P, P]),
            "gpma_query_edges": (st, [P, P, u64, P, P, P]),
            "gpma_query_neighbors": (st, [P, P, u64, P, P, P, u64, P, P]),
            "gpma_query_reachable": (st, [P, P, P, u64, P, P]),
            "gpma_bfs_init": (st, [P, u32, P, P]),
            "gpma_bfs_level": (st, [P, P, i32, P, P]),
            "gpma_cc_round": (st, [P, P, i32, P, P]),
            "gpma_pr_push": (st, [P, P, i32, P, P]),
            "gpma_pr_update": (st, [P, P, P, C.c_double, P, P]),
            "gpma_pr_update_rows": (st, [P, P, P, C.c_double, P, P]),
            "gpma_bfs_bits": (st, [P, P, i32, P, P]),
            "gpma_pr_update_rows_dev": (st, [P, P, P, C.c_double, P, P]),
            "gpma_validate_batch": (st, [P, P, P, u64, i32, P]),
            "gpma_bfs_merge": (st, [P, P, P, u32, i32, P]),
            "gpma_debug_profile": (st, [P, C.c_char_p]),
            "gpma_debug_profile_read": (st, [P, C.c_char_p, C.c_size_t]),
            "gpma_status_string": (C.c_char_p, [st]),
            "gpma_last_error": (C.c_char_p, [P]),
        }
        for name, (res, args) in sig.items():
            f = getattr(L, name)
            f.restype, f.argtypes = res, args
        _lib = L
    return _lib


EXPORTS = ["gpma_config_default", "gpma_create", "gpma_create_raw", "gpma_destroy", "gpma_update_batch",
           "gpma_bfs", "gpma_cc", "gpma_pagerank", "gpma_pagerank_f32", "gpma_export_csr", "gpma_stats",
           "gpma_debug_dump", "gpma_debug_set_trace", "gpma_debug_trace", "gpma_kernel_launches",
           "gpma_debug_profile", "gpma_debug_profile_read", "gpma_route", "gpma_bfs_init", "gpma_bfs_level",
           "gpma_cc_round", "gpma_pr_push", "gpma_pr_update", "gpma_pr_update_rows", "gpma_bfs_bits",
           "gpma_bfs_merge", "gpma_query_edges", "gpma_query_neighbors",
           "gpma_query_reachable", "gpma_debug_dump_aux", "gpma_dist_unique_id", "gpma_dist_create",
           "gpma_dist_info", "gpma_pr_update_rows_dev", "gpma_validate_batch", "gpma_stats_host",
           "gpma_status_string", "gpma_last_error"]


def _ptr(a):
    """Raw pointer of a torch tensor / numpy array (None passes NULL)."""
    if a is None:
        return None
    if hasattr(a, "data_ptr"):
        if not a.is_contiguous():
            raise ValueError("array must be contiguous")
        return a.data_ptr() or None
    if isinstance(a, np.ndarray):
        if not a.flags["C_CONTIGUOUS"]:
            raise ValueError("array must be contiguous")
        return a.ctypes.data or None
    raise TypeError(type(a))


def _numel(a) -> int:
    return int(a.numel()) if hasattr(a, "numel") else int(a.size)


def _itemsize(a) -> int:
    return int(a.element_size()) if hasattr(a, "element_size") else int(a.itemsize)


def _check_arr(a, itemsize: int, min_numel: int, what: str, device=None):
    """Reject arrays the C ABI would read out of bounds: wrong element size, too short, or on
    another device than the handle's (a host array is fine: the library stages it)."""
    if a is None:
        return
    if _itemsize(a) != itemsize:
        raise ValueError(f"{what}: element size {_itemsize(a)} B, expected {itemsize} B")
    if _numel(a) < min_numel:
        raise ValueError(f"{what}: {_numel(a)} elements, need at least {min_numel}")
    dev = getattr(a, "device", None) if hasattr(a, "data_ptr") else None     # torch tensors only
    if device is not None and dev is not None and dev.type == "cuda" and dev.index != device:
        raise ValueError(f"{what}: tensor on cuda:{dev.index}, handle on cuda:{device}")


_torch = None
_raw_stream = None


def _torch_mod():
    """torch (imported once) and its raw current-stream getter, or None without CUDA."""
    global _torch, _raw_stream
    if _torch is None:
        try:
            import torch
            _torch = torch
            if torch.cuda.is_available():
                _raw_stream = getattr(torch._C, "_cuda_getCurrentRawStream", None) or (
                    lambda d: torch.cuda.current_stream(d).cuda_stream)
        except Exception:
            _torch = False
    return _torch


def _stream(stream, device=None):
    if stream is None:
        _torch_mod()
        if _raw_stream is None:
            return None
        if device is None:
            device = _torch.cuda.current_device()
        return _raw_stream(device) or None
    if isinstance(stream, int):
        return stream or None
    return stream.cuda_stream or None


def _targ(a, itemsize: int, min_numel: int, what: str, device):
    """(pointer, numel) of an update / result array with _check_arr's checks, fast path for torch
    tensors (the per-call binding cost of the small-batch update path)."""
    if a is None:
        return None, 0
    T = _torch_mod()
    if T and type(a) is T.Tensor:
        n = a.numel()
        if a.element_size() != itemsize:
            raise ValueError(f"{what}: element size {a.element_size()} B, expected {itemsize} B")
        if n < min_numel:
            raise ValueError(f"{what}: {n} elements, need at least {min_numel}")
        if a.is_cuda and device is not None and a.get_device() != device:
            raise ValueError(f"{what}: tensor on cuda:{a.get_device()}, handle on cuda:{device}")
        if not a.is_contiguous():
            raise ValueError("array must be contiguous")
        return a.data_ptr() or None, n
    _check_arr(a, itemsize, min_numel, what, device)
    return _ptr(a), _numel(a)
    if isinstance(stream, int):
        return stream or None
    return stream.cuda_stream or None


def _update(*args):
    global _update
    _update = lib().gpma_update_batch       # bound once: the ctypes function itself
    return _update(*args)


class Gpma:
    """One GPMA+ store (one handle of the C ABI).  Method names follow gpma.h."""

    def __init__(self, handle, num_vertices, hooks=None):
        self._h = handle
        self.V = num_vertices
        self._hooks = hooks          # keeps the allocator callbacks alive for the handle's life
        try:
            import torch
            self.device = torch.cuda.current_device() if torch.cuda.is_available() else None
        except Exception:
            self.device = None

    # -- create / destroy -------------------------------------------------
    @classmethod
    def gpma_create(cls, num_vertices: int, init_keys=None, init_vals=None, *, leaf_slots: int = 0,
                    initial_capacity: int = 0, delete_mode: int = DELETE_LAZY, thresholds_bp=None,
                    init_density_bp: int = 6000, rows=None, algorithm: int = 0, stream=None,
                    torch_allocator: bool = False) -> "Gpma":
        cfg = gpma_config()
        lib().gpma_config_default(C.byref(cfg))
        hooks = None
        if torch_allocator:
            hooks = torch_allocator_hooks()
            cfg.alloc, cfg.free = hooks
        if init_keys is not None:
            _check_arr(init_keys, 8, 0, "init_keys")
            _check_arr(init_vals, 4, _numel(init_keys), "init_vals")
        cfg.algorithm = algorithm
        if rows is not None:
            cfg.row_begin, cfg.row_end = rows
        cfg.leaf_slots = leaf_slots
        cfg.initial_capacity = initial_capacity
        cfg.delete_mode = delete_mode
        cfg.init_density_bp = init_density_bp
        if thresholds_bp:
            cfg.rho_leaf_bp, cfg.rho_root_bp, cfg.tau_leaf_bp, cfg.tau_root_bp = thresholds_bp
        h = C.c_void_p()
        n = 0 if init_keys is None else _numel(init_keys)
        st = lib().gpma_create(num_vertices, _ptr(init_keys), _ptr(init_vals), n, C.byref(cfg),
                               _stream(stream), C.byref(h))
        if st != OK:
            raise GpmaError(st, "gpma_create")
        return cls(h, num_vertices, hooks)

    @classmethod
    def gpma_create_raw(cls, num_vertices: int, capacity: int, leaf_slots: int, keys, vals, *,
                        delete_mode: int = DELETE_LAZY, algorithm: int = 0, stream=None) -> "Gpma":
        cfg = gpma_config()
        lib().gpma_config_default(C.byref(cfg))
        cfg.delete_mode = delete_mode
        cfg.algorithm = algorithm
        h = C.c_void_p()
        st = lib().gpma_create_raw(num_vertices, capacity, leaf_slots, _ptr(keys), _ptr(vals), C.byref(cfg),
                                   _stream(stream), C.byref(h))
        if st != OK:
            raise GpmaError(st, "gpma_create_raw")
        return cls(h, num_vertices)

    def gpma_destroy(self):
        if self._h:
            lib().gpma_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.gpma_destroy()
        except Exception:
            pass

    def _check(self, st, what):
        if st != OK:
            msg = lib().gpma_last_error(self._h) if self._h else b""
            raise GpmaError(st, f"{what}: {msg.decode() if msg else ''}")

    # -- update -----------------------------------------------------------
    def gpma_update_batch(self, keys, vals=None, op: int = INSERT, stream=None, check: bool = True) -> int:
        kp, n = _targ(keys, 8, 0, "keys", self.device)
        vp, _ = _targ(vals, 4, n, "vals", self.device)
        st = _update(self._h, kp, vp, n, op, _stream(stream, self.device))
        if check and st != OK:
            self._check(st, "gpma_update_batch")
        return st

    def insert(self, keys, vals, stream=None):
        return self.gpma_update_batch(keys, vals, INSERT, stream)

    def delete(self, keys, stream=None):
        return self.gpma_update_batch(keys, None, DELETE, stream)

    # -- analytics --------------------------------------------------------
    def gpma_bfs(self, root: int, levels, stream=None):
        _check_arr(levels, 4, self.V, "levels", self.device)
        self._check(lib().gpma_bfs(self._h, root, _ptr(levels), _stream(stream)), "gpma_bfs")
        return levels

    def gpma_cc(self, labels, stream=None):
        _check_arr(labels, 4, self.V, "labels", self.device)
        self._check(lib().gpma_cc(self._h, _ptr(labels), _stream(stream)), "gpma_cc")
        return labels

    def gpma_pagerank(self, rank, warm_start: bool = False, damping: float = 0.85, tol_l1: float = 1e-3,
                      max_iter: int = 100, stream=None) -> int:
        it = C.c_int(0)
        if _itemsize(rank) not in (4, 8) or _numel(rank) < self.V:
            raise ValueError("rank: need V float64 (or float32) elements")
        f = lib().gpma_pagerank_f32 if str(getattr(rank, "dtype", "")).endswith("float32") else lib().gpma_pagerank
        self._check(f(self._h, _ptr(rank), int(warm_start), damping, tol_l1, max_iter, C.byref(it),
                      _stream(stream)), "gpma_pagerank")
        return it.value

    def gpma_export_csr(self, row_ptr=None, col=None, val=None, stream=None) -> int:
        nnz = C.c_uint64(0)
        cap = 0 if col is None else _numel(col)
        self._check(lib().gpma_export_csr(self._h, _ptr(row_ptr), _ptr(col), _ptr(val), cap, C.byref(nnz),
                                          _stream(stream)), "gpma_export_csr")
        return nnz.value

    # -- introspection ----------------------------------------------------
    def gpma_stats(self) -> dict:
        s = gpma_stats_t()
        self._check(lib().gpma_stats(self._h, C.byref(s)), "gpma_stats")
        return {f: getattr(s, f) for f, _ in s._fields_}

    def gpma_stats_host(self) -> dict:
        """gpma_stats without device work (live_edges / tombstones not counted)."""
        s = gpma_stats_t()
        self._check(lib().gpma_stats_host(self._h, C.byref(s)), "gpma_stats_host")
        return {f: getattr(s, f) for f, _ in s._fields_}

    def gpma_debug_dump(self, keys=None, vals=None, row_offset=None, leaf_live=None, heads=None, stream=None):
        self._check(lib().gpma_debug_dump(self._h, _ptr(keys), _ptr(vals), _ptr(row_offset), _ptr(leaf_live),
                                          _ptr(heads), _stream(stream)), "gpma_debug_dump")

    def gpma_debug_dump_aux(self, tomb_mask=None, leaf_guards=None, out_degree=None, stream=None):
        self._check(lib().gpma_debug_dump_aux(self._h, _ptr(tomb_mask), _ptr(leaf_guards), _ptr(out_degree),
                                              _stream(stream)), "gpma_debug_dump_aux")

    def gpma_dist_info(self) -> dict:
        r, n, rb, re = C.c_int(0), C.c_int(0), C.c_uint32(0), C.c_uint32(0)
        self._check(lib().gpma_dist_info(self._h, C.byref(r), C.byref(n), C.byref(rb), C.byref(re)), "gpma_dist_info")
        return {"rank": r.value, "nranks": n.value, "row_begin": rb.value, "row_end": re.value}

    @staticmethod
    def gpma_dist_unique_id() -> bytes:
        """The 128-byte NCCL unique id (call on one rank, broadcast it to the others)."""
        buf = C.create_string_buffer(128)
        st = lib().gpma_dist_unique_id(buf)
        if st != OK:
            raise GpmaError(st, "gpma_dist_unique_id (is NCCL loadable?)")
        return buf.raw

    @classmethod
    def gpma_dist_create(cls, uid: bytes, rank: int, nranks: int, num_vertices: int, init_keys=None,
                         init_vals=None, *, leaf_slots: int = 0, delete_mode: int = DELETE_LAZY,
                         stream=None) -> "Gpma":
        """Rank `rank` of a multi-GPU store (include/gpma.h "multi-GPU handle"): the library's
        NCCL communicator runs the routing / BFS / CC / PageRank exchanges; collective."""
        cfg = gpma_config()
        lib().gpma_config_default(C.byref(cfg))
        cfg.leaf_slots = leaf_slots
        cfg.delete_mode = delete_mode
        if init_keys is not None:
            _check_arr(init_keys, 8, 0, "init_keys")
            _check_arr(init_vals, 4, _numel(init_keys), "init_vals")
        h = C.c_void_p()
        n = 0 if init_keys is None else _numel(init_keys)
        idb = C.create_string_buffer(bytes(uid), 128)
        st = lib().gpma_dist_create(idb, rank, nranks, num_vertices, _ptr(init_keys), _ptr(init_vals), n,
                                    C.byref(cfg), _stream(stream), C.byref(h))
        if st != OK:
            raise GpmaError(st, "gpma_dist_create")
        return cls(h, num_vertices)

    def gpma_debug_set_trace(self, enable: bool):
        self._check(lib().gpma_debug_set_trace(self._h, int(enable)), "gpma_debug_set_trace")

    def gpma_debug_trace(self):
        n = C.c_uint64(0)
        lib().gpma_debug_trace(self._h, None, 0, C.byref(n))
        buf = np.zeros(4 * max(n.value, 1), np.uint64)
        lib().gpma_debug_trace(self._h, buf.ctypes.data, n.value, C.byref(n))
        return buf[: 4 * n.value].reshape(-1, 4)

    def gpma_debug_profile(self, kernel_filter: str | None):
        self._check(lib().gpma_debug_profile(self._h, kernel_filter.encode() if kernel_filter else None),
                    "gpma_debug_profile")

    def gpma_debug_profile_read(self) -> dict:
        buf = C.create_string_buffer(1 << 16)
        self._check(lib().gpma_debug_profile_read(self._h, buf, len(buf)), "gpma_debug_profile_read")
        out = {}
        for line in buf.value.decode().splitlines():
            name, n, ms = line.split("\t")
            out[name] = (int(n), float(ms))
        return out

    # -- query buffer ---------------------------------------------------------
    def gpma_query_edges(self, keys, vals=None, found=None, stream=None):
        self._check(lib().gpma_query_edges(self._h, _ptr(keys), _numel(keys), _ptr(vals), _ptr(found),
                                           _stream(stream)), "gpma_query_edges")

    def gpma_query_neighbors(self, verts, row_ptr=None, col=None, val=None, stream=None) -> int:
        nnz = C.c_uint64(0)
        cap = 0 if col is None else _numel(col)
        self._check(lib().gpma_query_neighbors(self._h, _ptr(verts), _numel(verts), _ptr(row_ptr), _ptr(col),
                                               _ptr(val), cap, C.byref(nnz), _stream(stream)),
                    "gpma_query_neighbors")
        return nnz.value

    def gpma_query_reachable(self, src, dst, out, stream=None):
        self._check(lib().gpma_query_reachable(self._h, _ptr(src), _ptr(dst), _numel(src), _ptr(out),
                                               _stream(stream)), "gpma_query_reachable")
        return out

    # -- sharded-store primitives (device tensors) ---------------------------
    def gpma_route(self, keys, vals, nranks: int, out_keys, out_vals, stream=None):
        counts = (C.c_uint64 * nranks)()
        self._check(lib().gpma_route(self._h, _ptr(keys), _ptr(vals), _numel(keys), nranks, _ptr(out_keys),
                                     _ptr(out_vals), counts, _stream(stream)), "gpma_route")
        return [int(c) for c in counts]

    def gpma_bfs_init(self, root: int, levels, stream=None):
        self._check(lib().gpma_bfs_init(self._h, root, _ptr(levels), _stream(stream)), "gpma_bfs_init")

    def gpma_bfs_level(self, levels, depth: int, stream=None) -> int:
        f = C.c_uint32(0)
        self._check(lib().gpma_bfs_level(self._h, _ptr(levels), depth, C.byref(f), _stream(stream)),
                    "gpma_bfs_level")
        return f.value

    def gpma_cc_round(self, labels, init: bool, stream=None) -> int:
        c = C.c_uint64(0)
        self._check(lib().gpma_cc_round(self._h, _ptr(labels), int(init), C.byref(c), _stream(stream)),
                    "gpma_cc_round")
        return c.value

    def gpma_pr_push(self, x, init: bool, y, stream=None):
        self._check(lib().gpma_pr_push(self._h, _ptr(x), int(init), _ptr(y), _stream(stream)), "gpma_pr_push")

    def gpma_pr_update(self, x, y, damping: float = 0.85, stream=None) -> float:
        e = C.c_double(0.0)
        self._check(lib().gpma_pr_update(self._h, _ptr(x), _ptr(y), damping, C.byref(e), _stream(stream)),
                    "gpma_pr_update")
        return e.value

    def gpma_pr_update_rows(self, x, y_rows, damping: float = 0.85, stream=None) -> float:
        e = C.c_double(0.0)
        self._check(lib().gpma_pr_update_rows(self._h, _ptr(x), _ptr(y_rows), damping, C.byref(e),
                                              _stream(stream)), "gpma_pr_update_rows")
        return e.value

    def gpma_pr_update_rows_dev(self, x, y_rows, err_dev, damping: float = 0.85, stream=None):
        self._check(lib().gpma_pr_update_rows_dev(self._h, _ptr(x), _ptr(y_rows), damping, _ptr(err_dev),
                                                  _stream(stream)), "gpma_pr_update_rows_dev")

    def gpma_validate_batch(self, keys, vals=None, op: int = INSERT, stream=None) -> int:
        """Status of a batch slice against the global vertex range (no mutation): 0 / 2 / 3."""
        return int(lib().gpma_validate_batch(self._h, _ptr(keys), _ptr(vals), _numel(keys), op, _stream(stream)))

    def gpma_bfs_bits(self, levels, depth: int, bitmap, stream=None):
        self._check(lib().gpma_bfs_bits(self._h, _ptr(levels), depth, _ptr(bitmap), _stream(stream)),
                    "gpma_bfs_bits")

    def gpma_bfs_merge(self, levels, bitmaps, nbitmaps: int, depth: int, stream=None):
        self._check(lib().gpma_bfs_merge(self._h, _ptr(levels), _ptr(bitmaps), nbitmaps, depth, _stream(stream)),
                    "gpma_bfs_merge")

    def gpma_kernel_launches(self) -> int:
        return int(lib().gpma_kernel_launches(self._h))
