"""CPU oracle for GPMA+ -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  The product path
(``paper_journals_pvldb_shalht17_b200``) never does: it shares no code with it.

The arithmetic lives in ``oracle/gpma_oracle.c`` (plain single-threaded C, -O2,
no SIMD intrinsics); this module is a ctypes wrapper plus numpy marshalling.
Each C function cites the PAPER.md passage it follows.  The root resize rule
(R6/R14) and the strict-delete layout, which no printed example reaches, are
pinned by hand-derived examples (tests/test_oracle_resize_pins.py) and
minimality properties; tools/oracle_mutations.sh shows each pin catching a
plausible mistake.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "gpma_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")

INSERT, DELETE = 0, 1
LAZY, REBALANCE = 0, 1
OK, INVALID, RANGE, RESERVED, OOM = 0, 1, 2, 3, 4
KEY_NONE = np.uint64(0xFFFFFFFFFFFFFFFF)
TOMB = np.uint32(0xFFFFFFFF)


def build(force: bool = False) -> str:
    """Compile the oracle (gcc -O2, single thread, no SIMD intrinsics)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        subprocess.check_call(["gcc", "-O2", "-shared", "-fPIC", "-o", _LIB, _SRC, "-lm"])
    return _LIB


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = C.CDLL(_LIB)
        P, u64, u32, i32 = C.c_void_p, C.c_uint64, C.c_uint32, C.c_int
        sig = {
            "orc_create": (P, [u32, P, P, u64, u32, u64, i32, P]),
            "orc_create_raw": (P, [u32, u64, u32, P, P, i32, P]),
            "orc_create_shard": (P, [u32, u32, u32, P, P, u64, u32, u64, i32, P]),
            "orc_destroy": (None, [P]),
            "orc_update": (i32, [P, P, P, u64, i32]),
            "orc_capacity": (u64, [P]),
            "orc_dump": (None, [P, P, P]),
            "orc_row_offset": (None, [P, P]),
            "orc_level_bounds": (None, [P, P, P]),
            "orc_stats": (None, [P, P]),
            "orc_trace": (u64, [P, P, u64]),
            "orc_export_csr": (u64, [P, P, P, P]),
            "orc_thresholds": (None, [u64, u32, u32, u32, u32, u32, P, P]),
            "orc_leaf_rule": (u32, [u64]),
            "orc_set_thresholds_bp": (None, [P, u32, u32, u32, u32]),
            "orc_bfs_csr": (None, [u32, P, P, u32, P]),
            "orc_set_algorithm": (None, [P, i32]),
            "orc_rounds_last": (u64, [P]),
            "orc_set_max_rounds": (None, [P, u64]),
            "orc_cc_csr": (None, [u32, P, P, P]),
            "orc_pagerank_csr": (i32, [u32, P, P, P, i32, C.c_double, C.c_double, i32]),
        }
        for name, (res, args) in sig.items():
            f = getattr(L, name)
            f.restype, f.argtypes = res, args
        _lib = L
    return _lib


def _p(a: np.ndarray | None):
    return None if a is None else a.ctypes.data


def _u64(a) -> np.ndarray:
    if hasattr(a, "numpy"):
        a = a.detach().cpu().numpy()
    a = np.asarray(a)
    if a.dtype == np.int64:
        a = a.view(np.uint64)
    elif a.dtype != np.uint64:
        a = a.astype(np.uint64)
    return np.ascontiguousarray(a)


def _u32(a) -> np.ndarray:
    if hasattr(a, "numpy"):
        a = a.detach().cpu().numpy()
    a = np.asarray(a)
    if a.dtype == np.int32:
        return np.ascontiguousarray(a.view(np.uint32))
    return np.ascontiguousarray(a.astype(np.uint32))


def thresholds(L: int, h: int, bp=(800, 4000, 9200, 8000)):
    mn = np.zeros(h + 1, np.uint64)
    mx = np.zeros(h + 1, np.uint64)
    lib().orc_thresholds(L, h, *bp, _p(mn), _p(mx))
    return mn.astype(np.int64).tolist(), mx.astype(np.int64).tolist()


def leaf_rule(cap0: int) -> int:
    return int(lib().orc_leaf_rule(cap0))


class OracleError(RuntimeError):
    def __init__(self, status):
        super().__init__(f"oracle status {status}")
        self.status = status


class Oracle:
    """One sequential GPMA+ store."""

    def __init__(self, V: int, keys=(), vals=(), *, leaf_slots: int = 0, capacity: int = 0,
                 delete_mode: int = LAZY, rows=None, algorithm: int = 0, _raw=None):
        st = C.c_int(0)
        if _raw is not None:
            cap, L, rk, rv = _raw
            rk, rv = _u64(rk), _u32(rv)
            self._h = lib().orc_create_raw(V, cap, L, _p(rk), _p(rv), delete_mode, C.byref(st))
        else:
            k, v = _u64(keys), _u32(vals)
            rb, re = rows if rows is not None else (0, 0)
            self._h = lib().orc_create_shard(V, rb, re, _p(k), _p(v), k.size, leaf_slots, capacity,
                                             delete_mode, C.byref(st))
        if st.value != OK:
            raise OracleError(st.value)
        self.V = V
        lib().orc_set_algorithm(self._h, algorithm)
        self.rb, self.nr = (rows[0], rows[1] - rows[0]) if rows is not None and rows[1] > rows[0] else (0, V)

    @classmethod
    def raw(cls, V, cap, L, keys, vals=None, delete_mode=LAZY, algorithm=0):
        vals = np.zeros(cap, np.uint32) if vals is None else vals
        return cls(V, _raw=(cap, L, keys, vals), delete_mode=delete_mode, algorithm=algorithm)

    @property
    def rounds(self) -> int:
        """GPMA (Alg. 1): retry rounds of the last insert batch."""
        return int(lib().orc_rounds_last(self._h))

    def set_max_rounds(self, r: int):
        """GPMA (Alg. 1) test hook: stop a batch after r rounds (0 = until every insertion took effect)."""
        lib().orc_set_max_rounds(self._h, r)

    def __del__(self):
        if getattr(self, "_h", None):
            lib().orc_destroy(self._h)
            self._h = None

    def update(self, keys, vals=None, op: int = INSERT) -> int:
        k = _u64(keys)
        v = None if vals is None else _u32(vals)
        return int(lib().orc_update(self._h, _p(k), _p(v), k.size, op))

    def insert(self, keys, vals):
        st = self.update(keys, vals, INSERT)
        if st:
            raise OracleError(st)

    def delete(self, keys):
        st = self.update(keys, None, DELETE)
        if st:
            raise OracleError(st)

    @property
    def capacity(self) -> int:
        return int(lib().orc_capacity(self._h))

    def stats(self) -> dict:
        out = np.zeros(16, np.uint64)
        lib().orc_stats(self._h, _p(out))
        names = ["cap", "L", "h", "V", "live", "tombstones", "guards", "slots_rewritten",
                 "windows_rewritten", "top_level", "pending", "resizes", "resizes_last", "row_begin", "rows"]
        return {n: int(out[i]) for i, n in enumerate(names)}

    def dump(self):
        cap = self.capacity
        k = np.zeros(cap, np.uint64)
        v = np.zeros(cap, np.uint32)
        lib().orc_dump(self._h, _p(k), _p(v))
        return k, v

    def row_offset(self):
        out = np.zeros(self.nr + 1, np.uint64)
        lib().orc_row_offset(self._h, _p(out))
        return out

    def level_bounds(self):
        h = self.stats()["h"]
        mn = np.zeros(h + 1, np.uint64)
        mx = np.zeros(h + 1, np.uint64)
        lib().orc_level_bounds(self._h, _p(mn), _p(mx))
        return mn.astype(np.int64).tolist(), mx.astype(np.int64).tolist()

    def trace(self):
        """Per-level (segment start slots, offsets incl. the closing one, flags) of the last batch."""
        n = int(lib().orc_trace(self._h, None, 0))
        buf = np.zeros(4 * max(n, 1), np.uint64)
        lib().orc_trace(self._h, _p(buf), n)
        levels = []
        for i in range(n):
            lvl, start, off, flag = (int(x) for x in buf[4 * i: 4 * i + 4])
            while len(levels) <= lvl:
                levels.append({"segments": [], "offsets": [], "flags": []})
            if flag == 2:
                levels[lvl]["offsets"].append(off)
            else:
                levels[lvl]["segments"].append(start)
                levels[lvl]["offsets"].append(off)
                levels[lvl]["flags"].append("Y" if flag else "N")
        return levels

    def export_csr(self):
        nnz = int(lib().orc_export_csr(self._h, None, None, None))
        rp = np.zeros(self.nr + 1, np.uint64)
        col = np.zeros(max(nnz, 1), np.uint32)
        val = np.zeros(max(nnz, 1), np.uint32)
        lib().orc_export_csr(self._h, _p(rp), _p(col), _p(val))
        return rp, col[:nnz], val[:nnz]

    # analytics on the exported CSR (the logical graph)
    def bfs(self, root: int):
        return bfs_csr(self.V, *self.export_csr()[:2], root)

    def cc(self):
        return cc_csr(self.V, *self.export_csr()[:2])

    def pagerank(self, x=None, damping=0.85, tol=1e-3, max_iter=100):
        return pagerank_csr(self.V, *self.export_csr()[:2], x=x, damping=damping, tol=tol,
                            max_iter=max_iter)


def bfs_csr(V, row_ptr, col, root):
    lv = np.zeros(V, np.int32)
    rp, cl = _u64(row_ptr), _u32(col)
    lib().orc_bfs_csr(V, _p(rp), _p(cl), root, _p(lv))
    return lv


def cc_csr(V, row_ptr, col):
    lab = np.zeros(V, np.uint32)
    rp, cl = _u64(row_ptr), _u32(col)
    lib().orc_cc_csr(V, _p(rp), _p(cl), _p(lab))
    return lab


def pagerank_csr(V, row_ptr, col, x=None, damping=0.85, tol=1e-3, max_iter=100):
    rp, cl = _u64(row_ptr), _u32(col)
    warm = x is not None
    xx = np.ascontiguousarray(np.array(x, dtype=np.float64)) if warm else np.zeros(V, np.float64)
    it = lib().orc_pagerank_csr(V, _p(rp), _p(cl), _p(xx), int(warm), damping, tol, max_iter)
    return xx, int(it)
