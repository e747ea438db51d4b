"""Independent checkers used by the tests (pure Python, small inputs only).

* ``Replay``      -- brute-force logical edge set: insert = map[key] := val, delete = erase
                     (the plain definition the method must reach).
* ``check_layout`` -- the structural invariants of SURVEY §8(c)-4 over a raw layout dump.
* ``SeqPMA``      -- a textbook sequential PMA insert (Ex. 1, [10,11]):
                     binary-search the leaf, place the entry at its rear, climb to the nearest
                     ancestor within the upper threshold, re-dispatch evenly.  GPMA+ with a
                     batch of one update must coincide with it.
None of this imports the oracle's arithmetic; thresholds come from the caller.
"""
from __future__ import annotations

import numpy as np

KEY_NONE = 0xFFFFFFFFFFFFFFFF
TOMB = 0xFFFFFFFF
GUARD = 0xFFFFFFFF


class Replay:
    def __init__(self, V, keys=(), vals=()):
        self.V = V
        self.m = {}
        for k, v in zip(keys, vals):
            self.m[int(k)] = int(v)

    def insert(self, keys, vals):
        for k, v in zip(keys, vals):
            self.m[int(k)] = int(v)

    def delete(self, keys):
        for k in keys:
            self.m.pop(int(k), None)

    def csr(self):
        items = sorted(self.m.items())
        rp = np.zeros(self.V + 1, np.uint64)
        for k, _ in items:
            rp[(k >> 32) + 1] += 1
        rp = np.cumsum(rp).astype(np.uint64)
        col = np.array([k & 0xFFFFFFFF for k, _ in items], np.uint32)
        val = np.array([v for _, v in items], np.uint32)
        return rp, col, val


def check_layout(keys, vals, L, V, mx0, row_offset=None, guards=True):
    """Invariants 1,2,3,5 of SURVEY §8(c)-4 on a raw dump. Returns the live count."""
    keys = [int(k) for k in keys]
    vals = [int(v) for v in vals]
    cap = len(keys)
    assert cap & (cap - 1) == 0 and cap >= 2 * L, "cap must be a power of two >= 2L"
    prev = -1
    guard_slot = {}
    live = 0
    for leaf in range(cap // L):
        seg = keys[leaf * L:(leaf + 1) * L]
        occ = [k != KEY_NONE for k in seg]
        n = sum(occ)
        assert occ == [True] * n + [False] * (L - n), f"leaf {leaf} not left-packed"
        assert n <= mx0, f"leaf {leaf} holds {n} > max_0 {mx0}"
        for p in range(n):
            k = seg[p]
            assert k > prev, f"slot {leaf * L + p}: keys not strictly increasing"
            prev = k
            s = leaf * L + p
            if (k & 0xFFFFFFFF) == GUARD:
                guard_slot[k >> 32] = s
            elif vals[s] != TOMB:
                live += 1
    if guards:
        assert sorted(guard_slot) == list(range(V)), "exactly one guard per vertex"
        if row_offset is not None:
            ro = [int(x) for x in row_offset]
            assert ro[0] == 0
            for u in range(V):
                assert ro[u + 1] == guard_slot[u], f"row_offset[{u + 1}] != slot(guard {u})"
            assert all(ro[i] <= ro[i + 1] for i in range(V))
    return live


def window_counts_ok(keys, vals, L, trace_levels, bounds, op_insert, cap_before, cap_after):
    """Invariant 4: every window rewritten (and not re-rewritten higher up) satisfies its bound,
    and every sub-window of it at level j satisfies count <= max_j."""
    mn, mx = bounds
    keys = [int(k) for k in keys]
    vals = [int(v) for v in vals]

    def count(s0, s1):
        return sum(1 for s in range(s0, s1) if keys[s] != KEY_NONE and vals[s] != TOMB)

    if cap_before != cap_after:
        return  # resized: the whole array was re-laid (checked by check_layout + root bound)
    accepted = []
    for lvl, rec in enumerate(trace_levels):
        for start, fl in zip(rec["segments"], rec["flags"]):
            if fl == "Y":
                accepted.append((lvl, start, start + (L << lvl)))
    for lvl, s0, s1 in accepted:
        if any(l2 > lvl and a <= s0 and s1 <= b for l2, a, b in accepted):
            continue
        n = count(s0, s1)
        if op_insert:
            assert n <= mx[lvl], f"window level {lvl} [{s0},{s1}) holds {n} > {mx[lvl]}"
        else:
            assert n >= mn[lvl], f"window level {lvl} [{s0},{s1}) holds {n} < {mn[lvl]}"
        for j in range(lvl):
            w = L << j
            for a in range(s0, s1, w):
                assert count(a, a + w) <= mx[j]


class SeqPMA:
    """Textbook sequential PMA of integer keys (no values) for the batch-size-1 pin."""

    def __init__(self, slots, L, mx):
        self.s = list(slots)
        self.L = L
        self.mx = mx  # per-level max entry counts

    def insert(self, k):
        L, s = self.L, self.s
        nleaf = len(s) // L
        # binary search: largest non-empty leaf whose first key <= k, else leaf 0
        heads = [(i, s[i * L]) for i in range(nleaf) if s[i * L] != KEY_NONE]
        lo, hi = 0, len(heads)
        while lo < hi:
            mid = (lo + hi) // 2
            if heads[mid][1] <= k:
                lo = mid + 1
            else:
                hi = mid
        leaf = heads[lo - 1][0] if lo else 0
        lvl = 0
        while True:
            w0 = (leaf >> lvl) << lvl
            a, b = w0 * L, (w0 + (1 << lvl)) * L
            ents = [x for x in s[a:b] if x != KEY_NONE]
            if len(ents) + 1 <= self.mx[lvl]:
                ents = sorted(ents + [k])
                nl = 1 << lvl
                N = len(ents)
                for l in range(nl):
                    lo_, hi_ = l * N // nl, (l + 1) * N // nl
                    for p in range(L):
                        s[a + l * L + p] = ents[lo_ + p] if p < hi_ - lo_ else KEY_NONE
                return lvl
            lvl += 1
            if (L << lvl) > len(s):
                raise RuntimeError("root overflow (not exercised)")
