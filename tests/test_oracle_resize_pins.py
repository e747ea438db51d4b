"""Pin the oracle's root rules -- R6 (the root is tested before any resize), R14 (how far to
double / halve) and the strict-delete dual (min_i) -- with hand-derived examples on
the Fig. 3-size PMA (32 slots, L = 4, h = 3; thresholds min 1,2,4,8 / max 3,6,12,24)
and with minimality properties over random runs.

Every expected layout below was derived by hand from Alg. 4 and the readings
R5/R7/R9/R14; the derivation is written next to each case.  A plausible mistake
in the oracle's resize / strict-delete code (doubling when level h-1 fails, one doubling only,
over-doubling, `<` for `<=` in a bound, halving one step too far or not at all) fails one of
them.  Thresholds of the other sizes used here, derived by hand from R4/R5 with L = 4:
  cap 16 (h=2):  rho .08 .24 .40 -> min 1,2,4;   tau .92 .86 .80 -> max 3,6,12
  cap 64 (h=4):  tau .92 .89 .86 .83 .80 -> raw 3,7,13,26,51 -> max 3,6,12,24,48
  cap 128 (h=5): tau .92 .896 .872 .848 .824 .80 -> raw 3,7,13,27,52,102 -> max 3,6,12,24,48,96
"""
import numpy as np
import pytest

import oracle as O
from gpma_gen import fig3_layout
from tests.brute import KEY_NONE, Replay, check_layout

NONE = -1


def _raw(leaves, L=4):
    keys = []
    for lf in leaves:
        keys += list(lf) + [NONE] * (L - len(lf))
    return np.array(keys, dtype=np.int64)


def _leaves(o, L=4):
    k, _ = o.dump()
    out = []
    for i in range(0, len(k), L):
        out.append([int(x) for x in k[i:i + L] if int(x) != KEY_NONE])
    return out


def _trace(o):
    return [(t["segments"], t["offsets"], t["flags"]) for t in o.trace()]


# ------------------------------------------------------------------ R6: root tested first
def test_root_accepts_without_resize():
    """Left half full (12 entries = max_2), right half 4 entries; insert 5 (R9: leaf 0).
    leaf 0: 3+1 > 3 N; [0,7]: 6+1 > 6 N; [0,15]: 12+1 > 12 N; root: 16+1 = 17 <= 24 Y.
    R7 over 8 leaves of 17 entries: counts 2,2,2,2,2,2,2,3.  The literal alternative of Alg. 4
    l.4 (double as soon as level h-1 fails) would give capacity 64 instead."""
    o = O.Oracle.raw(64, 32, 4, _raw([[10, 11, 12], [20, 21, 22], [30, 31, 32], [40, 41, 42],
                                      [50], [60], [70], [80]]))
    o.insert([5], [0])
    assert o.capacity == 32 and o.stats()["resizes_last"] == 0
    assert _leaves(o) == [[5, 10], [11, 12], [20, 21], [22, 30], [31, 32], [40, 41], [42, 50], [60, 70, 80]]
    assert _trace(o) == [([0], [0, 1], ["N"]), ([0], [0, 1], ["N"]), ([0], [0, 1], ["N"]),
                         ([0], [0, 1], ["Y"])]


# ------------------------------------------------------------------ R14: doubling
def _full_pma():
    """24 entries, 3 per leaf (= max_0 everywhere, = max_3 at the root): keys 10l+1..10l+3."""
    return O.Oracle.raw(128, 32, 4, _raw([[10 * l + 1, 10 * l + 2, 10 * l + 3] for l in range(8)]))


def test_root_rejects_then_one_doubling_layout():
    """Insert 4 into the full PMA: every level rejects (3+1>3, 6+1>6, 12+1>12, 24+1>24), so
    the root resizes with N = 25: 25 > max_3(32) = 24, 25 <= max_4(64) = 48 -> capacity 64.
    R7 over 16 leaves of 25 entries: floor(25(l+1)/16) - floor(25l/16) =
    1,2,1,2,1,2,1,2,2,1,2,1,2,1,2,2."""
    o = _full_pma()
    o.insert([4], [0])
    assert o.capacity == 64 and o.stats()["resizes_last"] == 1
    got = _leaves(o)
    assert [len(x) for x in got] == [1, 2, 1, 2, 1, 2, 1, 2, 2, 1, 2, 1, 2, 1, 2, 2]
    assert sum(got, []) == sorted([4] + [10 * l + j for l in range(8) for j in (1, 2, 3)])
    assert got[:3] == [[1], [2, 3], [4]]
    tr = o.trace()
    assert [t["flags"] for t in tr] == [["N"], ["N"], ["N"], ["N"]]


def test_doubling_boundary_is_inclusive():
    """24 + 24 new keys (10l+4..10l+6) -> N = 48 = max_4(64): exactly one doubling (`<=`)."""
    o = _full_pma()
    ks = [10 * l + j for l in range(8) for j in (4, 5, 6)]
    o.insert(ks, [0] * len(ks))
    assert o.capacity == 64
    assert [len(x) for x in _leaves(o)] == [3] * 16          # 48 over 16 leaves, R7


def test_doubling_repeats_until_it_fits():
    """24 + 25 new keys -> N = 49 > max_4(64) = 48, <= max_5(128) = 96: the root doubles twice
    in one batch (R14 'double repeatedly'); one doubling (P:983-984 read literally) would leave
    the root over its bound, and doubling once more than needed would give 256."""
    o = _full_pma()
    ks = [10 * l + j for l in range(8) for j in (4, 5, 6)] + [79]
    o.insert(ks, [0] * len(ks))
    assert o.capacity == 128 and o.stats()["resizes_last"] == 1
    # 49 entries over 32 leaves: floor(49(l+1)/32) - floor(49l/32); the first leaves 1,2,1,2
    assert [len(x) for x in _leaves(o)][:4] == [1, 2, 1, 2]
    assert sum(len(x) for x in _leaves(o)) == 49


# ------------------------------------------------------------------ strict deletes (dual, min_i)
def test_strict_delete_climbs_by_min_bounds():
    """Fig. 3 PMA (R26), strict deletes {2, 5, 8}.  Leaves: 2 -> 0, 5 and 8 -> 1.
    L0: leaf 0: 1-1 = 0 < min_0 = 1 N; leaf 1: 3-2 = 1 >= 1 Y -> [13].
    L1 [0,7]: (1+1)-1 = 1 < min_1 = 2 N.
    L2 [0,15]: (1+1+2+1)-1 = 4 >= min_2 = 4 Y (inclusive) -> {13,16,17,23} one per leaf."""
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), delete_mode=O.REBALANCE)
    o.delete([8, 2, 5])
    assert o.capacity == 32
    assert _leaves(o) == [[13], [16], [17], [23], [27, 28], [31], [34, 37, 42], [46, 51, 62]]
    assert _trace(o) == [([0, 4], [0, 1, 3], ["N", "Y"]), ([0], [0, 1], ["N"]), ([0], [0, 1], ["Y"])]


def test_strict_delete_reaches_root_and_halves():
    """Fig. 3 PMA, strict deletes of the 9 keys 16..42 (leaves 2,2,3,4,4,5,6,6,6).
    L0: every group empties its leaf (0 < 1) N N N N N.
    L1: [8,15] 3-3 = 0 N; [16,23] 3-3 = 0 N; [24,31] 6-3 = 3 >= 2 Y -> [46][51 62].
    L2: [0,15] 7-3 = 4 >= 4 Y -> [2][5][8][13]; [16,31] 6-3 = 3 < 4 N.
    L3 (root): 10-3 = 7 < 8 N -> resize with N = 7: 7 < min_3(32) = 8 and 7 <= max_2(16) = 12
    -> halve to 16; 7 >= min_2(16) = 4 -> stop.  R7: 7 over 4 leaves = 1,2,2,2."""
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), delete_mode=O.REBALANCE)
    o.delete([16, 17, 23, 27, 28, 31, 34, 37, 42])
    assert _trace(o) == [([8, 12, 16, 20, 24], [0, 2, 3, 5, 6, 9], ["N"] * 5),
                         ([8, 16, 24], [0, 3, 6, 9], ["N", "N", "Y"]),
                         ([0, 16], [0, 3, 6], ["Y", "N"]),
                         ([0], [0, 3], ["N"])]
    assert o.capacity == 16 and o.stats()["resizes_last"] == 1
    assert _leaves(o) == [[2], [5, 8], [13, 46], [51, 62]]


def test_strict_delete_halving_stops_at_min_bound():
    """Fig. 3 PMA, strict deletes of 12 keys leaving {2, 46, 51, 62}.
    L0: leaves 1..6 all empty out, N.  L1: [0,7] 4-3 = 1 < 2 N; [8,15] 0 N; [16,23] 0 N;
    [24,31] 6-3 = 3 >= 2 Y -> [46][51 62].  L2: [0,15] 7-6 = 1 < 4 N; [16,31] 6-3 = 3 < 4 N.
    Root: 13-9 = 4 < 8 N -> N = 4: halve to 16 (4 <= 12); at 16, 4 < min_2(16) = 4 is false
    -> stop at 16 (a `<=` would halve once more, to 8).  R7: one entry per leaf."""
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), delete_mode=O.REBALANCE)
    o.delete([5, 8, 13, 16, 17, 23, 27, 28, 31, 34, 37, 42])
    assert [t["flags"] for t in o.trace()] == [["N"] * 6, ["N", "N", "N", "Y"], ["N", "N"], ["N"]]
    assert o.capacity == 16
    assert _leaves(o) == [[2], [46], [51], [62]]


# ------------------------------------------------------------------ minimality over random runs
def _root_max(L, cap):
    h = int(np.log2(cap // L))
    return O.thresholds(L, h)[1][h]


def _root_min(L, cap):
    h = int(np.log2(cap // L))
    return O.thresholds(L, h)[0][h]


@pytest.mark.parametrize("seed", range(12))
def test_resize_minimality_random(seed):
    """After every resize: it happened only because the root window rejected (the last traced
    level is the root, flag N), and the new capacity is the one R14 names -- insert: the
    smallest power of two whose root holds N (N <= max_h(cap), N > max_h(cap/2)); strict
    delete: every halving was needed (N < min_h(2 cap)) and the last one stopped for a reason
    (N >= min_h(cap), cap = 2L, or the half could not hold N)."""
    rng = np.random.default_rng(900 + seed)
    V = 24
    o = O.Oracle(V, [], [], delete_mode=O.REBALANCE)
    ref = Replay(V)
    all_keys = [(s << 32) | d for s in range(V) for d in range(V)]
    rng.shuffle(all_keys)
    live = []
    pool = list(all_keys)
    seen_up = seen_down = 0
    for step in range(60):
        grow = step < 30
        cap0 = o.capacity
        h0 = o.stats()["h"]
        if grow:
            b = int(rng.integers(4, 40))
            ks = pool[:b]
            pool = pool[b:]
            o.insert(ks, [1] * len(ks))
            ref.insert(ks, [1] * len(ks))
            live += ks
        else:
            b = int(rng.integers(4, 40))
            ks = live[:b]
            live = live[b:]
            o.delete(ks)
            ref.delete(ks)
        st = o.stats()
        N = st["live"] + st["guards"]
        L, cap = st["L"], st["cap"]
        if st["resizes_last"]:
            tr = o.trace()
            assert len(tr) == h0 + 1 and tr[-1]["flags"] == ["N"]    # the root rejected (R6)
            if cap > cap0:
                seen_up += 1
                assert N <= _root_max(L, cap) and N > _root_max(L, cap // 2)
            else:
                seen_down += 1
                assert cap < cap0 and N < _root_min(L, 2 * cap)
                assert N >= _root_min(L, cap) or cap == 2 * L or N > _root_max(L, cap // 2)
        else:
            assert cap == cap0
        k, v = o.dump()
        mn, mx = o.level_bounds()
        assert check_layout(k, v, L, V, mx[0], o.row_offset()) == len(ref.m)
    assert seen_up and seen_down
