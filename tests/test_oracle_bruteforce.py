"""Pin the oracle's logical edge set and structural invariants by brute force (tiny graphs)."""
import numpy as np
import pytest

import oracle as O
from tests.brute import Replay, check_layout, window_counts_ok


def _keys(src, dst):
    return [(int(s) << 32) | int(d) for s, d in zip(src, dst)]


def _check(o, ref, V, op_insert, cap_before, mode):
    k, v = o.dump()
    st = o.stats()
    mn, mx = o.level_bounds()
    live = check_layout(k, v, st["L"], V, mx[0], o.row_offset())
    rp, col, val = o.export_csr()
    erp, ecol, evl = ref.csr()
    assert rp.tolist() == erp.tolist()
    assert col.tolist() == ecol.tolist()
    assert val.tolist() == evl.tolist()
    assert live == len(ref.m) == st["live"]
    if mode == O.REBALANCE:
        assert st["tombstones"] == 0
    window_counts_ok(k, v, st["L"], o.trace(), (mn, mx), op_insert, cap_before, st["cap"])
    if st["resizes_last"] and op_insert:
        assert st["live"] + st["guards"] <= mx[-1]


def _random_run(seed, mode, V=32, steps=40, maxb=24, pattern="random"):
    rng = np.random.default_rng(seed)
    init_n = int(rng.integers(0, 3 * V))
    src = rng.integers(0, V, init_n)
    dst = rng.integers(0, V, init_n)
    keys = _keys(src, dst)
    vals = rng.integers(0, 1 << 31, init_n).tolist()
    o = O.Oracle(V, keys, vals, delete_mode=mode)
    ref = Replay(V, keys, vals)
    _check(o, ref, V, True, o.capacity, mode)
    for step in range(steps):
        b = int(rng.integers(1, maxb))
        if pattern == "one_row":
            s = np.full(b, rng.integers(0, V))
            d = rng.integers(0, V, b)
        elif pattern == "ascending":
            base = int(rng.integers(0, V * V - b))
            ks = np.arange(base, base + b)
            s, d = ks // V, ks % V
        else:
            s = rng.integers(0, V, b)
            d = rng.integers(0, V, b)
        ks = _keys(s, d)
        if pattern == "reinsert" and ref.m and step % 2 == 1:
            ks = list(ref.m)[: b]
        cap0 = o.capacity
        if rng.random() < 0.5:
            vs = rng.integers(0, 1 << 31, len(ks)).tolist()
            if len(ks) > 2:  # duplicates inside the batch: the last occurrence wins (R10)
                ks.append(ks[0])
                vs.append(int(rng.integers(0, 1 << 31)))
            o.insert(ks, vs)
            ref.insert(ks, vs)
            _check(o, ref, V, True, cap0, mode)
        else:
            if ref.m and rng.random() < 0.7:  # mostly delete present keys
                present = list(ref.m)
                idx = rng.integers(0, len(present), min(len(ks), len(present)))
                ks = [present[i] for i in idx] + ks[: len(ks) // 3]
            o.delete(ks)
            ref.delete(ks)
            _check(o, ref, V, False, cap0, mode)
    return o


@pytest.mark.parametrize("seed", range(40))
def test_random_lazy(seed):
    _random_run(seed, O.LAZY)


@pytest.mark.parametrize("seed", range(40))
def test_random_rebalance(seed):
    _random_run(1000 + seed, O.REBALANCE)


@pytest.mark.parametrize("pattern", ["one_row", "ascending", "reinsert"])
@pytest.mark.parametrize("mode", [O.LAZY, O.REBALANCE])
def test_adversarial(pattern, mode):
    for seed in range(6):
        _random_run(77 + seed, mode, V=48, steps=30, maxb=40, pattern=pattern)


def test_grow_and_shrink_resize():
    """Doubling then halving (R14): invariants + logical set across many resizes."""
    V = 16
    o = O.Oracle(V, [], [], delete_mode=O.REBALANCE)
    ref = Replay(V)
    caps = [o.capacity]
    all_keys = [(s << 32) | d for s in range(V) for d in range(V)]
    rng = np.random.default_rng(3)
    rng.shuffle(all_keys)
    for i in range(0, len(all_keys), 16):
        ks = all_keys[i:i + 16]
        cap0 = o.capacity
        o.insert(ks, [1] * len(ks))
        ref.insert(ks, [1] * len(ks))
        _check(o, ref, V, True, cap0, O.REBALANCE)
        caps.append(o.capacity)
    assert max(caps) > caps[0]
    for i in range(0, len(all_keys), 16):
        ks = all_keys[i:i + 16]
        cap0 = o.capacity
        o.delete(ks)
        ref.delete(ks)
        _check(o, ref, V, False, cap0, O.REBALANCE)
        caps.append(o.capacity)
    assert caps[-1] < max(caps)
    assert o.stats()["live"] == 0


def test_lazy_tombstones_and_revive():
    V = 8
    keys = _keys([0, 0, 1, 2], [1, 2, 3, 4])
    o = O.Oracle(V, keys, [10, 11, 12, 13])
    o.delete([keys[1]])
    st = o.stats()
    assert st["tombstones"] == 1 and st["live"] == 3
    k, v = o.dump()
    slot = [i for i, x in enumerate(k) if int(x) == keys[1]][0]
    assert int(v[slot]) == 0xFFFFFFFF           # tombstone kept in place
    o.insert([keys[1]], [99])                    # revive in place (R12)
    k2, v2 = o.dump()
    assert int(v2[slot]) == 99 and (k2 == k).all()
    assert o.stats()["tombstones"] == 0
    o.delete([keys[1], keys[1], (7 << 32) | 7])  # duplicate + absent delete: no-ops beyond the first
    assert o.stats()["live"] == 3


@pytest.mark.parametrize("op", [O.INSERT, O.DELETE])
def test_validation_rejects_without_mutation(op):
    V = 8
    o = O.Oracle(V, _keys([0, 1], [1, 2]), [5, 6])
    before = o.dump()
    bad_range = [(1 << 32) | 2, (9 << 32) | 1]
    bad_guard = [(1 << 32) | 0xFFFFFFFF]
    vals = [1, 2]
    assert o.update(bad_range, vals if op == O.INSERT else None, op) == O.RANGE
    assert o.update(bad_guard, [1] if op == O.INSERT else None, op) == O.RESERVED
    if op == O.INSERT:
        assert o.update([(1 << 32) | 3], [0xFFFFFFFF], op) == O.RESERVED
    after = o.dump()
    assert (before[0] == after[0]).all() and (before[1] == after[1]).all()
    assert o.update([], None, op) == O.OK
