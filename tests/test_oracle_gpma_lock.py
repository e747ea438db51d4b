"""Pin the oracle's GPMA lock-based insertion (Alg. 1)."""
import numpy as np
import pytest

import oracle as O
from gpma_gen import fig3_layout
from tests.brute import KEY_NONE, Replay, SeqPMA, check_layout


def _occ(keys):
    return [int(k) for k in keys if int(k) != KEY_NONE]


def test_example2_round1_row(golden):
    """Fig. 4 Round1 row: the three round-1 winners land without conflicts."""
    g = golden("ex2_gpma_lock.json")
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), algorithm=1)
    o.insert(g["round1_winners"], [0] * 3)
    assert o.rounds == 1
    assert _occ(o.dump()[0]) == g["round1_row"]


def test_example2_full_batch_round1(golden):
    """The FULL batch {1,4,9,35,48}, stopped after round 1: the Fig. 4 Round1 row -- 1 beats
    4 for leaf 0 and 48 beats 35 for segment [24,31]; R28 reproduces both choices."""
    g = golden("ex2_gpma_lock.json")
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), algorithm=1)
    o.set_max_rounds(1)
    o.insert(g["batch"], [0] * 5)
    assert o.rounds == 1
    assert _occ(o.dump()[0]) == g["round1_row"]
    assert sorted(set(g["batch"]) - set(g["round1_row"])) == g["round1_losers"]


def test_example2_full_batch_two_rounds(golden):
    """The full batch needs a second round for the aborted insertions (4 and one of 35/48)."""
    g = golden("ex2_gpma_lock.json")
    o = O.Oracle.raw(64, 32, 4, fig3_layout(), algorithm=1)
    o.insert(g["batch"], [0] * 5)
    assert o.rounds == g["rounds"]
    assert _occ(o.dump()[0]) == sorted(set(g["round1_row"]) | set(g["batch"]))


def test_gpma_batch_of_one_is_sequential_pma():
    rng = np.random.default_rng(21)
    raw = [KEY_NONE if x == -1 else int(x) for x in fig3_layout().tolist()]
    o = O.Oracle.raw(4096, 32, 4, fig3_layout(), algorithm=1)
    _, mx = O.thresholds(4, 3)
    seq = SeqPMA(raw, 4, mx)
    present = set(_occ(raw))
    for _ in range(7):
        k = int(rng.integers(0, 4000))
        if k in present:
            continue
        present.add(k)
        seq.insert(k)
        o.insert([k], [0])
        assert [int(x) for x in o.dump()[0]] == seq.s


@pytest.mark.parametrize("seed", range(15))
def test_gpma_random_logical_set_and_invariants(seed):
    rng = np.random.default_rng(500 + seed)
    V = 40
    o = O.Oracle(V, [], [], algorithm=1)
    ref = Replay(V)
    for step in range(25):
        b = int(rng.integers(1, 60))
        ks = [int(a) << 32 | int(c) for a, c in zip(rng.integers(0, V // 4, b), rng.integers(0, V, b))]  # hot rows
        if rng.random() < 0.75:
            vs = rng.integers(0, 1 << 31, len(ks)).tolist()
            o.insert(ks, vs)
            ref.insert(ks, vs)
        else:
            o.delete(ks)
            ref.delete(ks)
        k, v = o.dump()
        st = o.stats()
        mn, mx = o.level_bounds()
        assert check_layout(k, v, st["L"], V, mx[0], o.row_offset()) == len(ref.m)
    rp, col, val = o.export_csr()
    erp, ecol, evl = ref.csr()
    assert col.tolist() == ecol.tolist() and val.tolist() == evl.tolist()
