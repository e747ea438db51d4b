"""Pin the CPU oracle to the values PAPER.md prints (goldens under tests/golden/)."""
import numpy as np
import pytest

import oracle as O
from gpma_gen import fig3_layout
from tests.brute import KEY_NONE, SeqPMA


def _occupied(keys):
    return [int(k) for k in keys if int(k) != KEY_NONE]


def test_fig3_threshold_table(golden):
    """Fig. 3 table: rho/tau decimals and min/max entry counts for sizes 4..32."""
    g = golden("fig3_thresholds.json")
    mn, mx = O.thresholds(4, 3)
    assert mn == g["min_entries"]
    assert mx == g["max_entries"]
    # the printed decimals are the linear rule rounded to 2 places (R4)
    h = 3
    for i in range(4):
        rho = (800 * (h - i) + 4000 * i) / (10000 * h)
        tau = (9200 * (h - i) + 8000 * i) / (10000 * h)
        assert round(rho + 1e-12, 2) == g["rho"][i]
        assert round(tau + 1e-12, 2) == g["tau"][i]


def test_fig3_table_rejects_raw_rounding():
    """R5: the raw ceil(rho*size)/floor(tau*size) would give 1,2,5,13 / 3,7,13,25 (not the table)."""
    mn, mx = O.thresholds(4, 3)
    assert mn != [1, 2, 5, 13] and mx != [3, 7, 13, 25]


@pytest.mark.parametrize("cap,L", [(16, 4), (32, 4), (1 << 14, 8), (1 << 25, 16), (1 << 28, 16),
                                   (1 << 31, 16)])
def test_leaf_rule(cap, L):
    """R3: L = max(4, 2^floor(log2 log2 cap)); Fig. 3 (32 -> 4), Fig. 5 (16 -> 4)."""
    assert O.leaf_rule(cap) == L


def test_example4_rounds(golden):
    """Ex. 4 / Fig. 6: every printed round of GPMA+ insertion."""
    g = golden("ex4_gpma_plus.json")
    o = O.Oracle.raw(64, g["capacity"], g["leaf_slots"], fig3_layout())
    k0, _ = o.dump()
    assert _occupied(k0) == g["original_sorted"]
    o.insert(g["insert"], [7] * len(g["insert"]))
    tr = o.trace()
    assert len(tr) == len(g["rounds"])
    for got, want in zip(tr, g["rounds"]):
        assert got["segments"] == want["segments"]
        assert got["offsets"] == want["offsets"]
        assert got["flags"] == want["flags"]
    k, _ = o.dump()
    assert _occupied(k) == g["rounds"][-1]["sorted_after"]


def test_example4_round0_content(golden):
    """Ex. 4 round 0 sorted contents: only the leaf-0 group is absorbed."""
    g = golden("ex4_gpma_plus.json")
    o = O.Oracle.raw(64, 32, 4, fig3_layout())
    o.insert([1, 4], [0, 0])  # the only group accepted in round 0
    k, _ = o.dump()
    assert _occupied(k) == g["rounds"][0]["sorted_after"]
    assert o.trace()[0]["flags"] == ["Y"]


def test_example1_single_insert(golden):
    """Ex. 1: 48 overflows its leaf (4 > 3) and lands in segment-[16,31]."""
    g = golden("ex1_pma_insert.json")
    o = O.Oracle.raw(64, 32, 4, fig3_layout())
    o.insert([g["insert"]], [0])
    tr = o.trace()
    assert tr[0]["flags"] == ["N"] and tr[1]["flags"] == ["N"] and tr[2]["flags"] == ["Y"]
    lvl = len(tr) - 1
    start = tr[lvl]["segments"][0]
    assert [start, start + (4 << lvl) - 1] == g["accepting_segment"]
    k, _ = o.dump()
    assert _occupied(k) == g["final_sorted"]


def test_batch_of_one_equals_sequential_pma():
    """GPMA+ with |U| = 1 coincides with the sequential PMA of Ex. 1 --
    checked over a random single-key insert sequence against tests/brute.SeqPMA."""
    rng = np.random.default_rng(5)
    raw = [int(x) for x in fig3_layout().tolist()]
    raw = [KEY_NONE if x == -1 else x for x in raw]
    o = O.Oracle.raw(4096, 32, 4, fig3_layout())
    _, mx = O.thresholds(4, 3)
    seq = SeqPMA(raw, 4, mx)
    present = set(_occupied(raw))
    for _ in range(7):  # stays below the root bound (24 entries)
        k = int(rng.integers(0, 4000))
        if k in present:
            continue
        present.add(k)
        seq.insert(k)
        o.insert([k], [0])
        got, _ = o.dump()
        assert [int(x) for x in got] == seq.s


def test_fig5_csr_on_gpma(golden):
    """Fig. 5: guards at slots 4, 8, 14; row offsets; export_csr arrays."""
    g = golden("fig5_csr.json")
    keys = [s << 32 | d for s, d, _ in g["edges"]]
    vals = [w for _, _, w in g["edges"]]
    o = O.Oracle(g["V"], keys, vals)
    st = o.stats()
    assert st["cap"] == g["capacity"] and st["L"] == g["leaf_slots"]
    k, v = o.dump()
    ents = []
    for x in _occupied(k):
        d = x & 0xFFFFFFFF
        ents.append([x >> 32, "inf" if d == 0xFFFFFFFF else d])
    assert ents == g["entries_in_order"]
    guard_slots = [i for i, x in enumerate(k) if int(x) != KEY_NONE and (int(x) & 0xFFFFFFFF) == 0xFFFFFFFF]
    assert guard_slots == g["guard_slots"]
    assert o.row_offset().tolist() == [0] + g["guard_slots"]
    rp, col, val = o.export_csr()
    assert rp.tolist() == g["csr_row_ptr"]
    assert col.tolist() == g["csr_col"]
    assert val.tolist() == g["csr_val"]
