"""Counter-based synthetic graph streams (shared input generator; no method arithmetic).

Recipe (SURVEY.md §8(d) "Synthetic inputs", R17):

* random bits: ``draw(seed, ctr) = splitmix64(splitmix64(seed) ^ ctr)`` -- a pure
  function of (seed, counter), identical on every device;
* RMAT (Graph500 a,b,c,d = .57,.19,.19,.05): one 16-bit uniform per recursion
  level (4 levels per 64-bit draw), compared against integer thresholds;
* uniform G(n,m): src = draw mod V, dst = draw mod V;
* self-loops dropped, endpoints >= V rejected (Pokec-shaped config), vertex ids
  scrambled by a seeded permutation (rank of draw(seed_perm, v));
* dedupe (set of unique keys), random timestamps ts = draw(seed_ts, key) --
  "we randomly set the timestamps of all edges"; the
  stream is the E unique edges with the smallest timestamps, in timestamp
  order;
* sliding window: the initial graph is the first half of the
  stream; slide s deletes the B oldest window edges, then inserts the next B.

Keys are int64 tensors holding ``src << 32 | dst`` (src, dst < 2**31, so the
signed and unsigned orders agree); values are int32 in [0, 2**31).
"""
from __future__ import annotations

import math
from dataclasses import dataclass, field

import torch

M64 = (1 << 64) - 1
KEY_NONE = M64                  # empty slot key (R2)
VAL_TOMB = 0xFFFFFFFF           # lazy-delete tombstone value (R12)
DST_GUARD = 0xFFFFFFFF          # guard column "infinity" (R1, Fig. 5)


def _i64(c: int) -> int:
    c &= M64
    return c - (1 << 64) if c >= (1 << 63) else c


_GOLDEN = _i64(0x9E3779B97F4A7C15)
_C1 = _i64(0xBF58476D1CE4E5B9)
_C2 = _i64(0x94D049BB133111EB)


def splitmix64_int(z: int) -> int:
    """Scalar splitmix64 on Python ints (used for seeds and to pin the tensor version)."""
    z = (z + 0x9E3779B97F4A7C15) & M64
    z = ((z ^ (z >> 30)) * 0xBF58476D1CE4E5B9) & M64
    z = ((z ^ (z >> 27)) * 0x94D049BB133111EB) & M64
    return z ^ (z >> 31)


def _srl(x: torch.Tensor, k: int) -> torch.Tensor:
    """Logical right shift of an int64 tensor viewed as u64."""
    return (x >> k) & ((1 << (64 - k)) - 1)


def splitmix64(z: torch.Tensor) -> torch.Tensor:
    """splitmix64 over an int64 tensor (wrapping arithmetic == u64 arithmetic)."""
    z = z + _GOLDEN
    z = (z ^ _srl(z, 30)) * _C1
    z = (z ^ _srl(z, 27)) * _C2
    return z ^ _srl(z, 31)


def draw(seed: int, ctr: torch.Tensor) -> torch.Tensor:
    """64 random bits (as int64) for each counter value: splitmix64(splitmix64(seed) ^ ctr)."""
    s = _i64(splitmix64_int(seed & M64))
    return splitmix64(ctr ^ s)


def _tag(seed: int, tag: int) -> int:
    return splitmix64_int((seed * 0x100000001B3 + tag) & M64)


def _scramble(V: int, seed: int, device) -> torch.Tensor:
    """Seeded vertex permutation new_id[v] (Graph500-style scramble)."""
    h = draw(_tag(seed, 0x5045524D), torch.arange(V, dtype=torch.int64, device=device))
    order = torch.argsort(h, stable=True)
    new_id = torch.empty(V, dtype=torch.int64, device=device)
    new_id[order] = torch.arange(V, dtype=torch.int64, device=device)
    return new_id


def rmat_edges(scale: int, ctr0: int, count: int, seed: int, abc=(0.57, 0.19, 0.19),
               device="cpu") -> tuple[torch.Tensor, torch.Tensor]:
    """Raw RMAT draws for candidate indices [ctr0, ctr0+count): (src, dst) in [0, 2**scale)."""
    a, b, c = abc
    ta, tab, tabc = int(a * 65536), int((a + b) * 65536), int((a + b + c) * 65536)
    e = torch.arange(ctr0, ctr0 + count, dtype=torch.int64, device=device)
    src = torch.zeros_like(e)
    dst = torch.zeros_like(e)
    w = None
    for lvl in range(scale):
        if lvl % 4 == 0:
            w = draw(_tag(seed, 0x524D4154 + lvl // 4), e)
        r = _srl(w, 16 * (lvl % 4)) & 0xFFFF
        sbit = (r >= tab).to(torch.int64)                    # quadrants c, d
        dbit = ((r >= ta) & (r < tab)) | (r >= tabc)          # quadrants b, d
        src = (src << 1) | sbit
        dst = (dst << 1) | dbit.to(torch.int64)
    return src, dst


def uniform_edges(V: int, ctr0: int, count: int, seed: int, device="cpu"):
    e = torch.arange(ctr0, ctr0 + count, dtype=torch.int64, device=device)
    src = _srl(draw(_tag(seed, 0x554E4953), e), 1) % V
    dst = _srl(draw(_tag(seed, 0x554E4944), e), 1) % V
    return src, dst


def edge_values(keys: torch.Tensor, seed: int) -> torch.Tensor:
    """Opaque u32 payload per edge (never the tombstone value): int32 in [0, 2**31)."""
    return (_srl(draw(_tag(seed, 0x56414C), keys), 33) & 0x7FFFFFFF).to(torch.int32)


_CUB_MAX = 1 << 30            # elements per sort/unique call (CUB takes < 2^31 items)


def make_stream(kind: str, V: int, E: int, seed: int, scale: int | None = None,
                device="cpu", sub_chunk: int = 1 << 27) -> torch.Tensor:
    """E unique edge keys (int64) in random-timestamp order.

    Draws candidates in rounds of max(E, 4096) until the set of unique, loop-free, in-range
    edges holds at least E keys; then orders that set by ts = draw(seed_ts, key) (signed
    int64 order, ties by key) and keeps the first E.  A round is generated in sub-chunks of
    `sub_chunk` candidates to bound memory, and the set is kept in source-range buckets of
    < 2^30 keys (sort limits at configs[4] scale, 2^31 edges); neither changes the stream.
    """
    new_id = _scramble(V, seed, device)
    chunk = max(E, 4096)
    nbk = 1
    while chunk * 2 // nbk > _CUB_MAX:                     # candidates per bucket per round
        nbk *= 2
    bnd = torch.tensor([((b * V) // nbk) << 32 for b in range(1, nbk)], dtype=torch.int64, device=device)
    buckets = [torch.empty(0, dtype=torch.int64, device=device) for _ in range(nbk)]
    ctr = 0
    while sum(b.numel() for b in buckets) < E:
        parts = [[b] for b in buckets]
        for c0 in range(ctr, ctr + chunk, sub_chunk):
            cn = min(sub_chunk, ctr + chunk - c0)
            if kind == "rmat":
                s, d = rmat_edges(scale, c0, cn, seed, device=device)
            elif kind == "uniform":
                s, d = uniform_edges(V, c0, cn, seed, device=device)
            else:
                raise ValueError(kind)
            ok = (s != d) & (s < V) & (d < V)
            s, d = new_id[s[ok]], new_id[d[ok]]
            u = torch.unique((s << 32) | d)                  # sorted
            del s, d, ok
            cut = [0] + torch.searchsorted(u, bnd).tolist() + [u.numel()]
            for b in range(nbk):
                parts[b].append(u[cut[b]:cut[b + 1]])
            del u
        ctr += chunk
        for b in range(nbk):                                 # one bucket's temporaries at a time
            buckets[b] = torch.unique(torch.cat(parts[b]))
            parts[b] = None
        del parts
        if ctr > 64 * chunk:
            raise RuntimeError("stream generator: too few unique edges")
    keys = buckets[0] if nbk == 1 else torch.cat(buckets)    # sorted: buckets are key ranges
    del buckets
    tseed = _tag(seed, 0x5453)
    if keys.numel() <= _CUB_MAX:
        ts = draw(tseed, keys)
        order = torch.argsort(ts, stable=True)               # keys are sorted -> ties broken by key
        return keys[order[:E]].contiguous()
    # above the sort limit: the 16 signed ranges of the top 4 bits of ts, in order, each sorted
    # stably on its own (its keys stay in key order, so ties still break by key); ts is drawn
    # in chunks and again per range, never held whole (its temporaries are 8 B per key each)
    top = torch.empty(keys.numel(), dtype=torch.int8, device=keys.device)
    for c0 in range(0, keys.numel(), _CUB_MAX // 4):
        top[c0:c0 + _CUB_MAX // 4] = ((draw(tseed, keys[c0:c0 + _CUB_MAX // 4]) >> 60) + 8).to(torch.int8)
    out = torch.empty(E, dtype=torch.int64, device=keys.device)
    pos = 0
    for b in range(16):
        idx = torch.nonzero(top == b).squeeze(1)
        if idx.numel() == 0:
            continue
        kr = keys[idx]
        del idx
        kb = kr[torch.argsort(draw(tseed, kr), stable=True)]
        del kr
        take = min(kb.numel(), E - pos)
        out[pos:pos + take] = kb[:take]
        pos += take
        del kb
        if pos == E:
            break
    return out


def weak_scaled(cfg_index: int, P: int) -> "StreamConfig":
    """Per-GPU work fixed as P grows (PAPER.md P:1700-1703 style): the RMAT scale grows by
    log2(P); V, E, window and the global batch all scale by P."""
    c = CONFIGS[cfg_index]
    lp = int(math.log2(P))
    assert 1 << lp == P, "P must be a power of two"
    return StreamConfig(f"{c.name}-x{P}", c.kind, c.V * P, c.E * P, c.window * P, c.batch * P, c.seed,
                        scale=None if c.scale is None else c.scale + lp, delete_mode=c.delete_mode)


@dataclass
class SlidingWindow:
    """Sliding-window schedule over a timestamp-ordered stream (R17)."""
    keys: torch.Tensor
    vals: torch.Tensor
    window: int
    batch: int

    @property
    def n_slides(self) -> int:
        return (self.keys.numel() - self.window) // self.batch

    def initial(self):
        return self.keys[: self.window], self.vals[: self.window]

    def slide(self, s: int):
        """(delete_keys, insert_keys, insert_vals) of slide s: expired first, then arrived."""
        B, W = self.batch, self.window
        dk = self.keys[s * B:(s + 1) * B]
        ik = self.keys[W + s * B: W + (s + 1) * B]
        iv = self.vals[W + s * B: W + (s + 1) * B]
        return dk, ik, iv

    def window_after(self, s: int):
        """Live window keys (stream order) after slide s (s = -1: the initial window)."""
        lo = (s + 1) * self.batch
        return self.keys[lo: lo + self.window]


@dataclass
class StreamConfig:
    name: str
    kind: str
    V: int
    E: int
    window: int
    batch: int
    seed: int
    scale: int | None = None
    delete_mode: str = "lazy"
    extra: dict = field(default_factory=dict)


# SURVEY.md §8(d) table; seeds 0x6D6100 + config index.
CONFIGS = {
    0: StreamConfig("rmat-s10", "rmat", 1024, 16384, 8192, 1024, 0x6D6100, scale=10),
    1: StreamConfig("pokec-shaped", "rmat", 1_600_000, 30_000_000, 15_000_000, 1_000_000,
                    0x6D6101, scale=21, extra={"batches": [100, 1000, 10_000, 100_000, 1_000_000]}),
    2: StreamConfig("graph500-s24-ef16", "rmat", 1 << 24, 1 << 28, 1 << 27, 1 << 20, 0x6D6102, scale=24),
    3: StreamConfig("uniform-16M-256M-resize", "uniform", 1 << 24, 1 << 28, 1 << 23, 1 << 20,
                    0x6D6103, delete_mode="rebalance"),
    4: StreamConfig("rmat-s27-sharded", "rmat", 1 << 27, 1 << 31, 1 << 30, 1 << 20, 0x6D6104, scale=27),
}


def config_stream(cfg: int | StreamConfig, seed: int | None = None, device="cpu", **over) -> SlidingWindow:
    c = CONFIGS[cfg] if isinstance(cfg, int) else cfg
    if over:
        c = StreamConfig(**{**c.__dict__, **over})
    sd = c.seed if seed is None else seed
    keys = make_stream(c.kind, c.V, c.E, sd, scale=c.scale, device=device)
    vals = edge_values(keys, sd)
    if torch.device(device).type == "cuda":
        # generated on torch's current stream; consumers may use other streams
        torch.cuda.synchronize(device)
    return SlidingWindow(keys, vals, c.window, c.batch)


def bfs_root(sw: SlidingWindow, seed: int, slide: int) -> int:
    """R18: src of window edge number draw(seed, slide) mod W (always has out-degree >= 1)."""
    w = sw.window_after(slide)
    idx = int(_srl(draw(_tag(seed, 0x524F4F54), torch.tensor([slide + 1], dtype=torch.int64)), 1)[0]) % w.numel()
    return int(w[idx].item()) >> 32


def fig3_layout():
    """PAPER.md Fig. 3 as reconstructed in SURVEY.md Appendix A.2 / R26.

    32 slots, leaf size 4; keys are the printed integers as (src=0, dst=k); an
    empty slot is KEY_NONE, i.e. -1 as int64.  Returned as an int64 tensor.
    """
    leaves = [[2], [5, 8, 13], [16, 17], [23], [27, 28], [31], [34, 37, 42], [46, 51, 62]]
    keys = []
    for lf in leaves:
        keys += lf + [-1] * (4 - len(lf))
    return torch.tensor(keys, dtype=torch.int64)


def fig5_edges():
    """PAPER.md Fig. 5: 3 vertices, 6 weighted edges (src, dst, weight)."""
    return [(0, 0, 1), (0, 2, 2), (1, 2, 3), (2, 0, 4), (2, 1, 5), (2, 2, 6)]
