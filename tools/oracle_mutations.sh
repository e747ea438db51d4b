#!/usr/bin/env bash
# Mutation check of the oracle pins (CPU only): apply one plausible mistake at a time to
# oracle/gpma_oracle.c and require that the pin tests FAIL; restores the source at the end.
# Usage: tools/oracle_mutations.sh   (prints one line per mutant: CAUGHT / MISSED)
set -u
cd "$(dirname "$0")/.."
SRC=oracle/gpma_oracle.c
cp "$SRC" /tmp/orc_orig.c
trap 'cp /tmp/orc_orig.c "$SRC"; rm -f oracle/liboracle.so' EXIT
TESTS="tests/test_oracle_resize_pins.py tests/test_oracle_gpma_lock.py tests/test_oracle_golden.py"
mut() {
  python - "$2" "$3" <<'EOF'
import sys
s = open('/tmp/orc_orig.c').read()
a, b = sys.argv[1], sys.argv[2]
assert a in s, a
open('oracle/gpma_oracle.c', 'w').write(s.replace(a, b, 1))
EOF
  rm -f oracle/liboracle.so
  if python -m pytest $TESTS -q -x >/dev/null 2>&1; then echo "MISSED  $1"; else echo "CAUGHT  $1"; fi
}
mut "R6: resize as soon as level h-1 fails" \
  'for (i = 0; i <= o->h && np > 0; i++) {               /* "while root' \
  'for (i = 0; i < o->h && np > 0; i++) {               /* "while root'
mut "R14: a single doubling" \
  'if (N <= mx[ilog2_u64(cap / o->L)]) break;
      cap *= 2;' 'cap *= 2; break;'
mut "R14: one doubling too many" \
  'if (N <= mx[ilog2_u64(cap / o->L)]) break;' \
  'if (N <= mx[ilog2_u64(cap / o->L)]) { if (cap != o->cap) cap *= 2; break; }'
mut "strict delete: > for >= min_i" \
  '(n >= u && n - u >= o->tmin[i])' '(n >= u && n - u > o->tmin[i])'
mut "halving: <= for < min_h" \
  'if (!(cap > 2ull * o->L && N < mn[hh])) break;' 'if (!(cap > 2ull * o->L && N <= mn[hh])) break;'
mut "halving: at most one halving" \
  'if (!(cap > 2ull * o->L && N < mn[hh])) break;' 'if (!(cap > 2ull * o->L && N < mn[hh]) || cap != o->cap) break;'
mut "R28: smallest key wins every segment" \
  'win = g0;
        }' 'win = g0;
        }
        win = g0;'
mut "R7: extras to the first leaves" \
  'uint64_t lo = l * N / nl, hi = (l + 1) * N / nl;' \
  'uint64_t lo = N - (nl - l) * N / nl, hi = N - (nl - l - 1) * N / nl;'
mut "R5: raw ceil/floor bounds without the 2*prev cap" \
  'mx[i] = raw_max < 2 * mx[i - 1] ? raw_max : 2 * mx[i - 1];' 'mx[i] = raw_max;'
