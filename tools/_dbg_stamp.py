"""Temporary globaltimer phase stamps in k_small_insert (tools only; restore update.cu with git
checkout afterwards).  Read with tools/_dbgprobe.py."""
p = 'paper_journals_pvldb_shalht17_b200/csrc/update.cu'
s = open(p).read()
s = s.replace('''template <int L>
__global__ void __launch_bounds__(SB_T) k_small_insert(''', '''__device__ unsigned long long gp_dbg_t[64];
__device__ __forceinline__ void dbg_stamp(int i) {
  if (threadIdx.x == 0) { unsigned long long t; asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t)); gp_dbg_t[i] = t; }
}
template <int L>
__global__ void __launch_bounds__(SB_T) k_small_insert(''', 1)
anchors = [('  // load + validate (RESERVED beats RANGE', 0),
           ('  // stable sort by key (the arrival index breaks ties), padding up to a power of two', 1),
           ('  // values and targets in key order, group heads\n  uint32_t f[2], sv_[2], st_[2];', 2),
           ('  uint32_t fe[2] = {f[0], f[1]}, ng = 0;', 3),
           ('  // the leaf groups, SB_ROWS at a time, each leaf in a shared-memory row', 4),
           ('  // the rejected new keys, in key order, with their targets: the pending list of level 1\n  uint32_t kf[2];', 20)]
for a, i in anchors:
    assert a in s, a
    s = s.replace(a, f"  dbg_stamp({i});\n" + a, 1)
old = '''      a_effs += o.effs;
    }
  }'''
assert old in s
s = s.replace(old, '''      a_effs += o.effs;
    }
    __syncthreads();
    dbg_stamp(5 + g0 / SB_ROWS);
  }''', 1)
old = '''    mirror_ctrl(c, c_host, seq);      // the control block, mirrored (zero-copy) for the host'''
assert old in s
s = s.replace(old, '''    dbg_stamp(21);
    mirror_ctrl(c, c_host, seq);
    dbg_stamp(22);''', 1)
s += '\nextern "C" void gp_dbg_times(unsigned long long *out) { cudaMemcpyFromSymbol(out, gp::gp_dbg_t, 64 * 8); }\n'
open(p, 'w').write(s)
