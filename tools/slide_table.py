import csv, collections, sys
rows=[r for r in csv.reader(open(sys.argv[1])) if len(r)>10]
h=rows[0]; ki=h.index("Kernel Name"); mi=h.index("Metric Name"); vi=h.index("Metric Value"); ii=h.index("ID")
L=collections.OrderedDict()
for r in rows[1:]:
    L.setdefault(r[ii], {"name": r[ki]})[r[mi]] = float(r[vi].replace(',',''))
seq=list(L.values())
starts=[i for i,x in enumerate(seq) if x["name"].startswith("void k_lazy_delete_r")]
def summarize(a,b):
    agg=collections.OrderedDict()
    for x in seq[a:b]:
        n=x["name"].split("(")[0].replace("void ","")
        e=agg.setdefault(n,[0,0.0,0.0])
        e[0]+=1; e[1]+=x["gpu__time_duration.sum"]/1e3; e[2]+=(x.get("dram__bytes_read.sum",0)+x.get("dram__bytes_write.sum",0))/1e6
    tot=sum(v[1] for v in agg.values())
    print(f"slide kernels total {tot:.1f} us, {sum(v[0] for v in agg.values())} launches")
    for k,v in sorted(agg.items(), key=lambda kv:-kv[1][1]): print(f"  {k:32s} {v[0]:3d} {v[1]:8.1f} us {v[2]:8.1f} MB")
for si in [int(x) for x in sys.argv[2:]]:
    print("slide", si); summarize(starts[si]-4, starts[si+1]-4)
