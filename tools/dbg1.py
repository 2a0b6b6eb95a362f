import sys, numpy as np, torch
sys.path.insert(0, '.')
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
g = Graph(1024, device=0)
s, d, w = wl.uniform_edges(1, 1, 4096, 1024)
print("insert", g.insert_edges(s, d, w, count=True), flush=True)
f, qw = g.query_edges(s, d)
print("query", int(f.sum()), flush=True)
print("delete", g.delete_edges(s, d, count=True), flush=True)
print(g.check_invariants())
