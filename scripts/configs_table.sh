# per-config numbers for DESIGN.md §6: one search at a time (latency view) and batched restarts
timeout 300 python scripts/probe.py --cfg C1,C2,C3,C4,C5
timeout 300 python scripts/probe_batch.py C1:148:1000 C2:50:2000 C3:50:400 C4:50:400 C5:8:3
